"""Thin ctypes binding of libppr.so (include/ppr.h) -- argument marshalling only.

Every step of the hot path runs in the library's CUDA kernels; there is no
fallback: if libppr.so is missing or no CUDA device is usable, the calls
raise.  Names follow the C ABI: ``Ppr.create`` -> ppr_create,
``Ppr.apply_batch`` -> ppr_apply_batch, ``Ppr.query`` -> ppr_query, ...
Device arrays may be passed as torch CUDA tensors (uint32 / float64), host
arrays as numpy arrays or CPU tensors.
"""
from __future__ import annotations

import ctypes
import os

import numpy as np

_PKG = os.path.dirname(os.path.abspath(__file__))
LIB_PATH = os.path.join(_PKG, "libppr.so")

PPR_OK, PPR_EINVAL, PPR_ERANGE, PPR_ENOENT, PPR_ENOMEM, PPR_ECUDA, PPR_EPOISONED, PPR_ENOCONV = \
    0, -1, -2, -3, -4, -5, -6, -7
MEM_HOST, MEM_DEVICE = 0, 1
MODE_OPT, MODE_EAGER, MODE_DUPDETECT, MODE_VANILLA, MODE_ASYNC, MODE_EAGER_SCAN, MODE_SHARED, \
    MODE_SORTAGG = 0, 1, 2, 3, 4, 5, 6, 7
MODES = {"opt": MODE_OPT, "eager": MODE_EAGER, "dupdetect": MODE_DUPDETECT, "vanilla": MODE_VANILLA,
         "async": MODE_ASYNC, "scan": MODE_EAGER_SCAN, "shared": MODE_SHARED, "sortagg": MODE_SORTAGG}
OPT_MODE, OPT_PUSH, OPT_MAX_ITERS, OPT_TIMING, OPT_FORCE_REBUILD = 1, 2, 3, 4, 5
OPT_RING_TAIL, OPT_RING_ALL, OPT_EDGE_CHAINS, OPT_GRAPHS, OPT_WAVE = 6, 7, 8, 9, 10
OPT_CHECK_ENQUEUE = 11
LAYOUT_ARRAYS, LAYOUT_PACKED = 0, 1


class Graph(ctypes.Structure):
    _fields_ = [("n", ctypes.c_uint32), ("m", ctypes.c_uint64),
                ("src", ctypes.POINTER(ctypes.c_uint32)), ("dst", ctypes.POINTER(ctypes.c_uint32)),
                ("undirected", ctypes.c_int)]


class Opts(ctypes.Structure):
    _fields_ = [("device", ctypes.c_int), ("cuda_stream", ctypes.c_void_p), ("mode", ctypes.c_int),
                ("slack", ctypes.c_double), ("min_cap", ctypes.c_uint32), ("relabel", ctypes.c_int),
                ("layout", ctypes.c_int), ("l2_persist", ctypes.c_int), ("pool_degrees", ctypes.c_int)]


class BatchStats(ctypes.Structure):
    _fields_ = [("iters_pos", ctypes.c_uint32), ("iters_neg", ctypes.c_uint32),
                ("pushes", ctypes.c_uint64), ("pushed_edges", ctypes.c_uint64),
                ("max_frontier", ctypes.c_uint64), ("touched", ctypes.c_uint64),
                ("num_arcs", ctypes.c_uint64), ("rebuilt", ctypes.c_uint32),
                ("kernel_launches", ctypes.c_uint32), ("h2d_bytes", ctypes.c_uint64),
                ("d2h_bytes", ctypes.c_uint64), ("ms_total", ctypes.c_float),
                ("ms_store", ctypes.c_float), ("ms_restore", ctypes.c_float),
                ("ms_push", ctypes.c_float), ("walk_edges", ctypes.c_uint64),
                ("ms_push_pos", ctypes.c_float), ("ms_push_neg", ctypes.c_float),
                ("entries", ctypes.c_uint64), ("dup_enqueues", ctypes.c_uint64)]

    def as_dict(self):
        return {k: getattr(self, k) for k, _ in self._fields_}


# every symbol include/ppr.h declares
EXPORTS = ["ppr_create", "ppr_apply_batch", "ppr_push", "ppr_query", "ppr_export_edges",
           "ppr_export_dout", "ppr_set_option", "ppr_reset", "ppr_device_bytes", "ppr_destroy",
           "ppr_reset_persisting_l2",
           "ppr_status_str", "ppr_last_error"]

_lib = None


def load(path: str = os.environ.get("PPR_LIB", LIB_PATH)):
    """Loads libppr.so (fails loudly if it has not been built)."""
    global _lib
    if _lib is not None:
        return _lib
    if not os.path.exists(path):
        raise RuntimeError(f"{path} not found: run `python -m paper_journals_pvldb_guolst17_b200.build`"
                           " (no CPU fallback exists)")
    lib = ctypes.CDLL(path)
    u32p = ctypes.POINTER(ctypes.c_uint32)
    vp = ctypes.c_void_p
    lib.ppr_create.argtypes = [ctypes.POINTER(Graph), u32p, ctypes.c_uint32, ctypes.c_double,
                               ctypes.c_double, ctypes.POINTER(Opts), ctypes.POINTER(vp),
                               ctypes.POINTER(BatchStats)]
    lib.ppr_apply_batch.argtypes = [vp, vp, vp, ctypes.c_uint64, vp, vp, ctypes.c_uint64,
                                    ctypes.c_int, ctypes.POINTER(BatchStats)]
    lib.ppr_push.argtypes = [vp, ctypes.POINTER(BatchStats)]
    lib.ppr_reset.argtypes = [vp]
    lib.ppr_query.argtypes = [vp, ctypes.c_uint32, vp, vp, ctypes.c_int]
    lib.ppr_export_edges.argtypes = [vp, u32p, u32p, ctypes.c_uint64, ctypes.POINTER(ctypes.c_uint64)]
    lib.ppr_export_dout.argtypes = [vp, u32p]
    lib.ppr_set_option.argtypes = [vp, ctypes.c_int, ctypes.c_int64]
    lib.ppr_reset_persisting_l2.argtypes = []
    lib.ppr_reset_persisting_l2.restype = ctypes.c_int
    lib.ppr_device_bytes.argtypes = [vp]
    lib.ppr_device_bytes.restype = ctypes.c_uint64
    lib.ppr_destroy.argtypes = [vp]
    lib.ppr_status_str.argtypes = [ctypes.c_int]
    lib.ppr_status_str.restype = ctypes.c_char_p
    lib.ppr_last_error.argtypes = [vp]
    lib.ppr_last_error.restype = ctypes.c_char_p
    for f in ("ppr_create", "ppr_apply_batch", "ppr_push", "ppr_query", "ppr_export_edges",
              "ppr_export_dout", "ppr_set_option", "ppr_reset", "ppr_destroy"):
        getattr(lib, f).restype = ctypes.c_int
    _lib = lib
    return lib


def reset_persisting_l2():
    """Return persisting L2 lines to normal status (call before an L2 flush)."""
    return load().ppr_reset_persisting_l2()


class PprError(RuntimeError):
    def __init__(self, code, msg):
        super().__init__(msg)
        self.code = code


def _host_u32(a):
    a = np.ascontiguousarray(np.asarray(a, dtype=np.uint32))
    return a, a.ctypes.data_as(ctypes.c_void_p)


def _ptr(a, mem):
    """(keepalive, pointer, length) for a host or device uint32 array."""
    if mem == MEM_DEVICE:
        import torch
        assert isinstance(a, torch.Tensor) and a.is_cuda and a.dtype in (torch.int32, torch.uint32)
        assert a.is_contiguous()
        return a, ctypes.c_void_p(a.data_ptr()), a.numel()
    if hasattr(a, "numpy") and not isinstance(a, np.ndarray):  # CPU torch tensor
        a = a.numpy()
    arr, p = _host_u32(a)
    return arr, p, len(arr)


class Ppr:
    """One PPR handle (one graph, S sources) on one GPU."""

    def __init__(self, n, src, dst, sources, alpha=0.15, eps=1e-9, mode="opt", device=0,
                 stream=None, undirected=False, slack=0.25, min_cap=4, relabel=-1,
                 layout=LAYOUT_ARRAYS, l2_persist=-1, pool_degrees=-1):
        lib = load()
        s, sp = _host_u32(src)
        d, dp = _host_u32(dst)
        assert len(s) == len(d)
        so, sop = _host_u32(sources)
        g = Graph(n=int(n), m=len(s), src=ctypes.cast(sp, ctypes.POINTER(ctypes.c_uint32)),
                  dst=ctypes.cast(dp, ctypes.POINTER(ctypes.c_uint32)), undirected=int(undirected))
        o = Opts(device=int(device), cuda_stream=stream, mode=MODES.get(mode, mode),
                 slack=float(slack), min_cap=int(min_cap), relabel=int(relabel),
                 layout=int(layout), l2_persist=int(l2_persist), pool_degrees=int(pool_degrees))
        h = ctypes.c_void_p()
        st = BatchStats()
        rc = lib.ppr_create(ctypes.byref(g), ctypes.cast(sop, ctypes.POINTER(ctypes.c_uint32)),
                            len(so), float(alpha), float(eps), ctypes.byref(o), ctypes.byref(h),
                            ctypes.byref(st))
        if rc != PPR_OK:
            raise PprError(rc, f"ppr_create: {lib.ppr_status_str(rc).decode()}")
        self._h = h
        self.n, self.S = int(n), len(so)
        self.sources = so.copy()
        self.alpha, self.eps = float(alpha), float(eps)
        self.create_stats = st.as_dict()

    def _check(self, rc, what):
        if rc != PPR_OK:
            lib = load()
            raise PprError(rc, f"{what}: {lib.ppr_status_str(rc).decode()}: "
                               f"{lib.ppr_last_error(self._h).decode()}")

    def close(self):
        if getattr(self, "_h", None):
            load().ppr_destroy(self._h)
            self._h = None

    def __del__(self):
        try:
            self.close()
        except Exception:
            pass

    def set_option(self, key, value):
        self._check(load().ppr_set_option(self._h, key, int(value)), "ppr_set_option")

    def apply_batch(self, ins_src=(), ins_dst=(), del_src=(), del_dst=(), mem=MEM_HOST,
                    raise_on_error=True):
        a, ap, na = _ptr(ins_src, mem)
        b, bp, nb = _ptr(ins_dst, mem)
        c, cp, nc = _ptr(del_src, mem)
        d, dp, nd = _ptr(del_dst, mem)
        assert na == nb and nc == nd
        st = BatchStats()
        rc = load().ppr_apply_batch(self._h, ap if na else None, bp if na else None, na,
                                    cp if nc else None, dp if nc else None, nc, mem,
                                    ctypes.byref(st))
        if raise_on_error:
            self._check(rc, "ppr_apply_batch")
            return st.as_dict()
        return rc, st.as_dict()

    def push(self):
        st = BatchStats()
        self._check(load().ppr_push(self._h, ctypes.byref(st)), "ppr_push")
        return st.as_dict()

    def reset(self):
        self._check(load().ppr_reset(self._h), "ppr_reset")

    def query(self, sidx=0, want_R=True):
        P = np.empty(self.n, dtype=np.float64)
        R = np.empty(self.n, dtype=np.float64) if want_R else None
        self._check(load().ppr_query(self._h, sidx, P.ctypes.data_as(ctypes.c_void_p),
                                     R.ctypes.data_as(ctypes.c_void_p) if want_R else None,
                                     MEM_HOST), "ppr_query")
        return (P, R) if want_R else P

    def query_device(self, sidx, P_out, R_out=None):
        """P_out / R_out: float64 CUDA tensors of n elements."""
        self._check(load().ppr_query(self._h, sidx, ctypes.c_void_p(P_out.data_ptr()),
                                     ctypes.c_void_p(R_out.data_ptr()) if R_out is not None else None,
                                     MEM_DEVICE), "ppr_query")

    def export_edges(self):
        lib = load()
        m = ctypes.c_uint64()
        rc = lib.ppr_export_edges(self._h, None, None, 0, ctypes.byref(m))
        if rc not in (PPR_OK, PPR_EINVAL):
            self._check(rc, "ppr_export_edges")
        src = np.empty(m.value, dtype=np.uint32)
        dst = np.empty(m.value, dtype=np.uint32)
        self._check(lib.ppr_export_edges(self._h, src.ctypes.data_as(ctypes.POINTER(ctypes.c_uint32)),
                                         dst.ctypes.data_as(ctypes.POINTER(ctypes.c_uint32)),
                                         m.value, ctypes.byref(m)), "ppr_export_edges")
        return src, dst

    def export_dout(self):
        d = np.empty(self.n, dtype=np.uint32)
        self._check(load().ppr_export_dout(self._h, d.ctypes.data_as(ctypes.POINTER(ctypes.c_uint32))),
                    "ppr_export_dout")
        return d

    @property
    def device_bytes(self):
        return int(load().ppr_device_bytes(self._h))
