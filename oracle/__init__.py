"""TEST INFRASTRUCTURE ONLY -- the independent CPU oracle.

Only ``tests/``, ``__graft_entry__.smoke()`` and ``bench.py``'s
``cpu_baseline`` / ``--impl reference`` legs may import this package.  It
shares no code with the CUDA product path (``paper_journals_pvldb_guolst17_b200``)
and never imports it; the only module both sides use is the seeded input
generator ``paper_journals_pvldb_guolst17_b200.workload``, which holds none of
the method's arithmetic.

Contents
--------
* ``Oracle``  -- ctypes wrapper over ``liboracle.so`` (``ppr_oracle.c``): the
  sequential local update scheme (Alg 1, Alg 2), CPU-Seq /
  CPU-Base batch processing and an Alg 3 round emulation
  (P:454-480), single-threaded fp64.
* ``exact``   -- numpy definitions used to check it: exact PPR by dense solve
  and power iteration, the Eq. 2 invariant checker, the error identity.
"""
from __future__ import annotations

import ctypes
import os
import subprocess

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_LIB_PATH = os.path.join(_HERE, "liboracle.so")
_SRC = os.path.join(_HERE, "ppr_oracle.c")

ORC_OK, ORC_EINVAL, ORC_ERANGE, ORC_ENOENT, ORC_ENOMEM = 0, -1, -2, -3, -4
SEQ, BASE, JACOBI = 0, 1, 2


def build(force: bool = False) -> str:
    """Compile liboracle.so (gcc, -O2 -ffp-contract=off: no FMA contraction)."""
    if force or not os.path.exists(_LIB_PATH) or (
        os.path.getmtime(_LIB_PATH) < max(os.path.getmtime(_SRC),
                                           os.path.getmtime(os.path.join(_HERE, "ppr_oracle.h")))
    ):
        cmd = ["gcc", "-O2", "-ffp-contract=off", "-std=c11", "-fPIC", "-shared",
               "-Wall", "-Wextra", "-o", _LIB_PATH, _SRC]
        subprocess.check_call(cmd)
    return _LIB_PATH


class _Stats(ctypes.Structure):
    _fields_ = [("pushes", ctypes.c_uint64), ("pushed_edges", ctypes.c_uint64),
                ("rounds_pos", ctypes.c_uint64), ("rounds_neg", ctypes.c_uint64)]


_lib = None


def _load():
    global _lib
    if _lib is None:
        lib = ctypes.CDLL(build())
        u32p = ctypes.POINTER(ctypes.c_uint32)
        f64p = ctypes.POINTER(ctypes.c_double)
        lib.oracle_create.argtypes = [ctypes.c_uint32, ctypes.c_uint64, u32p, u32p, u32p,
                                      ctypes.c_uint32, ctypes.c_double, ctypes.c_double,
                                      ctypes.POINTER(ctypes.c_void_p)]
        lib.oracle_create.restype = ctypes.c_int
        lib.oracle_destroy.argtypes = [ctypes.c_void_p]
        lib.oracle_destroy.restype = None
        lib.oracle_push.argtypes = [ctypes.c_void_p, ctypes.c_int, ctypes.c_int64]
        lib.oracle_push.restype = ctypes.c_int
        lib.oracle_apply.argtypes = [ctypes.c_void_p, u32p, u32p, ctypes.c_uint64, u32p, u32p,
                                     ctypes.c_uint64, ctypes.c_int, ctypes.c_int]
        lib.oracle_apply.restype = ctypes.c_int
        lib.oracle_set_state.argtypes = [ctypes.c_void_p, ctypes.c_uint32, f64p, f64p]
        lib.oracle_set_state.restype = ctypes.c_int
        lib.oracle_query.argtypes = [ctypes.c_void_p, ctypes.c_uint32, f64p, f64p]
        lib.oracle_query.restype = ctypes.c_int
        lib.oracle_num_arcs.argtypes = [ctypes.c_void_p]
        lib.oracle_num_arcs.restype = ctypes.c_uint64
        lib.oracle_export.argtypes = [ctypes.c_void_p, u32p, u32p]
        lib.oracle_export.restype = ctypes.c_uint64
        lib.oracle_dout.argtypes = [ctypes.c_void_p, u32p]
        lib.oracle_dout.restype = None
        lib.oracle_get_stats.argtypes = [ctypes.c_void_p, ctypes.POINTER(_Stats)]
        lib.oracle_get_stats.restype = None
        lib.oracle_reset_stats.argtypes = [ctypes.c_void_p]
        lib.oracle_reset_stats.restype = None
        _lib = lib
    return _lib


def _u32(a):
    a = np.ascontiguousarray(np.asarray(a, dtype=np.uint32))
    return a, a.ctypes.data_as(ctypes.POINTER(ctypes.c_uint32))


def _f64(a):
    a = np.ascontiguousarray(np.asarray(a, dtype=np.float64))
    return a, a.ctypes.data_as(ctypes.POINTER(ctypes.c_double))


class OracleError(RuntimeError):
    def __init__(self, code: int, what: str):
        super().__init__(f"{what}: oracle status {code}")
        self.code = code


class Oracle:
    """Sequential fp64 oracle for one graph and S sources (see ppr_oracle.h)."""

    def __init__(self, n, src, dst, sources, alpha, eps):
        lib = _load()
        self.n = int(n)
        self.sources = np.asarray(sources, dtype=np.uint32).copy()
        self.alpha, self.eps = float(alpha), float(eps)
        s, sp = _u32(src)
        d, dp = _u32(dst)
        so, sop = _u32(self.sources)
        h = ctypes.c_void_p()
        rc = lib.oracle_create(self.n, len(s), sp, dp, sop, len(so), self.alpha, self.eps,
                               ctypes.byref(h))
        if rc != ORC_OK:
            raise OracleError(rc, "oracle_create")
        self._h = h

    def close(self):
        if getattr(self, "_h", None):
            _load().oracle_destroy(self._h)
            self._h = None

    def __del__(self):
        try:
            self.close()
        except Exception:
            pass

    def push(self, mode=SEQ, max_steps=-1):
        rc = _load().oracle_push(self._h, mode, max_steps)
        if rc != ORC_OK:
            raise OracleError(rc, "oracle_push")

    def apply(self, ins_src=(), ins_dst=(), del_src=(), del_dst=(), mode=SEQ, do_push=True,
              raise_on_error=True):
        a, ap = _u32(ins_src)
        b, bp = _u32(ins_dst)
        c, cp = _u32(del_src)
        d, dp = _u32(del_dst)
        assert len(a) == len(b) and len(c) == len(d)
        rc = _load().oracle_apply(self._h, ap, bp, len(a), cp, dp, len(c), mode, int(do_push))
        if rc != ORC_OK and raise_on_error:
            raise OracleError(rc, "oracle_apply")
        return rc

    def set_state(self, sidx, P, R):
        p, pp = _f64(P)
        r, rp = _f64(R)
        assert len(p) == self.n and len(r) == self.n
        rc = _load().oracle_set_state(self._h, sidx, pp, rp)
        if rc != ORC_OK:
            raise OracleError(rc, "oracle_set_state")

    def query(self, sidx=0):
        P = np.empty(self.n, dtype=np.float64)
        R = np.empty(self.n, dtype=np.float64)
        rc = _load().oracle_query(self._h, sidx, P.ctypes.data_as(ctypes.POINTER(ctypes.c_double)),
                                  R.ctypes.data_as(ctypes.POINTER(ctypes.c_double)))
        if rc != ORC_OK:
            raise OracleError(rc, "oracle_query")
        return P, R

    @property
    def num_arcs(self):
        return int(_load().oracle_num_arcs(self._h))

    def export(self):
        """Arc multiset sorted by (dst, src): (src, dst) uint32 arrays."""
        m = self.num_arcs
        src = np.empty(m, dtype=np.uint32)
        dst = np.empty(m, dtype=np.uint32)
        k = _load().oracle_export(self._h, src.ctypes.data_as(ctypes.POINTER(ctypes.c_uint32)),
                                  dst.ctypes.data_as(ctypes.POINTER(ctypes.c_uint32)))
        assert k == m
        return src, dst

    def dout(self):
        d = np.empty(self.n, dtype=np.uint32)
        _load().oracle_dout(self._h, d.ctypes.data_as(ctypes.POINTER(ctypes.c_uint32)))
        return d

    def stats(self, reset=False):
        st = _Stats()
        _load().oracle_get_stats(self._h, ctypes.byref(st))
        if reset:
            _load().oracle_reset_stats(self._h)
        return {"pushes": st.pushes, "pushed_edges": st.pushed_edges,
                "rounds_pos": st.rounds_pos, "rounds_neg": st.rounds_neg}
