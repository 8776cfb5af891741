"""Seeded synthetic workloads shaped like the paper's sliding-window streams.

INPUT ONLY: this module holds none of the PPR method's arithmetic; it is the
one module both the CUDA path (tests, bench.py) and the CPU oracle consume.

Stream protocol: the edges of a graph get random
timestamps; the first 10% of the stream initialise a sliding window; each
slide of size k inserts the next k edges and deletes the k oldest.
The Orkut-shaped deletion-heavy variant and the Twitter-shaped resident
window are readings documented in DESIGN.md (Input recipe).
"""
from __future__ import annotations

import ctypes
import os
import subprocess
from dataclasses import dataclass, field

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SRC = os.path.join(_HERE, "rmat_stream.c")
_LIB = os.path.join(_HERE, "librmat.so")

GRAPH500 = (0.57, 0.19, 0.19)   # canonical Graph500 (a, b, c); d = 0.05
SHAPED = (0.50, 0.20, 0.20)     # "-shaped" configs; d = 0.10


def build(force=False):
    if force or not os.path.exists(_LIB) or os.path.getmtime(_LIB) < os.path.getmtime(_SRC):
        subprocess.check_call(["gcc", "-O3", "-fopenmp", "-std=c11", "-fPIC", "-shared", "-Wall",
                               "-o", _LIB, _SRC])
    return _LIB


_lib = None


def _load():
    global _lib
    if _lib is None:
        lib = ctypes.CDLL(build())
        lib.rmat_stream.argtypes = [ctypes.c_uint32, ctypes.c_uint64, ctypes.c_uint64,
                                    ctypes.c_double, ctypes.c_double, ctypes.c_double,
                                    ctypes.c_int, ctypes.POINTER(ctypes.c_uint32),
                                    ctypes.POINTER(ctypes.c_uint32)]
        lib.rmat_stream.restype = ctypes.c_int
        _lib = lib
    return _lib


def rmat_stream(n, m, seed=42, abc=SHAPED, undirected=False):
    """m unique arcs (or undirected edges) on [0, n), in stream order."""
    src = np.empty(m, dtype=np.uint32)
    dst = np.empty(m, dtype=np.uint32)
    rc = _load().rmat_stream(int(n), int(m), int(seed), float(abc[0]), float(abc[1]),
                             float(abc[2]), int(bool(undirected)),
                             src.ctypes.data_as(ctypes.POINTER(ctypes.c_uint32)),
                             dst.ctypes.data_as(ctypes.POINTER(ctypes.c_uint32)))
    if rc != 0:
        raise RuntimeError(f"rmat_stream failed ({rc}) for n={n} m={m}")
    return src, dst


def expand_undirected(src, dst):
    """Each undirected {u,v} becomes arcs u->v and v->u."""
    return np.concatenate([src, dst]), np.concatenate([dst, src])


def pick_sources(n, src, dst, band, count, seed=7):
    """`count` distinct sources drawn uniformly from the top-`band` vertices by
    out-degree in the initial window G0 (Table 2; reading R17)."""
    deg = np.bincount(np.asarray(src, dtype=np.int64), minlength=n)
    order = np.lexsort((np.arange(n), -deg))  # degree desc, id asc
    top = order[:min(band, n)]
    rng = np.random.default_rng(seed)
    return np.sort(rng.choice(top, size=count, replace=False)).astype(np.uint32)


@dataclass
class Stream:
    """A sliding window over a seeded stream.

    directed: window arcs are stream[lo:hi]; slide t inserts `ins_per_slide`
    new stream entries and deletes `del_per_slide` oldest ones.
    undirected: entries are edges; `arcs(...)` expands them."""
    n: int
    src: np.ndarray
    dst: np.ndarray
    w0: int
    ins_per_slide: int
    del_per_slide: int
    undirected: bool = False
    lo: int = field(default=0)
    hi: int = field(default=0)

    def __post_init__(self):
        self.lo, self.hi = 0, self.w0

    def window(self):
        s, d = self.src[self.lo:self.hi], self.dst[self.lo:self.hi]
        return expand_undirected(s, d) if self.undirected else (s.copy(), d.copy())

    def remaining_slides(self):
        a = (len(self.src) - self.hi) // max(self.ins_per_slide, 1) if self.ins_per_slide else 10**18
        b = (self.hi - self.lo) // max(self.del_per_slide, 1) if self.del_per_slide else 10**18
        return int(min(a, b))

    def next_batch(self):
        """(ins_src, ins_dst, del_src, del_dst) as arcs; advances the window."""
        i0, i1 = self.hi, self.hi + self.ins_per_slide
        d0, d1 = self.lo, self.lo + self.del_per_slide
        if i1 > len(self.src) or d1 > i0:
            raise StopIteration("stream exhausted")
        isrc, idst = self.src[i0:i1], self.dst[i0:i1]
        dsrc, ddst = self.src[d0:d1], self.dst[d0:d1]
        self.hi, self.lo = i1, d1
        if self.undirected:
            isrc, idst = expand_undirected(isrc, idst)
            dsrc, ddst = expand_undirected(dsrc, ddst)
        return (np.ascontiguousarray(isrc), np.ascontiguousarray(idst),
                np.ascontiguousarray(dsrc), np.ascontiguousarray(ddst))


# BASELINE.json configs -> concrete recipes (DESIGN.md Input recipe)
CONFIGS = {
    "tiny": dict(n=10_000, m=100_000, abc=GRAPH500, undirected=False, window=0.10,
                 ins=1_000, dele=1_000, eps=1e-7, band=1_000, sources=1, slides=50),
    "lj": dict(n=4_847_571, m=68_993_773, abc=SHAPED, undirected=False, window=0.10,
               ins=10_000, dele=10_000, eps=1e-9, band=1_000, sources=1, slides=100),
    "orkut": dict(n=3_072_441, m=117_185_083, abc=SHAPED, undirected=True, window=0.50,
                  ins=2_500, dele=7_500, eps=1e-9, band=1_000, sources=1, slides=100),
    "twitter": dict(n=41_652_230, m=1_500_000_000, abc=SHAPED, undirected=False, window=None,
                    ins=100_000, dele=100_000, eps=1e-9, band=1_000, sources=1, slides=10),
    "ms-lj": dict(n=4_847_571, m=68_993_773, abc=SHAPED, undirected=False, window=0.10,
                  ins=10_000, dele=10_000, eps=1e-9, band=1_000, sources=256, slides=100),
}


def make_stream(name, seed=42, **over):
    cfg = dict(CONFIGS[name])
    cfg.update(over)
    src, dst = rmat_stream(cfg["n"], cfg["m"], seed=seed, abc=cfg["abc"],
                           undirected=cfg["undirected"])
    if cfg["window"] is None:  # resident window: all but the insertions of 2*slides + 5 slides
        w0 = cfg["m"] - (2 * cfg["slides"] + 5) * cfg["ins"]
    else:
        w0 = int(round(cfg["window"] * cfg["m"]))
    st = Stream(cfg["n"], src, dst, w0, cfg["ins"], cfg["dele"], cfg["undirected"])
    return st, cfg
