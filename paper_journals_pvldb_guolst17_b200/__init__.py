"""B200-native batch-parallel Personalized PageRank maintenance on dynamic graphs.

Hot path (Guo, Li, Sha, Tan, PVLDB 11(1) 2017): graph-store apply -> invariant
restore -> two-phase frontier push to eps, all in hand-written sm_100a CUDA
behind the C ABI declared in include/ppr.h.  ``ppr`` is the thin ctypes
binding; ``workload`` is the seeded input generator.
"""
__all__ = ["ppr", "workload"]
