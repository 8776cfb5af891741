"""Multi-GPU plumbing for multi-source PPR.

Sources are independent unit-vector problems, so the
only exchange step is the edge batch: rank 0 owns the stream and broadcasts
each batch; every rank applies it to its own graph replica and maintains its
own shard of the sources.  These helpers are backend-agnostic (NCCL with CUDA
tensors in bench.py, gloo with CPU tensors in tests/test_dist_gloo.py); they
hold no PPR arithmetic.
"""
from __future__ import annotations

import hashlib

import numpy as np
import torch
import torch.distributed as dist


def partition_sources(sources, out_degree, world, rank):
    """Degree-dealt partition: sort the sources by G0 out-degree (descending,
    ties by id) and deal them round-robin, so every rank gets a similar mix of
    hub and non-hub sources (per-source work varies ~1000x with the degree
    band)."""
    sources = np.asarray(sources, dtype=np.int64)
    deg = np.asarray(out_degree)[sources]
    order = np.lexsort((sources, -deg))
    return np.sort(sources[order[rank::world]]).astype(np.uint32)


def pack_batch(ins_src, ins_dst, del_src, del_dst):
    """One flat int32 tensor [ins_src | ins_dst | del_src | del_dst] + counts."""
    parts = [np.asarray(x, dtype=np.uint32) for x in (ins_src, ins_dst, del_src, del_dst)]
    flat = np.concatenate(parts).view(np.int32)
    return torch.from_numpy(flat.copy()), (len(parts[0]), len(parts[2]))


def unpack_batch(flat, counts):
    """Views (ins_src, ins_dst, del_src, del_dst) of a packed batch tensor."""
    ni, nd = counts
    return (flat[0:ni], flat[ni:2 * ni], flat[2 * ni:2 * ni + nd], flat[2 * ni + nd:2 * ni + 2 * nd])


def broadcast_batch(flat, counts, group=None, src=0):
    """Broadcasts a packed batch from `src`; non-source ranks pass a tensor of
    the right size (or None) and get the data back."""
    if not dist.is_initialized() or dist.get_world_size() == 1:
        return flat
    device = flat.device if flat is not None else torch.device("cpu")
    n = 2 * (counts[0] + counts[1])
    if flat is None or flat.numel() != n:
        flat = torch.empty(n, dtype=torch.int32, device=device)
    dist.broadcast(flat, src, group=group)
    return flat


def max_over_ranks(x, device="cpu"):
    """Max of a float over all ranks (step time is the slowest rank's)."""
    t = torch.tensor([float(x)], dtype=torch.float64, device=device)
    if dist.is_initialized() and dist.get_world_size() > 1:
        dist.all_reduce(t, op=dist.ReduceOp.MAX)
    return float(t.item())


def sum_over_ranks(values, device="cpu"):
    t = torch.tensor([float(v) for v in values], dtype=torch.float64, device=device)
    if dist.is_initialized() and dist.get_world_size() > 1:
        dist.all_reduce(t, op=dist.ReduceOp.SUM)
    return [float(v) for v in t.tolist()]


def edge_set_digest(src, dst):
    """Order-independent 64-bit digest of an arc multiset (sorted (dst, src))."""
    key = (np.asarray(dst, dtype=np.uint64) << np.uint64(32)) | np.asarray(src, dtype=np.uint64)
    key = np.sort(key)
    return int.from_bytes(hashlib.blake2b(key.tobytes(), digest_size=8).digest(), "little") & ((1 << 62) - 1)


def replicas_agree(digest, device="cpu"):
    """True iff every rank's replica has the same arc multiset digest."""
    if not (dist.is_initialized() and dist.get_world_size() > 1):
        return True
    lo = torch.tensor([digest], dtype=torch.int64, device=device)
    hi = lo.clone()
    dist.all_reduce(lo, op=dist.ReduceOp.MIN)
    dist.all_reduce(hi, op=dist.ReduceOp.MAX)
    return int(lo.item()) == int(hi.item())
