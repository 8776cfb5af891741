"""The N > 1 host path with world_size 2 on CPU (gloo): source partition,
batch broadcast from rank 0, max-over-ranks timing, replica agreement.  The
per-rank compute is the oracle here (the CUDA path needs a GPU per rank);
what is tested is that every rank sees the same batches and that sharded
sources reproduce the single-process result exactly."""
import os
import socket
import tempfile

import numpy as np
import pytest
import torch
import torch.distributed as dist
import torch.multiprocessing as mp

import oracle
from paper_journals_pvldb_guolst17_b200 import dist as D, workload as W


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _worker(rank, world, port, outdir):
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        n = 400
        src, dst = W.rmat_stream(n, 6000, seed=11, abc=W.GRAPH500)
        st = W.Stream(n, src, dst, w0=1500, ins_per_slide=60, del_per_slide=90)
        g0s, g0d = st.window()
        deg = np.bincount(g0s, minlength=n)
        sources = W.pick_sources(n, g0s, g0d, band=50, count=6)
        mine = D.partition_sources(sources, deg, world, rank)
        o = oracle.Oracle(n, g0s, g0d, mine, 0.15, 1e-8)
        o.push(oracle.SEQ)
        times = []
        for t in range(4):
            if rank == 0:
                b = st.next_batch()
                flat, counts = D.pack_batch(*b)
            else:
                flat, counts = None, (60, 90)
            flat = D.broadcast_batch(flat, counts)
            ins_s, ins_d, del_s, del_d = (x.numpy().view(np.uint32) for x in D.unpack_batch(flat, counts))
            o.apply(ins_s, ins_d, del_s, del_d)
            times.append(D.max_over_ranks(1.0 + rank))
            es, ed = o.export()
            assert D.replicas_agree(D.edge_set_digest(es, ed))
        res = {int(s): o.query(i)[0] for i, s in enumerate(mine)}
        np.save(os.path.join(outdir, f"rank{rank}.npy"), {"P": res, "times": times}, allow_pickle=True)
    finally:
        dist.destroy_process_group()


def test_partition_is_a_degree_dealt_partition():
    deg = np.array([5, 1, 9, 3, 7, 2, 8, 0])
    srcs = np.array([0, 2, 3, 4, 6, 7])
    parts = [D.partition_sources(srcs, deg, 2, r) for r in range(2)]
    assert sorted(np.concatenate(parts).tolist()) == sorted(srcs.tolist())
    # by degree: 2(9) 6(8) 4(7) 0(5) 3(3) 7(0) -> rank0 {2,4,3}, rank1 {6,0,7}
    assert parts[0].tolist() == [2, 3, 4] and parts[1].tolist() == [0, 6, 7]


def test_pack_unpack_roundtrip():
    b = (np.array([1, 2], np.uint32), np.array([3, 4], np.uint32), np.array([5], np.uint32),
         np.array([6], np.uint32))
    flat, counts = D.pack_batch(*b)
    out = D.unpack_batch(flat, counts)
    for x, y in zip(b, out):
        np.testing.assert_array_equal(x, y.numpy().view(np.uint32))


def test_digest_is_order_independent():
    a = D.edge_set_digest([1, 2, 3], [4, 5, 6])
    b = D.edge_set_digest([3, 1, 2], [6, 4, 5])
    c = D.edge_set_digest([3, 1, 2], [6, 4, 4])
    assert a == b and a != c


def test_world2_gloo_sharded_sources_match_single_process():
    world = 2
    with tempfile.TemporaryDirectory() as d:
        mp.spawn(_worker, args=(world, _free_port(), d), nprocs=world, join=True)
        got = {}
        for r in range(world):
            x = np.load(os.path.join(d, f"rank{r}.npy"), allow_pickle=True).item()
            assert x["times"] == [2.0] * 4  # max over ranks
            got.update(x["P"])
    # single process, all sources, same stream
    n = 400
    src, dst = W.rmat_stream(n, 6000, seed=11, abc=W.GRAPH500)
    st = W.Stream(n, src, dst, w0=1500, ins_per_slide=60, del_per_slide=90)
    g0s, g0d = st.window()
    sources = W.pick_sources(n, g0s, g0d, band=50, count=6)
    assert sorted(got) == sorted(int(s) for s in sources)
    for s in sources:  # one source per handle: the sharded run must agree exactly
        o = oracle.Oracle(n, g0s, g0d, [s], 0.15, 1e-8)
        o.push(oracle.SEQ)
        st2 = W.Stream(n, src, dst, w0=1500, ins_per_slide=60, del_per_slide=90)
        st2.window()
        for _ in range(4):
            o.apply(*st2.next_batch())
        np.testing.assert_array_equal(o.query(0)[0], got[int(s)])
