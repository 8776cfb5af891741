"""Shared per-batch gates of the GPU parity tests:
arc multiset bit-exact vs the oracle, Eq. 2 at every vertex on the ORACLE's
arc multiset (reading R18), exact eps-termination, GPU vs oracle estimates
within 2 eps (reading R19).  Test infrastructure: imports the oracle."""
import numpy as np

from oracle import exact


def expand_undirected_arcs(src, dst):
    """{u, v} -> u->v and v->u, a self-loop {u, u} -> one arc u->u (P:868-870,
    ppr.h `undirected`): the oracle is fed arcs expanded here, independently of
    the library's own expansion."""
    src = np.asarray(src, dtype=np.uint32)
    dst = np.asarray(dst, dtype=np.uint32)
    loop = src == dst
    return (np.concatenate([src, dst[~loop]]), np.concatenate([dst, src[~loop]]))


def check_batch_state(h, o, sidx, s, eps, what, edges=None):
    """All per-batch gates for source number `sidx` (vertex s).  `edges`: the
    oracle's exported (src, dst), to reuse across sources of one batch."""
    P, R = h.query(sidx)
    Po, Ro = o.query(sidx)
    gs, gd = h.export_edges()
    os_, od = edges if edges is not None else o.export()
    np.testing.assert_array_equal(gd, od, err_msg=f"{what}: arc dst")
    np.testing.assert_array_equal(gs, os_, err_msg=f"{what}: arc src")
    assert exact.terminated(R, eps), (what, np.abs(R).max())
    ok, worst = exact.invariant_ok(h.n, os_, od, s, h.alpha, P, R)
    assert ok, (what, worst)
    assert np.max(np.abs(P - Po)) <= 2 * eps, (what, np.max(np.abs(P - Po)))
    return P, Po
