"""GPU parity on reduced versions of the BASELINE configs that the tiny tests
do not reach, each in the launch configuration bench.py uses for the full-size
config, every batch against the sequential oracle (tests/parity_util.py gates:
arc multiset bit-exact, Eq. 2 on the oracle's arcs, eps-termination, L_inf <=
2 eps).

* configs[2] Orkut-shaped: undirected edges expanded by the
  LIBRARY (ppr_graph.undirected = 1), 50% window, deletion-heavy
  slides (1/4 newest insertions + 3/4 oldest deletions), explicit self-loops and
  duplicate edges; dense (>= 8 arcs per vertex) so the Opt push runs on the
  ring from its seeds with 3 edge chains per lane.
* configs[2] k = 10^6 path: one deletion-heavy batch of > 2^18 arcs (the long
  radix-sort tiles with a separate scan kernel, a NEG-heavy push), in place and
  through the sort/merge rebuild.
* configs[3] Twitter-shaped: resident window, degree-relabelled
  ids, no persisting L2 window, ring from the seeds (the choices the library
  makes at full size, forced here at n = 2e6).
"""
import numpy as np
import pytest

import oracle
from oracle import exact
from paper_journals_pvldb_guolst17_b200 import ppr, workload as W
from tests.parity_util import check_batch_state, expand_undirected_arcs

pytestmark = pytest.mark.gpu

ALPHA = 0.15


@pytest.fixture(scope="module")
def orkut_small():
    """Orkut-shaped (R-MAT (0.5,0.2,0.2,0.1), 38.1 undirected edges per vertex)
    at n = 3e5, stream of unique undirected edges, window = first 50%."""
    n = 300_000
    m = int(n * 117_185_083 / 3_072_441)
    src, dst = W.rmat_stream(n, m, seed=42, abc=W.SHAPED, undirected=True)
    return n, src, dst, m // 2


def _undirected_handle(n, e0s, e0d, eps, **kw):
    arcs = expand_undirected_arcs(e0s, e0d)
    (s,) = W.pick_sources(n, arcs[0], arcs[1], 1000, 1)
    h = ppr.Ppr(n, e0s, e0d, [s], alpha=ALPHA, eps=eps, undirected=True, **kw)
    o = oracle.Oracle(n, arcs[0], arcs[1], [s], ALPHA, eps)
    o.push(oracle.SEQ)
    assert h.create_stats["num_arcs"] == len(arcs[0]) == o.num_arcs
    return h, o, int(s)


def _apply_both(h, o, ins, dels):
    """Undirected edge batch: the library expands it, the oracle gets arcs."""
    st = h.apply_batch(ins[0], ins[1], dels[0], dels[1])
    ia, da = expand_undirected_arcs(*ins), expand_undirected_arcs(*dels)
    o.apply(ia[0], ia[1], da[0], da[1])
    assert st["num_arcs"] == o.num_arcs
    return st


def test_orkut_reduced_undirected_library_expansion(orkut_small):
    n, src, dst, w0 = orkut_small
    eps = 1e-9
    h, o, s = _undirected_handle(n, src[:w0], dst[:w0], eps)
    check_batch_state(h, o, 0, s, eps, "orkut static")
    lo, hi = 0, w0
    rng = np.random.default_rng(3)
    loops = rng.choice(n, size=8, replace=False).astype(np.uint32)
    dup = rng.choice(w0, size=8, replace=False)
    k = 10_000
    for t in range(3):
        ni, nd = (k + 3) // 4, 3 * k // 4
        ins = [src[hi:hi + ni], dst[hi:hi + ni]]
        dels = [src[lo:lo + nd], dst[lo:lo + nd]]
        if t == 0:  # explicit self-loops and duplicate (multiset) edges, both orientations
            ins = [np.concatenate([ins[0], loops, src[dup], dst[dup[:4]]]),
                   np.concatenate([ins[1], loops, dst[dup], src[dup[:4]]])]
        if t == 2:  # delete a self-loop and one copy of a duplicated edge
            dels = [np.concatenate([dels[0], loops[:3], src[dup[-2:]]]),
                    np.concatenate([dels[1], loops[:3], dst[dup[-2:]]])]
        st = _apply_both(h, o, ins, dels)
        assert st["pushed_edges"] > 0
        hi, lo = hi + ni, lo + nd
        check_batch_state(h, o, 0, s, eps, f"orkut slide {t}")


def test_orkut_reduced_in_frontier_rounds(orkut_small):
    """The dense Orkut shape pushed in frontier rounds (ring schedule off)
    instead of on the ring: tiles of thousands of edges per CTA, double-buffered
    tiles claimed one ahead, the pipelined 2-chain walk on long in-lists."""
    n, src, dst, w0 = orkut_small
    eps = 1e-9
    h, o, s = _undirected_handle(n, src[:w0], dst[:w0], eps)
    h.set_option(ppr.OPT_RING_ALL, 0)
    h.set_option(ppr.OPT_RING_TAIL, 0)
    lo, hi = 0, w0
    k = 10_000
    for t in range(2):
        ni, nd = (k + 3) // 4, 3 * k // 4
        st = _apply_both(h, o, [src[hi:hi + ni], dst[hi:hi + ni]], [src[lo:lo + nd], dst[lo:lo + nd]])
        assert st["iters_pos"] > 2  # rounds, not the ring's single seed round
        hi, lo = hi + ni, lo + nd
        check_batch_state(h, o, 0, s, eps, f"orkut rounds slide {t}")


@pytest.mark.parametrize("rebuild", [False, True])
def test_orkut_big_deletion_heavy_batch(orkut_small, rebuild):
    """k = 2e5 undirected updates (5e4 insertions + 1.5e5 deletions) = 4e5 arcs
    per sort order, past the 2^18-key switch of the radix sort; the deletions
    dominate, so most of the push is the NEG phase."""
    n, src, dst, w0 = orkut_small
    eps = 1e-8
    h, o, s = _undirected_handle(n, src[:w0], dst[:w0], eps)
    if rebuild:
        h.set_option(ppr.OPT_FORCE_REBUILD, 1)
    k = 200_000
    ni, nd = k // 4, 3 * k // 4
    st = _apply_both(h, o, [src[w0:w0 + ni], dst[w0:w0 + ni]], [src[:nd], dst[:nd]])
    assert 2 * k > 2 ** 18
    assert st["rebuilt"] == (1 if rebuild else st["rebuilt"])
    assert st["iters_neg"] > 0 and st["ms_push_neg"] > 0
    check_batch_state(h, o, 0, s, eps, f"orkut big batch (rebuild={rebuild})")


def test_twitter_reduced_launch_configuration():
    """configs[3] protocol at n = 2e6: the window holds all but the last slides'
    insertions (resident), 12 arcs per vertex (dense), hub-band source;
    relabelling forced on, the persisting L2 window off and degree-carrying
    pool entries on, as the library chooses for the 41.6M-vertex shape
    (R + d_out = 500 MB)."""
    st, cfg = W.make_stream("twitter", n=2_000_000, m=24_000_000, ins=10_000, dele=10_000,
                            slides=3)
    eps = 1e-9
    g0s, g0d = st.window()
    (s,) = W.pick_sources(cfg["n"], g0s, g0d, cfg["band"], 1)
    h = ppr.Ppr(cfg["n"], g0s, g0d, [s], alpha=ALPHA, eps=eps, relabel=1, l2_persist=0,
                pool_degrees=1)
    o = oracle.Oracle(cfg["n"], g0s, g0d, [s], ALPHA, eps)
    o.push(oracle.SEQ)
    check_batch_state(h, o, 0, int(s), eps, "twitter static")
    for t in range(3):
        b = st.next_batch()
        stt = h.apply_batch(*b)
        o.apply(*b)
        # ring from the seeds: the seed round is the only round counted per phase
        assert stt["pushed_edges"] > 0 and stt["iters_pos"] <= 1 and stt["iters_neg"] <= 1
        check_batch_state(h, o, 0, int(s), eps, f"twitter slide {t}")
