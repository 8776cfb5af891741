"""GPU parity: the CUDA path (through the C ABI) against the CPU oracle and
the paper's printed values.  All tests need a B200 (`-m gpu`).

Gates per batch:
  * arc multiset: bit-exact vs the oracle after every batch;
  * Eq. 2 invariant at every vertex to 1e-12 relative (reading R18);
  * termination: -eps <= R <= eps exactly;
  * GPU vs oracle estimates: L_inf <= 2 eps (reading R19), L1 <= 1e-6 at
    eps = 1e-9 on the tiny config (reading R20);
  * Figs 1-3: bit-exact dyadic values in Vanilla (Alg 3) mode.
"""
import numpy as np
import pytest

import oracle
from oracle import exact
from paper_journals_pvldb_guolst17_b200 import ppr, workload as W
from tests import golden_figs as G
from tests.parity_util import check_batch_state, expand_undirected_arcs

pytestmark = pytest.mark.gpu

MODES = ["opt", "eager", "dupdetect", "vanilla", "async", "scan", "shared", "sortagg"]


def _fig_gpu(mode="vanilla", max_iters=0):
    h = ppr.Ppr(G.N, G.G0_SRC, G.G0_DST, [G.SOURCE], alpha=G.ALPHA, eps=G.EPS, mode=mode)
    return h


# ---------------------------------------------------------------- Figs 1-3 (bit-exact)

def test_fig3a_static_parallel_push_is_bit_exact():
    h = _fig_gpu("vanilla")
    P, R = h.query()
    np.testing.assert_array_equal(R, [1 / 16, 0, 0, 1 / 16])
    np.testing.assert_array_equal(P, [1 / 2, 1 / 4, 3 / 16, 1 / 16])
    st = h.create_stats
    assert st["iters_pos"] == 3 and st["pushes"] == 5  # Fig 3 caption


@pytest.mark.parametrize("mode", MODES)
def test_fig1_single_insertion(mode):
    h = _fig_gpu(mode)
    if mode != "vanilla":  # bring every mode to the Fig 1(a) state first
        h.close()
        h = _fig_gpu("vanilla")
        h.set_option(ppr.OPT_MODE, ppr.MODES[mode])
    h.set_option(ppr.OPT_PUSH, 0)
    h.apply_batch([0], [1])
    P, R = h.query()
    assert R[0] == 5 / 32  # Fig 1(b) 0.1562
    h.push()
    P, R = h.query()
    np.testing.assert_array_equal(R, [0, 5 / 64, 5 / 128, 1 / 16])   # Fig 1(d)
    np.testing.assert_array_equal(P, [37 / 64, 1 / 4, 3 / 16, 1 / 16])


def test_fig2_batch_restore_and_one_parallel_round():
    h = _fig_gpu("vanilla")
    h.set_option(ppr.OPT_PUSH, 0)
    h.apply_batch([0, 3], [1, 0])
    P, R = h.query()
    np.testing.assert_array_equal(R, [5 / 32, 0, 0, 7 / 32])        # Fig 2(b)
    st = h.push()
    assert st["iters_pos"] == 1
    P, R = h.query()
    np.testing.assert_array_equal(R, [7 / 128, 5 / 64, 5 / 128, 5 / 128])   # Fig 2(d)
    np.testing.assert_array_equal(P, [37 / 64, 1 / 4, 3 / 16, 11 / 64])
    blk = G.load()["fig2_d"]
    for v in range(4):
        assert G.matches_printed(P[v], blk["P"][v]) and G.matches_printed(R[v], blk["R"][v])


@pytest.mark.parametrize("rounds,Rw,Pw", [
    (1, [0, .5, .25, 0], [.5, 0, 0, 0]),                 # Fig 3 a(2)
    (2, [0, 0, .125, .125], [.5, .25, .125, 0]),         # Fig 3 a(3)
    (3, [.0625, 0, 0, .0625], [.5, .25, .1875, .0625]),  # Fig 3 a(4)
])
def test_fig3a_trace_rounds(rounds, Rw, Pw):
    h = _fig_gpu("vanilla")
    h.reset()                       # P = 0, R = e_s (Fig 3 a(1))
    P, R = h.query()
    np.testing.assert_array_equal(R, [1, 0, 0, 0])
    np.testing.assert_array_equal(P, [0, 0, 0, 0])
    h.set_option(ppr.OPT_MAX_ITERS, rounds)
    st = h.push()
    assert st["iters_pos"] == rounds
    P, R = h.query()
    np.testing.assert_array_equal(R, Rw)
    np.testing.assert_array_equal(P, Pw)


# ---------------------------------------------------------------- helpers

_check_batch_state = check_batch_state


def _run_stream(name, mode, slides, eps=None, sources=1, check_every=1, relabel=-1, options=None,
                layout=ppr.LAYOUT_ARRAYS, pool_degrees=-1, **over):
    """Streams `slides` batches through a handle and the oracle, checking the
    per-batch gates.  `options`: {ppr.OPT_*: value} set through ppr_set_option
    after create (schedule / kernel selection for the batches)."""
    st, cfg = W.make_stream(name, **over)
    eps = eps or cfg["eps"]
    g0s, g0d = st.window()
    srcs = W.pick_sources(cfg["n"], g0s, g0d, cfg["band"], sources)
    h = ppr.Ppr(cfg["n"], g0s, g0d, srcs, alpha=0.15, eps=eps, mode=mode,
                undirected=False, relabel=relabel, layout=layout, pool_degrees=pool_degrees)
    for k, v in (options or {}).items():
        h.set_option(k, v)
    o = oracle.Oracle(cfg["n"], g0s, g0d, srcs, 0.15, eps)
    o.push(oracle.SEQ)
    for i, s in enumerate(srcs):
        _check_batch_state(h, o, i, int(s), eps, "static")
    last = None
    for t in range(slides):
        b = st.next_batch()
        stats = h.apply_batch(*b)
        o.apply(*b, mode=oracle.SEQ)
        if t % check_every == check_every - 1 or t == slides - 1:
            for i, s in enumerate(srcs):
                last = _check_batch_state(h, o, i, int(s), eps, f"slide {t}")
        assert stats["num_arcs"] == o.num_arcs
    return h, o, last


# ---------------------------------------------------------------- tiny config (configs[0])

@pytest.mark.parametrize("mode", MODES)
def test_tiny_config_all_modes_track_oracle(mode):
    _run_stream("tiny", mode, slides=12)


@pytest.mark.parametrize("mode", MODES)
def test_wide_pool_entries_track_oracle(mode):
    # ppr_opts.pool_degrees = 1: in-list entries carry (d_out(u), u), refreshed after
    # every restore (the format the library picks for DRAM-resident residuals)
    _run_stream("tiny", mode, slides=8, pool_degrees=1, sources=3 if mode == "shared" else 1)


@pytest.mark.parametrize("rebuild", [0, 1])
def test_wide_pool_entries_rebuild_and_relabel(rebuild):
    _run_stream("tiny", "opt", slides=6, pool_degrees=1, relabel=1,
                options={ppr.OPT_FORCE_REBUILD: rebuild, ppr.OPT_RING_ALL: 1})
    with pytest.raises(ppr.PprError) as ex:  # the packed records keep u32 in-list entries
        _run_stream("tiny", "opt", slides=1, pool_degrees=1, layout=ppr.LAYOUT_PACKED)
    assert ex.value.code == ppr.PPR_EINVAL


@pytest.mark.parametrize("tail,ring_all", [(0, 0), (16384, 0), (16384, 1), (64, 0)])
def test_opt_schedules_track_oracle(tail, ring_all):
    # Opt rounds only / rounds with the ring tail / ring from the seeds (DESIGN.md
    # "Hybrid tail"), selected through ppr_set_option: every schedule meets the same gates
    opts = {ppr.OPT_RING_TAIL: tail, ppr.OPT_RING_ALL: ring_all}
    _run_stream("tiny", "opt", slides=6, options=opts)
    _run_stream("tiny", "opt", slides=3, sources=3, options=opts)


@pytest.mark.parametrize("tail,ring_all", [(0, 0), (16384, 0), (16384, 1), (64, 0)])
def test_opt_enqueues_each_entry_exactly_once(tail, ring_all):
    """SURVEY 8(a) correctness note on the fused self-update: with
    PPR_OPT_CHECK_ENQUEUE every enqueue sets an in-queue flag and every dequeue
    clears it before the entry's exchange, so an entry enqueued while queued is
    counted -- exactly-once enqueue means the count stays 0 on every batch, for
    every schedule (rounds, ring tail, ring from the seeds with lazy
    done-accounting), single- and multi-source (the check is its own build of
    the 2-chain Opt push, push_chk.cu)."""
    for sources, slides in ((1, 8), (3, 4)):
        st, cfg = W.make_stream("tiny")
        g0s, g0d = st.window()
        srcs = W.pick_sources(cfg["n"], g0s, g0d, cfg["band"], sources)
        h = ppr.Ppr(cfg["n"], g0s, g0d, srcs, alpha=0.15, eps=cfg["eps"], mode="opt")
        for k, v in {ppr.OPT_RING_TAIL: tail, ppr.OPT_RING_ALL: ring_all,
                     ppr.OPT_CHECK_ENQUEUE: 1}.items():
            h.set_option(k, v)
        o = oracle.Oracle(cfg["n"], g0s, g0d, srcs, 0.15, cfg["eps"])
        o.push(oracle.SEQ)
        total = 0
        for t in range(slides):
            b = st.next_batch()
            stats = h.apply_batch(*b)
            o.apply(*b, mode=oracle.SEQ)
            assert stats["dup_enqueues"] == 0, f"slide {t}: {stats['dup_enqueues']} duplicate enqueues"
            total += stats["pushes"]
        for i, s in enumerate(srcs):
            _check_batch_state(h, o, i, int(s), cfg["eps"], "after the checked slides")
        assert total > 0
        h.close()


def test_opt_enqueue_check_lj_full_size():
    """The exactly-once check on the LJ shape in the bench's configuration
    (ring from the seeds, lazy done-accounting, 592 CTAs): 0 duplicates."""
    st, cfg = W.make_stream("lj")
    g0s, g0d = st.window()
    (s,) = W.pick_sources(cfg["n"], g0s, g0d, cfg["band"], 1)
    h = ppr.Ppr(cfg["n"], g0s, g0d, [s], alpha=0.15, eps=cfg["eps"], mode="opt")
    h.set_option(ppr.OPT_CHECK_ENQUEUE, 1)
    for t in range(3):
        stats = h.apply_batch(*st.next_batch())
        assert stats["pushed_edges"] > 10**6
        assert stats["dup_enqueues"] == 0, f"slide {t}: {stats['dup_enqueues']} duplicate enqueues"
    h.close()


@pytest.mark.parametrize("tail,ring_all", [(0, 0), (16384, 1)])
def test_opt_three_edge_chains_track_oracle(tail, ring_all):
    # the Opt push compiled with 3 edge chains per lane (push_u3.cu, chosen for
    # dense graphs) forced on the tiny config, rounds and ring schedules
    opts = {ppr.OPT_EDGE_CHAINS: 3, ppr.OPT_RING_TAIL: tail, ppr.OPT_RING_ALL: ring_all}
    _run_stream("tiny", "opt", slides=6, options=opts)
    _run_stream("tiny", "opt", slides=3, sources=3, options=opts)


@pytest.mark.parametrize("mode,ring_all,relabel", [("opt", 0, -1), ("opt", 1, 1),
                                                   ("eager", 0, -1), ("vanilla", 0, 1)])
def test_packed_vertex_records_track_oracle(mode, ring_all, relabel):
    # single-source handles in the packed layout (one 32-byte {R, P, slab, d_out}
    # record per vertex): same gates as the arrays
    _run_stream("tiny", mode, slides=8, relabel=relabel, layout=ppr.LAYOUT_PACKED,
                options={ppr.OPT_RING_ALL: ring_all})


@pytest.mark.parametrize("n_arcs", [32768, 32769, 2 ** 18, 2 ** 18 + 1])
def test_radix_sort_tile_switch(n_arcs):
    # batches at the radix sort's switches and one key past each: <= 64 tiles of
    # 512 keys (chained passes: the scatter builds the next pass's histogram),
    # more tiles with a scan kernel, and past 2^18 keys 4096-key tiles; with
    # duplicates and an insert/delete pair of the same arc
    n = 200_000
    src, dst = W.rmat_stream(n, 1_000_000, seed=9, abc=W.SHAPED)
    w0 = 500_000
    (s,) = W.pick_sources(n, src[:w0], dst[:w0], 1000, 1)
    h = ppr.Ppr(n, src[:w0], dst[:w0], [s], alpha=0.15, eps=1e-8)
    o = oracle.Oracle(n, src[:w0], dst[:w0], [s], 0.15, 1e-8)
    o.push(oracle.SEQ)
    ni = n_arcs // 2
    nd = n_arcs - ni
    ins = (np.concatenate([src[w0:w0 + ni - 3], src[:2], [7]]), np.concatenate([dst[w0:w0 + ni - 3], dst[:2], [8]]))
    dels = (np.concatenate([src[:nd - 1], [7]]), np.concatenate([dst[:nd - 1], [8]]))
    h.apply_batch(*ins, *dels)
    o.apply(*ins, *dels)
    _check_batch_state(h, o, 0, int(s), 1e-8, f"batch of {n_arcs} arcs")


@pytest.mark.parametrize("mode", ["opt", "scan", "vanilla"])
def test_tiny_config_degree_relabelled(mode):
    # internal degree-ordered ids: every id at the boundary must stay external
    _run_stream("tiny", mode, slides=8, relabel=1)


def test_tiny_config_multi_source_relabelled():
    _run_stream("tiny", "opt", slides=4, sources=3, relabel=1)


def test_fig2_bit_exact_with_relabelling():
    h = ppr.Ppr(G.N, G.G0_SRC, G.G0_DST, [G.SOURCE], alpha=G.ALPHA, eps=G.EPS, mode="vanilla",
                relabel=1)
    h.apply_batch([0, 3], [1, 0])
    P, R = h.query()
    np.testing.assert_array_equal(R, [7 / 128, 5 / 64, 5 / 128, 5 / 128])
    np.testing.assert_array_equal(P, [37 / 64, 1 / 4, 3 / 16, 11 / 64])
    d = h.export_dout()
    np.testing.assert_array_equal(d, [2, 1, 2, 2])


def test_tiny_config_full_50_slides_opt():
    _run_stream("tiny", "opt", slides=50, check_every=5)


def test_tiny_config_eps_1e9_l1_gate():
    # reading R20: L1 <= 1e-6 at eps = 1e-9 on the tiny config
    h, o, (P, Po) = _run_stream("tiny", "opt", slides=20, eps=1e-9, check_every=10)
    assert np.sum(np.abs(P - Po)) <= 1e-6


def test_tiny_config_multi_source():
    _run_stream("tiny", "opt", slides=6, sources=4, check_every=3)


@pytest.mark.parametrize("sources", [3, 32, 40, 70])
def test_tiny_config_multi_source_shared(sources):
    # PPR_MODE_SHARED (DESIGN.md K-SHARED): one full group, partial groups
    # (S = 40: lanes 8..31 of group 1 idle), several groups; every source of
    # every batch against the sequential oracle
    _run_stream("tiny", "shared", slides=5, sources=sources, check_every=1)


def test_shared_statistics_are_per_call():
    # walk_edges / entries are the push's own counts for each call (round 1 left
    # walk_edges accumulating across calls): a call without a push reports 0
    st, cfg = W.make_stream("tiny")
    g0s, g0d = st.window()
    srcs = W.pick_sources(cfg["n"], g0s, g0d, cfg["band"], 40)
    h = ppr.Ppr(cfg["n"], g0s, g0d, srcs, alpha=0.15, eps=1e-8, mode="shared")
    s1 = h.apply_batch(*st.next_batch())
    assert 0 < s1["walk_edges"] <= s1["pushed_edges"] and 0 < s1["entries"] <= s1["pushes"]
    s2 = h.apply_batch(*st.next_batch())
    assert s2["walk_edges"] <= s2["pushed_edges"] and s2["entries"] <= s2["pushes"]
    h.set_option(ppr.OPT_PUSH, 0)
    s3 = h.apply_batch(*st.next_batch())
    assert s3["walk_edges"] == 0 and s3["entries"] == 0 and s3["pushed_edges"] == 0
    ho = ppr.Ppr(cfg["n"], g0s, g0d, srcs[:1], alpha=0.15, eps=1e-8)
    so = ho.apply_batch(*st.next_batch())
    assert so["entries"] == so["pushes"] and so["walk_edges"] == so["pushed_edges"]


@pytest.mark.parametrize("wave", [32, 64])
def test_tiny_config_multi_source_shared_waves(wave):
    # PPR_OPT_WAVE: one push launch per wave of source groups after the shared
    # store/restore; 70 sources = 2 full groups + a partial one
    _run_stream("tiny", "shared", slides=4, sources=70, check_every=1,
                options={ppr.OPT_WAVE: wave})


def test_tiny_config_multi_source_shared_relabelled_rebuild():
    st, cfg = W.make_stream("tiny")
    g0s, g0d = st.window()
    srcs = W.pick_sources(cfg["n"], g0s, g0d, cfg["band"], 36)
    h = ppr.Ppr(cfg["n"], g0s, g0d, srcs, alpha=0.15, eps=1e-8, mode="shared", relabel=1)
    o = oracle.Oracle(cfg["n"], g0s, g0d, srcs, 0.15, 1e-8)
    o.push(oracle.SEQ)
    h.set_option(ppr.OPT_FORCE_REBUILD, 1)
    for t in range(3):
        b = st.next_batch()
        stt = h.apply_batch(*b)
        assert stt["rebuilt"] == 1 and stt["walk_edges"] <= stt["pushed_edges"]
        o.apply(*b)
        for i, s in enumerate(srcs):
            _check_batch_state(h, o, i, int(s), 1e-8, f"shared rebuild slide {t} source {i}")


def test_shared_full_scan_push_matches_static():
    # ppr_reset + ppr_push (seed_all) recomputes static PPR for all sources
    st, cfg = W.make_stream("tiny")
    g0s, g0d = st.window()
    srcs = W.pick_sources(cfg["n"], g0s, g0d, cfg["band"], 33)
    h = ppr.Ppr(cfg["n"], g0s, g0d, srcs, alpha=0.15, eps=1e-8, mode="shared")
    h.reset()
    h.push()
    gs, gd = h.export_edges()
    for i in (0, 17, 32):
        P, R = h.query(i)
        assert exact.terminated(R, 1e-8)
        Pstar = exact.ppr_power(cfg["n"], gs, gd, int(srcs[i]), 0.15)
        assert np.max(np.abs(P - Pstar)) <= 1e-8 * (1 + 1e-6)


# ---------------------------------------------------------------- sort-and-aggregate (NEXT-4)

def _tiny_static(mode, eps, sources=1, relabel=0):
    st, cfg = W.make_stream("tiny")
    g0s, g0d = st.window()
    srcs = W.pick_sources(cfg["n"], g0s, g0d, cfg["band"], sources)
    h = ppr.Ppr(cfg["n"], g0s, g0d, srcs, alpha=0.15, eps=eps, mode=mode, relabel=relabel)
    o = oracle.Oracle(cfg["n"], g0s, g0d, srcs, 0.15, eps)
    return st, cfg, srcs, h, o


@pytest.mark.parametrize("eps,sources", [(1e-7, 1), (1e-9, 1), (1e-8, 3)])
def test_sortagg_static_push_bit_exact_vs_alg3_oracle(eps, sources):
    # PPR_MODE_SORTAGG applies each round's increments to R(v) in ascending-u
    # order, exactly the oracle's Alg 3 emulation: same rounds,
    # same pushes, and P, R equal bit for bit from P = 0, R = e_s
    st, cfg, srcs, h, o = _tiny_static("sortagg", eps, sources)
    o.push(oracle.JACOBI)
    so, sg = o.stats(), h.create_stats
    assert sg["pushes"] == so["pushes"] and sg["pushed_edges"] == so["pushed_edges"]
    for i in range(sources):
        P, R = h.query(i)
        Po, Ro = o.query(i)
        np.testing.assert_array_equal(R, Ro)
        np.testing.assert_array_equal(P, Po)
    if sources == 1:
        assert sg["iters_pos"] == so["rounds_pos"] and sg["iters_neg"] == so["rounds_neg"]


@pytest.mark.parametrize("rounds", [1, 4, 17])
def test_sortagg_round_by_round_bit_exact(rounds):
    # budgeted Alg 3 (max_iters rounds per phase) from P = 0, R = e_s
    st, cfg, srcs, h, o = _tiny_static("sortagg", 1e-9)
    h.reset()
    h.set_option(ppr.OPT_MAX_ITERS, rounds)
    stt = h.push()
    assert stt["iters_pos"] == rounds
    o2 = oracle.Oracle(cfg["n"], *st.window(), srcs, 0.15, 1e-9)
    o2.set_state(0, np.zeros(cfg["n"]), np.eye(1, cfg["n"], int(srcs[0]))[0])
    o2.push(oracle.JACOBI, max_steps=rounds)
    P, R = h.query()
    Po, Ro = o2.query()
    np.testing.assert_array_equal(R, Ro)
    np.testing.assert_array_equal(P, Po)


def test_sortagg_bit_reproducible_across_runs():
    # no atomics: two handles fed the same stream agree bit for bit after every
    # batch (restore, store and push), also with degree-relabelled ids
    st, cfg = W.make_stream("tiny")
    g0s, g0d = st.window()
    srcs = W.pick_sources(cfg["n"], g0s, g0d, cfg["band"], 2)
    hs = [ppr.Ppr(cfg["n"], g0s, g0d, srcs, alpha=0.15, eps=1e-9, mode="sortagg", relabel=1)
          for _ in range(2)]
    for t in range(6):
        b = st.next_batch()
        for h in hs:
            h.apply_batch(*b)
        for i in range(2):
            (P1, R1), (P2, R2) = hs[0].query(i), hs[1].query(i)
            np.testing.assert_array_equal(P1, P2)
            np.testing.assert_array_equal(R1, R2)


def test_tiny_against_power_iteration():
    st, cfg = W.make_stream("tiny")
    g0s, g0d = st.window()
    (s,) = W.pick_sources(cfg["n"], g0s, g0d, cfg["band"], 1)
    h = ppr.Ppr(cfg["n"], g0s, g0d, [s], alpha=0.15, eps=cfg["eps"])
    for _ in range(3):
        h.apply_batch(*st.next_batch())
    P, R = h.query()
    gs, gd = h.export_edges()
    Pstar = exact.ppr_power(cfg["n"], gs, gd, int(s), 0.15)
    assert np.max(np.abs(P - Pstar)) <= cfg["eps"] * (1 + 1e-6)


# ---------------------------------------------------------------- restore (Lemma 3 vs Alg 1 x k)

def _restore_term_scale(n, alpha, s, P, R, dout0, b):
    """Per-vertex magnitude of the terms either evaluation sums: the batch
    closed form (Lemma 3 proof: |r0| + (sum_j |op_j|(1-a)|P(v_j)| +
    |S0|(a 1[u=s] + |P(u)| + a|r0|)) / (a d_k), or 1[u=s] + |P(u)|/a when d_k = 0,
    reading R4) and the oracle's k sequential Alg 1 calls (the
    largest intermediate |R(u)| and update term, with the intermediate
    degrees).  Both evaluations are exact up to a few ulps of this scale."""
    isrc, idst, dsrc, ddst = (np.asarray(x, dtype=np.int64) for x in b)
    u = np.concatenate([isrc, dsrc])
    v = np.concatenate([idst, ddst])
    op = np.concatenate([np.ones(len(isrc)), -np.ones(len(dsrc))])
    S0 = np.bincount(u, weights=op, minlength=n)
    A1 = np.bincount(u, weights=(1 - alpha) * np.abs(P[v]), minlength=n)
    dk = dout0.astype(np.float64) + S0
    one = np.zeros(n)
    one[s] = 1.0
    with np.errstate(divide="ignore", invalid="ignore"):
        t = np.abs(R) + (A1 + np.abs(S0) * (alpha * one + np.abs(P) + alpha * np.abs(R))) / (alpha * dk)
    scale = np.where(dk > 0, t, one + np.abs(P) / alpha)
    # the sequential path: insertions then deletions, in order (oracle CPU-Seq)
    d = dout0.astype(np.int64).copy()
    r = np.array(R, dtype=np.float64)
    for uu, vv, o in zip(u.tolist(), v.tolist(), op.tolist()):
        d[uu] += int(o)
        if d[uu] > 0:
            term = ((1 - alpha) * abs(P[vv]) + abs(P[uu]) + alpha * abs(r[uu]) + alpha * one[uu]) / (alpha * d[uu])
            r[uu] += o * ((1 - alpha) * P[vv] - P[uu] - alpha * r[uu] + alpha * one[uu]) / (alpha * d[uu])
        else:
            term = one[uu] + abs(P[uu]) / alpha
            r[uu] = one[uu] - P[uu] / alpha
        scale[uu] = max(scale[uu], term, abs(r[uu]))
    return scale


def test_restore_closed_form_matches_sequential_alg1():
    st, cfg = W.make_stream("tiny")
    g0s, g0d = st.window()
    srcs = W.pick_sources(cfg["n"], g0s, g0d, cfg["band"], 2)
    h = ppr.Ppr(cfg["n"], g0s, g0d, srcs, alpha=0.15, eps=1e-7)
    o = oracle.Oracle(cfg["n"], g0s, g0d, srcs, 0.15, 1e-7)
    for sidx in range(2):  # start both from the GPU's converged state
        P, R = h.query(sidx)
        o.set_state(sidx, P, R)
    h.set_option(ppr.OPT_PUSH, 0)
    for t in range(3):
        b = st.next_batch()
        before = [h.query(sidx) for sidx in range(2)]
        dout0 = h.export_dout()
        stt = h.apply_batch(*b)
        assert stt["ms_restore"] > 0  # device-clock time of the restore kernel
        o.apply(*b, do_push=False)
        touched = np.zeros(h.n, dtype=bool)
        touched[np.concatenate([b[0], b[2]])] = True
        for sidx in range(2):
            P, R = h.query(sidx)
            Po, Ro = o.query(sidx)
            np.testing.assert_array_equal(P, Po)
            np.testing.assert_array_equal(R[~touched], Ro[~touched])  # restore touches only u
            scale = _restore_term_scale(h.n, h.alpha, int(srcs[sidx]), *before[sidx], dout0, b)
            d, sc = np.abs(R - Ro)[touched], scale[touched]
            assert np.all(d[sc == 0] == 0)  # all terms zero: both sides exactly 0
            err = d[sc > 0] / sc[sc > 0]
            assert np.max(err) <= 1e-12, (sidx, np.max(err))
        np.testing.assert_array_equal(h.export_dout(), o.dout())
        # continue from identical states
        h.push()
        for sidx in range(2):
            P, R = h.query(sidx)
            o.set_state(sidx, P, R)


# ---------------------------------------------------------------- edge cases

def _small(mode="opt", eps=1e-9):
    src = [0, 1, 2, 2, 3, 0]
    dst = [3, 0, 0, 1, 2, 1]
    h = ppr.Ppr(4, src, dst, [0], alpha=0.15, eps=eps, mode=mode)
    o = oracle.Oracle(4, src, dst, [0], 0.15, eps)
    o.push(oracle.SEQ)
    return h, o


def test_empty_batch_is_noop():
    h, _ = _small()
    P0, R0 = h.query()
    st = h.apply_batch()
    assert st["kernel_launches"] == 0
    P1, R1 = h.query()
    np.testing.assert_array_equal(P0, P1)
    np.testing.assert_array_equal(R0, R1)


def test_absent_deletion_enoent_state_unchanged():
    h, _ = _small()
    P0, R0 = h.query()
    e0 = h.export_edges()
    rc, _ = h.apply_batch([1], [3], [3, 1], [1, 2], raise_on_error=False)
    assert rc == ppr.PPR_ENOENT
    P1, R1 = h.query()
    np.testing.assert_array_equal(P0, P1)
    np.testing.assert_array_equal(R0, R1)
    e1 = h.export_edges()
    np.testing.assert_array_equal(e0[0], e1[0])
    np.testing.assert_array_equal(e0[1], e1[1])
    h.apply_batch([1], [3])  # the handle stays usable


def test_out_of_range_erange_state_unchanged():
    h, _ = _small()
    P0, R0 = h.query()
    rc, _ = h.apply_batch([1], [4], raise_on_error=False)
    assert rc == ppr.PPR_ERANGE
    rc, _ = h.apply_batch([], [], [9], [0], raise_on_error=False)
    assert rc == ppr.PPR_ERANGE
    P1, R1 = h.query()
    np.testing.assert_array_equal(P0, P1)
    np.testing.assert_array_equal(R0, R1)


def test_insert_then_delete_same_arc_cancels_exactly():
    h, _ = _small()
    P0, R0 = h.query()
    h.apply_batch([1], [3], [1], [3])
    P1, R1 = h.query()
    np.testing.assert_array_equal(P0, P1)
    np.testing.assert_array_equal(R0, R1)


def test_delete_last_out_arc_and_multiset_semantics():
    h, o = _small()
    for b in [([0, 0], [3, 3], [], []),        # multiplicity 3 on 0->3
              ([], [], [3], [2]),              # vertex 3 loses its only out-arc
              ([2, 2], [2, 2], [0, 0], [3, 1]),  # self-loops, deletions
              ([1, 3], [1, 0], [2], [2])]:
        h.apply_batch(*b)
        o.apply(*b)
        _check_batch_state(h, o, 0, 0, 1e-9, str(b))


@pytest.mark.parametrize("mode", MODES)
def test_forced_rebuild_path(mode):
    st, cfg = W.make_stream("tiny")
    g0s, g0d = st.window()
    srcs = W.pick_sources(cfg["n"], g0s, g0d, cfg["band"], 1)
    h = ppr.Ppr(cfg["n"], g0s, g0d, srcs, alpha=0.15, eps=1e-7, mode=mode)
    o = oracle.Oracle(cfg["n"], g0s, g0d, srcs, 0.15, 1e-7)
    o.push(oracle.SEQ)
    h.set_option(ppr.OPT_FORCE_REBUILD, 1)
    for t in range(3):
        b = st.next_batch()
        stt = h.apply_batch(*b)
        assert stt["rebuilt"] == 1
        o.apply(*b)
        _check_batch_state(h, o, 0, int(srcs[0]), 1e-7, f"rebuild slide {t}")


def test_growing_graph_rebuilds_with_replayed_batch_graphs():
    # insert-only batches of one shape: the batch's CUDA graph is replayed while
    # rebuilds flip the active pool and the spare pool is regrown to a different
    # size; the rebuild must check the capacity of the pool that is spare on the
    # device at replay time (not the one captured)
    n = 2000
    src, dst = W.rmat_stream(n, 12_000, seed=21, abc=W.GRAPH500)
    w0 = 2000
    (s,) = W.pick_sources(n, src[:w0], dst[:w0], 100, 1)
    h = ppr.Ppr(n, src[:w0], dst[:w0], [s], alpha=0.15, eps=1e-9, min_cap=1, slack=0.0)
    o = oracle.Oracle(n, src[:w0], dst[:w0], [s], 0.15, 1e-9)
    o.push(oracle.SEQ)
    rebuilt = 0
    for t in range(10):
        b = (src[w0 + 1000 * t:w0 + 1000 * (t + 1)], dst[w0 + 1000 * t:w0 + 1000 * (t + 1)], [], [])
        stt = h.apply_batch(*b)
        rebuilt += stt["rebuilt"]
        o.apply(*b)
        _check_batch_state(h, o, 0, int(s), 1e-9, f"growing slide {t}")
    assert rebuilt >= 2


def test_device_memory_batches():
    import torch
    st, cfg = W.make_stream("tiny")
    g0s, g0d = st.window()
    srcs = W.pick_sources(cfg["n"], g0s, g0d, cfg["band"], 1)
    h = ppr.Ppr(cfg["n"], g0s, g0d, srcs, alpha=0.15, eps=1e-7)
    o = oracle.Oracle(cfg["n"], g0s, g0d, srcs, 0.15, 1e-7)
    o.push(oracle.SEQ)
    for t in range(3):
        b = st.next_batch()
        tb = [torch.from_numpy(x.astype(np.int32)).cuda() for x in b]
        torch.cuda.synchronize()
        h.apply_batch(*tb, mem=ppr.MEM_DEVICE)
        o.apply(*b)
        _check_batch_state(h, o, 0, int(srcs[0]), 1e-7, f"device slide {t}")


def test_undirected_stream():
    n = 3000
    src, dst = W.rmat_stream(n, 20000, seed=5, abc=W.GRAPH500, undirected=True)
    st = W.Stream(n, src, dst, w0=10000, ins_per_slide=250, del_per_slide=750, undirected=True)
    g0s, g0d = st.window()  # already expanded to arcs
    srcs = W.pick_sources(n, g0s, g0d, 100, 1)
    h = ppr.Ppr(n, g0s, g0d, srcs, alpha=0.15, eps=1e-8)
    o = oracle.Oracle(n, g0s, g0d, srcs, 0.15, 1e-8)
    o.push(oracle.SEQ)
    for t in range(4):
        b = st.next_batch()
        h.apply_batch(*b)
        o.apply(*b)
        _check_batch_state(h, o, 0, int(srcs[0]), 1e-8, f"undirected slide {t}")


# ---------------------------------------------------------------- full BASELINE sizes

def test_lj_full_size_against_oracle():
    """configs[1] at full size in the bench's launch configuration (Opt mode,
    degree relabelling on): the static state and two 10^4+10^4 slides, every
    vertex checked -- arc multiset bit-exact, Eq. 2, termination, L_inf <= 2 eps
    against the sequential oracle."""
    st, cfg = W.make_stream("lj")
    g0s, g0d = st.window()
    (s,) = W.pick_sources(cfg["n"], g0s, g0d, cfg["band"], 1)
    h = ppr.Ppr(cfg["n"], g0s, g0d, [s], alpha=0.15, eps=cfg["eps"], mode="opt")
    o = oracle.Oracle(cfg["n"], g0s, g0d, [s], 0.15, cfg["eps"])
    o.push(oracle.SEQ)
    _check_batch_state(h, o, 0, int(s), cfg["eps"], "lj static")
    for t in range(2):
        b = st.next_batch()
        stats = h.apply_batch(*b)
        o.apply(*b)
        assert stats["pushed_edges"] > 10**6  # a real hub-band workload
        _check_batch_state(h, o, 0, int(s), cfg["eps"], f"lj slide {t}")


def test_orkut_full_size_properties():
    """configs[2] shape at full size (undirected, 50% window, deletion-heavy
    k = 10^4): the arc multiset equals the expansion of the window's stream
    edges (computed here, independently of the GPU), termination and Eq. 2 at
    every vertex on those arcs."""
    st, cfg = W.make_stream("orkut")
    e0s, e0d = st.src[st.lo:st.hi].copy(), st.dst[st.lo:st.hi].copy()
    arcs = expand_undirected_arcs(e0s, e0d)
    (s,) = W.pick_sources(cfg["n"], arcs[0], arcs[1], cfg["band"], 1)
    h = ppr.Ppr(cfg["n"], e0s, e0d, [s], alpha=0.15, eps=cfg["eps"], undirected=True)
    assert h.create_stats["num_arcs"] == len(arcs[0])
    for t in range(2):
        i0, i1, d0, d1 = st.hi, st.hi + cfg["ins"], st.lo, st.lo + cfg["dele"]
        stats = h.apply_batch(st.src[i0:i1], st.dst[i0:i1], st.src[d0:d1], st.dst[d0:d1])
        st.hi, st.lo = i1, d1
        assert stats["num_arcs"] == 2 * (st.hi - st.lo)
    P, R = h.query()
    assert exact.terminated(R, cfg["eps"])
    es, ed = expand_undirected_arcs(st.src[st.lo:st.hi], st.dst[st.lo:st.hi])
    order = np.lexsort((es, ed))  # (dst, src) order of ppr_export_edges
    es, ed = es[order], ed[order]
    gs, gd = h.export_edges()
    np.testing.assert_array_equal(gd, ed)
    np.testing.assert_array_equal(gs, es)
    ok, worst = exact.invariant_ok(cfg["n"], es, ed, int(s), 0.15, P, R)
    assert ok, worst


def test_lj_multi_source_shared_full_size():
    """configs[4] shape (LJ-shaped, hub-band sources) in the bench's launch
    configuration for several sources per rank (PPR_MODE_SHARED, relabelled):
    two 10^4+10^4 slides with S = 64; termination for every source, Eq. 2 for
    sampled sources, and one source against the sequential oracle (every
    vertex, L_inf <= 2 eps)."""
    st, cfg = W.make_stream("lj")
    g0s, g0d = st.window()
    srcs = W.pick_sources(cfg["n"], g0s, g0d, cfg["band"], 64)
    h = ppr.Ppr(cfg["n"], g0s, g0d, srcs, alpha=0.15, eps=cfg["eps"], mode="shared")
    k = 37  # the oracle follows one source of the second group
    o = oracle.Oracle(cfg["n"], g0s, g0d, [srcs[k]], 0.15, cfg["eps"])
    o.push(oracle.SEQ)
    for t in range(2):
        b = st.next_batch()
        stats = h.apply_batch(*b)
        o.apply(*b)
        assert stats["walk_edges"] < stats["pushed_edges"]  # in-lists really shared
    gs, gd = h.export_edges()
    os_, od = o.export()
    np.testing.assert_array_equal(gd, od)
    np.testing.assert_array_equal(gs, os_)
    for i in range(64):
        P, R = h.query(i)
        assert exact.terminated(R, cfg["eps"]), i
        if i in (0, 31, 32, k, 63):
            ok, worst = exact.invariant_ok(cfg["n"], gs, gd, int(srcs[i]), 0.15, P, R)
            assert ok, (i, worst)
        if i == k:
            Po, _ = o.query(0)
            assert np.max(np.abs(P - Po)) <= 2 * cfg["eps"]
