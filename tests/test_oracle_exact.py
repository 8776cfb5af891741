"""Pins for the oracle and for its exact checkers, against closed forms and
brute force -- nothing here compares the oracle with itself.

* exact.ppr_dense is pinned by closed forms derived by hand (directed cycle,
  complete digraph, empty graph) and by the undirected reversibility identity
  linking it to the literal Eq. 1 solve.
* exact.ppr_power is pinned to ppr_dense.
* exact.invariant_residual is pinned by exact states (zero residual) and by
  perturbed states (must fail).
* The oracle's pushes (SEQ / JACOBI / BASE) are pinned to P* within eps,
  Eq. 2 and termination on random graphs and batches.
"""
import numpy as np
import pytest

import oracle
from oracle import exact
from paper_journals_pvldb_guolst17_b200 import workload as W


# ---------------------------------------------------------------- closed forms

def test_dense_solve_empty_graph():
    # no arcs: P* = alpha e_s (Eq. 2 with every sum empty)
    P = exact.ppr_dense(5, [], [], 2, 0.15)
    np.testing.assert_allclose(P, [0, 0, 0.15, 0, 0], atol=1e-16)


@pytest.mark.parametrize("L,alpha", [(3, 0.15), (7, 0.5), (12, 0.2)])
def test_dense_solve_directed_cycle(L, alpha):
    # cycle v -> v+1 (mod L): P*(v) = alpha (1-alpha)^dist(v->s) / (1 - (1-alpha)^L)
    src = list(range(L))
    dst = [(v + 1) % L for v in range(L)]
    s = 1
    P = exact.ppr_dense(L, src, dst, s, alpha)
    want = [alpha * (1 - alpha) ** ((s - v) % L) / (1 - (1 - alpha) ** L) for v in range(L)]
    np.testing.assert_allclose(P, want, rtol=1e-13, atol=1e-16)


@pytest.mark.parametrize("n,alpha", [(2, 0.15), (5, 0.15), (9, 0.3)])
def test_dense_solve_complete_digraph(n, alpha):
    # K_n: P*(s) = a(1+a(n-2)) / (1+a(n-2)-(1-a)^2); P*(v!=s) = (1-a)P*(s)/(1+a(n-2))
    src = [u for u in range(n) for v in range(n) if u != v]
    dst = [v for u in range(n) for v in range(n) if u != v]
    s = 0
    a = alpha
    P = exact.ppr_dense(n, src, dst, s, alpha)
    ps = a * (1 + a * (n - 2)) / (1 + a * (n - 2) - (1 - a) ** 2)
    po = (1 - a) * ps / (1 + a * (n - 2))
    np.testing.assert_allclose(P, [ps] + [po] * (n - 1), rtol=1e-13)


def _random_graph(n, m, seed, undirected=False):
    rng = np.random.default_rng(seed)
    src = rng.integers(0, n, m)
    dst = rng.integers(0, n, m)
    keep = src != dst
    src, dst = src[keep], dst[keep]
    if undirected:
        src, dst = np.concatenate([src, dst]), np.concatenate([dst, src])
    return src.astype(np.uint32), dst.astype(np.uint32)


@pytest.mark.parametrize("seed", [1, 2, 3])
def test_dense_solve_undirected_reversibility(seed):
    # On an undirected graph pi_s(v) (literal Eq. 1) = P*(v) d(v) / d(s).
    # A transposed operand or a wrong normalisation in ppr_dense fails this.
    n = 40
    src, dst = _random_graph(n, 120, seed, undirected=True)
    d = np.bincount(src, minlength=n)
    s = int(np.argmax(d))
    rev = exact.ppr_dense(n, src, dst, s, 0.15)
    fwd = exact.forward_ppr(n, src, dst, s, 0.15)
    np.testing.assert_allclose(fwd, rev * d / d[s], rtol=1e-12, atol=1e-16)


@pytest.mark.parametrize("seed", [4, 5])
def test_power_iteration_matches_dense_solve(seed):
    n = 60
    src, dst = _random_graph(n, 200, seed)
    for s in (0, 17):
        np.testing.assert_allclose(exact.ppr_power(n, src, dst, s, 0.15),
                                   exact.ppr_dense(n, src, dst, s, 0.15), atol=1e-14)


def test_invariant_checker_accepts_fixed_point_and_rejects_perturbations():
    n = 30
    src, dst = _random_graph(n, 90, 6)
    s, a = 3, 0.15
    P = exact.ppr_dense(n, src, dst, s, a)
    R = np.zeros(n)
    assert exact.invariant_ok(n, src, dst, s, a, P, R)[0]
    # P = 0, R = e_s is also exact (Fig 3 a(1))
    R0 = np.zeros(n)
    R0[s] = 1
    assert exact.invariant_ok(n, src, dst, s, a, np.zeros(n), R0)[0]
    # any single perturbation must be caught
    for v in (0, s, n - 1):
        Pb = P.copy()
        Pb[v] += 1e-9
        assert not exact.invariant_ok(n, src, dst, s, a, Pb, R)[0]
        Rb = R.copy()
        Rb[v] -= 1e-9
        assert not exact.invariant_ok(n, src, dst, s, a, P, Rb)[0]
    # wrong source is caught
    assert not exact.invariant_ok(n, src, dst, (s + 1) % n, a, P, R)[0]


def test_error_identity_on_arbitrary_consistent_state():
    # Any (P, R) with R := ((1-a)D^-1 A P + a e_s - P)/a satisfies Eq. 2, and
    # then P* - P = a (I - (1-a) D^-1 A)^-1 R exactly.
    n = 25
    src, dst = _random_graph(n, 70, 7)
    s, a = 2, 0.2
    rng = np.random.default_rng(0)
    P = rng.random(n) * 0.1
    T = exact.transition_rev(n, src, dst)
    e = np.zeros(n)
    e[s] = 1
    R = ((1 - a) * T @ P + a * e - P) / a
    assert exact.invariant_ok(n, src, dst, s, a, P, R)[0]
    np.testing.assert_allclose(exact.ppr_dense(n, src, dst, s, a) - P,
                               exact.error_from_residual(n, src, dst, R, a), atol=1e-14)


# ---------------------------------------------------------------- oracle pushes

def _check_state(o, sidx, s, tol_eps=True):
    P, R = o.query(sidx)
    src, dst = o.export()
    assert exact.terminated(R, o.eps)
    ok, worst = exact.invariant_ok(o.n, src, dst, s, o.alpha, P, R)
    assert ok, worst
    if tol_eps:
        Pstar = exact.ppr_dense(o.n, src, dst, s, o.alpha)
        assert np.max(np.abs(P - Pstar)) <= o.eps * (1 + 1e-9)
    return P, R


@pytest.mark.parametrize("mode", [oracle.SEQ, oracle.JACOBI])
@pytest.mark.parametrize("seed", [11, 12, 13])
def test_static_push_is_eps_accurate(mode, seed):
    n = 80
    src, dst = _random_graph(n, 300, seed)
    sources = [0, 5, 41]
    o = oracle.Oracle(n, src, dst, sources, 0.15, 1e-6)
    o.push(mode)
    for i, s in enumerate(sources):
        _check_state(o, i, s)


@pytest.mark.parametrize("mode", [oracle.SEQ, oracle.BASE, oracle.JACOBI])
def test_sliding_window_batches_stay_eps_accurate(mode):
    n = 120
    src, dst = W.rmat_stream(n, 1500, seed=3, abc=W.GRAPH500)
    st = W.Stream(n, src, dst, w0=300, ins_per_slide=40, del_per_slide=40)
    g0s, g0d = st.window()
    srcs = W.pick_sources(n, g0s, g0d, band=10, count=2, seed=7)
    o = oracle.Oracle(n, g0s, g0d, srcs, 0.15, 1e-7)
    o.push(oracle.SEQ if mode == oracle.BASE else mode)
    for _ in range(6):
        o.apply(*st.next_batch(), mode=mode)
        for i, s in enumerate(srcs):
            _check_state(o, i, int(s))


def test_restore_alone_re_establishes_eq2_everywhere():
    # Alg 1 only (no push): Eq. 2 must hold at every vertex after the batch.
    n = 100
    src, dst = W.rmat_stream(n, 1200, seed=5, abc=W.GRAPH500)
    st = W.Stream(n, src, dst, w0=400, ins_per_slide=60, del_per_slide=60)
    g0s, g0d = st.window()
    o = oracle.Oracle(n, g0s, g0d, [7], 0.15, 1e-6)
    o.push(oracle.SEQ)
    for _ in range(4):
        o.apply(*st.next_batch(), do_push=False)
        P, R = o.query()
        s2, d2 = o.export()
        ok, worst = exact.invariant_ok(n, s2, d2, 7, 0.15, P, R)
        assert ok, worst
        o.push(oracle.SEQ)


def test_seq_vs_jacobi_within_2eps():
    n = 200
    src, dst = W.rmat_stream(n, 3000, seed=9, abc=W.GRAPH500)
    st1 = W.Stream(n, src, dst, w0=600, ins_per_slide=50, del_per_slide=50)
    st2 = W.Stream(n, src, dst, w0=600, ins_per_slide=50, del_per_slide=50)
    g0s, g0d = st1.window()
    eps = 1e-8
    a = oracle.Oracle(n, g0s, g0d, [int(np.argmax(np.bincount(g0s, minlength=n)))], 0.15, eps)
    b = oracle.Oracle(n, g0s, g0d, a.sources, 0.15, eps)
    a.push(oracle.SEQ)
    b.push(oracle.JACOBI)
    for _ in range(5):
        a.apply(*st1.next_batch(), mode=oracle.SEQ)
        b.apply(*st2.next_batch(), mode=oracle.JACOBI)
        Pa, _ = a.query()
        Pb, _ = b.query()
        assert np.max(np.abs(Pa - Pb)) <= 2 * eps


# ---------------------------------------------------------------- semantics (readings R4, R8)

def _small():
    src = [0, 1, 2, 2, 3, 0]
    dst = [3, 0, 0, 1, 2, 1]
    o = oracle.Oracle(4, src, dst, [0], 0.15, 1e-9)
    o.push(oracle.SEQ)
    return o


def test_absent_deletion_is_enoent_and_changes_nothing():
    o = _small()
    P0, R0 = o.query()
    e0 = o.export()
    rc = o.apply([1], [3], [3, 1], [1, 2], raise_on_error=False)  # 3->1 absent
    assert rc == oracle.ORC_ENOENT
    P1, R1 = o.query()
    np.testing.assert_array_equal(P0, P1)
    np.testing.assert_array_equal(R0, R1)
    np.testing.assert_array_equal(e0[0], o.export()[0])


def test_out_of_range_is_erange_and_changes_nothing():
    o = _small()
    P0, R0 = o.query()
    assert o.apply([1], [4], raise_on_error=False) == oracle.ORC_ERANGE
    assert o.apply([], [], [9], [0], raise_on_error=False) == oracle.ORC_ERANGE
    P1, R1 = o.query()
    np.testing.assert_array_equal(P0, P1)
    np.testing.assert_array_equal(R0, R1)


def test_deletion_may_match_an_insertion_of_the_same_batch():
    o = _small()
    P0, R0 = o.query()
    assert o.apply([1], [3], [1], [3], do_push=False) == 0  # insert then delete 1->3
    P1, R1 = o.query()
    np.testing.assert_array_equal(P0, P1)
    np.testing.assert_allclose(R1, R0, atol=1e-15)
    assert o.num_arcs == 6


def test_multiset_insertions():
    o = _small()
    o.apply([0, 0], [3, 3])  # 0->3 now has multiplicity 3
    s, d = o.export()
    assert int(np.sum((s == 0) & (d == 3))) == 3
    assert o.dout()[0] == 4
    _check_state(o, 0, 0)


def test_deleting_last_out_arc_sets_residual_from_empty_sum():
    # reading R4: d_out(u) = 0 after the update -> R(u) = 1[u=s] - P(u)/alpha
    o = _small()
    P0, _ = o.query()
    o.apply([], [], [3], [2], do_push=False)  # vertex 3's only out-arc
    P1, R1 = o.query()
    assert o.dout()[3] == 0
    assert R1[3] == 0.0 - P0[3] / 0.15
    o.apply([], [], [0, 0], [3, 1], do_push=False)  # the source loses both out-arcs
    P2, R2 = o.query()
    assert R2[0] == 1.0 - P0[0] / 0.15
    o.push(oracle.SEQ)
    _check_state(o, 0, 0)


# ---------------------------------------------------------------- tiny config (BASELINE configs[0])

def test_tiny_config_oracle_tracks_power_iteration():
    """configs[0] shape (n=1e4, 10% window of a 1e5-arc Graph500 stream,
    1e3+1e3 slides), a hub source: the oracle stays within eps of the exact
    reverse PPR (power iteration, pinned above) after every checked slide."""
    cfg = W.CONFIGS["tiny"]
    st, cfg = W.make_stream("tiny")
    g0s, g0d = st.window()
    (s,) = W.pick_sources(cfg["n"], g0s, g0d, cfg["band"], 1)
    o = oracle.Oracle(cfg["n"], g0s, g0d, [s], 0.15, cfg["eps"])
    o.push(oracle.SEQ)
    for t in range(6):
        o.apply(*st.next_batch(), mode=oracle.SEQ)
        if t % 2 == 1:
            P, R = o.query()
            src, dst = o.export()
            assert exact.terminated(R, cfg["eps"])
            ok, worst = exact.invariant_ok(cfg["n"], src, dst, int(s), 0.15, P, R)
            assert ok, worst
            Pstar = exact.ppr_power(cfg["n"], src, dst, int(s), 0.15)
            assert np.max(np.abs(P - Pstar)) <= cfg["eps"] * (1 + 1e-6)
