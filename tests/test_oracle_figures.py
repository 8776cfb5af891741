"""Pins the oracle to the paper's worked example (Figs 1-3), bit for bit.

Every printed state is checked two ways: (1) the oracle's fp64 value truncated
to 4 decimals equals the printed value (the figures' own printing rule), and
(2) the exact dyadic value that the decoded algorithms produce (DESIGN.md
readings) -- all states are dyadic rationals, so fp64 is exact.
"""
import numpy as np
import pytest

import oracle
from oracle import exact
from tests import golden_figs as G

BLOCKS = G.load()


def _oracle():
    return oracle.Oracle(G.N, G.G0_SRC, G.G0_DST, [G.SOURCE], G.ALPHA, G.EPS)


def _check_printed(name, P, R):
    blk = BLOCKS[name]
    for v in range(G.N):
        assert G.matches_printed(R[v], blk["R"][v]), (name, "R", v, R[v], blk["R"][v])
        if v in blk["typo"]:
            continue
        assert G.matches_printed(P[v], blk["P"][v]), (name, "P", v, P[v], blk["P"][v])


def test_golden_file_parses():
    assert len(BLOCKS) == 13
    for blk in BLOCKS.values():
        assert blk["cite"].startswith("P:")
        assert None not in blk["R"] and None not in blk["P"]


def test_reconstructed_g0_satisfies_eq2_at_every_printed_g0_state():
    # The reconstructed G0 must make Eq. 2 hold at the exact dyadic states
    # behind Fig 3 (a1..a4, b2..b5); this is what pins the reconstruction.
    exact_states = {
        "fig3_a1": ([1, 0, 0, 0], [0, 0, 0, 0]),
        "fig3_a2": ([0, .5, .25, 0], [.5, 0, 0, 0]),
        "fig3_a3": ([0, 0, .125, .125], [.5, .25, .125, 0]),
        "fig3_a4": ([.0625, 0, 0, .0625], [.5, .25, .1875, .0625]),
        "fig3_b3": ([0, 0, .375, 0], [.5, .25, 0, 0]),
        "fig3_b4": ([0, 0, 0, .1875], [.5, .25, .1875, 0]),
        "fig3_b5": ([.09375, 0, 0, 0], [.5, .25, .1875, .09375]),
    }
    for name, (R, P) in exact_states.items():
        _check_printed(name, P, R)
        ok, worst = exact.invariant_ok(G.N, G.G0_SRC, G.G0_DST, G.SOURCE, G.ALPHA, P, R)
        assert ok, (name, worst)


@pytest.mark.parametrize("rounds,name", [(0, "fig3_a1"), (1, "fig3_a2"), (2, "fig3_a3"),
                                         (3, "fig3_a4")])
def test_fig3a_parallel_push_trace(rounds, name):
    o = _oracle()
    if rounds:
        o.push(oracle.JACOBI, rounds)
    P, R = o.query()
    _check_printed(name, P, R)


def test_fig3a_converges_in_three_rounds_with_five_pushes():
    # Fig 3 caption: the parallel push pushes {v1, v2, v3, v3, v4}.
    o = _oracle()
    o.push(oracle.JACOBI, -1)
    st = o.stats()
    assert st["rounds_pos"] == 3 and st["rounds_neg"] == 0
    assert st["pushes"] == 5
    P, R = o.query()
    np.testing.assert_array_equal(R, [1 / 16, 0, 0, 1 / 16])
    np.testing.assert_array_equal(P, [1 / 2, 1 / 4, 3 / 16, 1 / 16])


@pytest.mark.parametrize("pushes,name", [(0, "fig3_a1"), (1, "fig3_b2"), (2, "fig3_b3"),
                                         (3, "fig3_b4"), (4, "fig3_b5")])
def test_fig3b_sequential_push_trace(pushes, name):
    o = _oracle()
    if pushes:
        o.push(oracle.SEQ, pushes)
    P, R = o.query()
    _check_printed(name, P, R)


def test_fig3b_converges_with_four_pushes():
    # Fig 3 caption: the sequential push pushes {v1, v2, v3, v4}.
    o = _oracle()
    o.push(oracle.SEQ, -1)
    assert o.stats()["pushes"] == 4
    P, R = o.query()
    np.testing.assert_array_equal(R, [3 / 32, 0, 0, 0])
    np.testing.assert_array_equal(P, [1 / 2, 1 / 4, 3 / 16, 3 / 32])


def _fig1a_state():
    o = _oracle()
    o.push(oracle.JACOBI, -1)  # Fig 1(a) == Fig 3 a(4)
    P, R = o.query()
    _check_printed("fig1_a", P, R)
    return o


def test_fig1_single_insertion_restore_then_push():
    o = _fig1a_state()
    o.apply([0], [1], mode=oracle.SEQ, do_push=False)  # e1 = v1 -> v2
    P, R = o.query()
    _check_printed("fig1_b", P, R)
    assert R[0] == 5 / 32
    o.push(oracle.SEQ, -1)
    P, R = o.query()
    _check_printed("fig1_d", P, R)
    np.testing.assert_array_equal(R, [0, 5 / 64, 5 / 128, 1 / 16])
    np.testing.assert_array_equal(P, [37 / 64, 1 / 4, 3 / 16, 1 / 16])
    # the misprinted P1(1) of Fig 1(d) is the 0.5781 of Fig 2(d)
    assert G.matches_printed(P[0], BLOCKS["fig2_d"]["P"][0])


def test_fig2_batch_restore_then_one_parallel_round():
    o = _fig1a_state()
    o.apply([0, 3], [1, 0], mode=oracle.JACOBI, do_push=False)  # e1 = v1->v2, e2 = v4->v1
    P, R = o.query()
    _check_printed("fig2_b", P, R)
    assert R[0] == 5 / 32 and R[3] == 7 / 32
    o.stats(reset=True)
    o.push(oracle.JACOBI, -1)
    assert o.stats()["rounds_pos"] == 1  # "achieves convergence in one iteration"
    P, R = o.query()
    _check_printed("fig2_d", P, R)
    np.testing.assert_array_equal(R, [7 / 128, 5 / 64, 5 / 128, 5 / 128])
    np.testing.assert_array_equal(P, [37 / 64, 1 / 4, 3 / 16, 11 / 64])


def test_fig_states_satisfy_eq2_after_updates():
    o = _fig1a_state()
    o.apply([0, 3], [1, 0], mode=oracle.JACOBI, do_push=True)
    P, R = o.query()
    src, dst = o.export()
    ok, worst = exact.invariant_ok(G.N, src, dst, G.SOURCE, G.ALPHA, P, R)
    assert ok, worst
    # the converged state is within eps of the exact reverse PPR (reading R1) ...
    Pstar = exact.ppr_dense(G.N, src, dst, G.SOURCE, G.ALPHA)
    assert np.max(np.abs(P - Pstar)) <= G.EPS
    # ... and the error identity P* - P = alpha (I-(1-alpha)D^-1 A)^-1 R holds
    err = exact.error_from_residual(G.N, src, dst, R, G.ALPHA)
    np.testing.assert_allclose(Pstar - P, err, atol=1e-15)


def test_fig_example_rejects_forward_reading():
    # Reading R1: the literal Eq. 1 (W = A^T D^-1) is NOT the fixed point of
    # the push; on the example it lies > eps from the converged state.
    o = _oracle()
    o.push(oracle.JACOBI, -1)
    P, _ = o.query()
    fwd = exact.forward_ppr(G.N, G.G0_SRC, G.G0_DST, G.SOURCE, G.ALPHA)
    rev = exact.ppr_dense(G.N, G.G0_SRC, G.G0_DST, G.SOURCE, G.ALPHA)
    assert np.max(np.abs(P - rev)) <= G.EPS
    assert np.max(np.abs(P - fwd)) > G.EPS
