"""TEST INFRASTRUCTURE ONLY -- exact definitions used to pin the oracle and to
check every batch (see oracle/__init__.py for who may import this).

Notation (Table 1): A is the adjacency (multiset counts,
A[u, v] = multiplicity of arc u -> v), d = d_out, alpha the teleport
probability, s the source.

Reading R1: the fixed point of Eq. 2 / Lemma 1 / Algs 1-4 is
    P* = alpha (I - (1-alpha) D^-1 A)^-1 e_s
(D^-1 A, a zero row for d(u) = 0 -- reading R5), i.e. Eq. 1 with W read as
the W^T = D^-1 A of Lemma 1.  ``forward_ppr`` computes Eq. 1 with its
literal W = A^T D^-1 -- used only for the undirected reversibility
pin, never as a target.
"""
from __future__ import annotations

import numpy as np


def adjacency(n, src, dst):
    """Dense A with multiplicity: A[u, v] = #arcs u -> v."""
    A = np.zeros((n, n), dtype=np.float64)
    np.add.at(A, (np.asarray(src, dtype=np.int64), np.asarray(dst, dtype=np.int64)), 1.0)
    return A


def transition_rev(n, src, dst):
    """D^-1 A (row-substochastic; zero rows at d_out = 0)."""
    A = adjacency(n, src, dst)
    d = A.sum(axis=1)
    inv = np.divide(1.0, d, out=np.zeros_like(d), where=d > 0)
    return A * inv[:, None]


def ppr_dense(n, src, dst, s, alpha):
    """P* = alpha (I - (1-alpha) D^-1 A)^-1 e_s by a dense LU solve (numpy)."""
    M = np.eye(n) - (1.0 - alpha) * transition_rev(n, src, dst)
    e = np.zeros(n)
    e[s] = 1.0
    return alpha * np.linalg.solve(M, e)


def error_from_residual(n, src, dst, R, alpha):
    """alpha (I - (1-alpha) D^-1 A)^-1 R -- equals P* - P whenever Eq. 2 holds."""
    M = np.eye(n) - (1.0 - alpha) * transition_rev(n, src, dst)
    return alpha * np.linalg.solve(M, np.asarray(R, dtype=np.float64))


def ppr_power(n, src, dst, s, alpha, tol=1e-15, max_iter=100000):
    """Power iteration x <- alpha e_s + (1-alpha) D^-1 A x until ||dx||_inf < tol.
    Sparse mat-vec written with numpy scatter-add (A x)(u) = sum_{u->v} x(v)."""
    src = np.asarray(src, dtype=np.int64)
    dst = np.asarray(dst, dtype=np.int64)
    d = np.bincount(src, minlength=n).astype(np.float64)
    inv = np.divide(1.0, d, out=np.zeros_like(d), where=d > 0)
    x = np.zeros(n)
    x[s] = alpha
    for _ in range(max_iter):
        ax = np.zeros(n)
        np.add.at(ax, src, x[dst])
        xn = (1.0 - alpha) * inv * ax
        xn[s] += alpha
        if np.max(np.abs(xn - x)) < tol:
            return xn
        x = xn
    raise RuntimeError("power iteration did not converge")


def forward_ppr(n, src, dst, s, alpha):
    """Eq. 1 literally: pi = alpha e_s + (1-alpha) A^T D^-1 pi."""
    A = adjacency(n, src, dst)
    d = A.sum(axis=1)
    inv = np.divide(1.0, d, out=np.zeros_like(d), where=d > 0)
    W = A.T * inv[None, :]
    e = np.zeros(n)
    e[s] = 1.0
    return alpha * np.linalg.solve(np.eye(n) - (1.0 - alpha) * W, e)


def invariant_residual(n, src, dst, s, alpha, P, R):
    """Eq. 2 at every vertex v:
        lhs(v) = P(v) + alpha R(v)
        rhs(v) = (1-alpha)/d(v) * sum_{x in N_out(v)} P(x) + alpha 1[v=s]
    summed in long double.  Returns (|lhs - rhs|, scale) where
        scale(v) = |P(v)| + alpha|R(v)| + (1-alpha)/d(v) sum |P(x)| + alpha 1[v=s]
    (reading R18: pass iff |lhs-rhs| <= 1e-12 * max(scale, alpha))."""
    ld = np.longdouble
    src = np.asarray(src, dtype=np.int64)
    dst = np.asarray(dst, dtype=np.int64)
    P = np.asarray(P, dtype=np.float64).astype(ld)
    R = np.asarray(R, dtype=np.float64).astype(ld)
    a = ld(alpha)
    d = np.bincount(src, minlength=n).astype(ld)
    sumP = np.zeros(n, dtype=ld)
    np.add.at(sumP, src, P[dst])
    sumAbs = np.zeros(n, dtype=ld)
    np.add.at(sumAbs, src, np.abs(P[dst]))
    safe = np.where(d > 0, d, ld(1))
    ones = np.zeros(n, dtype=ld)
    ones[s] = ld(1)
    rhs = np.where(d > 0, (ld(1) - a) * sumP / safe, ld(0)) + a * ones
    lhs = P + a * R
    scale = np.abs(P) + a * np.abs(R) + np.where(d > 0, (ld(1) - a) * sumAbs / safe, ld(0)) + a * ones
    return np.abs(lhs - rhs).astype(np.float64), scale.astype(np.float64)


def invariant_ok(n, src, dst, s, alpha, P, R, rel=1e-12):
    err, scale = invariant_residual(n, src, dst, s, alpha, P, R)
    bound = rel * np.maximum(scale, alpha)
    return bool(np.all(err <= bound)), float(np.max(err / bound)) if n else 0.0


def terminated(R, eps):
    """Termination condition of Alg 2/3 (reading R10): -eps <= R <= eps."""
    R = np.asarray(R)
    return bool(np.all(R <= eps) and np.all(R >= -eps))
