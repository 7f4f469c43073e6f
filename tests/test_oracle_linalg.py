"""Pins for oracle/linalg.py against closed forms, brute force and LAPACK (numpy/scipy, tests only)."""

import itertools

import numpy as np
import pytest
import scipy.linalg as sla

from oracle.linalg import (RankDeficientError, back_substitution, dlarfg, householder_qr,
                           qrcp_truncated, rows_orth)


@pytest.mark.parametrize("x", [[3.0, 4.0], [-3.0, 4.0, 12.0], [0.0, 1.0, 1.0], [2.0, 0.0, 0.0], [5.0]])
def test_dlarfg_reflects_to_beta_e1(x):
    x = np.array(x)
    beta, tau, v = dlarfg(x)
    H = np.eye(x.size) - tau * np.outer(v, v)
    np.testing.assert_allclose(H @ x, np.r_[beta, np.zeros(x.size - 1)], atol=1e-14)
    np.testing.assert_allclose(H @ H.T, np.eye(x.size), atol=1e-14)
    assert abs(abs(beta) - np.linalg.norm(x)) < 1e-14
    if np.linalg.norm(x[1:]) > 0:
        assert np.sign(beta) == -np.sign(x[0] if x[0] != 0 else 1.0)   # LAPACK: beta = -sign(alpha)||x||


@pytest.mark.parametrize("m,n", [(7, 7), (40, 9), (300, 31), (5, 1)])
def test_householder_qr_matches_lapack_and_invariants(m, n):
    rng = np.random.default_rng(m * 100 + n)
    X = rng.standard_normal((m, n))
    Q, R = householder_qr(X)
    assert Q.shape == (m, n) and R.shape == (n, n)
    np.testing.assert_allclose(Q.T @ Q, np.eye(n), atol=20 * n * 2.2e-16)
    np.testing.assert_allclose(Q @ R, X, atol=20 * n * 2.2e-16 * np.abs(X).max())
    assert np.all(np.diag(R) > 0) and np.allclose(R, np.triu(R))
    Ql, Rl = np.linalg.qr(X)
    d = np.sign(np.diag(Rl))
    np.testing.assert_allclose(Q, Ql * d, atol=1e-12)
    np.testing.assert_allclose(R, Rl * d[:, None], atol=1e-12)


def test_householder_qr_exact_on_permutation_matrix():
    """A column permutation of the identity has the closed-form QR (Q = that matrix, R = I)."""
    P = np.eye(6)[:, [3, 0, 5, 1, 4, 2]]
    Q, R = householder_qr(P)
    np.testing.assert_array_equal(R, np.eye(6))
    np.testing.assert_array_equal(Q, P)


def test_rows_orth_equals_cholqr_definition():
    """CholQR: G = X X^T, Rbar^T Rbar = G, Q = Rbar^{-T} X.  On a well-conditioned
    short-wide X the oracle's Householder LQ factor equals this closed form."""
    rng = np.random.default_rng(3)
    X = rng.standard_normal((12, 200))
    Qx, Rbar = rows_orth(X)
    Lc = np.linalg.cholesky(X @ X.T)                  # lower, positive diagonal
    np.testing.assert_allclose(Rbar, Lc.T, rtol=1e-12, atol=1e-12)
    np.testing.assert_allclose(Qx, np.linalg.solve(Lc, X), atol=1e-12)
    np.testing.assert_allclose(Qx @ Qx.T, np.eye(12), atol=1e-14)
    np.testing.assert_allclose(Rbar.T @ Qx, X, atol=1e-12)


def _brute_force_pivots(B, k):
    """At each step, each remaining column's residual against span(chosen columns),
    computed from scratch; argmax (ties -> lowest index)."""
    chosen = []
    n = B.shape[1]
    for _ in range(k):
        best, bi = -1.0, -1
        if chosen:
            Qc, _ = np.linalg.qr(B[:, chosen])
        for c in range(n):
            if c in chosen:
                continue
            r = B[:, c] - (Qc @ (Qc.T @ B[:, c]) if chosen else 0.0)
            nr = np.linalg.norm(r)
            if nr > best:
                best, bi = nr, c
        chosen.append(bi)
    return chosen


@pytest.mark.parametrize("seed", range(6))
def test_qrcp_pivots_match_brute_force(seed):
    rng = np.random.default_rng(seed)
    B = rng.standard_normal((6, 14)) * (1.0 + np.arange(14))[None, :] ** 0.3
    perm, Rhat, gaps = qrcp_truncated(B, 5)
    assert list(perm[:5]) == _brute_force_pivots(B, 5)
    assert np.all(gaps >= 0)


@pytest.mark.parametrize("shape,k", [((20, 60), 12), ((110, 400), 100), ((30, 30), 30)])
def test_qrcp_matches_lapack_dgeqp3(shape, k):
    """Same pivots as LAPACK dgeqp3 (scipy qr(pivoting=True)) on tie-free matrices, and the
    same |R| rows (Householder signs may differ row-wise)."""
    rng = np.random.default_rng(shape[0])
    B = rng.standard_normal(shape) @ np.diag(np.exp(-np.linspace(0, 6, shape[1])))
    B = B[:, rng.permutation(shape[1])]
    perm, Rhat, gaps = qrcp_truncated(B, k)
    _, Rl, pl = sla.qr(B, pivoting=True, mode="economic")
    assert list(perm[:k]) == list(pl[:k])
    # trailing permutation follows the same LAPACK swap semantics
    assert list(perm) == list(pl) or k < shape[1]
    np.testing.assert_allclose(np.abs(Rhat[:, :k]), np.abs(Rl[:k, :k]), atol=1e-11)
    # R̂ times P^T reproduces B's projection: B P = Q̂ R̂ on the first k columns
    Qh, _ = np.linalg.qr(B[:, perm[:k]])
    np.testing.assert_allclose(np.abs(Qh.T @ B[:, perm]), np.abs(Rhat), atol=1e-10)


def test_qrcp_rank_deficient_raises():
    B = np.zeros((4, 10))
    B[:, 0] = 1.0
    with pytest.raises(RankDeficientError):
        qrcp_truncated(B, 2)


def test_qrcp_tie_breaks_to_lowest_original_index():
    B = np.eye(3)[:, [0, 1, 2, 0]] * np.array([1.0, 2.0, 2.0, 1.0])   # cols 1 and 2 tie
    perm, _, _ = qrcp_truncated(B, 2)
    assert perm[0] == 1 and perm[1] == 2


def test_back_substitution_exact_and_lstsq():
    U = np.triu(np.array([[1, 2, -1], [0, 1, 3], [0, 0, 1]], dtype=float))
    X = np.array([[1, -2], [0, 5], [3, 1]], dtype=float)
    np.testing.assert_array_equal(back_substitution(U, U @ X), X)   # small integers: exact
    rng = np.random.default_rng(5)
    B = rng.standard_normal((30, 80))
    perm, Rhat, _ = qrcp_truncated(B, 20)
    T = back_substitution(Rhat[:, :20], Rhat[:, 20:])
    np.testing.assert_allclose(T, sla.solve_triangular(Rhat[:, :20], Rhat[:, 20:]), atol=1e-12)
    # T is the least-squares coefficient (B P_1)^+ B P_2, for l > k too:
    # B P_1 = Q1 R11, B P_2 = Q1 R12 + Q2 R22 with Q1 ⟂ Q2, so (B P_1)^+ B P_2 = R11^{-1} R12.
    Tl = np.linalg.lstsq(B[:, perm[:20]], B[:, perm[20:]], rcond=None)[0]
    np.testing.assert_allclose(T, Tl, atol=1e-9 * max(1, np.abs(Tl).max()))
