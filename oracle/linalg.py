"""Oracle building blocks: Householder QR, truncated QRCP, back substitution.

TEST INFRASTRUCTURE ONLY (see oracle/__init__.py).  Plain numpy, float64,
one column / one pivot step at a time, in the order the paper's algorithms
(and the LAPACK routines it names) perform them.  Vector-matrix products go
through the oracle's own fixed-order GEMM (``oracle.gemm.matmul``); 2-norms are
sqrt(sum of squares); nothing is blocked, fused or reordered.
"""

from __future__ import annotations

import numpy as np

from .gemm import matmul


class RankDeficientError(ValueError):
    """A QRCP step found every remaining residual column norm equal to zero."""


def dlarfg(x: np.ndarray):
    """Householder reflector H = I - tau v v^T with H x = (beta, 0, ..., 0)^T.

    LAPACK dlarfg convention (the reflector used by QP3):
    beta = -sign(alpha) * ||x||, tau = (beta - alpha)/beta, v = (1, x[1:]/(alpha - beta)),
    and tau = 0 (H = I) when x[1:] = 0.  sign(0) = +1 (Fortran SIGN).
    """
    x = np.asarray(x, dtype=np.float64)
    alpha = float(x[0])
    xnorm = float(np.sqrt(np.sum(x[1:] * x[1:]))) if x.size > 1 else 0.0
    v = np.zeros_like(x)
    v[0] = 1.0
    if xnorm == 0.0:
        return alpha, 0.0, v
    h = float(np.hypot(alpha, xnorm))
    beta = -h if alpha >= 0.0 else h
    tau = (beta - alpha) / beta
    v[1:] = x[1:] / (alpha - beta)
    return beta, tau, v


def householder_qr(X: np.ndarray):
    """Thin QR X = Q R (m x n, m >= n) by Householder reflections [8],
    sign-normalised so that R has a positive diagonal -- the unique QR factor
    that CholQR also defines ("R upper-triangular with non-negative diagonal",
    P:L476-481, Sec. 4).  Returns (Q m x n with orthonormal columns, R n x n).
    """
    A = np.array(X, dtype=np.float64, copy=True)
    m, n = A.shape
    if m < n:
        raise ValueError("householder_qr needs m >= n")
    vs, taus = [], []
    for j in range(n):
        beta, tau, v = dlarfg(A[j:, j])
        if tau != 0.0 and j + 1 < n:
            w = matmul(v, A[j:, j + 1:])
            A[j:, j + 1:] -= tau * np.outer(v, w)
        A[j, j] = beta
        A[j + 1:, j] = 0.0
        vs.append(v)
        taus.append(tau)
    R = np.triu(A[:n, :n])
    Q = np.zeros((m, n))
    Q[:n, :n] = np.eye(n)
    for j in reversed(range(n)):          # Q = H_0 H_1 ... H_{n-1} [I; 0]
        v, tau = vs[j], taus[j]
        if tau != 0.0:
            w = matmul(v, Q[j:, :])
            Q[j:, :] -= tau * np.outer(v, w)
    d = np.where(np.diag(R) < 0.0, -1.0, 1.0)
    return Q * d[None, :], R * d[:, None]


def rows_orth(X: np.ndarray):
    """QR(B) of Fig. 2(a) lines 5/10 for a short-wide l x n matrix (l <= n).

    The paper applies CholQR "to compute the LQ factorization of the
    short-wide matrix" (P:L470-481 and footnote 3): X = Rbar^T Qx
    with Rbar upper-triangular, non-negative diagonal, Qx orthonormal rows.
    That factor is unique for full-rank X; the oracle computes it by the stable
    Householder QR of X^T (reading R3).  Returns (Qx, Rbar).
    """
    Q, R = householder_qr(np.asarray(X).T)
    return Q.T.copy(), R


def qrcp_truncated(B: np.ndarray, k: int, *, return_trailing: bool = False):
    """Truncated QRCP (QP3 stopped after k columns, Sec. 2) of B (l x n).

    Step j = 0..k-1: (i) residual norms ||W[j:, c]||, c >= j, RECOMPUTED from
    the current columns (reading R5: the exact quantity that downdating
    approximates); (ii) pivot = the largest, ties to the
    lowest original column index; (iii) LAPACK swap of columns j and p;
    (iv) dlarfg reflector on W[j:, j] applied to the trailing columns.

    Returns perm (int64[n]; perm[:k] are the pivots P_{1:k}), Rhat (k x n,
    upper trapezoidal: Rhat[:, :k] = R̂_{1:k}, Rhat[:, k:] = R̂_{k+1:n} of
    P:L238-253) and the relative pivot gaps (best - second)/best per step.
    """
    W = np.array(B, dtype=np.float64, copy=True)
    l, n = W.shape
    if not 1 <= k <= min(l, n):
        raise ValueError("need 1 <= k <= min(l, n)")
    perm = np.arange(n, dtype=np.int64)
    gaps = []
    for j in range(k):
        norms = np.sqrt(np.sum(W[j:, j:] ** 2, axis=0))
        best = norms.max()
        if best == 0.0:
            raise RankDeficientError(f"zero residual norm at QRCP step {j}")
        cand = np.nonzero(norms == best)[0]
        p = j + int(cand[np.argmin(perm[j + cand])])
        rest = np.delete(norms, p - j)
        second = rest.max() if rest.size else 0.0
        gaps.append((best - second) / best)
        if p != j:
            W[:, [j, p]] = W[:, [p, j]]
            perm[[j, p]] = perm[[p, j]]
        beta, tau, v = dlarfg(W[j:, j])
        if tau != 0.0 and j + 1 < n:
            w = matmul(v, W[j:, j + 1:])
            W[j:, j + 1:] -= tau * np.outer(v, w)
        W[j, j] = beta
        W[j + 1:, j] = 0.0
    Rhat = np.triu(W[:k, :])
    if return_trailing:
        return perm, Rhat, np.array(gaps), W[k:, k:].copy()
    return perm, Rhat, np.array(gaps)


def back_substitution(U: np.ndarray, Y: np.ndarray) -> np.ndarray:
    """X = U^{-1} Y for upper-triangular U (k x k), row by row from the bottom
    (the triangular solve T := R̂_{1:k}^{-1} R̂_{k+1:n} of Fig. 2(b) line 9)."""
    U = np.asarray(U, dtype=np.float64)
    X = np.array(Y, dtype=np.float64, copy=True)
    k = U.shape[0]
    for i in reversed(range(k)):
        if i + 1 < k:
            X[i] -= matmul(U[i, i + 1:], X[i + 1:])
        X[i] /= U[i, i]
    return X
