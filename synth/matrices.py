"""Synthetic test matrices A = U diag(sigma) V^T (the paper's A := X Sigma Y).

Recipe:

* sigma follows one of the laws below, 0-based i = 0..n-1 (Table 1, P:L636-640,
  reading R6: no floor, 0-based index).
* V is Haar-random n x n (QR of a Gaussian, sign-fixed).
* U (m x n, orthonormal columns):
  - if n divides m: "stacked" U = sqrt(n/m) [D_1 Pi_1 Q0; ...; D_b Pi_b Q0] with Q0
    Haar n x n, Pi_b random row permutations and D_b random +-1 diagonals.  This
    is exactly orthonormal, costs O(mn) and lets each GPU build its own row
    block on the device (Gaussian Omega is rotation invariant, so the
    statistics of B, P, T, e do not depend on U's structure);
  - otherwise a dense Haar U from the QR of an m x n Gaussian (small m only).
* A is returned column-major (Fortran order), the LAPACK/MAGMA layout the
  library expects.
"""

from __future__ import annotations

import math

import numpy as np

LAWS = ("exp-paper", "exp-k", "power", "power2", "slow", "rank-k")


def singular_values(law: str, n: int, k: int) -> np.ndarray:
    """sigma_i, i = 0..n-1.

    exp-paper  10^(-i/10)      Table 1 "exponent"
    power      (i+1)^-3        Table 1 "power"
    exp-k      10^(-5 i / k)   keeps sigma_k/sigma_0 = 1e-5 like Table 1 at any k
                               (equals exp-paper at k = 50)
    power2     (i+1)^-2        fallback slow law
    slow       (i+1)^-1/2      slowly decaying spectrum (HMT-bound checks)
    rank-k     1 for i < k, 0 otherwise (exact-recovery special case)
    """
    i = np.arange(n, dtype=np.float64)
    if law == "exp-paper":
        return 10.0 ** (-i / 10.0)
    if law == "exp-k":
        return 10.0 ** (-5.0 * i / k)
    if law == "power":
        return (i + 1.0) ** -3.0
    if law == "power2":
        return (i + 1.0) ** -2.0
    if law == "slow":
        return (i + 1.0) ** -0.5
    if law == "rank-k":
        return np.where(i < k, 1.0, 0.0)
    raise ValueError(f"unknown law {law!r}")


def haar_orthogonal(n: int, rng: np.random.Generator, m: int | None = None) -> np.ndarray:
    """m x n (default n x n) matrix with Haar-distributed orthonormal columns."""
    m = n if m is None else m
    G = rng.standard_normal((m, n))
    Q, R = np.linalg.qr(G)
    return Q * np.where(np.diag(R) < 0, -1.0, 1.0)[None, :]


def _factors(m: int, n: int, law: str, k: int, seed: int):
    rng = np.random.default_rng(seed)
    sigma = singular_values(law, n, k)
    V = haar_orthogonal(n, rng)
    if m % n == 0 and m >= n:
        Q0 = haar_orthogonal(n, rng)
        M0 = (Q0 * sigma[None, :]) @ V.T                 # n x n
        nb = m // n
        rows = np.concatenate([rng.permutation(n) for _ in range(nb)]).astype(np.int64)
        signs = rng.choice(np.array([-1.0, 1.0]), size=m)
        factor = signs * math.sqrt(n / m)                 # exact: +-1 times a double
        return dict(kind="stacked", sigma=sigma, M0=M0, rows=rows, factor=factor)
    r = min(m, n)
    U = haar_orthogonal(r, rng, m)                        # m x r
    return dict(kind="dense", sigma=sigma, A=(U * sigma[None, :r]) @ V[:, :r].T)


def make_matrix(m: int, n: int, law: str = "exp-k", k: int = 50, seed: int = 2015,
                rows: tuple[int, int] | None = None):
    """Return (A, sigma): A float64 column-major, rows[0]:rows[1] of the global
    m x n matrix (default: all rows), and its exact singular values."""
    f = _factors(m, n, law, k, seed)
    r0, r1 = (0, m) if rows is None else rows
    if f["kind"] == "stacked":
        A = f["factor"][r0:r1, None] * f["M0"][f["rows"][r0:r1], :]
    else:
        A = f["A"][r0:r1]
    return np.asfortranarray(A), f["sigma"]


def make_matrix_torch(m: int, n: int, law: str = "exp-k", k: int = 50, seed: int = 2015,
                      rows: tuple[int, int] | None = None, device="cuda", chunk_rows: int = 1 << 17):
    """Same matrix as :func:`make_matrix`, built on ``device`` (only the n x n
    core goes over PCIe).  Returns (At, sigma) where ``At`` is an (m_local, n)
    view with strides (1, m_local) -- i.e. column-major, lda = m_local."""
    import torch

    f = _factors(m, n, law, k, seed)
    r0, r1 = (0, m) if rows is None else rows
    ml = r1 - r0
    if f["kind"] != "stacked":
        A = np.asfortranarray(f["A"][r0:r1])
        At = torch.empty((n, ml), dtype=torch.float64, device=device)
        At.copy_(torch.from_numpy(np.ascontiguousarray(A.T)))
        return At.t(), f["sigma"]
    M0T = torch.from_numpy(np.ascontiguousarray(f["M0"].T)).to(device)        # n x n, M0T[c, r] = M0[r, c]
    rows_t = torch.from_numpy(f["rows"][r0:r1]).to(device)
    fac_t = torch.from_numpy(f["factor"][r0:r1]).to(device)
    At = torch.empty((n, ml), dtype=torch.float64, device=device)             # column-major storage of A
    for s in range(0, ml, chunk_rows):
        e = min(ml, s + chunk_rows)
        At[:, s:e] = torch.index_select(M0T, 1, rows_t[s:e]) * fac_t[None, s:e]
    return At.t(), f["sigma"]


# BASELINE.json configs (SURVEY §8d laws; seeds recorded in every bench line)
CONFIGS = {
    "cfg1": dict(m=500, n=200, k=20, p=10, q=0, law="exp-paper"),
    "cfg2": dict(m=50_000, n=5_000, k=100, p=10, q=1, law="exp-k"),
    "cfg3": dict(m=100_000, n=10_000, k=200, p=20, q=2, law="power"),
    "cfg4": dict(m=1_000_000, n=5_000, k=100, p=10, q=1, law="exp-k"),
    "cfg5": dict(m=200_000, n=8_000, k=100, p=10, q=1, law="exp-k"),
}
MATRIX_SEED = 2015
OMEGA_SEED = 0x5C15


def matrix_spec(name: str) -> dict:
    return dict(CONFIGS[name])


def config_variant(name: str, **over) -> dict:
    """A BASELINE config with overrides (e.g. the cfg5 k / q sweep)."""
    c = dict(CONFIGS[name])
    c.update(over)
    return c
