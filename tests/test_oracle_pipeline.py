"""Pins for oracle/pipeline.py (Fig. 2) against the paper's printed values, closed forms,
special cases that reduce to LAPACK, and bounds."""

import json
import os

import numpy as np
import pytest
import scipy.linalg as sla

from oracle import pipeline as PL
from oracle.linalg import qrcp_truncated
from oracle.philox import omega
from synth.matrices import make_matrix, singular_values


def test_table1_singular_value_laws(golden_dir):
    """Table 1: sigma_0, the printed "sigma_{k+1}" (= sigma[49], reading R6) and
    kappa(A) (= sigma_0 / sigma[49]) for the "power" and "exponent" laws, n = 500, k = 50."""
    g = json.load(open(os.path.join(golden_dir, "paper_values.json")))["table1"]
    for name, law in (("power", "power"), ("exponent", "exp-paper")):
        s = singular_values(law, g["n"], g["k"])
        assert s[0] == g[name]["sigma0"]
        assert abs(s[49] - g[name]["sigma_k1"]) <= 0.05 * g[name]["sigma_k1"]     # printed to 2 digits
        assert abs(s[0] / s[49] - g[name]["kappa"]) <= 0.05 * g[name]["kappa"]


def test_synth_matrix_has_the_prescribed_singular_values():
    for (m, n, law) in [(600, 200, "exp-paper"), (500, 200, "power"), (1000, 250, "exp-k")]:
        A, s = make_matrix(m, n, law, 50, seed=1)
        sv = np.linalg.svd(A, compute_uv=False)
        np.testing.assert_allclose(sv, s, atol=1e-14 * n)


def test_sample_is_partition_invariant():
    """B = sum_i Omega(i) A(i) over a 1-D row partition equals Omega A."""
    A, _ = make_matrix(400, 100, "exp-k", 20, seed=2)
    B = PL.sample(A, 25, seed=9)
    parts = [(0, 133), (133, 134), (134, 301), (301, 400)]
    Bs = sum(PL.sample(A[r0:r1], 25, seed=9, row_offset=r0) for r0, r1 in parts)
    np.testing.assert_allclose(Bs, B, atol=1e-13 * np.abs(B).max())
    ref = omega(25, 0, 400, 9) @ A  # BLAS (another summation order), test-only
    np.testing.assert_allclose(B, ref, atol=1e-14 * np.abs(ref).max())


def test_power_iteration_spans_omega_A_AtA_q():
    """POWER (Fig. 2(a)) only re-mixes rows, so rowspace(B_q) = rowspace(Omega A (A^T A)^q)
    (P:L287-291), and C after line 10 has orthonormal rows."""
    A, _ = make_matrix(300, 80, "slow", 10, seed=4)
    B0 = PL.sample(A, 12, seed=5)
    Bq, C = PL.power_iterate(A, B0, 2, return_C=True)
    Z = B0 @ A.T @ A @ A.T @ A
    Qz, _ = np.linalg.qr(Z.T)
    resid = Bq.T - Qz @ (Qz.T @ Bq.T)
    assert np.linalg.norm(resid) <= 1e-10 * np.linalg.norm(Bq)
    np.testing.assert_allclose(C @ C.T, np.eye(12), atol=1e-13)
    assert PL.power_iterate(A, B0, 0) is B0


def test_omega_identity_reduces_to_truncated_qp3():
    """Special case Omega = I (l = m, via the B override), q = 0: Fig. 2(b) is then truncated
    QP3 of A itself -- pivots = LAPACK dgeqp3 pivots, Rbar = |R̂_11| row signs, R rows = QP3's."""
    rng = np.random.default_rng(8)
    A = rng.standard_normal((24, 60)) @ np.diag(np.exp(-np.linspace(0, 4, 60)))
    k = 8
    res = PL.rs_lowrank(A, k, 24 - k, 0, seed=0, B_override=A)
    Ql, Rl, pl = sla.qr(A, pivoting=True, mode="economic")
    assert list(res.perm[:k]) == list(pl[:k])
    # R in original column order vs dgeqp3's first k rows in original order (rows fixed after k steps)
    R_orig = np.empty_like(res.R)
    R_orig[:, res.perm] = res.R
    Rl_orig = np.empty((k, 60))
    Rl_orig[:, pl] = Rl[:k]
    np.testing.assert_allclose(np.abs(R_orig), np.abs(Rl_orig), atol=1e-12)
    np.testing.assert_allclose(np.abs(res.Q), np.abs(Ql[:, :k]), atol=1e-12)


@pytest.mark.parametrize("q,p", [(0, 5), (1, 0), (2, 0)])
def test_exact_recovery_when_rank_is_k(q, p):
    """rank(A) = k: the approximation is exact (e at rounding level)."""
    A, _ = make_matrix(400, 100, "rank-k", 10, seed=3)
    res = PL.rs_lowrank(A, 10, p, q, seed=1)
    assert res.err <= 1e-13


@pytest.mark.parametrize("law", ["exp-paper", "power", "slow"])
@pytest.mark.parametrize("q", [0, 1])
def test_error_between_eckart_young_and_column_id_bound(law, q):
    """Lower bound: Eckart-Young, e >= (sum_{j>=k} sigma_j^2)^{1/2} / ||A||_F.
    Upper bound (deterministic): with Pi the projector on rowspace(B),
    ||A P_2 - A P_1 T|| <= (||A||_2 / sigma_l(B)) ||R̂_22|| + (1 + ||T||_2^2)^{1/2} ||A (I - Pi)||."""
    m, n, k, p = 600, 150, 15, 10
    A, s = make_matrix(m, n, law, k, seed=6)
    res = PL.rs_lowrank(A, k, p, q, seed=2)
    nrmA = np.sqrt(np.sum(s ** 2))
    ey = np.sqrt(np.sum(s[k:] ** 2)) / nrmA
    assert res.err >= ey * (1 - 1e-10)
    # e is the column-ID error: the first k columns of A P are reproduced exactly
    D1 = A[:, res.perm[:k]] - res.Q @ res.R[:, :k]
    assert np.linalg.norm(D1) <= 1e-12 * nrmA
    D2 = A[:, res.perm[k:]] - A[:, res.perm[:k]] @ res.T
    np.testing.assert_allclose(res.err, np.linalg.norm(D2) / nrmA, rtol=1e-8, atol=1e-15)
    Qb, _ = np.linalg.qr(res.B.T)
    eps_rf = np.linalg.norm(A - (A @ Qb) @ Qb.T, 2)
    _, _, _, R22 = qrcp_truncated(res.B, k, return_trailing=True)
    sl = np.linalg.svd(res.B, compute_uv=False)[-1]
    bound = s[0] / sl * np.linalg.norm(R22, 2) + np.sqrt(1 + np.linalg.norm(res.T, 2) ** 2) * eps_rf
    assert np.linalg.norm(D2, 2) <= bound * (1 + 1e-8)


def test_range_finder_hmt_frobenius_bound():
    """HMT [9] Thm 10.5 (cited at P:L292-296): E||(I - Pi_B) A^T||_F <= (1 + k/(p-1))^{1/2}
    (sum_{j>=k} sigma_j^2)^{1/2} for q = 0; asserted on a 5-seed mean with the exact constant."""
    m, n, k, p = 500, 250, 20, 8
    A, s = make_matrix(m, n, "slow", k, seed=12)
    tail = np.sqrt(np.sum(s[k:] ** 2))
    vals = []
    for seed in range(5):
        B = PL.sample(A, k + p, seed=100 + seed)
        Qb, _ = np.linalg.qr(B.T)
        vals.append(np.linalg.norm(A - (A @ Qb) @ Qb.T))
    assert np.mean(vals) <= np.sqrt(1 + k / (p - 1)) * tail
    assert np.mean(vals) >= tail * (1 - 1e-12)


def test_power_iteration_reduces_error_monotonically_in_median():
    """error ~ c^{1/(2q+1)} sigma_{k+1} -> decreases with q (median of seeds)."""
    A, s = make_matrix(800, 200, "slow", 20, seed=13)
    med = []
    for q in (0, 1, 2):
        med.append(np.median([PL.rs_lowrank(A, 20, 5, q, seed=40 + t).err for t in range(5)]))
    assert med[0] > med[1] > med[2]


@pytest.mark.slow
def test_fig6_statistical_reproduction(golden_dir):
    """Figure 6: medians over 5 seeds within +-30% of the printed errors for the
    Table 1 matrices (n = 500, k = 50, p = 10; m = 1000 suffices by rotation invariance of a
    Gaussian Omega)."""
    g = json.load(open(os.path.join(golden_dir, "paper_values.json")))["fig6"]
    for name, law in (("power", "power"), ("exponent", "exp-paper")):
        errs = {"QP3": [], "q0": [], "q1": [], "q2": []}
        for seed in range(5):
            A, _ = make_matrix(1000, 500, law, 50, seed=500 + seed)
            errs["QP3"].append(PL.qp3_baseline(A, 50)[2])
            for q in (0, 1, 2):
                errs[f"q{q}"].append(PL.rs_lowrank(A, 50, 10, q, seed=700 + seed).err)
        for key, vals in errs.items():
            med = float(np.median(vals))
            want = g[name][key]
            assert abs(med - want) <= 0.30 * want, (name, key, med, want)


def test_scaling_by_power_of_two_is_exact():
    """A -> 2A gives B -> 2B, R -> 2R bitwise and Q unchanged (every step is homogeneous)."""
    A, _ = make_matrix(200, 60, "exp-paper", 8, seed=21)
    r1 = PL.rs_lowrank(A, 8, 4, 1, seed=3)
    r2 = PL.rs_lowrank(2 * A, 8, 4, 1, seed=3)
    np.testing.assert_array_equal(r2.B0, 2 * r1.B0)
    np.testing.assert_array_equal(r2.perm, r1.perm)
    np.testing.assert_array_equal(r2.R, 2 * r1.R)
    np.testing.assert_array_equal(r2.Q, r1.Q)
