"""Pins for oracle/adaptive.py (Fig. 3, the fixed-accuracy adaptive scheme)."""

import math

import numpy as np
import pytest

from oracle import adaptive as AD
from oracle import pipeline as PL
from oracle.linalg import rows_orth
from synth.matrices import make_matrix


def _proj(B):
    return B.T @ B


def test_bcgs2_makes_rows_orthogonal():
    rng = np.random.default_rng(0)
    X, _ = rows_orth(rng.standard_normal((5, 40)))
    Y = rng.standard_normal((3, 40)) + 1e3 * X[:3]          # nearly in span(X): needs the second pass
    Z = AD.bcgs2(X, Y)
    assert np.abs(Z @ X.T).max() <= 1e-12 * np.abs(Y).max()
    np.testing.assert_array_equal(AD.bcgs2(np.zeros((0, 40)), Y), Y)


def test_borth_qr_equals_qr_of_the_projection():
    """R17: in exact arithmetic the two-pass form is QR(Y - Y X^T X); the rows are orthonormal and
    orthogonal to X, and the positive-diagonal LQ factor ties the result to one basis."""
    rng = np.random.default_rng(1)
    X, _ = rows_orth(rng.standard_normal((6, 50)))
    Y = rng.standard_normal((4, 50))
    Z = AD.borth_qr(X, Y)
    np.testing.assert_allclose(Z @ Z.T, np.eye(4), atol=1e-14)
    assert np.abs(Z @ X.T).max() <= 1e-14
    P = np.eye(50) - X.T @ X                      # textbook projector, then one Householder QR
    Zt, _ = rows_orth(Y @ P)
    np.testing.assert_allclose(Z, Zt, atol=1e-13)
    np.testing.assert_allclose(AD.borth_qr(np.zeros((0, 50)), Y), rows_orth(Y)[0], atol=0)


def test_basis_stays_orthonormal_past_the_numerical_rank():
    """Exponent matrix (sigma_i = 10^(-i/10)) sampled to l = 256 > numerical rank ~160 with
    l_inc = 32: every block past the rank is rounding noise, yet B B^T = I to O(u) (R17)."""
    A, _ = make_matrix(1500, 600, "exp-paper", 50, seed=8)
    res = AD.adaptive_sample(A, eps=0.0, ell_inc=32, q=0, seed=3, ell_max=256)
    assert res.ell == 256
    assert np.abs(res.B @ res.B.T - np.eye(256)).max() <= 1e-13


def test_single_round_q0_equals_fixed_rank_orthonormal_sample():
    """One round with l_inc = l: B = QR(Omega[0:l] A), the fixed-rank sample (R16)."""
    A, _ = make_matrix(300, 80, "exp-paper", 10, seed=1)
    res = AD.adaptive_sample(A, eps=0.0, ell_inc=12, q=0, seed=7, ell_max=12)
    Bf, _ = rows_orth(PL.sample(A, 12, 7))
    np.testing.assert_allclose(res.B, Bf, atol=1e-13)
    assert res.ell == 12 and not res.converged


@pytest.mark.parametrize("q", [0, 1])
def test_blocks_are_orthonormal_and_q0_span_matches(q):
    A, _ = make_matrix(400, 120, "exp-paper", 10, seed=2)
    res = AD.adaptive_sample(A, eps=0.0, ell_inc=8, q=q, seed=3, ell_max=40)
    assert res.ell == 40
    np.testing.assert_allclose(res.B @ res.B.T, np.eye(40), atol=1e-13)
    if q == 0:  # block Gram-Schmidt does not change the span of Omega[0:l] A
        Bf, _ = rows_orth(PL.sample(A, 40, 3))
        np.testing.assert_allclose(_proj(res.B), _proj(Bf), atol=1e-11)


def test_estimator_bounds_the_range_error():
    """Bound (4) (HMT eq. (4.3), c_ad = 10): ||A - A B^T B||_2 <= 10 sqrt(2/pi) eps~,
    with failure probability <= min(m, n) 10^-l_inc; and eps~ never falls below the true error of
    the projected Gaussian test vectors' expectation by more than chance (eps~ > 0)."""
    A, s = make_matrix(600, 200, "exp-paper", 20, seed=4)
    res = AD.adaptive_sample(A, eps=1e-6, ell_inc=8, q=0, seed=5, ell_max=160)
    assert res.converged
    est = res.history[-1][1]
    err = np.linalg.norm(A - (A @ res.B.T) @ res.B, 2)
    assert err <= 10 * math.sqrt(2 / math.pi) * est
    assert est <= 1e-6
    # the rank found is close to where sigma drops below eps (10^(-i/10) = 1e-6 at i = 60)
    assert 56 <= res.ell <= 96


def test_error_estimates_decrease_with_power_iteration():
    """The paper's Fig. 16: with q > 0 the same accuracy is reached with fewer vectors."""
    A, _ = make_matrix(600, 300, "power", 20, seed=6)
    r0 = AD.adaptive_sample(A, eps=1e-5, ell_inc=8, q=0, seed=9, ell_max=200)
    r1 = AD.adaptive_sample(A, eps=1e-5, ell_inc=8, q=1, seed=9, ell_max=200)
    assert r0.converged and r1.converged
    assert r1.ell <= r0.ell


@pytest.mark.slow
def test_fig16_exponent_matrix_reaches_1e12_near_l_120_160():
    """Fig. 16: exponent matrix, eps = 1e-12, l_init = l_inc = 8,
    q = 0 reaches eps~ < 1e-12 at l ~ 120-160 (n = 500 suffices by rotation invariance)."""
    A, _ = make_matrix(1000, 500, "exp-paper", 50, seed=7)
    res = AD.adaptive_sample(A, eps=1e-12, ell_inc=8, q=0, seed=11, ell_max=400)
    assert res.converged
    assert 112 <= res.ell <= 176
    ests = [e for _, e in res.history]
    assert ests[-1] <= 1e-12 and ests[0] > 1e-2


def test_interp_increment_rule():
    """R19b on a closed form: log10 eps~ linear in l (slope -0.1 per vector, as sigma_i = 10^(-i/10))
    predicts l* exactly; the increment is rounded up to a multiple of 8."""
    hist = [(8, 1e-1), (16, 10 ** -1.8)]          # slope -0.1 / vector
    # eps = 1e-6 -> l* = 16 + (-6 + 1.8) / -0.1 = 58; at l = 24: need 34 -> 40
    assert AD.next_inc("interp", hist, 24, 8, 1e-6) == 40
    assert AD.next_inc("interp", hist, 24, 8, 10 ** -2.0) == 8      # l* = 18 < l: minimum 8
    assert AD.next_inc("interp", hist[:1], 24, 16, 1e-6) == 16      # one estimate: unchanged
    assert AD.next_inc("interp", [(8, 1e-3), (16, 1e-2)], 24, 16, 1e-6) == 16  # no decrease
    assert AD.next_inc("interp", hist, 24, 8, 0.0) == 8             # eps = 0: unchanged
    assert AD.next_inc("static", hist, 24, 8, 1e-6) == 8


def test_interp_policy_reaches_tolerance_in_fewer_rounds():
    """Fig. 17 "adapt. linc": on the exponent matrix the interpolated increment needs fewer rounds
    than the static l_inc = 8 and still meets eps (bound (4) holds for the final basis)."""
    A, s = make_matrix(1000, 400, "exp-paper", 50, seed=12)
    r_s = AD.adaptive_sample(A, 1e-10, 8, 0, 5, 400)
    r_i = AD.adaptive_sample(A, 1e-10, 8, 0, 5, 400, inc_policy="interp")
    assert r_s.converged and r_i.converged
    assert len(r_i.history) < len(r_s.history)
    assert r_i.history[-1][1] <= 1e-10
    err = np.linalg.norm(A - (A @ r_i.B.T) @ r_i.B, 2)
    assert err <= 10 * math.sqrt(2 / math.pi) * r_i.history[-1][1]
    np.testing.assert_allclose(r_i.B @ r_i.B.T, np.eye(r_i.ell), atol=1e-13)
