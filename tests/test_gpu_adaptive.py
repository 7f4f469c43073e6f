"""GPU parity of the adaptive fixed-accuracy scheme (Fig. 3) against oracle/adaptive.py."""

import numpy as np
import pytest
import torch

from tests.gpu_helpers import pivots_comparable, rel, to_dev, to_np

pytestmark = pytest.mark.gpu
if not torch.cuda.is_available():  # pragma: no cover
    pytest.skip("needs a GPU", allow_module_level=True)

import paper_conf_sc_maryykltd15_b200 as rs  # noqa: E402
from oracle import adaptive as AD  # noqa: E402
from oracle import pipeline as OPL  # noqa: E402
from synth.matrices import make_matrix  # noqa: E402

SEED = 0x5C15


def _eps_between(hist, idx):
    """A tolerance strictly between the oracle's estimates idx-1 and idx (robust stopping round)."""
    return float(np.sqrt(hist[idx - 1][1] * hist[idx][1]))


@pytest.mark.parametrize("q,inc,law", [(0, 8, "exp-paper"), (1, 16, "exp-paper"), (0, 24, "power")])
def test_adaptive_matches_oracle(q, inc, law):
    m, n, lmax = 3000, 500, 160
    A, _ = make_matrix(m, n, law, 50, seed=21 + q)
    probe = AD.adaptive_sample(A, 0.0, inc, q, SEED, lmax)          # full history to place eps
    stop = min(4, len(probe.history) - 1)
    eps = _eps_between(probe.history, stop)
    o = AD.adaptive_sample(A, eps, inc, q, SEED, lmax)
    assert o.converged
    Ad = to_dev(A)
    h = rs.create(m, m, 0, n, lmax, 0, SEED)
    try:
        ell, est, hist = rs.sample_adaptive(h, Ad, eps, inc, q)
        assert ell == o.ell
        assert len(hist) == len(o.history)
        for (lg, eg), (lo, eo) in zip(hist, o.history):
            assert lg == lo and abs(eg - eo) <= 1e-8 * max(eo, 1e-300) + 1e-14
        B = to_np(rs.get_sample(h))
        assert B.shape == (ell, n)
        assert rel(B, o.B) <= 1e-8, rel(B, o.B)   # per-block CholQR2+BCGS2 vs Householder+BCGS2
        np.testing.assert_allclose(B @ B.T, np.eye(ell), atol=1e-13)
        # Steps 2-3 on the adaptive sample with k = l
        perm = torch.empty(n, dtype=torch.int64, device="cuda")
        rs.pivot(h, perm)
        Q = rs.empty_colmajor(m, lmax)
        R = rs.empty_colmajor(lmax, n)
        rs.factor(h, Ad, Q, R)
        perm = perm.cpu().numpy()
        Qn, Rn = to_np(Q)[:, :ell], to_np(R)[:ell]
    finally:
        rs.destroy(h)
    perm_o, Rhat_o, T_o, gaps_o = OPL.pivot(o.B, ell)
    kc = pivots_comparable(gaps_o, ell)
    assert list(perm[:kc]) == list(perm_o[:kc])
    e_gpu = OPL.approx_error(A, perm, Qn, Rn)
    Qo, Rbo, Ro = OPL.factor(A, perm_o, T_o, ell)
    e_or = OPL.approx_error(A, perm_o, Qo, Ro)
    assert abs(e_gpu - e_or) <= 1e-12 + 1e-6 * e_or
    assert np.abs(Qn.T @ Qn - np.eye(ell)).max() <= 1e-13


@pytest.mark.parametrize("inc0,q", [(8, 0), (16, 1)])
def test_adaptive_interp_policy_matches_oracle(inc0, q):
    """R19b: the interpolated increments, the estimates and the final basis match
    the oracle run with the same policy."""
    m, n, lmax = 3000, 500, 200
    A, _ = make_matrix(m, n, "exp-paper", 50, seed=41 + q)
    eps = 1e-6    # final l ~ 72-112 stays inside the numerical rank (basis unique)
    o = AD.adaptive_sample(A, eps, inc0, q, SEED, lmax, inc_policy="interp")
    assert o.converged
    Ad = to_dev(A)
    h = rs.create(m, m, 0, n, lmax, 0, SEED)
    try:
        ell, est, hist = rs.sample_adaptive(h, Ad, eps, inc0, q, inc_policy="interp")
        B = to_np(rs.get_sample(h))
    finally:
        rs.destroy(h)
    assert [lg for lg, _ in hist] == [lo for lo, _ in o.history]
    assert ell == o.ell
    for (_, eg), (_, eo) in zip(hist, o.history):
        assert abs(eg - eo) <= 1e-8 * eo + 1e-14
    # the rows of the last (large) block are fixed only to u ||A|| / sigma_min(block) ~ 1e-5
    # (reading R17: a re-mixing inside the block); all earlier blocks match element-wise, the
    # whole basis through the range error it leaves
    lp = hist[-2][0]
    assert rel(B[:lp], o.B[:lp]) <= 1e-8
    e_g = np.linalg.norm(A - (A @ B.T) @ B)
    e_o = np.linalg.norm(A - (A @ o.B.T) @ o.B)
    assert abs(e_g - e_o) <= 1e-6 * e_o + 1e-13 * np.linalg.norm(A)
    np.testing.assert_allclose(B @ B.T, np.eye(ell), atol=1e-13)


def test_adaptive_reports_not_converged_at_lmax():
    m, n = 2000, 400
    A, _ = make_matrix(m, n, "slow", 20, seed=3)
    Ad = to_dev(A)
    h = rs.create(m, m, 0, n, 32, 0, SEED)
    try:
        with pytest.raises(rs.RSError) as ei:
            rs.sample_adaptive(h, Ad, 1e-12, 8, 0)
        assert ei.value.name == "RS_ERR_NOT_CONVERGED"
        ell, est, hist = rs.sample_adaptive(h, Ad, 1e-12, 8, 0, raise_on_max=False)
        assert ell == 32 and est > 1e-12
        o = AD.adaptive_sample(A, 1e-12, 8, 0, SEED, 32)
        assert not o.converged and o.ell == 32
        assert rel(to_np(rs.get_sample(h)), o.B) <= 1e-9
    finally:
        rs.destroy(h)


def test_adaptive_argument_checks():
    A, _ = make_matrix(500, 100, "slow", 10, seed=1)
    Ad = to_dev(A)
    h = rs.create(500, 500, 0, 100, 24, 8, SEED)   # p != 0
    try:
        with pytest.raises(rs.RSError) as ei:
            rs.sample_adaptive(h, Ad, 1e-3, 8, 0)
        assert ei.value.name == "RS_ERR_INVALID_ARG"
    finally:
        rs.destroy(h)
    h = rs.create(500, 500, 0, 100, 24, 0, SEED)
    try:
        with pytest.raises(rs.RSError):
            rs.sample_adaptive(h, Ad, 1e-3, 12, 0)          # not a multiple of 8
    finally:
        rs.destroy(h)
