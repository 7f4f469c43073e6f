"""GPU: CholQR breakdown fallbacks (R20).

The exponent law sigma_i = 10^(-i/10) at l = 110 with q = 1 makes CholQR2 break down in the power
iteration (kappa(C) ~ sigma_1 / sigma_l = 1e11, kappa^2 u >> 1) and in the factor step
(kappa(A P_1) ~ 1e10).  The library then redoes the power iteration with shifted CholQR and the
factor with shifted CholQR4/6; the oracle (Householder throughout) never breaks down, so the
comparison is on what is unique: the pivots where the oracle's gaps separate them, the
approximation error, and the orthonormality of Q."""

import numpy as np
import pytest
import torch

from tests.gpu_helpers import pivots_comparable, to_dev, to_np

pytestmark = pytest.mark.gpu
if not torch.cuda.is_available():  # pragma: no cover
    pytest.skip("needs a GPU", allow_module_level=True)

import paper_conf_sc_maryykltd15_b200 as rs  # noqa: E402
from oracle import pipeline as OPL  # noqa: E402
from synth.matrices import make_matrix  # noqa: E402

SEED = 0x5C15


@pytest.mark.parametrize("m,n,k,p,q", [(3000, 500, 100, 10, 1), (4000, 600, 120, 8, 2)])
def test_breakdown_fallback_matches_oracle(m, n, k, p, q):
    A, s = make_matrix(m, n, "exp-paper", 50, seed=31 + q)
    Ad = to_dev(A)
    perm, Q, R, h = rs.rs_lowrank.rs_lowrank(Ad, k, p, q, SEED)
    try:
        robust_iters, factor_shifts = rs.get_fallbacks(h)
        B = to_np(rs.get_sample(h))
    finally:
        rs.destroy(h)
    assert robust_iters >= 1 and factor_shifts >= 2, (robust_iters, factor_shifts)
    perm, Qn, Rn = perm.cpu().numpy(), to_np(Q), to_np(R)
    o = OPL.rs_lowrank(A, k, p, q, SEED)
    kc = pivots_comparable(o.gaps, k)
    assert kc >= 20
    assert list(perm[:kc]) == list(o.perm[:kc])
    # B spans what the oracle's B spans, along its well-determined leading directions
    Ub = np.linalg.svd(B, full_matrices=False)[2][:40]
    Uo = np.linalg.svd(o.B, full_matrices=False)[2][:40]
    assert np.linalg.norm(Ub.T @ Ub - Uo.T @ Uo, 2) <= 1e-8
    e_gpu = OPL.approx_error(A, perm, Qn, Rn)
    # both errors are at the sigma_{k+1} level of a rank-revealing choice (||.||_F normalised)
    sk1 = s[k] / np.linalg.norm(s)
    assert e_gpu <= 50 * sk1 and o.err <= 50 * sk1, (e_gpu, o.err, sk1)
    assert np.abs(Qn.T @ Qn - np.eye(k)).max() <= 1e-13
    # A P_{1:k} = Q R_{:, 1:k} to working accuracy
    Ap = A[:, perm[:k]]
    assert np.linalg.norm(Ap - Qn @ Rn[:, :k]) <= 1e-13 * np.linalg.norm(Ap)


def test_no_fallback_on_well_conditioned_input():
    A, _ = make_matrix(2000, 300, "exp-k", 20, seed=3)
    perm, Q, R, h = rs.rs_lowrank.rs_lowrank(to_dev(A), 20, 10, 1, SEED)
    try:
        assert rs.get_fallbacks(h) == (0, 0)
    finally:
        rs.destroy(h)
