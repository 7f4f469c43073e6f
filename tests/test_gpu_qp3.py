"""GPU parity of the truncated QP3 baseline (rs_qp3_truncated) against
oracle.linalg.qrcp_truncated (Sec. 2).

The GPU version downdates column norms (LAPACK cancellation test, exact recomputation on
failure) where the oracle recomputes them exactly (reading R5); pivots are compared where the
oracle's relative gap at every step so far is >= 1e-10, as for the QRCP of B."""

import numpy as np
import pytest
import torch

from tests.gpu_helpers import pivots_comparable, rel, to_dev, to_np

pytestmark = pytest.mark.gpu
if not torch.cuda.is_available():  # pragma: no cover
    pytest.skip("needs a GPU", allow_module_level=True)

import paper_conf_sc_maryykltd15_b200 as rs  # noqa: E402
from oracle import linalg as OL  # noqa: E402
from oracle import pipeline as OPL  # noqa: E402
from synth.matrices import make_matrix  # noqa: E402


def _q_from_reflectors(W, tau, k):
    """Q (m x k) = H_0 ... H_{k-1} I[:, :k] from the LAPACK-layout reflectors (test-side check)."""
    m = W.shape[0]
    Q = np.eye(m, k)
    for j in reversed(range(k)):
        v = np.zeros(m)
        v[j] = 1.0
        v[j + 1:] = W[j + 1:, j]
        Q -= tau[j] * np.outer(v, v @ Q)
    return Q


@pytest.mark.parametrize("m,n,k,law", [
    (500, 200, 20, "exp-paper"),       # BASELINE configs[0] shape
    (3001, 777, 70, "exp-k"),          # three panels, odd m, n
    (6145, 400, 33, "power"),          # GEMV row chunks + ragged tail, one column past a panel
    (300, 1000, 100, "exp-k"),         # wide (m < n)
    (4000, 500, 100, "exp-paper"),     # norms fall 10^10 within the run: downdating cancellations
])
def test_qp3_matches_oracle(m, n, k, law):
    A, _ = make_matrix(m, n, law, min(k, 50), seed=m + n + k)
    W = to_dev(A)
    perm, tau, res = rs.qp3_truncated(W, k, residual=True)
    perm, tau, Wn = perm.cpu().numpy(), tau.cpu().numpy(), to_np(W)
    perm_o, Rhat_o, gaps_o, R22_o = OL.qrcp_truncated(A, k, return_trailing=True)
    kc = pivots_comparable(gaps_o, k)
    assert kc >= min(k, 10)
    assert list(perm[:kc]) == list(perm_o[:kc])
    assert sorted(perm) == list(range(n))
    R = np.triu(Wn[:k])
    if kc == k:
        assert list(perm) == list(perm_o)
        assert rel(R, Rhat_o) <= 1e-11, rel(R, Rhat_o)
        assert abs(res - np.linalg.norm(R22_o)) <= 1e-9 * np.linalg.norm(A)
    # whatever the pivots: A P_{1:k} = Q R_{:, 1:k} and the trailing residual is R22
    Q = _q_from_reflectors(Wn, tau, k)
    np.testing.assert_allclose(Q.T @ Q, np.eye(k), atol=1e-13)
    Ap = A[:, perm]
    assert np.linalg.norm(Ap[:, :k] - Q @ R[:, :k]) <= 1e-13 * np.linalg.norm(A)
    assert np.linalg.norm(Ap[:, k:] - Q @ R[:, k:]) <= 1.01 * res + 1e-13 * np.linalg.norm(A)


def test_qp3_error_matches_fig6_column():
    """Fig. 6's "QP3" column is ||R22||_F / ||A||_F: the GPU residual equals the oracle's."""
    A, _ = make_matrix(2000, 300, "power", 30, seed=4)
    W = to_dev(A)
    _, _, res = rs.qp3_truncated(W, 30, residual=True)
    _, _, e_o = OPL.qp3_baseline(A, 30)
    assert abs(res / np.linalg.norm(A) - e_o) <= 1e-12 + 1e-9 * e_o


def test_qp3_rejects_bad_arguments():
    A = to_dev(np.zeros((10, 8)))
    with pytest.raises(rs.RSError):
        rs.qp3_truncated(A, 9)
    with pytest.raises(rs.RSError):
        rs.qp3_truncated(A, 0)
