"""Shared helpers for the -m gpu parity tests (CUDA path via the C ABI vs the CPU oracle)."""

import numpy as np
import torch

U = 2.0 ** -53


def to_dev(A: np.ndarray, device="cuda", ld=None) -> torch.Tensor:
    from paper_conf_sc_maryykltd15_b200 import empty_colmajor

    m, n = A.shape
    t = empty_colmajor(m, n, device=device, ld=ld)
    t.copy_(torch.from_numpy(np.asarray(A, dtype=np.float64)))
    return t


def to_np(t: torch.Tensor) -> np.ndarray:
    return t.detach().cpu().numpy().astype(np.float64)


def rel(x, y) -> float:
    y = np.asarray(y)
    d = np.linalg.norm(np.asarray(x) - y)
    ny = np.linalg.norm(y)
    return float(d / ny) if ny > 0 else float(d)


def pivots_comparable(gaps, k, thresh=1e-10):
    """Number of leading pivot steps whose oracle gap is >= thresh."""
    for j, g in enumerate(gaps[:k]):
        if g < thresh:
            return j
    return k


def q_tolerance(Rbar) -> float:
    """Q parity tolerance: 1e-11 when kappa(Rbar) <= 2e5, else 50 kappa u (reading R9)."""
    kap = np.linalg.cond(Rbar)
    return max(1e-11, 50.0 * kap * U)
