"""The library's NCCL code path (allreduce of B and of every Gram matrix) at world size 1 on the
GPU: ncclAllReduce is called whenever a communicator is attached (counted through the "comm"
profiling scope), and results must be bitwise identical to the communicator-free run (a 1-rank
allreduce is a copy) -- through the phases and through the CUDA-graph-captured rs_lowrank_run."""

import os

import numpy as np
import pytest
import torch

from tests.gpu_helpers import rel, to_dev, to_np

pytestmark = pytest.mark.gpu
if not torch.cuda.is_available():  # pragma: no cover
    pytest.skip("needs a GPU", allow_module_level=True)

import paper_conf_sc_maryykltd15_b200 as rs  # noqa: E402
from synth.matrices import make_matrix  # noqa: E402


def test_nccl_world_size_one_matches_no_comm():
    from paper_conf_sc_maryykltd15_b200 import build

    build.build()
    uid = rs.rs_lowrank.comm_get_unique_id()
    comm = rs.rs_lowrank.comm_init(1, uid, 0)
    try:
        A, _ = make_matrix(6000, 500, "exp-k", 40, seed=3)
        Ad = to_dev(A)
        outs = []
        for c in (None, comm):
            h = rs.create(6000, 6000, 0, 500, 40, 10, 0x5C15, nccl_comm=c)
            rs.set_profiling(h, True)
            perm, Q, R, _ = rs.rs_lowrank.rs_lowrank(Ad, 40, 10, 1, 0x5C15, h=h)
            prof = rs.get_profile(h)
            ncomm = prof.get("comm", {}).get("launches", 0)
            # B after the sample and after the power pass, 2 Grams of C, 2 k x k Grams of the factor
            assert ncomm == (6 if c is not None else 0), prof.get("comm")
            outs.append((to_np(rs.get_sample(h)), perm.cpu().numpy(), to_np(Q), to_np(R)))
            for _ in range(2):   # capture, then replay
                rs.run(h, Ad, 1, perm, Q, R)
            outs.append((to_np(rs.get_sample(h)), perm.cpu().numpy(), to_np(Q), to_np(R)))
            rs.destroy(h)
        for o in outs[1:]:
            for x, y in zip(outs[0], o):
                np.testing.assert_array_equal(x, y)
    finally:
        rs.rs_lowrank.comm_destroy(comm)


def test_run_host_matches_device_api():
    """rs_lowrank_run_host (host buffers, the e2e entry point) = device-buffer calls."""
    m, n, k, p, q = 3000, 400, 30, 10, 1
    A, _ = make_matrix(m, n, "exp-k", k, seed=8)
    Ad = to_dev(A)
    perm, Q, R, h = rs.rs_lowrank.rs_lowrank(Ad, k, p, q, 0x5C15)
    Ah = rs.empty_colmajor(m, n, device="cpu", pin=True)
    Ah.copy_(torch.from_numpy(A))
    Adev = rs.empty_colmajor(m, n)
    Qh = rs.empty_colmajor(m, k, device="cpu", pin=True)
    Rh = rs.empty_colmajor(k, n, device="cpu", pin=True)
    ph = torch.empty(n, dtype=torch.int64, pin_memory=True)
    Qd, Rd = rs.empty_colmajor(m, k), rs.empty_colmajor(k, n)
    rs.run_host(h, Ah, Adev, q, ph, Qh, Rh, Qd, Rd)
    rs.destroy(h)
    np.testing.assert_array_equal(ph.numpy(), perm.cpu().numpy())
    np.testing.assert_array_equal(Qh.numpy(), to_np(Q))
    np.testing.assert_array_equal(Rh.numpy(), to_np(R))
