"""Multi-rank path on ONE GPU: N ranks' handles (1-D row partition) run the whole
pipeline concurrently in N host threads, with the library's reductions (allreduce of B and of every
Gram matrix) routed through rs_lowrank_set_allreduce_hook to an in-process sum over the
N handles' device buffers instead of NCCL.  Every CUDA kernel of the N > 1 code path runs exactly
as it does under NCCL; only the transport differs.  Results are compared with the CPU oracle
(same tolerances as tests/test_gpu_parity.py) and with the single-rank GPU run."""

import os
import threading

import numpy as np
import pytest
import torch

from tests.gpu_helpers import pivots_comparable, q_tolerance, rel, to_dev, to_np

pytestmark = pytest.mark.gpu

if not torch.cuda.is_available():  # pragma: no cover
    pytest.skip("needs a GPU", allow_module_level=True)

import paper_conf_sc_maryykltd15_b200 as rs  # noqa: E402
from oracle import pipeline as OPL  # noqa: E402
from paper_conf_sc_maryykltd15_b200.partition import row_split  # noqa: E402
from synth.matrices import make_matrix  # noqa: E402

SEED = 0x5C15
_SERIAL = os.environ.get("RS_MR_SERIAL") == "1"  # debugging: serialise the ranks' library calls


@pytest.fixture(scope="module", autouse=True)
def _built():
    from paper_conf_sc_maryykltd15_b200 import build

    build.build()
    rs.load_library()


class _DevBuf:
    """__cuda_array_interface__ view of `count` doubles at a raw device pointer."""

    def __init__(self, ptr, count):
        self.__cuda_array_interface__ = {"shape": (count,), "typestr": "<f8", "data": (ptr, False),
                                         "version": 3, "strides": None}


class InProcessAllreduce:
    """Sum over N handles in one process.  Every rank syncs its stream and parks its buffer; rank 0
    copies the N buffers to the host, sums them in rank order (deterministic, plain numpy) and writes
    the sum back to every buffer before any rank continues.  Between reductions the N ranks' kernels
    run concurrently on the one GPU (their streams overlap); RS_MR_SERIAL=1 serialises the ranks'
    library calls with a token instead (debugging aid; DESIGN.md §7 has the history of the r01
    overlap finding and the r02 evidence that it does not occur with the current library)."""

    def __init__(self, nranks):
        self.n = nranks
        self.bufs = [None] * nranks
        self.barrier = threading.Barrier(nranks, timeout=300)
        self.calls = [0] * nranks
        self.token = threading.Lock()

    def hook(self, rank, stream):
        def fn(buf, count, stream_ptr):
            stream.synchronize()
            self.bufs[rank] = (buf, count)
            self.calls[rank] += 1
            if _SERIAL:
                self.token.release()
            self.barrier.wait()
            if rank == 0:
                counts = {c for _, c in self.bufs}
                assert len(counts) == 1, f"ranks disagree on the reduction size: {self.bufs}"
                torch.cuda.synchronize()
                views = [torch.as_tensor(_DevBuf(b, count), device="cuda") for b, _ in self.bufs]
                parts = [v.cpu().numpy() for v in views]
                total = parts[0].copy()
                for x in parts[1:]:
                    total += x
                src = torch.from_numpy(total)
                for v in views:
                    v.copy_(src)
                torch.cuda.synchronize()
            self.barrier.wait()
            if _SERIAL:
                self.token.acquire()

        return fn


def _run_ranks(A, nranks, k, p, q):
    m, n = A.shape
    comm = InProcessAllreduce(nranks)
    out = [None] * nranks
    errs = [None] * nranks
    dev = torch.device("cuda", 0)

    def work(r):
        if _SERIAL:
            comm.token.acquire()
        try:
            torch.cuda.set_device(dev)
            r0, r1 = row_split(m, nranks, r)
            stream = torch.cuda.Stream(device=dev)
            with torch.cuda.stream(stream):
                Ad = to_dev(np.asfortranarray(A[r0:r1]))
                stream.synchronize()
                h = rs.create(m, r1 - r0, r0, n, k, p, SEED, device=dev, stream=stream)
                try:
                    rs.rs_lowrank.set_allreduce_hook(h, nranks, r, comm.hook(r, stream))
                    perm = torch.empty(n, dtype=torch.int64, device=dev)
                    Q = rs.empty_colmajor(r1 - r0, k, device=dev)
                    R = rs.empty_colmajor(k, n, device=dev)
                    rs.sample(h, Ad)
                    rs.power_iterate(h, Ad, q)
                    rs.pivot(h, perm)
                    rs.factor(h, Ad, Q, R)
                    stream.synchronize()
                    B = to_np(rs.get_sample(h))
                    out[r] = dict(r0=r0, r1=r1, B=B, perm=perm.cpu().numpy(), Q=to_np(Q), R=to_np(R),
                                  fallbacks=rs.get_fallbacks(h))
                finally:
                    rs.destroy(h)
        except BaseException as e:  # noqa: BLE001
            errs[r] = e
            comm.barrier.abort()
        finally:
            if _SERIAL:
                comm.token.release()

    ts = [threading.Thread(target=work, args=(r,)) for r in range(nranks)]
    for t in ts:
        t.start()
    for t in ts:
        t.join()
    for e in errs:
        if e is not None:
            raise e
    assert len(set(comm.calls)) == 1 and comm.calls[0] > 0, comm.calls
    return out, comm.calls[0]


@pytest.mark.parametrize("m,n,k,p,q,nranks", [
    (20000, 1000, 50, 10, 1, 2),
    (20005, 700, 40, 10, 2, 3),     # ragged split: row offsets 6669, 13337 (Philox blocks straddle ranks)
    (30000, 5000, 100, 10, 1, 4),   # cfg2/cfg4's (n, k, p, q); QRCP on the grid kernel
])
def test_multirank_pipeline_matches_oracle(m, n, k, p, q, nranks):
    A, _ = make_matrix(m, n, "exp-k", k, seed=m + 7 * nranks)
    ranks, ncalls = _run_ranks(A, nranks, k, p, q)
    # allreduces: B after the sample and after each power pass, 2 Grams of C per pass, 2 k x k Grams
    assert ncalls >= 1 + 3 * q + 2, ncalls
    o = OPL.rs_lowrank(A, k, p, q, SEED)
    kc = pivots_comparable(o.gaps, k)
    r0 = ranks[0]
    # replicated outputs are bitwise identical on every rank (identical allreduced inputs)
    for r in ranks[1:]:
        assert np.array_equal(r["B"], r0["B"]) and np.array_equal(r["perm"], r0["perm"]) and np.array_equal(r["R"], r0["R"])
    Q = np.vstack([r["Q"] for r in ranks])
    assert rel(r0["B"], o.B) <= 1e-11, (rel(r0["B"], o.B), [r["fallbacks"] for r in ranks])
    assert list(r0["perm"][:kc]) == list(o.perm[:kc])
    if kc == k:
        assert list(r0["perm"]) == list(o.perm)
        assert rel(r0["R"], o.R) <= 1e-11
        assert rel(Q, o.Q) <= q_tolerance(o.Rbar)
        e = OPL.approx_error(A, r0["perm"], Q, r0["R"])
        assert abs(e - o.err) <= 1e-12, (e, o.err)
    assert float(np.abs(Q.T @ Q - np.eye(k)).max()) <= 1e-13


def test_multirank_equals_single_rank_up_to_summation_order():
    """N = 3 vs N = 1 on the GPU: same pivots, B / Q / R within summation-order rounding."""
    m, n, k, p, q = 12001, 600, 30, 10, 1
    A, _ = make_matrix(m, n, "exp-k", k, seed=99)
    ranks, _ = _run_ranks(A, 3, k, p, q)
    perm1, Q1, R1, h = rs.rs_lowrank.rs_lowrank(to_dev(A), k, p, q, SEED)
    try:
        B1 = to_np(rs.get_sample(h))
    finally:
        rs.destroy(h)
    assert np.array_equal(ranks[0]["perm"], perm1.cpu().numpy())
    assert rel(ranks[0]["B"], B1) <= 1e-13
    assert rel(ranks[0]["R"], to_np(R1)) <= 1e-12
    assert rel(np.vstack([r["Q"] for r in ranks]), to_np(Q1)) <= 1e-11


def test_allreduce_hook_state_checks():
    h = rs.create(64, 64, 0, 64, 8, 2, SEED)
    try:
        with pytest.raises(rs.RSError):
            rs.rs_lowrank.set_allreduce_hook(h, 2, 2, lambda *a: None)   # rank out of range
        A = to_dev(np.eye(64))
        rs.sample(h, A)
        with pytest.raises(rs.RSError):
            rs.rs_lowrank.set_allreduce_hook(h, 2, 0, lambda *a: None)   # not directly after create
    finally:
        rs.destroy(h)
