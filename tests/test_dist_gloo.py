"""World-size-2 (and 3) gloo tests of the N > 1 host logic on CPU.

Each rank holds its row block A(r) (paper_conf_sc_maryykltd15_b200.partition.row_split)
and runs the distributed schedule the CUDA library runs: local partial products +
allreduce of B, distributed CholQR2 of the row-distributed C through allreduced Gram matrices
 with the second R^{-T} applied to the small product, replicated QRCP, and the
distributed CholQR2 of A(r) P_{1:k}.  The numpy arithmetic stands in for the kernels; the
collectives are real torch.distributed (gloo) calls.  Results must match the single-process oracle.
"""

import os
import socket

import numpy as np
import pytest
import torch
import torch.distributed as dist
import torch.multiprocessing as mp

from paper_conf_sc_maryykltd15_b200.partition import all_splits, row_split


def _free_port():
    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    p = s.getsockname()[1]
    s.close()
    return p


def _allreduce(x: np.ndarray) -> np.ndarray:
    t = torch.from_numpy(np.ascontiguousarray(x))
    dist.all_reduce(t)
    return t.numpy()


def _cholqr_rows_dist(X):
    """CholQR of the rows of a column-distributed short-wide X (l x m_local): G = sum X X^T."""
    G = _allreduce(X @ X.T)
    L = np.linalg.cholesky(G)
    return np.linalg.solve(L, X), L


def _worker(rank, world, port, cfg, out_q):
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        from oracle import pipeline as OPL
        from oracle.linalg import back_substitution, qrcp_truncated
        from synth.matrices import make_matrix

        m, n, k, p, q, seed = cfg
        A, _ = make_matrix(m, n, "exp-k", k, seed=11)
        r0, r1 = row_split(m, world, rank)
        Ar = np.asfortranarray(A[r0:r1])
        ell = k + p
        B = _allreduce(OPL.sample(Ar, ell, 0x5C15, row_offset=r0))
        for _ in range(q):
            # replicated CholQR2 of B (identical on every rank)
            Bt = B
            for _ in range(2):
                L = np.linalg.cholesky(Bt @ Bt.T)
                Bt = np.linalg.solve(L, Bt)
            C = Bt @ Ar.T                       # l x m_local
            C1, _ = _cholqr_rows_dist(C)
            G2 = _allreduce(C1 @ C1.T)
            L2 = np.linalg.cholesky(G2)
            B1 = _allreduce(C1 @ Ar)            # sum_r C1(r) A(r)
            B = np.linalg.solve(L2, B1)         # = C2 A with C2 = L2^{-1} C1
        perm, Rhat, gaps = qrcp_truncated(B, k)
        T = back_substitution(Rhat[:, :k], Rhat[:, k:])
        X = Ar[:, perm[:k]]
        Rb = np.eye(k)
        for _ in range(2):
            L = np.linalg.cholesky(_allreduce(X.T @ X))
            X = np.linalg.solve(L, X.T).T
            Rb = L.T @ Rb
        R = Rb @ np.hstack([np.eye(k), T])
        out_q.put((rank, B, perm, R, X, r0, r1))
    finally:
        dist.destroy_process_group()


def _run(world, cfg):
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = _free_port()
    procs = [ctx.Process(target=_worker, args=(r, world, port, cfg, q)) for r in range(world)]
    for pr in procs:
        pr.start()
    res = [q.get(timeout=240) for _ in range(world)]
    for pr in procs:
        pr.join(timeout=60)
        assert pr.exitcode == 0
    return sorted(res, key=lambda t: t[0])


def test_row_split_covers_rows_in_order():
    for m, nr in [(10, 3), (1_000_000, 8), (7, 7), (5, 8), (0, 2)]:
        sp = all_splits(m, nr)
        assert sp[0][0] == 0 and sp[-1][1] == m
        assert all(sp[i][1] == sp[i + 1][0] for i in range(nr - 1))
        sizes = [b - a for a, b in sp]
        assert max(sizes) - min(sizes) <= 1 and sizes == sorted(sizes, reverse=True)
    with pytest.raises(ValueError):
        row_split(10, 2, 2)


@pytest.mark.parametrize("world,cfg", [(2, (1203, 240, 20, 8, 1, 0)), (3, (900, 150, 12, 6, 2, 0))])
def test_distributed_schedule_matches_single_process_oracle(world, cfg):
    from oracle import pipeline as OPL
    from synth.matrices import make_matrix

    m, n, k, p, q, _ = cfg
    res = _run(world, cfg)
    A, _ = make_matrix(m, n, "exp-k", k, seed=11)
    o = OPL.rs_lowrank(A, k, p, q, 0x5C15)
    B0 = res[0][1]
    for r in res[1:]:
        np.testing.assert_array_equal(r[1], B0)          # replicated B is bitwise identical
        np.testing.assert_array_equal(r[2], res[0][2])   # so are the pivots
    assert np.linalg.norm(B0 - o.B) <= 1e-11 * np.linalg.norm(o.B)
    assert list(res[0][2][:k]) == list(o.perm[:k])
    R = res[0][3]
    assert np.linalg.norm(R - o.R) <= 1e-10 * np.linalg.norm(o.R)
    Q = np.vstack([r[4] for r in res])                   # row blocks in rank order
    assert np.abs(Q.T @ Q - np.eye(k)).max() <= 1e-13
    e = OPL.approx_error(A, res[0][2], Q, R)
    assert abs(e - o.err) <= 1e-12
