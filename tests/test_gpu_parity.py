"""GPU parity: the CUDA path (through the C ABI) against the CPU oracle, element by element.

Tolerances (BASELINE.json north_star, DESIGN.md §2 R9): Omega bit-exact; B, R normwise relative
<= 1e-11 at every conditioning; T <= 1e-11 kappa-scaled by kappa(R^_11) above 2e5 and Q <= 1e-11
kappa-scaled by kappa(Rbar) above 2e5 (the only two quantities that inherit a condition number,
SURVEY §8c-4); pivots identical where every step's oracle gap >= 1e-10; |e_gpu - e_oracle| <= 1e-12
on the normalised error.  Every case's achieved errors are printed (and appended to $RS_PARITY_LOG
when set), so tolerance decisions rest on data."""

import json
import math
import os

import numpy as np
import pytest
import torch

from tests.gpu_helpers import pivots_comparable, q_tolerance, rel, to_dev, to_np

pytestmark = pytest.mark.gpu

cuda = pytest.importorskip("torch").cuda
if not cuda.is_available():  # pragma: no cover
    pytest.skip("needs a GPU", allow_module_level=True)

import paper_conf_sc_maryykltd15_b200 as rs  # noqa: E402
from oracle import philox as OP  # noqa: E402
from oracle import pipeline as OPL  # noqa: E402
from synth.matrices import make_matrix  # noqa: E402

SEED = 0x5C15


@pytest.fixture(scope="module", autouse=True)
def _built():
    from paper_conf_sc_maryykltd15_b200 import build

    build.build()
    rs.load_library()


# ------------------------------------------------------------------------------------------
# Omega: bit-exact against the oracle's Philox + RS-BM32
# ------------------------------------------------------------------------------------------
@pytest.mark.parametrize("j0,ncols", [(0, 64), (3, 1001), (123457, 517), (2**33 + 5, 40)])
def test_omega_bit_exact(j0, ncols):
    ell = 37
    h = rs.create(64, 64, 0, 64, 30, 7, SEED)
    try:
        got = to_np(rs.omega(h, j0, ncols))
        want = OP.omega(ell, j0, j0 + ncols, SEED)
        assert got.shape == want.shape
        np.testing.assert_array_equal(got, want)
    finally:
        rs.destroy(h)


def test_omega_bit_exact_large_sample():
    """1.85 M values (37 rows x 50 000 columns, odd start) against the oracle, bit for bit."""
    h = rs.create(64, 64, 0, 64, 30, 7, SEED)
    try:
        got = to_np(rs.omega(h, 7, 50000))
        np.testing.assert_array_equal(got, OP.omega(37, 7, 50007, SEED))
    finally:
        rs.destroy(h)


# ------------------------------------------------------------------------------------------
# Step 1: B = Omega A (fused Philox GEMM + split-K)
# ------------------------------------------------------------------------------------------
@pytest.mark.parametrize("m,n,k,p", [(500, 200, 20, 10), (1237, 301, 13, 6), (20000, 1000, 50, 10), (64, 130, 8, 0)])
def test_sample_parity(m, n, k, p):
    A, _ = make_matrix(m, n, "exp-k", k, seed=m + n)
    Ad = to_dev(A)
    h = rs.create(m, m, 0, n, k, p, SEED)
    try:
        rs.sample(h, Ad)
        B = to_np(rs.get_sample(h))
    finally:
        rs.destroy(h)
    Bo = OPL.sample(A, k + p, SEED)
    assert rel(B, Bo) <= 1e-13


@pytest.mark.parametrize("m,n,k,p", [
    (40000, 130, 8, 4),      # l = 12 (one 16-row M tile), 2 N tiles: groups of 2 members
    (30000, 300, 100, 28),   # l = 128 (MFW = 8), 3 N tiles
    (2048, 700, 20, 10),     # m_local at the ring threshold (8 chunks of 256 rows)
    (1000003, 129, 30, 2),   # m = 1e6 + 3 rows (A's tail inside the last chunk), 2 N tiles (129 = 128 + 1)
])
def test_sample_ring_shapes(m, n, k, p):
    """The ring sample GEMM (m_local >= 2048, l <= 128) at its edges: tiny and full M tiles, a
    ragged last N tile, the smallest K it takes, and a K tail inside a chunk -- B = Omega A
    against the oracle's fixed-order product."""
    rng = np.random.default_rng(m + n)
    A = np.asfortranarray(rng.standard_normal((m, n)))
    B = _sample_gpu(A, k, p)
    assert rel(B, OPL.sample(A, k + p, SEED)) <= 1e-13


@pytest.mark.parametrize("m,n,k,p", [
    (60000, 1032, 100, 10),   # n % 128 = 8 (cfg2/cfg4's tail width), l = 110: 8 full N tiles share it
    (50000, 1036, 60, 4),     # tail of 12 columns: the second tail n8 block is ragged; l = 64 (MFW 4)
    (40000, 1040, 120, 8),    # tail of 16 (cfg3's width), l = 128 (MFW 8)
    (3000, 1288, 100, 10),    # K = 3 000 rows: units with fewer K stages than N tiles (some get no tail stage)
])
def test_sample_narrow_last_tile(m, n, k, p):
    """Ring sample GEMM with a last N tile of 8 / 12 / 16 columns (the widths the KC tail fold takes
    in B := C~ A; the ring kernel keeps its own narrow tile) -- B = Omega A against the oracle."""
    rng = np.random.default_rng(m + 7 * n)
    A = np.asfortranarray(rng.standard_normal((m, n)))
    B = _sample_gpu(A, k, p)
    Bo = OPL.sample(A, k + p, SEED)
    assert rel(B, Bo) <= 1e-13
    # the tail columns on their own (an error confined to them would hide in the global norm)
    t0 = (n // 128) * 128
    assert rel(B[:, t0:], Bo[:, t0:]) <= 1e-13


def _sample_gpu(A, k, p):
    m, n = A.shape
    h = rs.create(m, m, 0, n, k, p, SEED)
    try:
        rs.sample(h, to_dev(A))
        return to_np(rs.get_sample(h))
    finally:
        rs.destroy(h)


@pytest.mark.parametrize("m,split", [(3001, 1499), (10001, 4999)])
def test_sample_row_offset_partition_sums_to_whole(m, split):
    """Two row blocks (offset not a multiple of 4) computed by two handles sum to the 1-rank B --
    on the cluster sample kernel (m_local < 2048) and on the ring sample kernel (m_local >= 2048,
    Philox blocks straddling the chunk and rank boundaries)."""
    n, k, p = 257, 16, 8
    A, _ = make_matrix(m, n, "exp-k", k, seed=7)
    parts = [(0, split), (split, m)]
    Bs = []
    for r0, r1 in parts:
        h = rs.create(m, r1 - r0, r0, n, k, p, SEED)
        try:
            rs.sample(h, to_dev(np.asfortranarray(A[r0:r1])))
            Bs.append(to_np(rs.get_sample(h)))
        finally:
            rs.destroy(h)
    Bo = OPL.sample(A, k + p, SEED)
    assert rel(Bs[0] + Bs[1], Bo) <= 1e-13
    assert rel(Bs[0], OPL.sample(np.asfortranarray(A[:split]), k + p, SEED)) <= 1e-13


@pytest.mark.parametrize("m,n,k,p", [(3001, 257, 16, 8), (20000, 1000, 100, 10), (500, 64, 5, 3)])
def test_sample_columns_parity(m, n, k, p):
    """Column sampling B_c = Omega_c A^T (Fig. 8(b)); Omega_c keyed by column index, tag 1."""
    A, _ = make_matrix(m, n, "exp-k", k, seed=m + 7)
    h = rs.create(m, m, 0, n, k, p, SEED)
    try:
        Bc = to_np(rs.sample_columns(h, to_dev(A)))
    finally:
        rs.destroy(h)
    want = OP.omega(k + p, 0, n, SEED, 1) @ A.T
    assert Bc.shape == (k + p, m)
    assert rel(Bc, want) <= 1e-13


def test_sample_columns_row_partition_is_local():
    """Each rank's rows of A give exactly its own columns of B_c (no reduction)."""
    m, n, k, p = 2001, 300, 12, 4
    A, _ = make_matrix(m, n, "exp-k", k, seed=9)
    want = OP.omega(k + p, 0, n, SEED, 1) @ A.T
    for r0, r1 in [(0, 1000), (1000, m)]:
        h = rs.create(m, r1 - r0, r0, n, k, p, SEED)
        try:
            Bc = to_np(rs.sample_columns(h, to_dev(np.asfortranarray(A[r0:r1]))))
        finally:
            rs.destroy(h)
        assert rel(Bc, want[:, r0:r1]) <= 1e-13


def test_sample_with_padded_leading_dimension():
    m, n, k, p = 777, 150, 10, 5
    A, _ = make_matrix(m, n, "exp-k", k, seed=3)
    Ad = to_dev(A, ld=800)
    assert Ad.stride(1) == 800
    h = rs.create(m, m, 0, n, k, p, SEED)
    try:
        rs.sample(h, Ad)
        assert rel(to_np(rs.get_sample(h)), OPL.sample(A, k + p, SEED)) <= 1e-13
    finally:
        rs.destroy(h)


# ------------------------------------------------------------------------------------------
# The whole pipeline
# ------------------------------------------------------------------------------------------
def _run_gpu(A, k, p, q, seed=SEED, *, graph=False):
    """The C-ABI phases (sample, power_iterate, pivot, factor), or with graph=True the whole step
    through rs_lowrank_run (captured once, then replayed: the second call's result is returned)."""
    Ad = to_dev(A)
    if graph:
        m, n = A.shape
        h = rs.create(m, m, 0, n, k, p, seed)
        perm = torch.empty(n, dtype=torch.int64, device="cuda")
        Q = rs.empty_colmajor(m, k)
        R = rs.empty_colmajor(k, n)
        rs.run(h, Ad, q, perm, Q, R)
        rs.run(h, Ad, q, perm, Q, R)
    else:
        perm, Q, R, h = rs.rs_lowrank.rs_lowrank(Ad, k, p, q, seed)
    try:
        B = to_np(rs.get_sample(h))
        T, Rhat, gaps = rs.get_pivot_data(h)
        out = dict(B=B, perm=perm.cpu().numpy(), Q=to_np(Q), R=to_np(R), T=to_np(T), Rhat=to_np(Rhat),
                   gaps=np.array(gaps))
    finally:
        rs.destroy(h)
    return out


def _log(case, errs, tol):
    rec = {"case": case, "errs": errs, "tol": tol}
    print("PARITY " + json.dumps(rec, default=float))
    path = os.environ.get("RS_PARITY_LOG")
    if path:
        with open(path, "a") as fh:
            fh.write(json.dumps(rec, default=float) + "\n")


def _compare(A, k, p, q, seed=SEED, *, law=None, graph=False):
    g = _run_gpu(A, k, p, q, seed, graph=graph)
    o = OPL.rs_lowrank(A, k, p, q, seed)
    kc = pivots_comparable(o.gaps, k)
    errs = {"B": rel(g["B"], o.B), "pivots_equal": list(g["perm"][:kc]) == list(o.perm[:kc]), "kc": kc}
    tol = {"B": 1e-11}
    if kc == k:
        errs["perm_all_equal"] = list(g["perm"]) == list(o.perm)
        errs["T"] = rel(g["T"], o.T)
        errs["Rhat"] = rel(np.abs(g["Rhat"]), np.abs(o.Rhat))
        errs["R"] = rel(g["R"], o.R)
        errs["Q"] = rel(g["Q"], o.Q)
        # same evaluator for both factorizations
        errs["e_gpu"] = OPL.approx_error(A, g["perm"], g["Q"], g["R"])
        errs["e_oracle"] = o.err
        # T = R̂11^{-1} R̂12 inherits kappa(R̂11) and Q inherits kappa(Rbar) (reading R9);
        # R = Rbar [I T] does not (two correct pipelines agree on R to ~1e-15 at every kappa): 1e-11
        kap11 = np.linalg.cond(o.Rhat[:, :k])
        errs["kappa_R11"] = float(kap11)
        errs["kappa_Rbar"] = float(np.linalg.cond(o.Rbar))
        tol.update({"T": max(1e-11, 50 * kap11 * 2.0 ** -53), "Rhat": 1e-11, "R": 1e-11, "Q": q_tolerance(o.Rbar)})
    Qg = g["Q"]
    errs["orth"] = float(np.abs(Qg.T @ Qg - np.eye(k)).max())
    _log(dict(m=A.shape[0], n=A.shape[1], k=k, p=p, q=q, graph=graph), errs, tol)
    msg = f"errs={errs} tol={tol}"
    assert errs["pivots_equal"], msg
    for key, t in tol.items():
        assert errs[key] <= t, msg
    if kc == k:
        assert errs["perm_all_equal"], msg
        assert abs(errs["e_gpu"] - errs["e_oracle"]) <= 1e-12, msg
    assert errs["orth"] <= 1e-13, msg
    return g, o


@pytest.mark.parametrize("q", [0, 1, 2])
def test_pipeline_cfg1(q):
    """BASELINE configs[0]: m=500, n=200, k=20, p=10, exp-paper decay (plus q = 1, 2)."""
    A, _ = make_matrix(500, 200, "exp-paper", 20, seed=2015)
    _compare(A, 20, 10, q)


@pytest.mark.parametrize("m,n,k,p,q,law", [
    (1237, 301, 13, 6, 1, "exp-k"),       # ragged: l = 19 (pads to 24), m, n not tile multiples
    (3000, 600, 40, 10, 2, "power"),
    (20000, 1000, 50, 10, 1, "exp-k"),    # several N tiles, split-K
    (2000, 400, 120, 8, 1, "exp-k"),      # l = 128: full M tile
    (4000, 500, 150, 10, 0, "exp-k"),     # l = 160 > 128: two M tiles, k > 128
    (6000, 900, 400, 10, 1, "exp-k"),     # cfg5's largest k: l = 410, four M tiles, Cholesky n > 128
    (8000, 1000, 200, 20, 2, "power"),    # cfg3 law and (k, p, q) at reduced m, n
    # KC tail fold in B := C~ A (n % 128 = 8 / 12 / 16: the last N % 128 columns computed by the
    # producer warpgroup's tail warps on every (n / 128)-th K stage); the last with few K stages
    # per split (N tiles without a tail stage)
    (30000, 1032, 100, 10, 1, "exp-k"),
    (20000, 1292, 50, 14, 2, "power"),
    (2500, 1040, 100, 10, 1, "exp-k"),
    # m / 128 >= 8 x 148 tiles: the short-K applies (C1 = L^-1 C, Q1 = X R^-1) run on the persistent
    # MC kernel (resident operand, balanced triangular fragment / box sets)
    (160000, 300, 50, 10, 1, "exp-k"),
    (152000, 400, 100, 10, 1, "exp-k"),   # cfg2/cfg4's (k, p): l = 110, MFW 7 apply, k = 100 factor
])
def test_pipeline_ragged_and_multitile(m, n, k, p, q, law):
    A, _ = make_matrix(m, n, law, k, seed=m + 3 * n)
    _compare(A, k, p, q)


@pytest.mark.parametrize("m,n,k,p,q,law", [
    (50000, 5000, 100, 10, 1, "exp-k"),      # BASELINE configs[1] (cfg2) exactly
    (100000, 10000, 200, 20, 2, "power"),   # BASELINE configs[2] (cfg3) exactly: l = 220, q = 2
    (1000000, 600, 100, 10, 1, "exp-k"),    # m = 1e6 (cfg4's m, k, p, q): 7 813 persistent tiles, long split-K
])
def test_pipeline_baseline_shapes(m, n, k, p, q, law):
    """The benchmarked shapes against the oracle (the cfg4 bench shape itself is checked on
    sampled outputs in test_cfg4_full_size_sampled)."""
    A, _ = make_matrix(m, n, law, k, seed=2015)
    _compare(A, k, p, q)


@pytest.mark.parametrize("m,n,k,p,q,law", [
    (20000, 1000, 50, 10, 1, "exp-k"),
    (152000, 400, 100, 10, 1, "exp-k"),
    (3000, 600, 40, 10, 2, "power"),
])
def test_pipeline_graph_run_parity(m, n, k, p, q, law):
    """rs_lowrank_run (the step captured as one CUDA graph and replayed) against the oracle."""
    A, _ = make_matrix(m, n, law, k, seed=m + 3 * n)
    _compare(A, k, p, q, graph=True)


def test_graph_run_equals_phases_bitwise():
    A, _ = make_matrix(30000, 700, "exp-k", 60, seed=12)
    g1 = _run_gpu(A, 60, 10, 1)
    g2 = _run_gpu(A, 60, 10, 1, graph=True)
    for key in ("B", "Q", "R", "T", "Rhat", "perm", "gaps"):
        np.testing.assert_array_equal(g1[key], g2[key])


@pytest.mark.parametrize("own_stream", [False, True])
def test_graph_run_is_captured_once_and_replayed(own_stream):
    """The first rs_lowrank_run captures (the library's launchers run during the capture), later
    calls replay the graph (no launcher runs: the launch counter stands still) -- on the legacy
    default stream as well as on a caller's stream -- and reproduce the first result bitwise."""
    m, n, k, p, q = 20000, 600, 40, 10, 1
    A, _ = make_matrix(m, n, "exp-k", k, seed=21)
    st = torch.cuda.Stream() if own_stream else torch.cuda.default_stream()
    with torch.cuda.stream(st):
        Ad = to_dev(A)
        h = rs.create(m, m, 0, n, k, p, SEED, stream=st)
        try:
            perm = torch.empty(n, dtype=torch.int64, device="cuda")
            Q, R = rs.empty_colmajor(m, k), rs.empty_colmajor(k, n)
            n0 = rs.kernel_launches()
            rs.run(h, Ad, q, perm, Q, R)
            n1 = rs.kernel_launches()
            Q1, R1 = to_np(Q), to_np(R)
            for _ in range(3):
                rs.run(h, Ad, q, perm, Q, R)
            n2 = rs.kernel_launches()
            assert n1 > n0 and n2 == n1, (n0, n1, n2)
            np.testing.assert_array_equal(to_np(Q), Q1)
            np.testing.assert_array_equal(to_np(R), R1)
        finally:
            rs.destroy(h)


def test_cfg4_full_size_sampled():
    """BASELINE configs[3] at full size (m = 1e6, n = 5 000, k = 100, p = 10, q = 1) in the launch
    configuration bench.py times (rs_lowrank_run).  The sample B = Omega A is compared entry by
    entry with the oracle on sampled (row, column) pairs -- each a length-1e6 dot product of the
    oracle's Omega row with a column of A, in the oracle's fixed order; the rest through properties
    that hold at any size: Q^T Q = I, A P_1 = Q Rbar (the first k columns of R reproduce A's pivot
    columns exactly), and the error between Eckart-Young and 5x it."""
    from oracle.gemm import matmul
    from oracle.philox import omega
    from synth.matrices import make_matrix_torch

    m, n, k, p, q = 1_000_000, 5000, 100, 10, 1
    A, sigma = make_matrix_torch(m, n, "exp-k", k, seed=2015, rows=(0, m), device="cuda")
    h = rs.create(m, m, 0, n, k, p, SEED)
    try:
        rs.sample(h, A)
        B0 = to_np(rs.get_sample(h))
        rows = [0, 37, 109]
        cols = [0, 1, 2500, 4097, 4999]
        Om = omega(k + p, 0, m, SEED, rows=rows)
        Ac = A[:, cols].cpu().numpy()
        ref = matmul(Om, Ac)
        got = B0[np.ix_(rows, cols)]
        err = float(np.linalg.norm(got - ref) / np.linalg.norm(ref))
        _log(dict(m=m, n=n, k=k, p=p, q=q, what="B0 sampled"), {"B0": err}, {"B0": 1e-11})
        assert err <= 1e-11, err
        perm = torch.empty(n, dtype=torch.int64, device="cuda")
        Q = rs.empty_colmajor(m, k)
        R = rs.empty_colmajor(k, n)
        rs.run(h, A, q, perm, Q, R)
        orth = float((Q.T @ Q - torch.eye(k, dtype=torch.float64, device="cuda")).abs().max())
        AP1 = A[:, perm[:k]]
        rel1 = float(torch.linalg.norm(AP1 - Q @ R[:, :k]) / torch.linalg.norm(AP1))
        D2 = torch.zeros((), dtype=torch.float64, device="cuda")
        A2 = torch.zeros((), dtype=torch.float64, device="cuda")
        for c0 in range(0, n, 500):
            D = A[:, perm[c0:c0 + 500]] - Q @ R[:, c0:c0 + 500]
            D2 += (D * D).sum()
            A2 += (A[:, c0:c0 + 500] ** 2).sum()
        e = math.sqrt(float(D2) / float(A2))
        ey = math.sqrt(float((sigma[k:] ** 2).sum()) / float((sigma ** 2).sum()))
        _log(dict(m=m, n=n, k=k, p=p, q=q, what="properties"), {"orth": orth, "AP1": rel1, "e": e, "e_EY": ey},
             {"orth": 1e-13, "AP1": 1e-13})
        assert orth <= 1e-13 and rel1 <= 1e-13
        assert ey <= e <= 5 * ey, (e, ey)   # r01 bench: e = 2.32e-5, Eckart-Young 1.0e-5
    finally:
        rs.destroy(h)


@pytest.mark.parametrize("m,n,k,p,q", [
    (2000, 5000, 100, 10, 0),   # cfg2/cfg4's n, k, p: 8 lanes per column, 79 CTAs
    (1500, 5000, 60, 10, 1),   # (n % m != 0: a Gaussian U, no tied column norms)
    (600, 9500, 30, 10, 0),     # n > 148 x 64: 4 lanes per column, 75 CTAs
])
def test_pipeline_wide_n_grid_qrcp(m, n, k, p, q):
    """n > 2048: the truncated QRCP runs on the flag-synchronised grid kernel (not the single-
    cluster one).  A = (n x m matrix with the exp-k law)^T: same singular values, cheap to build."""
    At, _ = make_matrix(n, m, "exp-k", k, seed=m + 3 * n)
    A = np.asfortranarray(At.T)
    _compare(A, k, p, q)


def test_pipeline_is_bitwise_deterministic():
    A, _ = make_matrix(5000, 400, "exp-k", 30, seed=5)
    g1 = _run_gpu(A, 30, 10, 1)
    g2 = _run_gpu(A, 30, 10, 1)
    for key in ("B", "Q", "R", "T"):
        np.testing.assert_array_equal(g1[key], g2[key])
    np.testing.assert_array_equal(g1["perm"], g2["perm"])


@pytest.mark.parametrize("m,n,k,p,q", [(20000, 1032, 60, 10, 1), (3000, 600, 40, 10, 2)])
def test_power_of_two_scaling_is_exact(m, n, k, p, q):
    """SURVEY 8(c) invariance: A -> 4 A gives B -> 4 B, R -> 4 R bit for bit and Q, T, perm
    unchanged -- every step (split-K and tail-fold sums, CholQR2, QRCP, TRSM) is homogeneous and
    scaling by a power of two is exact in IEEE arithmetic (sqrt of 16^s exact, no over/underflow
    here), so any stray constant, mis-scaled shift or wrong term in a kernel would show."""
    A, _ = make_matrix(m, n, "exp-k", k, seed=m + n)
    g1 = _run_gpu(A, k, p, q)
    g4 = _run_gpu(np.asfortranarray(4.0 * A), k, p, q)
    np.testing.assert_array_equal(g4["perm"], g1["perm"])
    np.testing.assert_array_equal(g4["B"], 4.0 * g1["B"])
    np.testing.assert_array_equal(g4["R"], 4.0 * g1["R"])
    np.testing.assert_array_equal(g4["Q"], g1["Q"])
    np.testing.assert_array_equal(g4["T"], g1["T"])


def test_column_permutation_permutes_pivots():
    """SURVEY 8(c) invariance: A -> A Pi (tie-free) selects the same columns, in Pi's labels, with
    the same R up to rounding (columns moved into / out of the 8-column KC tail fold are summed in
    another order, so the comparison is normwise, not bitwise)."""
    m, n, k, p, q = 20000, 1032, 60, 10, 1
    A, _ = make_matrix(m, n, "exp-k", k, seed=77)
    pi = np.random.default_rng(3).permutation(n)
    g1 = _run_gpu(A, k, p, q)
    g2 = _run_gpu(np.asfortranarray(A[:, pi]), k, p, q)
    np.testing.assert_array_equal(pi[g2["perm"][:k]], g1["perm"][:k])
    # R's first k columns (the pivot columns) in pivot order; the rest compared after undoing pi
    assert rel(g2["R"][:, :k], g1["R"][:, :k]) <= 1e-12
    inv = np.empty(n, dtype=np.int64)
    inv[pi] = np.arange(n)
    R1 = np.zeros_like(g1["R"])
    R2 = np.zeros_like(g2["R"])
    R1[:, g1["perm"]] = g1["R"]
    R2[:, pi[g2["perm"]]] = g2["R"]
    assert rel(R2, R1) <= 1e-12


def test_omega_identity_special_case_is_truncated_qp3():
    """set_sample(B := A) with l = m, q = 0: pivots = LAPACK dgeqp3's; |R| rows = QP3's."""
    import scipy.linalg as sla

    rng = np.random.default_rng(8)
    A = np.asfortranarray(rng.standard_normal((24, 60)) @ np.diag(np.exp(-np.linspace(0, 4, 60))))
    k = 8
    Ad = to_dev(A)
    h = rs.create(24, 24, 0, 60, k, 16, SEED)
    try:
        rs.set_sample(h, Ad)
        perm = torch.empty(60, dtype=torch.int64, device="cuda")
        rs.pivot(h, perm)
        Q = rs.empty_colmajor(24, k)
        R = rs.empty_colmajor(k, 60)
        rs.factor(h, Ad, Q, R)
        perm = perm.cpu().numpy()
        R = to_np(R)
    finally:
        rs.destroy(h)
    _, Rl, pl = sla.qr(A, pivoting=True, mode="economic")
    assert list(perm[:k]) == list(pl[:k])
    R_orig = np.empty_like(R)
    R_orig[:, perm] = R
    Rl_orig = np.empty((k, 60))
    Rl_orig[:, pl] = Rl[:k]
    np.testing.assert_allclose(np.abs(R_orig), np.abs(Rl_orig), atol=1e-12)


def test_exact_recovery_rank_k():
    A, _ = make_matrix(3000, 300, "rank-k", 12, seed=4)
    g = _run_gpu(A, 12, 6, 0)
    e = OPL.approx_error(A, g["perm"], g["Q"], g["R"])
    assert e <= 1e-13


# ------------------------------------------------------------------------------------------
# errors and state machine
# ------------------------------------------------------------------------------------------
@pytest.mark.parametrize("graph", [False, True])
def test_rank_deficient_power_iteration_falls_back_and_recovers_exactly(graph):
    """rank(A) = k < l with q >= 1: Gram(C) is singular, so CholQR2 breaks down;
    power_iterate only flags it on the device, pivot redoes the iteration with shifted CholQR
    (R20) -- through the phases or after the graph replay of rs_lowrank_run -- and rank(A) <= k is
    still recovered exactly (||A P - Q R|| at rounding level)."""
    A, _ = make_matrix(2000, 200, "rank-k", 10, seed=9)
    Ad = to_dev(A)
    if graph:
        h = rs.create(2000, 2000, 0, 200, 10, 8, SEED)
        perm = torch.empty(200, dtype=torch.int64, device="cuda")
        Q, R = rs.empty_colmajor(2000, 10), rs.empty_colmajor(10, 200)
        rs.run(h, Ad, 1, perm, Q, R)
    else:
        perm, Q, R, h = rs.rs_lowrank.rs_lowrank(Ad, 10, 8, 1, SEED)
    try:
        assert rs.get_fallbacks(h)[0] == 1
        assert rs.get_info(h)[0] == 0
    finally:
        rs.destroy(h)
    e = OPL.approx_error(A, perm.cpu().numpy(), to_np(Q), to_np(R))
    assert e <= 1e-13


def test_zero_matrix_reports_rank_deficient():
    A = np.zeros((300, 100), order="F")
    Ad = to_dev(A)
    h = rs.create(300, 300, 0, 100, 5, 3, SEED)
    try:
        rs.sample(h, Ad)
        with pytest.raises(rs.RSError) as ei:
            rs.pivot(h, None)
        assert ei.value.name == "RS_ERR_RANK_DEFICIENT"
    finally:
        rs.destroy(h)


def test_state_machine_and_argument_checks():
    A, _ = make_matrix(300, 100, "exp-k", 5, seed=1)
    Ad = to_dev(A)
    h = rs.create(300, 300, 0, 100, 5, 3, SEED)
    try:
        with pytest.raises(rs.RSError) as ei:
            rs.pivot(h, None)
        assert ei.value.name == "RS_ERR_BAD_STATE"
        with pytest.raises(rs.RSError):
            rs.factor(h, Ad, rs.empty_colmajor(300, 5), rs.empty_colmajor(5, 100))
        odd = torch.empty((100, 301), dtype=torch.float64, device="cuda")[:, :300].t()
        with pytest.raises(rs.RSError) as ei:
            rs.sample(h, odd)   # ld = 301 is odd
        assert ei.value.name == "RS_ERR_INVALID_ARG"
        rs.sample(h, Ad)
        rs.power_iterate(h, Ad, 1)
        with pytest.raises(rs.RSError) as ei:
            rs.power_iterate(h, Ad, 1)   # at most once per sample (the sample is kept for a replay)
        assert ei.value.name == "RS_ERR_BAD_STATE"
        rs.pivot(h, None)
        with pytest.raises(rs.RSError) as ei:
            rs.power_iterate(h, Ad, 1)
        assert ei.value.name == "RS_ERR_BAD_STATE"
    finally:
        rs.destroy(h)
