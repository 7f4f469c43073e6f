"""Pins for oracle/philox.py: the Gaussian sampling matrix Omega (Fig. 2(b) line 2)."""

import math
import os

import numpy as np
import pytest

from oracle import philox as P


def _kat_rows(golden_dir):
    rows = []
    with open(os.path.join(golden_dir, "philox_kat.txt")) as fh:
        for line in fh:
            if line.strip() and not line.startswith("#"):
                rows.append([int(w, 16) for w in line.split()])
    return rows


def test_philox_known_answer_vectors(golden_dir):
    """Random123 KAT vectors (external, published values)."""
    rows = _kat_rows(golden_dir)
    assert len(rows) == 3
    for c0, c1, c2, c3, k0, k1, *want in rows:
        got = [int(v) for v in P.philox4x32_10(c0, c1, c2, c3, k0, k1)]
        assert got == want


def test_philox_vectorised_matches_scalar_rounds():
    """Array evaluation equals per-element evaluation (no cross-lane mixing)."""
    rng = np.random.default_rng(7)
    c = rng.integers(0, 2**32, size=(4, 50), dtype=np.uint64)
    k0, k1 = 0x12345678, 0x9ABCDEF0
    vec = P.philox4x32_10(c[0], c[1], c[2], c[3], k0, k1)
    for j in range(50):
        one = P.philox4x32_10(int(c[0, j]), int(c[1, j]), int(c[2, j]), int(c[3, j]), k0, k1)
        assert [int(v[j]) for v in vec] == [int(v) for v in one]


def _uv(x, y):
    u = (2.0 * (x.astype(np.float64) // 512) + 1.0) * 2.0 ** -24
    v = (y.astype(np.float64) // 256) * 2.0 ** -24
    return u, v


EDGE_X = np.array([0, 1, 511, 512, 0x7FFFFFFF, 0x80000000, 0xFFFFFE00, 0xFFFFFFFF], dtype=np.uint32)
EDGE_Y = np.array([0, 0xFF, 0x20000000, 0x3FFFFF00, 0x40000000, 0x80000000, 0xC0000000, 0xFFFFFFFF],
                  dtype=np.uint32)


def test_log_and_sincos_against_libm():
    """The binary32 polynomials reproduce ln, cos, sin (libm, float64) to a few binary32 ulp
    over a dense random grid plus the edge words (u = 2^-24, u -> 1, quadrant boundaries)."""
    rng = np.random.default_rng(11)
    x = np.concatenate([rng.integers(0, 2**32, 400_000, dtype=np.uint64).astype(np.uint32), EDGE_X])
    y = np.concatenate([rng.integers(0, 2**32, 400_000, dtype=np.uint64).astype(np.uint32), EDGE_Y])
    u, v = _uv(x, y)
    L = P._ln_uniform(x).astype(np.float64)
    assert np.all(np.abs(L - np.log(u)) <= 3e-7 * np.abs(np.log(u)) + 1e-12)
    c, s = P._sincos_turn(y)
    assert np.max(np.abs(c - np.cos(2 * np.pi * v))) <= 2e-7
    assert np.max(np.abs(s - np.sin(2 * np.pi * v))) <= 2e-7
    z0, z1 = P.gaussian_pair(x, y)
    rho = np.sqrt(-2.0 * np.log(u))
    assert np.max(np.abs(z0 - rho * np.cos(2 * np.pi * v))) <= 1e-6
    assert np.max(np.abs(z1 - rho * np.sin(2 * np.pi * v))) <= 1e-6
    # exact special points: v = 0 gives (rho, +0); quarter turn gives (0, rho) up to sign of zero
    z0, z1 = P.gaussian_pair(np.array([0x80000000], np.uint32), np.array([0], np.uint32))
    assert z1[0] == 0.0 and z0[0] > 0
    z0, z1 = P.gaussian_pair(np.array([0x80000000], np.uint32), np.array([0x40000000], np.uint32))
    assert z0[0] == 0.0 and z1[0] > 0


def test_omega_is_standard_normal():
    """Omega entries are N(0, 1): moments and a KS test on 2.2e6 draws."""
    from scipy import stats

    om = P.omega(110, 0, 20_000, 0x5C15)
    assert om.shape == (110, 20_000)
    z = om.ravel()
    assert abs(z.mean()) < 5 * 1 / math.sqrt(z.size)
    assert abs(z.var() - 1.0) < 5 * math.sqrt(2 / z.size)
    assert abs(stats.skew(z)) < 0.01 and abs(stats.kurtosis(z)) < 0.02
    assert stats.kstest(z, "norm").pvalue > 1e-3
    # rows (different counters c1) are uncorrelated
    cc = np.corrcoef(om[:8])
    assert np.max(np.abs(cc - np.eye(8))) < 5 / math.sqrt(om.shape[1])


def test_omega_is_partition_invariant():
    """Omega is keyed by global row index j: any column block equals the slice of the whole
    (1-D block-column distribution of Omega), incl. blocks not aligned to 4."""
    full = P.omega(13, 0, 1001, 99)
    for j0, j1 in [(0, 1), (3, 4), (5, 17), (400, 1001), (998, 1001), (7, 7)]:
        np.testing.assert_array_equal(P.omega(13, j0, j1, 99), full[:, j0:j1])
    # the 64-bit counter split: j >= 2^34 uses c3
    hi = P.omega(2, 2**34, 2**34 + 8, 99)
    lo = P.omega(2, 0, 8, 99)
    assert not np.array_equal(hi, lo)


def test_omega_seed_and_tag_change_stream():
    a = P.omega(4, 0, 64, 1)
    assert not np.array_equal(a, P.omega(4, 0, 64, 2))
    assert not np.array_equal(a, P.omega(4, 0, 64, 1, tag=1))
    assert not np.array_equal(a, P.omega(4, 0, 64, 1 + (1 << 32)))


def test_omega_golden_regression(golden_dir):
    """First values of Omega for the default seed, frozen by scripts/make_golden.py
    (which calls only oracle/)."""
    path = os.path.join(golden_dir, "omega_seed5C15_4x16.txt")
    want = np.loadtxt(path)
    got = P.omega(4, 0, 16, 0x5C15)
    np.testing.assert_array_equal(got, want)


def test_omega_row_subset_equals_full_rows():
    """omega(..., rows=R) generates only the rows R of the same Omega (per-entry counters)."""
    from oracle.philox import omega

    full = omega(40, 3, 700, 0x5C15)
    np.testing.assert_array_equal(omega(40, 3, 700, 0x5C15, rows=[39, 0, 17]), full[[39, 0, 17]])
