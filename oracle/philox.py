"""Oracle: the Gaussian sampling matrix Omega = PRNG(l, m) (Fig. 2(b) line 2).

TEST INFRASTRUCTURE ONLY (see oracle/__init__.py).

Paper: "we used NVIDIA's cuRAND library to generate a Gaussian matrix Omega
(matrix whose entries follow the standard normal distribution N(0,1) ...)"
(Sec. 4).  The paper is silent on the generator, the seed and the
normal transform; DESIGN.md §3 fixes them (reading R1):

* Philox4x32-10 (Salmon et al., Random123) with the published multipliers and
  Weyl constants, 10 rounds, key bumped before rounds 2..10.  Pinned by the
  Random123 known-answer vectors (tests/golden/philox_kat.txt).
* Counter for Omega[i, j] (i < l the sample row, j < m_global the GLOBAL row
  of A): (c0, c1, c2, c3) = (floor(j/4) mod 2^32, i, tag, floor(j/4) >> 32);
  key = (seed mod 2^32, seed >> 32).  Output words (x0, x1) -> Omega[i, 4t],
  Omega[i, 4t+1]; (x2, x3) -> Omega[i, 4t+2], Omega[i, 4t+3].
* RS-BM32: a Box-Muller transform written only with IEEE-754 binary32
  correctly-rounded +, -, *, /, sqrt (no fused multiply-add, no library
  transcendental), so that any conforming implementation reproduces it bit for
  bit.  The result is widened exactly to binary64.

Everything here is plain numpy on uint32/uint64/float32 arrays, evaluated in
exactly the order DESIGN.md §3 writes down.
"""

from __future__ import annotations

import math

import numpy as np

# Random123 Philox4x32 constants (Salmon, Moraes, Dror, Shaw, SC11).
PHILOX_M0 = np.uint64(0xD2511F53)
PHILOX_M1 = np.uint64(0xCD9E8D57)
PHILOX_W0 = 0x9E3779B9
PHILOX_W1 = 0xBB67AE85
MASK32 = np.uint64(0xFFFFFFFF)


def philox4x32_10(c0, c1, c2, c3, k0: int, k1: int):
    """Philox4x32 with 10 rounds on arrays of 32-bit counters.

    One round: (hi0, lo0) = M0*c0, (hi1, lo1) = M1*c2 (32x32 -> 64 products);
    c' = (hi1 ^ c1 ^ k0, lo1, hi0 ^ c3 ^ k1, lo0).  Key bump between rounds:
    k0 += W0, k1 += W1 (mod 2^32).  Returns four uint32 arrays.
    """
    x0 = np.asarray(c0, dtype=np.uint64) & MASK32
    x1 = np.asarray(c1, dtype=np.uint64) & MASK32
    x2 = np.asarray(c2, dtype=np.uint64) & MASK32
    x3 = np.asarray(c3, dtype=np.uint64) & MASK32
    x0, x1, x2, x3 = np.broadcast_arrays(x0, x1, x2, x3)
    ka, kb = k0 & 0xFFFFFFFF, k1 & 0xFFFFFFFF
    for r in range(10):
        if r > 0:
            ka = (ka + PHILOX_W0) & 0xFFFFFFFF
            kb = (kb + PHILOX_W1) & 0xFFFFFFFF
        p0 = PHILOX_M0 * x0            # exact: < 2^64
        p1 = PHILOX_M1 * x2
        hi0, lo0 = p0 >> np.uint64(32), p0 & MASK32
        hi1, lo1 = p1 >> np.uint64(32), p1 & MASK32
        x0, x1, x2, x3 = (hi1 ^ x1 ^ np.uint64(ka), lo1,
                          hi0 ^ x3 ^ np.uint64(kb), lo0)
    return tuple(a.astype(np.uint32) for a in (x0, x1, x2, x3))


# ---- RS-BM32 constants, each written as its mathematical definition --------
# (the CUDA side types its own copies; a bit-exact GPU test compares them)
F32 = np.float32
_SQRT2 = F32(math.sqrt(2.0))
_LN2_HI = F32(0.693145751953125)                 # 0x3F317200: few bits, exact products
_LN2_LO = F32(math.log(2.0) - 0.693145751953125)
# 2*atanh(s) = 2s + s^3 * (2/3 + s^2*(2/5 + s^2*(2/7 + s^2*(2/9 + s^2*2/11))))
_LOG_C = [F32(2.0 / d) for d in (3, 5, 7, 9, 11)]
# sin(pi/2 x) = x * sum_{n odd <= 9} s_n x^(n-1),  s_n = (-1)^((n-1)/2) (pi/2)^n / n!
_SIN_C = [F32((-1) ** ((n - 1) // 2) * (math.pi / 2) ** n / math.factorial(n)) for n in (1, 3, 5, 7, 9)]
# cos(pi/2 x) = 1 + sum_{2 <= n even <= 10} c_n x^n,  c_n = (-1)^(n/2) (pi/2)^n / n!
_COS_C = [F32((-1) ** (n // 2) * (math.pi / 2) ** n / math.factorial(n)) for n in (2, 4, 6, 8, 10)]


def _ln_uniform(x):
    """ln(u) for u = (2*(x>>9)+1) * 2^-24, in binary32 (DESIGN.md §3 step 1-2)."""
    a = (x.astype(np.uint32) >> np.uint32(9)).astype(np.int64)
    v = 2 * a + 1                                   # odd integer in [1, 2^24)
    _, ex = np.frexp(v.astype(np.float64))          # v = mant * 2^ex, mant in [1/2, 1): exact
    e = ex.astype(np.int64) - 1                     # 2^e <= v < 2^(e+1)
    f = (v.astype(F32) * np.ldexp(np.ones(e.shape), -e).astype(F32)).astype(F32)  # v*2^-e in [1,2): exact
    big = f >= _SQRT2
    f = np.where(big, f * F32(0.5), f).astype(F32)  # exact
    e = np.where(big, e + 1, e)
    E = (e - 24).astype(F32)                        # u = 2^(e-24) * f, f in [sqrt2/2, sqrt2)
    s = ((f - F32(1.0)) / (f + F32(1.0))).astype(F32)
    s2 = (s * s).astype(F32)
    t = _LOG_C[4]
    for c in (_LOG_C[3], _LOG_C[2], _LOG_C[1], _LOG_C[0]):
        t = ((t * s2).astype(F32) + c).astype(F32)
    r = ((s * s2).astype(F32) * t).astype(F32)
    lnf = ((s + s).astype(F32) + r).astype(F32)
    L = ((E * _LN2_HI).astype(F32) + ((E * _LN2_LO).astype(F32) + lnf).astype(F32)).astype(F32)
    return L


def _sincos_turn(y):
    """(cos 2*pi*v, sin 2*pi*v) for v = (y>>8) * 2^-24, binary32 (DESIGN.md §3 step 3)."""
    b = y.astype(np.uint32) >> np.uint32(8)
    quad = (b >> np.uint32(22)).astype(np.int64)
    r = (b & np.uint32(0x3FFFFF)).astype(np.int64)
    flip = r > (1 << 21)                             # angle > pi/4 in the quadrant
    rr = np.where(flip, (1 << 22) - r, r)
    x = (rr.astype(F32) * F32(2.0 ** -22)).astype(F32)  # exact, x in [0, 1/2]
    x2 = (x * x).astype(F32)
    ps = _SIN_C[4]
    for c in (_SIN_C[3], _SIN_C[2], _SIN_C[1], _SIN_C[0]):
        ps = ((ps * x2).astype(F32) + c).astype(F32)
    S = (x * ps).astype(F32)
    pc = _COS_C[4]
    for c in (_COS_C[3], _COS_C[2], _COS_C[1], _COS_C[0]):
        pc = ((pc * x2).astype(F32) + c).astype(F32)
    C = ((pc * x2).astype(F32) + F32(1.0)).astype(F32)
    cq = np.where(flip, S, C).astype(F32)           # cos of the in-quadrant angle
    sq = np.where(flip, C, S).astype(F32)
    cos_t = np.select([quad == 0, quad == 1, quad == 2], [cq, -sq, -cq], sq).astype(F32)
    sin_t = np.select([quad == 0, quad == 1, quad == 2], [sq, cq, -sq], -cq).astype(F32)
    return cos_t, sin_t


def gaussian_pair(x, y):
    """RS-BM32: two N(0,1) binary32 values from two uint32 words (radius from x, angle from y)."""
    L = _ln_uniform(np.asarray(x, dtype=np.uint32))
    w = (-(L + L)).astype(F32)                       # -2 ln u >= 0
    rho = np.sqrt(w).astype(F32)                     # IEEE sqrt
    c, s = _sincos_turn(np.asarray(y, dtype=np.uint32))
    return (rho * c).astype(F32), (rho * s).astype(F32)


def omega(ell: int, j0: int, j1: int, seed: int, tag: int = 0, rows=None) -> np.ndarray:
    """Omega[:, j0:j1] (l x (j1-j0), float64): the Gaussian sampling matrix of
    Step 1, B = Omega A (Fig. 2(b) line 2), columns indexed
    by GLOBAL row j of A so every row-block partition sees the same Omega
    (1-D block-column layout of Omega).  ``rows`` (optional) selects
    the Omega rows to generate (default 0..l-1): each entry depends only on its
    own (row, column) counter."""
    nrow = ell if rows is None else len(rows)
    if j1 <= j0:
        return np.zeros((nrow, 0))
    t0, t1 = j0 // 4, (j1 + 3) // 4
    t = np.arange(t0, t1, dtype=np.uint64)[None, :]
    i = (np.arange(ell, dtype=np.uint64) if rows is None else np.asarray(rows, dtype=np.uint64))[:, None]
    x0, x1, x2, x3 = philox4x32_10(t & MASK32, i, np.uint64(tag), t >> np.uint64(32),
                                   seed & 0xFFFFFFFF, (seed >> 32) & 0xFFFFFFFF)
    z0, z1 = gaussian_pair(x0, x1)
    z2, z3 = gaussian_pair(x2, x3)
    full = np.stack([z0, z1, z2, z3], axis=-1).reshape(nrow, -1).astype(np.float64)
    return full[:, j0 - 4 * t0: j1 - 4 * t0]
