"""Pins of the oracle's own fixed-order GEMM (oracle/gemm.py, oracle/csrc/gemm.c; SURVEY §8(c)
c-1 step 2: "a triple loop with one level of cache blocking over K; each output accumulated
sequentially in increasing K, so the sum order is defined and identical for any thread count")."""

import numpy as np
import pytest

from oracle.gemm import matmul


def _int_mat(rng, shape, lo=-8, hi=8):
    return rng.integers(lo, hi + 1, size=shape).astype(np.float64)


@pytest.mark.parametrize("M,N,K", [(1, 1, 1), (3, 7, 5), (130, 300, 260), (5, 513, 129), (110, 40, 1000)])
def test_exact_on_small_integers(M, N, K):
    """Every product and partial sum is an integer < 2^53: the result is exact in any order, so it
    must equal integer arithmetic bit for bit (catches a dropped term, a wrong index, a transposed
    operand, a tile edge)."""
    rng = np.random.default_rng(M * 1000 + N + K)
    X, Y = _int_mat(rng, (M, K)), _int_mat(rng, (K, N))
    ref = (X.astype(np.int64) @ Y.astype(np.int64)).astype(np.float64)
    assert np.array_equal(matmul(X, Y), ref)
    assert np.array_equal(matmul(np.asfortranarray(X), np.asfortranarray(Y)), ref)
    assert np.array_equal(matmul(Y.T, X.T), ref.T)


def test_summation_order_is_increasing_k():
    """c <- c + a_k b_k for k = 0, 1, ... (product rounded, then sum rounded, no FMA): a column
    where the order decides the result, and random data, both equal to a scalar Python loop."""
    X = np.array([[1.0, 1.0, 1.0, 1.0]])
    Y = np.array([[1e16], [1.0], [-1e16], [1.0]])
    # increasing k: ((1e16 + 1) - 1e16) + 1 = 0 + 1 = 1 (1e16 + 1 rounds back to 1e16)
    assert matmul(X, Y)[0, 0] == 1.0
    # decreasing k: ((1 - 1e16) + 1) + 1e16 = (-1e16 + 1) + 1e16 = -1e16 + 1e16 = 0 (each +1 rounds away)
    assert matmul(X[:, ::-1].copy(), Y[::-1].copy())[0, 0] == 0.0
    # FMA would keep a*b unrounded: a*b = 1 + 2^-30 + 2^-60 rounds to 1 + 2^-30, the sum with
    # -(1 + 2^-30) is then exactly 0; an FMA gives 2^-60
    a = 1.0 + 2.0 ** -30
    X = np.array([[1.0, a]])
    Y = np.array([[-(1.0 + 2.0 ** -29)], [a]])
    assert matmul(X, Y)[0, 0] == (1.0 * -(1.0 + 2.0 ** -29)) + (a * a)
    rng = np.random.default_rng(3)
    for (M, N, K) in [(2, 300, 270), (131, 3, 140)]:
        X, Y = rng.standard_normal((M, K)), rng.standard_normal((K, N))
        C = matmul(X, Y)
        for i in range(M):
            for j in range(N):
                c = 0.0
                for k in range(K):
                    c = c + float(X[i, k]) * float(Y[k, j])
                assert C[i, j] == c


def test_thread_count_and_layout_invariance():
    rng = np.random.default_rng(11)
    X, Y = rng.standard_normal((150, 700)), rng.standard_normal((700, 530))
    C1 = matmul(X, Y, nthreads=1)
    for nt in (2, 5, 8):
        assert np.array_equal(matmul(X, Y, nthreads=nt), C1)
    assert np.array_equal(matmul(np.asfortranarray(X), Y), C1)
    assert np.array_equal(matmul(X, np.asfortranarray(Y)), C1)
    Xb = np.zeros((150, 1400))
    Xb[:, ::2] = X
    assert np.array_equal(matmul(Xb[:, ::2], Y), C1)          # strided view


def test_vector_semantics_and_empty():
    rng = np.random.default_rng(5)
    X, v = rng.standard_normal((9, 6)), rng.standard_normal(6)
    assert matmul(X, v).shape == (9,) and matmul(v[:6], X.T).shape == (9,)
    assert np.isclose(matmul(v, v), float(np.sum(v * v)), rtol=1e-15)
    assert matmul(np.zeros((0, 4)), np.zeros((4, 3))).shape == (0, 3)
    assert np.array_equal(matmul(np.zeros((2, 0)), np.zeros((0, 3))), np.zeros((2, 3)))


def test_agrees_with_blas_to_rounding():
    """Test-only cross-check against numpy's BLAS product (another summation order)."""
    rng = np.random.default_rng(7)
    X, Y = rng.standard_normal((110, 3000)), rng.standard_normal((3000, 400))
    C = matmul(X, Y)
    ref = X @ Y
    scale = np.abs(X) @ np.abs(Y)
    assert float(np.max(np.abs(C - ref) / scale)) <= 3000 * 2.0 ** -53
    assert float(np.linalg.norm(C - ref) / np.linalg.norm(ref)) <= 1e-14
