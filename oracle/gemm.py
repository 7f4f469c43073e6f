"""Oracle matrix product: the definition C[i, j] = sum_k A[i, k] B[k, j] with a fixed summation
order (every output accumulates its terms one at a time in increasing k, product rounded then sum
rounded, no FMA) -- SURVEY.md §8(c) c-1 step 2, the north star's "its own naive GEMM".

TEST INFRASTRUCTURE ONLY (see oracle/__init__.py).  The arithmetic is the plain C loop nest in
``oracle/csrc/gemm.c`` (OpenMP over output tiles only, so the result does not depend on the thread
count).  It shares no code with the CUDA path.  Pinned by tests/test_oracle_gemm.py: exact on
small-integer inputs, the per-output summation order checked against a pure-Python loop, thread- and
layout-invariance, and (test-only) agreement with numpy's BLAS ``@`` to rounding.
"""

from __future__ import annotations

import ctypes
import hashlib
import os
import subprocess
import threading

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SRC = os.path.join(_HERE, "csrc", "gemm.c")
_LIBDIR = os.path.join(_HERE, "lib")
_LIB = os.path.join(_LIBDIR, "liboracle_gemm.so")
_STAMP = _LIB + ".stamp"
_lock = threading.Lock()
_lib = None


def _cpu_flags() -> str:
    try:
        with open("/proc/cpuinfo") as fh:
            for line in fh:
                if line.startswith("flags"):
                    return line
    except OSError:
        pass
    return ""


def _digest() -> str:
    h = hashlib.sha256()
    with open(_SRC, "rb") as fh:
        h.update(fh.read())
    h.update(_cpu_flags().encode())  # -march=native: rebuilt on a host with other ISA extensions
    return h.hexdigest()


def build(force: bool = False) -> str:
    """Compile oracle/csrc/gemm.c into oracle/lib/liboracle_gemm.so (gcc, OpenMP)."""
    digest = _digest()
    if not force and os.path.exists(_LIB) and os.path.exists(_STAMP) and open(_STAMP).read() == digest:
        return _LIB
    os.makedirs(_LIBDIR, exist_ok=True)
    tmp = f"{_LIB}.{os.getpid()}.tmp"
    cmd = ["gcc", "-O3", "-march=native", "-ffp-contract=off", "-fno-fast-math", "-fopenmp", "-shared", "-fPIC",
           _SRC, "-o", tmp]
    r = subprocess.run(cmd, capture_output=True, text=True)
    if r.returncode != 0:
        raise RuntimeError(f"oracle gemm build failed:\n{r.stderr}")
    os.replace(tmp, _LIB)
    with open(_STAMP + f".{os.getpid()}", "w") as fh:
        fh.write(digest)
    os.replace(_STAMP + f".{os.getpid()}", _STAMP)
    return _LIB


def _load():
    global _lib
    with _lock:
        if _lib is None:
            lib = ctypes.CDLL(build())
            i64, p = ctypes.c_int64, ctypes.c_void_p
            lib.oracle_gemm.argtypes = [i64, i64, i64, p, i64, i64, p, i64, p, i64, ctypes.c_int]
            lib.oracle_gemm.restype = None
            _lib = lib
    return _lib


def default_threads() -> int:
    v = os.environ.get("RS_ORACLE_THREADS")
    return int(v) if v else (os.cpu_count() or 1)


def _unit_cols(X: np.ndarray) -> bool:
    """X[k, j] at X[k*ld + j] for some ld >= 0 (elements, not bytes)."""
    return X.shape[1] <= 1 or X.strides[1] == 8 and X.strides[0] % 8 == 0 and X.strides[0] >= 0


def _strided(X: np.ndarray) -> bool:
    return all(s % 8 == 0 and s >= 0 for s in X.strides)


def matmul(X, Y, nthreads: int | None = None) -> np.ndarray:
    """X @ Y (float64) in the oracle's fixed order.  1-D operands follow numpy's rules."""
    X = np.asarray(X, dtype=np.float64)
    Y = np.asarray(Y, dtype=np.float64)
    xv, yv = X.ndim == 1, Y.ndim == 1
    X2 = X[None, :] if xv else X
    Y2 = Y[:, None] if yv else Y
    M, K = X2.shape
    K2, N = Y2.shape
    if K != K2:
        raise ValueError(f"shape mismatch {X.shape} @ {Y.shape}")
    nt = default_threads() if nthreads is None else nthreads
    lib = _load()
    if M == 0 or N == 0 or K == 0:  # empty sum = +0.0
        C = np.zeros((M, N))
    elif not _strided(X2) or not _strided(Y2):
        return matmul(np.ascontiguousarray(X), np.ascontiguousarray(Y), nthreads)
    elif _unit_cols(Y2):  # C = X Y: X is the scalar operand, Y rows are vectors
        C = np.empty((M, N))
        lib.oracle_gemm(M, N, K, X2.ctypes.data, X2.strides[0] // 8, X2.strides[1] // 8, Y2.ctypes.data,
                        Y2.strides[0] // 8 if K > 1 else 0, C.ctypes.data, N, nt)
    elif _unit_cols(X2.T):  # C^T = Y^T X^T: X^T rows (columns of X) are contiguous
        Ct = np.empty((N, M))
        Xt, Yt = X2.T, Y2.T
        lib.oracle_gemm(N, M, K, Yt.ctypes.data, Yt.strides[0] // 8, Yt.strides[1] // 8, Xt.ctypes.data,
                        Xt.strides[0] // 8 if K > 1 else 0, Ct.ctypes.data, M, nt)
        C = Ct.T
    else:  # neither operand has a unit-stride output dimension: copy the smaller one
        if Y2.size <= X2.size:
            return matmul(X, np.ascontiguousarray(Y), nthreads)
        return matmul(np.asfortranarray(X), Y, nthreads)
    if xv and yv:
        return np.float64(C[0, 0])
    if xv:
        return np.ascontiguousarray(C[0])
    if yv:
        return np.ascontiguousarray(C[:, 0])
    return np.ascontiguousarray(C)
