"""Thin Python binding of the C ABI in ``include/rs_lowrank.h`` (argument marshalling only).

Every step of the path runs in the CUDA library ``lib/librs_lowrank.so``; this module only
converts torch tensors to (pointer, leading dimension) pairs, checks layouts and maps status codes
to exceptions.  There is no CPU fallback: if the library is missing, importing a function that
needs it raises.

Matrices are column-major: an m x n matrix is a torch tensor of shape (m, n) with strides
(1, ld), ld >= m and even (use :func:`empty_colmajor`).
"""

from __future__ import annotations

import ctypes
import os
from dataclasses import dataclass

import torch

_PKG = os.path.dirname(os.path.abspath(__file__))
LIB_PATH = os.path.join(_PKG, "lib", "librs_lowrank.so")

STATUS = {0: "RS_OK", 1: "RS_ERR_INVALID_ARG", 2: "RS_ERR_BAD_STATE", 3: "RS_ERR_CUDA", 4: "RS_ERR_NCCL",
          5: "RS_ERR_NOT_SPD", 6: "RS_ERR_RANK_DEFICIENT", 7: "RS_ERR_WORKSPACE", 8: "RS_ERR_UNSUPPORTED",
          9: "RS_ERR_NOT_CONVERGED"}

ABI_FUNCTIONS = (
    "rs_lowrank_workspace_bytes", "rs_lowrank_create", "rs_lowrank_sample", "rs_lowrank_power_iterate",
    "rs_lowrank_pivot", "rs_lowrank_factor", "rs_lowrank_run", "rs_lowrank_run_host", "rs_lowrank_sample_adaptive",
    "rs_lowrank_destroy",
    "rs_lowrank_get_sample", "rs_lowrank_set_sample", "rs_lowrank_get_pivot_data", "rs_lowrank_omega",
    "rs_lowrank_get_info", "rs_lowrank_get_fallbacks", "rs_lowrank_set_profiling", "rs_lowrank_get_profile", "rs_lowrank_reset_profile",
    "rs_lowrank_kernel_launches", "rs_qp3_workspace_bytes", "rs_qp3_truncated", "rs_lowrank_sample_columns",
    "rs_lowrank_last_error", "rs_lowrank_set_allreduce_hook", "rs_comm_get_unique_id", "rs_comm_init", "rs_comm_destroy",
    "rs_comm_info",
)


# rs_allreduce_fn: int (*)(void* ctx, double* buf, int64_t count, void* cuda_stream)
ALLREDUCE_FN = ctypes.CFUNCTYPE(ctypes.c_int, ctypes.c_void_p, ctypes.c_void_p, ctypes.c_int64, ctypes.c_void_p)


class RSError(RuntimeError):
    def __init__(self, code: int, msg: str):
        super().__init__(f"{STATUS.get(code, code)}: {msg}")
        self.code = code
        self.name = STATUS.get(code, str(code))


_lib = None


def load_library(path: str = LIB_PATH):
    """Load (once) the CUDA library; raises if it is missing -- no fallback."""
    global _lib
    if _lib is not None:
        return _lib
    if not os.path.exists(path):
        raise RuntimeError(f"CUDA library {path} is missing: run `python -m paper_conf_sc_maryykltd15_b200.build` "
                           "(or __graft_entry__.build()); there is no CPU fallback")
    lib = ctypes.CDLL(path)
    P, I64, I32, U64, SZ = ctypes.c_void_p, ctypes.c_int64, ctypes.c_int32, ctypes.c_uint64, ctypes.c_size_t
    D = ctypes.POINTER(ctypes.c_double)
    sig = {
        "rs_lowrank_workspace_bytes": (SZ, [I64, I64, I32, I32, I32]),
        "rs_lowrank_create": (ctypes.c_int, [ctypes.POINTER(P), I64, I64, I64, I64, I32, I32, U64, P, SZ, P, P]),
        "rs_lowrank_sample": (ctypes.c_int, [P, P, I64]),
        "rs_lowrank_power_iterate": (ctypes.c_int, [P, P, I64, I32]),
        "rs_lowrank_pivot": (ctypes.c_int, [P, P]),
        "rs_lowrank_factor": (ctypes.c_int, [P, P, I64, P, I64, P, I64]),
        "rs_lowrank_run": (ctypes.c_int, [P, P, I64, I32, P, P, I64, P, I64]),
        "rs_lowrank_run_host": (ctypes.c_int, [P, P, I64, P, I64, I32, P, P, I64, P, I64, P, I64, P, I64]),
        "rs_lowrank_sample_adaptive": (ctypes.c_int, [P, P, I64, ctypes.c_double, I32, I32, I32, ctypes.POINTER(I32),
                                                      D, D, I32]),
        "rs_lowrank_destroy": (ctypes.c_int, [P]),
        "rs_lowrank_get_sample": (ctypes.c_int, [P, P, I64]),
        "rs_lowrank_set_sample": (ctypes.c_int, [P, P, I64]),
        "rs_lowrank_get_pivot_data": (ctypes.c_int, [P, P, I64, P, I64, D]),
        "rs_lowrank_omega": (ctypes.c_int, [P, I64, I64, P, I64]),
        "rs_lowrank_get_info": (ctypes.c_int, [P, ctypes.POINTER(I64)]),
        "rs_lowrank_get_fallbacks": (ctypes.c_int, [P, ctypes.POINTER(I32)]),
        "rs_lowrank_set_profiling": (ctypes.c_int, [P, I32]),
        "rs_lowrank_get_profile": (ctypes.c_int, [P, ctypes.c_char_p, D, ctypes.POINTER(I64), D]),
        "rs_lowrank_reset_profile": (ctypes.c_int, [P]),
        "rs_lowrank_kernel_launches": (I64, []),
        "rs_lowrank_set_allreduce_hook": (ctypes.c_int, [P, I32, I32, ALLREDUCE_FN, P]),
        "rs_qp3_workspace_bytes": (SZ, [I64, I64, I32]),
        "rs_lowrank_sample_columns": (ctypes.c_int, [P, P, I64, P, I64]),
        "rs_qp3_truncated": (ctypes.c_int, [I64, I64, I32, P, I64, P, P, D, P, SZ, P]),
        "rs_lowrank_last_error": (ctypes.c_char_p, [P]),
        "rs_comm_get_unique_id": (ctypes.c_int, [ctypes.c_char_p]),
        "rs_comm_init": (ctypes.c_int, [ctypes.POINTER(P), I32, ctypes.c_char_p, I32]),
        "rs_comm_destroy": (ctypes.c_int, [P]),
        "rs_comm_info": (ctypes.c_int, [P, ctypes.POINTER(I32), ctypes.POINTER(I32)]),
    }
    for name, (res, args) in sig.items():
        fn = getattr(lib, name)
        fn.restype = res
        fn.argtypes = args
    _lib = lib
    return lib


# ---------------------------------------------------------------------------------------------
# layout helpers
# ---------------------------------------------------------------------------------------------
def empty_colmajor(m: int, n: int, device="cuda", dtype=torch.float64, ld: int | None = None, pin: bool = False):
    """Uninitialised m x n column-major tensor (strides (1, ld)), ld >= m rounded up to even."""
    ld = max(m, 1) if ld is None else ld
    ld += ld & 1
    if device == "cpu" or (isinstance(device, torch.device) and device.type == "cpu"):
        store = torch.empty((n, ld), dtype=dtype, pin_memory=pin)
    else:
        store = torch.empty((n, ld), dtype=dtype, device=device)
    return store[:, :m].t()


def colmajor_ld(t: torch.Tensor, name: str = "matrix") -> int:
    if t.dim() != 2:
        raise ValueError(f"{name} must be 2-D")
    if t.dtype != torch.float64:
        raise ValueError(f"{name} must be float64 (the paper's precision, P:L666-667)")
    m, n = t.shape
    if n > 1 and t.stride(0) != 1:
        raise ValueError(f"{name} must be column-major (stride(0) == 1), got strides {t.stride()}")
    ld = t.stride(1) if n > 1 else max(m, 1)
    return ld


def _check(code: int, h=None):
    if code != 0:
        msg = load_library().rs_lowrank_last_error(h).decode() if h else ""
        raise RSError(code, msg)


def _stream_ptr(stream) -> int:
    if stream is None:
        stream = torch.cuda.current_stream()
    return stream.cuda_stream


# ---------------------------------------------------------------------------------------------
# ABI-named functions
# ---------------------------------------------------------------------------------------------
def workspace_bytes(m_local: int, n: int, k: int, p: int, nranks: int = 1) -> int:
    return int(load_library().rs_lowrank_workspace_bytes(m_local, n, k, p, nranks))


@dataclass
class Handle:
    ptr: ctypes.c_void_p
    workspace: torch.Tensor
    m_global: int
    m_local: int
    row_offset: int
    n: int
    k: int
    p: int
    seed: int
    stream: torch.cuda.Stream
    adaptive_ell: int = 0  # set by sample_adaptive (then pivot/factor use k = l = adaptive_ell)

    @property
    def ell(self) -> int:
        return self.adaptive_ell or (self.k + self.p)

    @property
    def k_eff(self) -> int:
        return self.adaptive_ell or self.k


def create(m_global: int, m_local: int, row_offset: int, n: int, k: int, p: int, seed: int = 0x5C15, *,
           device=None, stream=None, nccl_comm=None) -> Handle:
    lib = load_library()
    device = torch.device("cuda", torch.cuda.current_device()) if device is None else torch.device(device)
    nbytes = workspace_bytes(m_local, n, k, p)
    if nbytes == 0:
        raise RSError(1, "invalid sizes")
    ws = torch.empty(nbytes, dtype=torch.uint8, device=device)
    stream = torch.cuda.current_stream(device) if stream is None else stream
    h = ctypes.c_void_p()
    code = lib.rs_lowrank_create(ctypes.byref(h), m_global, m_local, row_offset, n, k, p, seed & (2**64 - 1),
                                 ws.data_ptr(), nbytes, stream.cuda_stream, nccl_comm)
    _check(code)
    return Handle(h, ws, m_global, m_local, row_offset, n, k, p, seed, stream)


def sample(h: Handle, A: torch.Tensor):
    _check(load_library().rs_lowrank_sample(h.ptr, A.data_ptr(), colmajor_ld(A, "A")), h.ptr)
    h.adaptive_ell = 0


def power_iterate(h: Handle, A: torch.Tensor, q: int):
    _check(load_library().rs_lowrank_power_iterate(h.ptr, A.data_ptr(), colmajor_ld(A, "A"), q), h.ptr)


def pivot(h: Handle, perm: torch.Tensor | None = None):
    if perm is not None and (perm.dtype != torch.int64 or not perm.is_cuda):
        raise ValueError("perm must be a CUDA int64 tensor")
    _check(load_library().rs_lowrank_pivot(h.ptr, perm.data_ptr() if perm is not None else None), h.ptr)


def factor(h: Handle, A: torch.Tensor, Q: torch.Tensor, R: torch.Tensor):
    _check(load_library().rs_lowrank_factor(h.ptr, A.data_ptr(), colmajor_ld(A, "A"), Q.data_ptr(),
                                            colmajor_ld(Q, "Q"), R.data_ptr(), colmajor_ld(R, "R")), h.ptr)


def run(h: Handle, A: torch.Tensor, q: int, perm: torch.Tensor | None, Q: torch.Tensor, R: torch.Tensor):
    """The whole step (rs_lowrank_run): sample -> power_iterate(q) -> pivot -> factor, replayed as one
    CUDA graph after the first call with the same buffers."""
    if perm is not None and (perm.dtype != torch.int64 or not perm.is_cuda):
        raise ValueError("perm must be a CUDA int64 tensor")
    _check(load_library().rs_lowrank_run(h.ptr, A.data_ptr(), colmajor_ld(A, "A"), q,
                                         perm.data_ptr() if perm is not None else None, Q.data_ptr(),
                                         colmajor_ld(Q, "Q"), R.data_ptr(), colmajor_ld(R, "R")), h.ptr)
    h.adaptive_ell = 0


def run_host(h: Handle, A_host: torch.Tensor, A_dev: torch.Tensor, q: int, perm_host: torch.Tensor,
             Q_host: torch.Tensor, R_host: torch.Tensor, Q_dev: torch.Tensor, R_dev: torch.Tensor):
    _check(load_library().rs_lowrank_run_host(
        h.ptr, A_host.data_ptr(), colmajor_ld(A_host, "A_host"), A_dev.data_ptr(), colmajor_ld(A_dev, "A_dev"), q,
        perm_host.data_ptr(), Q_host.data_ptr(), colmajor_ld(Q_host, "Q_host"), R_host.data_ptr(),
        colmajor_ld(R_host, "R_host"), Q_dev.data_ptr(), colmajor_ld(Q_dev, "Q_dev"), R_dev.data_ptr(),
        colmajor_ld(R_dev, "R_dev")), h.ptr)


INC_POLICIES = {"static": 0, "interp": 1}


def sample_adaptive(h: Handle, A: torch.Tensor, eps: float, ell_inc: int, q: int = 0, *, inc_policy="static",
                    raise_on_max=True):
    """Fig. 3 adaptive sampling; returns (l, eps~, [(l, eps~) per round]).  The handle must have
    been created with k = l_max and p = 0.  inc_policy: "static" or "interp"."""
    ell = ctypes.c_int32()
    est = ctypes.c_double()
    hist = (ctypes.c_double * 2048)()
    code = load_library().rs_lowrank_sample_adaptive(h.ptr, A.data_ptr(), colmajor_ld(A, "A"), eps, ell_inc, q,
                                                     INC_POLICIES[inc_policy], ctypes.byref(ell),
                                                     ctypes.byref(est), hist, 1024)
    rounds = []
    for r in range(1024):
        if hist[2 * r] == 0:
            break
        rounds.append((int(hist[2 * r]), hist[2 * r + 1]))
    if code in (0, 9):
        h.adaptive_ell = int(ell.value)
    if code == 9 and not raise_on_max:
        return int(ell.value), est.value, rounds
    _check(code, h.ptr)
    return int(ell.value), est.value, rounds


def sample_columns(h: Handle, A: torch.Tensor, Bc: torch.Tensor | None = None) -> torch.Tensor:
    """Column sampling B_c = Omega_c A^T (l x m_local, Fig. 8(b)); returns B_c."""
    if Bc is None:
        Bc = empty_colmajor(h.k + h.p, h.m_local, device=h.workspace.device)
    _check(load_library().rs_lowrank_sample_columns(h.ptr, A.data_ptr(), colmajor_ld(A, "A"), Bc.data_ptr(),
                                                    colmajor_ld(Bc, "B_c")), h.ptr)
    return Bc


def destroy(h: Handle):
    if h.ptr:
        _check(load_library().rs_lowrank_destroy(h.ptr))
        h.ptr = ctypes.c_void_p()


def get_sample(h: Handle) -> torch.Tensor:
    B = empty_colmajor(h.ell, h.n, device=h.workspace.device)
    _check(load_library().rs_lowrank_get_sample(h.ptr, B.data_ptr(), colmajor_ld(B)), h.ptr)
    return B


def set_sample(h: Handle, B: torch.Tensor):
    _check(load_library().rs_lowrank_set_sample(h.ptr, B.data_ptr(), colmajor_ld(B, "B")), h.ptr)
    h.adaptive_ell = 0


def get_pivot_data(h: Handle):
    """(T k x (n-k), R̂ k x n in pivot order, gaps[k]) after pivot."""
    dev = h.workspace.device
    k = h.k_eff
    T = empty_colmajor(k, max(h.n - k, 1), device=dev)
    Rh = empty_colmajor(k, h.n, device=dev)
    gaps = (ctypes.c_double * k)()
    _check(load_library().rs_lowrank_get_pivot_data(h.ptr, T.data_ptr(), colmajor_ld(T), Rh.data_ptr(),
                                                    colmajor_ld(Rh), gaps), h.ptr)
    return T[:, : h.n - k], Rh, list(gaps)


def set_allreduce_hook(h: Handle, nranks: int, rank: int, fn) -> None:
    """Route this handle's reductions through `fn(buf_ptr, count, stream_ptr) -> None` instead of
    NCCL (rs_lowrank_set_allreduce_hook).  The ctypes callback is kept alive on the handle."""
    def _cb(ctx, buf, count, stream):
        try:
            fn(int(buf), int(count), int(stream) if stream else 0)
            return 0
        except Exception:  # noqa: BLE001 -- reported to the library as a failed reduction
            import traceback

            traceback.print_exc()
            return 1

    cb = ALLREDUCE_FN(_cb)
    h._ar_cb = cb
    _check(load_library().rs_lowrank_set_allreduce_hook(h.ptr, nranks, rank, cb, None), h.ptr)


def omega(h: Handle, j0: int, ncols: int) -> torch.Tensor:
    out = empty_colmajor(h.ell, max(ncols, 1), device=h.workspace.device)
    _check(load_library().rs_lowrank_omega(h.ptr, j0, ncols, out.data_ptr(), colmajor_ld(out)), h.ptr)
    return out[:, :ncols]


def get_info(h: Handle):
    arr = (ctypes.c_int64 * 2)()
    _check(load_library().rs_lowrank_get_info(h.ptr, arr), h.ptr)
    return int(arr[0]), int(arr[1])


def get_fallbacks(h: Handle):
    """(power iterations redone with shifted CholQR, shifted passes of the last factor)."""
    arr = (ctypes.c_int32 * 2)()
    _check(load_library().rs_lowrank_get_fallbacks(h.ptr, arr), h.ptr)
    return int(arr[0]), int(arr[1])


def set_profiling(h: Handle, enable: bool = True):
    _check(load_library().rs_lowrank_set_profiling(h.ptr, 1 if enable else 0), h.ptr)


PROFILE_NAMES = ("gemm_sample", "gemm_power_c", "gemm_power_b", "gram", "apply", "chol", "qrcp", "factor",
                 "reduce", "comm", "other")


def get_profile(h: Handle) -> dict:
    lib = load_library()
    out = {}
    for nm in PROFILE_NAMES:
        ms, fl = ctypes.c_double(), ctypes.c_double()
        nl = ctypes.c_int64()
        _check(lib.rs_lowrank_get_profile(h.ptr, nm.encode(), ctypes.byref(ms), ctypes.byref(nl), ctypes.byref(fl)),
               h.ptr)
        out[nm] = {"ms": ms.value, "launches": int(nl.value), "flops": fl.value}
    return out


def reset_profile(h: Handle):
    _check(load_library().rs_lowrank_reset_profile(h.ptr), h.ptr)


def kernel_launches() -> int:
    return int(load_library().rs_lowrank_kernel_launches())


class Qp3:
    """Workspace for the truncated QP3 baseline of an m x n matrix (rs_qp3_truncated)."""

    def __init__(self, m: int, n: int, k: int, device=None):
        device = torch.device("cuda", torch.cuda.current_device()) if device is None else torch.device(device)
        self.m, self.n, self.k = m, n, k
        nbytes = int(load_library().rs_qp3_workspace_bytes(m, n, k))
        if nbytes == 0:
            raise RSError(1, "invalid sizes")
        self.workspace = torch.empty(nbytes, dtype=torch.uint8, device=device)
        self.perm = torch.empty(n, dtype=torch.int64, device=device)
        self.tau = torch.empty(max(k, 1), dtype=torch.float64, device=device)

    def run(self, A: torch.Tensor, *, residual: bool = False, stream=None):
        """Overwrites A (LAPACK layout: R in rows < k, reflectors below).  Returns ||R22||_F when
        residual=True (synchronises), else None."""
        res = ctypes.c_double(-1.0)
        code = load_library().rs_qp3_truncated(
            self.m, self.n, self.k, A.data_ptr(), colmajor_ld(A, "A"), self.perm.data_ptr(), self.tau.data_ptr(),
            ctypes.byref(res) if residual else None, self.workspace.data_ptr(), self.workspace.numel(),
            _stream_ptr(stream))
        _check(code)
        return res.value if residual else None


def qp3_truncated(A: torch.Tensor, k: int, *, residual: bool = False):
    """Truncated QP3 of A (overwritten).  Returns (perm, tau, ||R22||_F or None)."""
    m, n = A.shape
    q = Qp3(m, n, k, device=A.device)
    res = q.run(A, residual=residual)
    return q.perm, q.tau, res


def last_error(h: Handle) -> str:
    return load_library().rs_lowrank_last_error(h.ptr).decode()


def comm_get_unique_id() -> bytes:
    buf = ctypes.create_string_buffer(128)
    _check(load_library().rs_comm_get_unique_id(buf))
    return buf.raw


def comm_init(nranks: int, uid: bytes, rank: int) -> int:
    c = ctypes.c_void_p()
    _check(load_library().rs_comm_init(ctypes.byref(c), nranks, uid, rank))
    return c.value


def comm_info(comm: int) -> tuple[int, int]:
    """(nranks, rank) of an NCCL communicator made by comm_init."""
    n, r = ctypes.c_int32(), ctypes.c_int32()
    _check(load_library().rs_comm_info(comm, ctypes.byref(n), ctypes.byref(r)))
    return int(n.value), int(r.value)


def comm_destroy(comm: int):
    _check(load_library().rs_comm_destroy(comm))


# ---------------------------------------------------------------------------------------------
# convenience: the whole Fig. 2(b) on one rank's block
# ---------------------------------------------------------------------------------------------
def rs_lowrank(A: torch.Tensor, k: int, p: int, q: int, seed: int = 0x5C15, *, m_global: int | None = None,
               row_offset: int = 0, nccl_comm=None, h: Handle | None = None):
    """Run sample -> power_iterate(q) -> pivot -> factor.  Returns (perm, Q, R, handle)."""
    m_local, n = A.shape
    m_global = m_local if m_global is None else m_global
    own = h is None
    if own:
        h = create(m_global, m_local, row_offset, n, k, p, seed, device=A.device, nccl_comm=nccl_comm)
    perm = torch.empty(n, dtype=torch.int64, device=A.device)
    Q = empty_colmajor(m_local, k, device=A.device)
    R = empty_colmajor(k, n, device=A.device)
    sample(h, A)
    power_iterate(h, A, q)
    pivot(h, perm)
    factor(h, A, Q, R)
    return perm, Q, R, h
