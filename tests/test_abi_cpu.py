"""CPU-side checks of the boundary: the C-ABI library builds, loads and exports every symbol that
include/rs_lowrank.h declares; host-only entry points behave (no compute calls without a GPU)."""

import ctypes
import os
import re
import subprocess

import pytest

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
HEADER = os.path.join(ROOT, "include", "rs_lowrank.h")


def _declared():
    src = open(HEADER).read()
    return sorted(set(re.findall(r"^RS_API\s+[\w\s\*]+?\b(rs_\w+)\s*\(", src, flags=re.M)))


@pytest.fixture(scope="module")
def lib():
    from paper_conf_sc_maryykltd15_b200 import build

    build.build()
    from paper_conf_sc_maryykltd15_b200.rs_lowrank import load_library

    return load_library()


def test_header_declares_the_north_star_entry_points():
    names = _declared()
    for fn in ("create", "sample", "power_iterate", "pivot", "factor", "destroy"):
        assert f"rs_lowrank_{fn}" in names
    assert len(names) >= 20


def test_library_exports_every_declared_symbol(lib):
    from paper_conf_sc_maryykltd15_b200.rs_lowrank import ABI_FUNCTIONS, LIB_PATH

    declared = _declared()
    assert sorted(ABI_FUNCTIONS) == declared
    out = subprocess.run(["nm", "-D", "--defined-only", LIB_PATH], capture_output=True, text=True).stdout
    exported = set(re.findall(r"\bT (rs_\w+)", out))
    missing = [d for d in declared if d not in exported]
    assert not missing, missing
    for d in declared:
        assert getattr(lib, d) is not None


def test_library_is_sm100a_only(lib):
    from paper_conf_sc_maryykltd15_b200.rs_lowrank import LIB_PATH

    out = subprocess.run(["cuobjdump", "--list-elf", LIB_PATH], capture_output=True, text=True).stdout
    archs = set(re.findall(r"sm_(\d+a?)", out))
    assert archs == {"100a"}, archs
    sass = subprocess.run(["cuobjdump", "-sass", LIB_PATH], capture_output=True, text=True).stdout
    assert "DMMA.8x8x4" in sass          # FP64 tensor-core tiles
    assert "UTMALDG" in sass             # TMA loads


def test_workspace_bytes_is_host_only_and_monotone(lib):
    from paper_conf_sc_maryykltd15_b200 import workspace_bytes

    a = workspace_bytes(50_000, 5_000, 100, 10)
    b = workspace_bytes(100_000, 5_000, 100, 10)
    assert 0 < a < b
    assert workspace_bytes(500, 200, 20, 10) > 0
    assert workspace_bytes(-1, 10, 1, 0) == 0 and workspace_bytes(10, 10, 0, 0) == 0


def test_create_rejects_bad_arguments_without_touching_a_device(lib):
    h = ctypes.c_void_p()
    ws = ctypes.c_void_p(0)
    # l = k + p > n  -> RS_ERR_INVALID_ARG before any CUDA call
    assert lib.rs_lowrank_create(ctypes.byref(h), 100, 100, 0, 10, 8, 4, 1, ws, 0, None, None) == 1
    assert lib.rs_lowrank_create(ctypes.byref(h), 100, 50, 60, 30, 4, 4, 1, ws, 0, None, None) == 1
    assert lib.rs_lowrank_create(None, 100, 100, 0, 30, 4, 4, 1, ws, 0, None, None) == 1
    assert lib.rs_lowrank_destroy(None) == 1


def test_no_runtime_development_switches(lib):
    """A/B switches are compile-time only (-DRS_DEV_*): the shipped library reads no RS_* variable."""
    from paper_conf_sc_maryykltd15_b200.rs_lowrank import LIB_PATH

    strs = subprocess.run(["strings", LIB_PATH], capture_output=True, text=True).stdout
    for name in ("RS_PHILOX_GENMODE", "RS_PHILOX_CLUSTER", "RS_KC_NO_PWG", "RS_MC_NO_PWG", "RS_MC_WM",
                 "RS_MC_NO_TMA3D", "RS_MC_NO_PERSIST", "RS_QRCP_SMEM", "RS_QRCP_TIMING", "RS_QRCP_BARRIER",
                 "RS_CHOL_BLOCKED", "RS_CHOL_TPT", "RS_CHOL_SMEM_MAX_N"):
        assert name not in strs, name
