"""compute-sanitizer over one small rank-k approximation that runs every kernel family of the
fixed-rank path (Philox sample GEMM, KC/MC GEMMs, SYRK, the tall-skinny triangular applies,
Cholesky, QRCP, TRSM, split-K reduce, gather): memcheck, synccheck, initcheck and racecheck must
report nothing (SURVEY §5 "race detection / sanitizers")."""

import os
import re
import shutil
import subprocess
import sys

import pytest
import torch

pytestmark = pytest.mark.gpu
if not torch.cuda.is_available():  # pragma: no cover
    pytest.skip("needs a GPU", allow_module_level=True)

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
SAN = shutil.which("compute-sanitizer") or "/usr/local/cuda/bin/compute-sanitizer"


@pytest.fixture(scope="module", autouse=True)
def _built():
    from paper_conf_sc_maryykltd15_b200 import build

    build.build()


@pytest.mark.parametrize("tool", ["memcheck", "synccheck", "initcheck", "racecheck"])
def test_sanitizer_clean(tool):
    cmd = [SAN, "--tool", tool, "--error-exitcode", "17"]
    if tool == "racecheck":
        cmd += ["--racecheck-report", "analysis"]
    cmd += [sys.executable, os.path.join(ROOT, "scripts", "sanitize_run.py"), "--m", "3000", "--n", "600", "--k",
            "50", "--p", "10", "--q", "1"]
    r = subprocess.run(cmd, capture_output=True, text=True, timeout=1500, cwd=ROOT)
    out = r.stdout + r.stderr
    if r.returncode == 86 and "closed" in out:
        # the GPU pool's compute-sanitizer wrapper refuses to run (operator decision); the r02
        # runs of this test before the closure are in profiles/r02_summary.md
        pytest.skip("compute-sanitizer is closed on this GPU pool: " + out.strip().splitlines()[0][:200])
    assert r.returncode == 0, out[-4000:]
    assert "ok " in out, out[-2000:]
    m = re.search(r"(ERROR|RACECHECK) SUMMARY: (\d+)", out)
    assert m and m.group(2) == "0", out[-4000:]
