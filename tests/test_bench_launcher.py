"""bench.py --gpus N outside torchrun re-launches itself with N ranks (torch.distributed.run on
127.0.0.1) and rank 0 prints exactly one JSON line carrying the max over ranks.  Exercised on CPU
through the launcher self-test (gloo, no GPU): rank r reports 10 + r ms."""

import json
import os
import subprocess
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


def _run(n):
    env = {k: v for k, v in os.environ.items() if k not in ("WORLD_SIZE", "RANK", "LOCAL_RANK", "MASTER_ADDR",
                                                              "MASTER_PORT")}
    r = subprocess.run([sys.executable, os.path.join(ROOT, "bench.py"), "--gpus", str(n), "--launcher-selftest",
                        "--steps", "2"], capture_output=True, text=True, env=env, timeout=300, cwd=ROOT)
    assert r.returncode == 0, r.stderr[-2000:]
    lines = [x for x in r.stdout.splitlines() if x.startswith("{")]
    assert len(lines) == 1, r.stdout
    return json.loads(lines[0])


def test_launcher_spawns_n_ranks_and_reports_max():
    j = _run(3)
    assert j["n_gpus"] == 3 and j["ms_per_step"] == 12.0 and j["steps"] == 2


def test_single_rank_runs_in_process():
    j = _run(1)
    assert j["n_gpus"] == 1 and j["ms_per_step"] == 10.0
