"""The CPU oracle on a FULL workload (default cfg4: m = 1e6, n = 5 000, k = 100, p = 10, q = 1), timed
phase by phase on the host's cores -- the measured (not extrapolated) oracle time that bench.py's
bounded cpu_baseline sample stands in for.  One JSON line.  Needs ~50 GB of host memory at cfg4.

  python scripts/oracle_full.py --cfg cfg4
"""
import argparse
import json
import os
import platform
import sys
import time

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

from oracle import gemm as OG  # noqa: E402
from oracle import pipeline as OPL  # noqa: E402
from synth.matrices import CONFIGS, MATRIX_SEED, OMEGA_SEED, make_matrix  # noqa: E402


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--cfg", default="cfg4")
    args = ap.parse_args()
    c = CONFIGS[args.cfg]
    m, n, k, p, q = c["m"], c["n"], c["k"], c["p"], c["q"]
    t0 = time.perf_counter()
    A, _ = make_matrix(m, n, c["law"], k, seed=MATRIX_SEED)
    t_gen = time.perf_counter() - t0
    t = {}
    t0 = time.perf_counter()
    B = OPL.sample(A, k + p, OMEGA_SEED)
    t["sample"] = time.perf_counter() - t0
    t0 = time.perf_counter()
    B = OPL.power_iterate(A, B, q)
    t["power"] = time.perf_counter() - t0
    t0 = time.perf_counter()
    perm, Rhat, T, gaps = OPL.pivot(B, k)
    t["pivot"] = time.perf_counter() - t0
    t0 = time.perf_counter()
    Q, Rbar, R = OPL.factor(A, perm, T, k)
    t["factor"] = time.perf_counter() - t0
    cpu = ""
    try:
        with open("/proc/cpuinfo") as fh:
            cpu = next(line.split(":", 1)[1].strip() for line in fh if line.startswith("model name"))
    except (OSError, StopIteration):
        cpu = platform.processor()
    print(json.dumps({"cfg": args.cfg, "m": m, "n": n, "k": k, "p": p, "q": q, "law": c["law"],
                      "seconds_total": sum(t.values()), "phases_s": t, "matrix_build_s": t_gen,
                      "threads": OG.default_threads(), "cpu": cpu, "host": platform.node(),
                      "what": "oracle/ pipeline (fixed-order C GEMM + numpy Householder) on the full matrix; "
                              "error evaluation not timed"}), flush=True)


if __name__ == "__main__":
    main()
