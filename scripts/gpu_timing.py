"""Quick per-phase timing of the CUDA pipeline (development aid; bench.py is the contract)."""
import argparse
import json
import os
import sys
import time

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import torch  # noqa: E402

import paper_conf_sc_maryykltd15_b200 as rs  # noqa: E402
from synth.matrices import CONFIGS, make_matrix_torch  # noqa: E402


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--cfg", default="cfg2")
    ap.add_argument("--reps", type=int, default=3)
    ap.add_argument("--m", type=int, default=0)
    ap.add_argument("--n", type=int, default=0)
    ap.add_argument("--k", type=int, default=0)
    ap.add_argument("--q", type=int, default=-1)
    args = ap.parse_args()
    c = dict(CONFIGS[args.cfg])
    if args.m:
        c["m"] = args.m
    if args.n:
        c["n"] = args.n
    if args.k:
        c["k"] = args.k
    if args.q >= 0:
        c["q"] = args.q
    m, n, k, p, q = c["m"], c["n"], c["k"], c["p"], c["q"]
    t0 = time.time()
    A, _ = make_matrix_torch(m, n, c["law"], k, seed=2015, device="cuda")
    torch.cuda.synchronize()
    print(f"matrix {m}x{n} built in {time.time() - t0:.1f}s", flush=True)
    h = rs.create(m, m, 0, n, k, p, 0x5C15)
    perm = torch.empty(n, dtype=torch.int64, device="cuda")
    Q = rs.empty_colmajor(m, k)
    R = rs.empty_colmajor(k, n)
    for rep in range(args.reps + 1):
        if rep == 1:
            rs.reset_profile(h)
            rs.set_profiling(h, True)
        s = torch.cuda.current_stream()
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        e0.record(s)
        rs.sample(h, A)
        rs.power_iterate(h, A, q)
        rs.pivot(h, perm)
        rs.factor(h, A, Q, R)
        e1.record(s)
        torch.cuda.synchronize()
        print(f"rep {rep}: {e0.elapsed_time(e1):.3f} ms", flush=True)
    prof = rs.get_profile(h)
    ell = k + p
    out = {"cfg": args.cfg, "m": m, "n": n, "k": k, "p": p, "q": q}
    for nm, v in prof.items():
        if v["launches"]:
            v["ms_per_rep"] = v["ms"] / max(args.reps, 1)
            v["tflops"] = v["flops"] / (v["ms"] * 1e9) if v["ms"] > 0 else 0
            out[nm] = v
    gemm_ms = sum(prof[x]["ms"] for x in ("gemm_sample", "gemm_power_c", "gemm_power_b")) / max(args.reps, 1)
    gemm_fl = 2.0 * ell * m * n * (1 + 2 * q)
    out["gemm_tflops"] = gemm_fl / (gemm_ms * 1e9) if gemm_ms > 0 else None
    print(json.dumps(out, indent=1))
    rs.destroy(h)


if __name__ == "__main__":
    main()
