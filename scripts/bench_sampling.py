"""Sampling rates (Fig. 8): row sampling B = Omega A (Philox fused into the DMMA GEMM)
and column sampling B_c = Omega_c A^T, for l = 32 ... 512 on the paper's 50 000 x 2 500 matrix.
Device time with CUDA events (median of --reps); TF/s = 2 l m n / t.  Prints one JSON line per l."""

import argparse
import json
import os
import statistics
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import torch  # noqa: E402

import paper_conf_sc_maryykltd15_b200 as rs  # noqa: E402
from synth.matrices import make_matrix_torch  # noqa: E402


def timed(fn, reps):
    s = torch.cuda.current_stream()
    out = []
    for _ in range(reps):
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        e0.record(s)
        fn()
        e1.record(s)
        torch.cuda.synchronize()
        out.append(e0.elapsed_time(e1))
    return statistics.median(out)


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--m", type=int, default=50_000)
    ap.add_argument("--n", type=int, default=2_500)
    ap.add_argument("--ells", default="8,16,32,64,128,256,512")
    ap.add_argument("--reps", type=int, default=7)
    args = ap.parse_args()
    m, n = args.m, args.n
    A, _ = make_matrix_torch(m, n, "exp-paper", 50, seed=2015, device="cuda")
    for ell in [int(x) for x in args.ells.split(",")]:
        h = rs.create(m, m, 0, n, ell, 0, 0x5C15)
        Bc = rs.empty_colmajor(ell, m)
        rs.sample(h, A)
        rs.sample_columns(h, A, Bc)
        t_row = timed(lambda: rs.sample(h, A), args.reps)
        t_col = timed(lambda: rs.sample_columns(h, A, Bc), args.reps)
        rs.destroy(h)
        fl = 2.0 * ell * m * n
        print(json.dumps({"experiment": "sampling rate (Fig. 8)", "m": m, "n": n, "l": ell,
                          "row_ms": round(t_row, 4), "row_tflops": round(fl / (t_row * 1e9), 2),
                          "col_ms": round(t_col, 4), "col_tflops": round(fl / (t_col * 1e9), 2),
                          "hbm_floor_ms": round(8.0 * m * n / 6.54e12 * 1e3, 4)}), flush=True)


if __name__ == "__main__":
    main()
