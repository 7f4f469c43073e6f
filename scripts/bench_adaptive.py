"""Adaptive fixed-accuracy scheme on the GPU: the paper's Sec. 10 experiment (Figs. 16-18).

Exponent matrix 50 000 x 2 500 (sigma_i = 10^(-i/10)), eps = 1e-12, q = 0, l_inc in {8, 16, 32, 64}
(P:L1045-1064, L1138-1215).  Reports per l_inc: the final l, the (l, eps~) history, the sampling
time, the GEMM rate of the small-l_inc products (Fig. 18) and the time of the whole Steps 1-3.
Prints one JSON line per l_inc."""

import argparse
import json
import os
import sys
import time

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import torch  # noqa: E402

import paper_conf_sc_maryykltd15_b200 as rs  # noqa: E402
from synth.matrices import make_matrix_torch  # noqa: E402


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--m", type=int, default=50_000)
    ap.add_argument("--n", type=int, default=2_500)
    ap.add_argument("--eps", type=float, default=1e-12)
    ap.add_argument("--q", type=int, default=0)
    ap.add_argument("--lmax", type=int, default=400)
    ap.add_argument("--incs", default="8,16,32,64")
    ap.add_argument("--policies", default="static,interp")
    args = ap.parse_args()
    A, sigma = make_matrix_torch(args.m, args.n, "exp-paper", 50, seed=2015, device="cuda")
    runs = [(pol, int(x)) for pol in args.policies.split(",") for x in args.incs.split(",")]
    for pol, inc in runs:
        h = rs.create(args.m, args.m, 0, args.n, args.lmax, 0, 0x5C15)
        rs.sample_adaptive(h, A, args.eps, inc, args.q, inc_policy=pol, raise_on_max=False)  # warm-up
        torch.cuda.synchronize()
        rs.reset_profile(h)
        rs.set_profiling(h, True)
        s = torch.cuda.current_stream()
        e0, e1, e2 = (torch.cuda.Event(enable_timing=True) for _ in range(3))
        e0.record(s)
        ell, est, hist = rs.sample_adaptive(h, A, args.eps, inc, args.q, inc_policy=pol, raise_on_max=False)
        e1.record(s)
        perm = torch.empty(args.n, dtype=torch.int64, device="cuda")
        Q = rs.empty_colmajor(args.m, args.lmax)
        R = rs.empty_colmajor(args.lmax, args.n)
        rs.pivot(h, perm)
        factor_status = "ok"
        try:  # CholQR2 of A P_{1:l} breaks down when kappa(A P_{1:l})^2 u >> 1
            rs.factor(h, A, Q, R)
        except rs.RSError as ex:
            factor_status = ex.name
        e2.record(s)
        torch.cuda.synchronize()
        prof = rs.get_profile(h)
        k = ell
        Qk, Rk = Q[:, :k], R[:k]
        fac_err = float(torch.linalg.norm(A[:, perm] - Qk @ Rk) / torch.linalg.norm(A))  # check only
        q_orth = float((Qk.T @ Qk - torch.eye(k, device="cuda", dtype=torch.float64)).abs().max())
        gm = prof["gemm_sample"]
        line = {
            "experiment": "adaptive fixed-accuracy (Fig. 3 / Figs. 16-18)",
            "m": args.m, "n": args.n, "eps": args.eps, "q": args.q, "inc_policy": pol, "l_inc": inc, "l": ell, "eps_est": est,
            "history": hist,
            "sample_ms": e0.elapsed_time(e1), "total_ms": e0.elapsed_time(e2), "factor_status": factor_status,
            "factor_rel_err_F": fac_err, "q_orth": q_orth,
            "sampling_gemm_tflops": gm["flops"] / (gm["ms"] * 1e9) if gm["ms"] else None,
            "phases_ms": {k: round(v["ms"], 3) for k, v in prof.items() if v["launches"]},
            "phases_launches": {k: v["launches"] for k, v in prof.items() if v["launches"]},
        }
        print(json.dumps(line), flush=True)
        rs.destroy(h)


if __name__ == "__main__":
    main()
