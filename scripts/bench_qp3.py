"""Random sampling vs the truncated QP3 baseline on the same B200 (the paper's Fig. 7 / 11-14
comparison; 12.8x (q = 0) / 6.6x (q = 1) on one K40c).

Default workload: n = 2 500, m in {2 500, 10 000, 20 000, 50 000}, k = 54, p = 10, q in {0, 1},
exponent-law singular values.  Both sides start from A resident in HBM; QP3 works
in place on a copy made outside the timed region (LAPACK semantics).  Device time with CUDA
events, median of --reps runs.  Prints one JSON line per (m, q)."""

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
        torch.cuda.synchronize()
        e0.record(s)
        fn()
        e1.record(s)
        torch.cuda.synchronize()
        out.append(e0.elapsed_time(e1))
    return statistics.median(out)


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--n", type=int, default=2500)
    ap.add_argument("--ms", default="2500,10000,20000,50000")
    ap.add_argument("--k", type=int, default=54)
    ap.add_argument("--p", type=int, default=10)
    ap.add_argument("--qs", default="0,1")
    ap.add_argument("--law", default="exp-paper")
    ap.add_argument("--reps", type=int, default=5)
    args = ap.parse_args()
    n, k, p = args.n, args.k, args.p
    for m in [int(x) for x in args.ms.split(",")]:
        A, _ = make_matrix_torch(m, n, args.law, 50, seed=2015, device="cuda")
        W = rs.empty_colmajor(m, n)
        qp3 = rs.Qp3(m, n, k)

        def run_qp3():
            qp3.run(W)

        def prep():
            W.copy_(A)

        # QP3: copy outside the timed region
        ts = []
        for _ in range(args.reps + 1):
            prep()
            ts.append(timed(run_qp3, 1))
        t_qp3 = statistics.median(ts[1:])
        W.copy_(A)
        res = qp3.run(W, residual=True)
        normA = float(torch.linalg.norm(A))
        for q in [int(x) for x in args.qs.split(",")]:
            h = rs.create(m, m, 0, n, k, p, 0x5C15)
            perm = torch.empty(n, dtype=torch.int64, device="cuda")
            Q = rs.empty_colmajor(m, k)
            R = rs.empty_colmajor(k, n)

            def run_rs():
                rs.sample(h, A)
                rs.power_iterate(h, A, q)
                rs.pivot(h, perm)
                rs.factor(h, A, Q, R)

            run_rs()
            t_rs = timed(run_rs, args.reps)
            err_rs = float(torch.linalg.norm(A[:, perm] - Q @ R) / normA)  # check only
            rs.reset_profile(h)
            rs.set_profiling(h, True)
            for _ in range(args.reps):
                run_rs()
            torch.cuda.synchronize()
            rs.set_profiling(h, False)
            phases = {nm: round(v["ms"] / args.reps, 4) for nm, v in rs.get_profile(h).items() if v["launches"]}
            rs.destroy(h)
            print(json.dumps({
                "experiment": "RS vs truncated QP3 (Fig. 7)", "m": m, "n": n, "k": k, "p": p, "q": q,
                "law": args.law, "rs_ms": round(t_rs, 4), "qp3_ms": round(t_qp3, 4),
                "speedup_rs_over_qp3": round(t_qp3 / t_rs, 3),
                "qp3_GBps_trailing_reads": round(8.0 * m * sum(n - j for j in range(k)) / (t_qp3 * 1e6), 1),
                "err_rs": err_rs, "err_qp3": res / normA, "rs_phases_ms": phases}), flush=True)


if __name__ == "__main__":
    main()
