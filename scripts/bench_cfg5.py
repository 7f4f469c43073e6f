"""BASELINE configs[4] sweep on one B200: m = 200 000, n = 8 000, k in {50, 100, 200, 400}, p = 10,
q in {0, 1, 2}, exp-k singular values.  Per (k, q): RS time (sample -> factor, CUDA events, median),
accuracy e = ||A P - Q R||_F / ||A||_F against the Eckart-Young optimum e_EY = ||sigma_{k+1:}||_2 /
||sigma||_2 and against sigma_{k+1}, and the truncated QP3 of A on the same GPU (rs_qp3_truncated,
the paper's baseline, with its own error ||R22||_F / ||A||_F).  One JSON line per (k, q).

(The configuration names 8 GPUs; the driver's scaling runs use bench.py.  This script measures
the per-GPU work of the sweep and the RS-vs-QP3 comparison the config asks for.)"""

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


def timed(fn, reps, prep=None):
    s = torch.cuda.current_stream()
    out = []
    for _ in range(reps):
        if prep:
            prep()
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
    ap.add_argument("--m", type=int, default=200_000)
    ap.add_argument("--n", type=int, default=8_000)
    ap.add_argument("--ks", default="50,100,200,400")
    ap.add_argument("--qs", default="0,1,2")
    ap.add_argument("--p", type=int, default=10)
    ap.add_argument("--reps", type=int, default=3)
    ap.add_argument("--no-qp3", action="store_true")
    args = ap.parse_args()
    m, n, p = args.m, args.n, args.p
    for k in [int(x) for x in args.ks.split(",")]:
        A, sigma = make_matrix_torch(m, n, "exp-k", k, seed=2015, device="cuda")
        sig = torch.as_tensor(sigma, dtype=torch.float64)
        normA = float(torch.linalg.norm(A))
        e_ey = float(torch.sqrt(torch.sum(sig[k:] ** 2)) / torch.sqrt(torch.sum(sig ** 2)))
        qp3 = {}
        if not args.no_qp3:
            W = rs.empty_colmajor(m, n)
            q3 = rs.Qp3(m, n, k)
            t_qp3 = timed(lambda: q3.run(W), args.reps, prep=lambda: W.copy_(A))
            W.copy_(A)
            res = q3.run(W, residual=True)
            qp3 = {"qp3_ms": round(t_qp3, 3), "qp3_err": res / normA}
            del W, q3
            torch.cuda.empty_cache()
        for q in [int(x) for x in args.qs.split(",")]:
            h = rs.create(m, m, 0, n, k, p, 0x5C15)
            perm = torch.empty(n, dtype=torch.int64, device="cuda")
            Q = rs.empty_colmajor(m, k)
            R = rs.empty_colmajor(k, n)

            def run():
                rs.sample(h, A)
                rs.power_iterate(h, A, q)
                rs.pivot(h, perm)
                rs.factor(h, A, Q, R)

            run()
            t = timed(run, args.reps)
            fb = rs.get_fallbacks(h)
            rs.destroy(h)
            err = float(torch.linalg.norm(A[:, perm] - Q @ R) / normA)  # check only (torch matmul)
            line = {"experiment": "cfg5 sweep (1 GPU)", "m": m, "n": n, "k": k, "p": p, "q": q, "law": "exp-k",
                    "rs_ms": round(t, 3), "err": err, "e_EY": e_ey, "err_over_eEY": err / e_ey,
                    "sigma_k1_rel": float(sig[k] / torch.sqrt(torch.sum(sig ** 2))), "fallbacks": fb,
                    "gemm_tflops_effective": 2.0 * (k + p) * m * n * (1 + 2 * q) / (t * 1e9)}
            line.update(qp3)
            if qp3:
                line["speedup_rs_over_qp3"] = round(qp3["qp3_ms"] / t, 2)
            print(json.dumps(line), flush=True)
            del Q, R
        del A
        torch.cuda.empty_cache()


if __name__ == "__main__":
    main()
