"""Per-rank slice of a multi-GPU run on ONE GPU (the 8-GPU box is not reachable from this
environment): the work rank 0 does for N ranks -- m_local = ceil(m / N) rows of cfg4's A, the
replicated small factorisations, and every reduction point as a real ncclAllReduce on a 1-rank
communicator (launch and synchronisation cost included, no transfer) -- timed as the bench times
its step (rs_lowrank_run, CUDA-graph replay, CUDA events).  One JSON line per N.

  python scripts/rank_slice.py --cfg cfg4 --ranks 1 2 4 8
"""
import argparse
import json
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)

import torch  # noqa: E402

import paper_conf_sc_maryykltd15_b200 as rs  # noqa: E402
from paper_conf_sc_maryykltd15_b200.partition import row_split  # noqa: E402
from synth.matrices import CONFIGS, make_matrix_torch  # noqa: E402


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--cfg", default="cfg4")
    ap.add_argument("--ranks", type=int, nargs="+", default=[1, 2, 4, 8])
    ap.add_argument("--reps", type=int, default=5)
    args = ap.parse_args()
    c = dict(CONFIGS[args.cfg])
    m, n, k, p, q = c["m"], c["n"], c["k"], c["p"], c["q"]
    ell = k + p
    rs.load_library()
    uid = rs.rs_lowrank.comm_get_unique_id()
    comm = rs.rs_lowrank.comm_init(1, uid, 0)
    for N in args.ranks:
        r0, r1 = row_split(m, N, 0)
        ml = r1 - r0
        A, _ = make_matrix_torch(m, n, c["law"], k, seed=2015, rows=(r0, r1), device="cuda")
        st = torch.cuda.Stream()
        h = rs.create(m, ml, r0, n, k, p, 0x5C15, stream=st, nccl_comm=comm if N > 1 else None)
        perm = torch.empty(n, dtype=torch.int64, device="cuda")
        Q = rs.empty_colmajor(ml, k)
        R = rs.empty_colmajor(k, n)
        rs.set_profiling(h, True)
        for _ in range(3):
            rs.run(h, A, q, perm, Q, R)
        torch.cuda.synchronize()
        rs.reset_profile(h)
        e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
        e0.record(st)
        for _ in range(args.reps):
            rs.run(h, A, q, perm, Q, R)
        e1.record(st)
        torch.cuda.synchronize()
        ms = e0.elapsed_time(e1) / args.reps
        prof = rs.get_profile(h)
        phases = {nm: round(v["ms"] / args.reps, 4) for nm, v in prof.items() if v["launches"]}
        gemm = sum(prof[g]["ms"] for g in ("gemm_sample", "gemm_power_c", "gemm_power_b")) / args.reps
        # allreduce messages of one step: B (l x n) after the sample and after each power pass, two
        # l x l Grams per pass, two k x k Grams in the factor
        msgs = [8 * ell * n] * (1 + q) + [8 * ell * ell] * (2 * q) + [8 * k * k] * 2
        print(json.dumps({"cfg": args.cfg, "ranks": N, "m_local": ml, "ms_per_step": ms, "gemm_ms": gemm,
                          "gemm_tflops": 2.0 * ell * ml * n * (1 + 2 * q) / (gemm * 1e9),
                          "phases_ms": phases, "allreduce_bytes": msgs,
                          "comm_launches_per_step": prof.get("comm", {}).get("launches", 0) / args.reps}),
              flush=True)
        rs.destroy(h)
        del A, Q, R
        torch.cuda.empty_cache()
    rs.rs_lowrank.comm_destroy(comm)


if __name__ == "__main__":
    main()
