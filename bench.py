"""Benchmark: FP64 rank-k approximation (random sampling, Mary et al. SC15) on 1..8 B200.

One "step" = one whole rank-k approximation of the workload matrix through the C ABI:
sample (B = Omega A) -> power_iterate(q) -> pivot (truncated QRCP of B, T) -> factor (CholQR2 of
A P_{1:k}, R = Rbar [I T]).  A is resident in HBM and row-block partitioned over the ranks
(P:L535-541); total work is fixed as N grows ("strong" scaling, like the paper's Fig. 15).

    python bench.py [--gpus N] [--steps K] [--warmup W] [--workload cfg4] [--impl ours|reference]

Prints ONE JSON line on rank 0.  With --gpus N > 1 and no torchrun environment (WORLD_SIZE unset)
the script re-launches itself under torch.distributed.run with N ranks on 127.0.0.1.  The timed
step is rs_lowrank_run (the whole step replayed as one CUDA graph).  --impl reference times the CPU
oracle (the only reference this paper has: it ships no code) on a bounded row sample of the same
workload.
"""

from __future__ import annotations

import argparse
import json
import math
import os
import subprocess
import sys
import threading
import time

ROOT = os.path.dirname(os.path.abspath(__file__))
sys.path.insert(0, ROOT)

METRIC = "FP64 rank-k approx time (s) & sampling TFLOP/s vs FP64 peak at 1/2/4/8 B200"
FP64_PEAK_TFLOPS = 37.1   # measured DMMA.8x8x4 register-only probe (profiles/r01_probe_fp64_peak.jsonl)
FP64_NOMINAL_TFLOPS = 148 * 64 * 2 * 1.965e9 / 1e12   # 148 SM x 64 FP64 FMA/clk x 2 x 1.965 GHz = 37.2


def workload(name: str) -> dict:
    from synth.matrices import CONFIGS, MATRIX_SEED, OMEGA_SEED

    c = dict(CONFIGS[name])
    c.update(name=name, matrix_seed=MATRIX_SEED, omega_seed=OMEGA_SEED)
    return c


def describe(c: dict) -> str:
    return f"{c['name']}: m={c['m']} n={c['n']} k={c['k']} p={c['p']} q={c['q']} sigma={c['law']}"


def row_split(m: int, nranks: int, rank: int):
    from paper_conf_sc_maryykltd15_b200.partition import row_split as _rs

    return _rs(m, nranks, rank)


def gemm_flops(c: dict) -> float:
    return 2.0 * (c["k"] + c["p"]) * c["m"] * c["n"] * (1 + 2 * c["q"])


# --------------------------------------------------------------------------------------------
# clocks sampled with nvidia-smi during the timed region
# --------------------------------------------------------------------------------------------
class ClockSampler:
    FIELDS = ("clocks.sm", "clocks.max.sm", "power.draw", "clocks_event_reasons.active",
              "clocks_event_reasons.hw_slowdown", "clocks_event_reasons.hw_thermal_slowdown",
              "clocks_event_reasons.sw_thermal_slowdown", "clocks_event_reasons.sw_power_cap")

    def __init__(self, gpu_index: int):
        self.idx = gpu_index
        self.rows = []
        self._stop = threading.Event()
        self._t = None

    def _run(self):
        cmd = ["nvidia-smi", "-i", str(self.idx), f"--query-gpu={','.join(self.FIELDS)}", "--format=csv,noheader,nounits"]
        while not self._stop.is_set():
            try:
                out = subprocess.run(cmd, capture_output=True, text=True, timeout=5).stdout.strip()
                if out:
                    self.rows.append([x.strip() for x in out.split(",")])
            except Exception:  # noqa: BLE001
                pass
            self._stop.wait(0.2)

    def __enter__(self):
        self._t = threading.Thread(target=self._run, daemon=True)
        self._t.start()
        return self

    def __exit__(self, *a):
        self._stop.set()
        if self._t:
            self._t.join(timeout=10)

    def summary(self) -> dict:
        if not self.rows:
            return {"sm_mhz": None, "sm_max_mhz": None, "reasons": ["unsampled"], "samples": 0}
        sm = sorted(float(r[0]) for r in self.rows if r[0].replace(".", "").isdigit())
        mx = max(float(r[1]) for r in self.rows if r[1].replace(".", "").isdigit())
        names = ["hw_slowdown", "hw_thermal_slowdown", "sw_thermal_slowdown", "sw_power_cap"]
        reasons = sorted({names[i] for r in self.rows for i in range(4) if len(r) > 4 + i and r[4 + i] == "Active"})
        return {"sm_mhz": sm[len(sm) // 2] if sm else None, "sm_max_mhz": mx, "reasons": reasons,
                "samples": len(self.rows), "power_w_max": max(float(r[2]) for r in self.rows
                                                               if r[2].replace(".", "").isdigit())}


# --------------------------------------------------------------------------------------------
# CPU oracle on a bounded row sample (cpu_baseline / --impl reference)
# --------------------------------------------------------------------------------------------
def oracle_sample_run(c: dict, m_s: int) -> dict:
    """Oracle pipeline on the first m_s rows (a multiple of n: same stacked structure) of the
    workload; m-linear phases are extrapolated to the full m, the m-independent QRCP is not."""
    import numpy as np

    from oracle import pipeline as OPL
    from synth.matrices import make_matrix

    A, _ = make_matrix(m_s, c["n"], c["law"], c["k"], seed=c["matrix_seed"])
    ell = c["k"] + c["p"]
    t = {}
    t0 = time.perf_counter()
    B = OPL.sample(A, ell, c["omega_seed"])
    t["sample"] = time.perf_counter() - t0
    t0 = time.perf_counter()
    B = OPL.power_iterate(A, B, c["q"])
    t["power"] = time.perf_counter() - t0
    t0 = time.perf_counter()
    perm, Rhat, T, gaps = OPL.pivot(B, c["k"])
    t["pivot"] = time.perf_counter() - t0
    t0 = time.perf_counter()
    OPL.factor(A, perm, T, c["k"])
    t["factor"] = time.perf_counter() - t0
    scale = c["m"] / m_s
    full = (t["sample"] + t["power"] + t["factor"]) * scale + t["pivot"]
    return {"seconds_sample": sum(t.values()), "seconds_extrapolated": full, "phases": t, "m_sample": m_s}


def full_oracle_reference(c: dict):
    """The oracle timed once on the FULL workload (scripts/oracle_full.py, stored under profiles/):
    context for the bounded in-run sample above, not re-measured here."""
    path = os.path.join(ROOT, "profiles", f"r02_oracle_full_{c['name']}.json")
    if not os.path.exists(path):
        return None
    try:
        j = json.loads(open(path).read().strip().splitlines()[-1])
    except (OSError, ValueError, IndexError):
        return None
    if (j.get("m"), j.get("n"), j.get("k"), j.get("p"), j.get("q")) != (c["m"], c["n"], c["k"], c["p"], c["q"]):
        return None
    return {"value": j["seconds_total"], "unit": "s", "threads": j.get("threads"), "phases_s": j.get("phases_s"),
            "source": os.path.relpath(path, ROOT)}


def cpu_threads() -> int:
    """Threads the oracle's C GEMM (OpenMP over output tiles) runs with."""
    from oracle.gemm import default_threads

    return default_threads()


def oracle_m_sample(c: dict) -> int:
    # ~10-20 s of oracle work per sample on the 16-core GPU host; a multiple of n keeps the stacked U
    return max(c["n"], min(c["m"], 16 * c["n"]) // c["n"] * c["n"])


def run_reference(args, c):
    rank = int(os.environ.get("RANK", "0"))
    if rank != 0:
        return
    m_s = oracle_m_sample(c)
    for _ in range(args.warmup):
        oracle_sample_run(c, m_s)
    vals, samp = [], []
    for _ in range(args.steps):
        r = oracle_sample_run(c, m_s)
        vals.append(r["seconds_extrapolated"])
        samp.append(r["seconds_sample"])
    v = sum(vals) / len(vals)
    cores = cpu_threads()
    line = {
        "impl": "reference", "metric": METRIC, "value": v, "unit": "s", "n_gpus": args.gpus, "steps": args.steps,
        "warmup": args.warmup, "ms_per_step": 1e3 * sum(samp) / len(samp), "higher_is_better": False,
        "scaling": "strong", "vs_baseline": None, "dtype": "f64", "data": "synthetic",
        "config": {"workload": describe(c), "m": c["m"], "n": c["n"], "k": c["k"], "p": c["p"], "q": c["q"],
                   "law": c["law"], "parallelism": "cpu oracle (fixed-order C GEMM, OpenMP over output tiles; numpy Householder)"},
        "cpu_baseline": {"value": v, "unit": "s", "cores": cores, "kind": "oracle",
                         "sample": f"oracle pipeline on the first {m_s} of {c['m']} rows per step; sample/power/"
                                   f"factor time scaled by m/{m_s}, QRCP time unscaled"},
        "e2e": {"value": v, "unit": "s", "h2d_bytes_per_step": 0, "d2h_bytes_per_step": 0},
    }
    print(json.dumps(line), flush=True)


# --------------------------------------------------------------------------------------------
# launcher: N ranks on one node
# --------------------------------------------------------------------------------------------
def _free_port() -> int:
    import socket

    s = socket.socket()
    s.bind(("127.0.0.1", 0))
    port = s.getsockname()[1]
    s.close()
    return port


def spawn_command(nproc: int, argv: list[str], port: int) -> list[str]:
    return [sys.executable, "-m", "torch.distributed.run", "--nnodes=1", f"--nproc-per-node={nproc}",
            "--master-addr", "127.0.0.1", "--master-port", str(port), os.path.abspath(__file__), *argv]


def maybe_spawn(args, argv: list[str]) -> None:
    """--gpus N > 1 outside torchrun: re-exec this script under torch.distributed.run (one rank per
    GPU); rank 0 prints the one JSON line.  Exits with the launcher's return code."""
    if args.gpus <= 1 or "WORLD_SIZE" in os.environ or args.impl == "reference":
        return
    raise SystemExit(subprocess.call(spawn_command(args.gpus, argv, _free_port())))


def max_over_ranks(vals: list[float], device) -> list[float]:
    """Element-wise max over the ranks (device-timed numbers: the job is as slow as its slowest rank)."""
    import torch
    import torch.distributed as dist

    t = torch.tensor(vals, dtype=torch.float64, device=device)
    if dist.is_initialized() and dist.get_world_size() > 1:
        dist.all_reduce(t, op=dist.ReduceOp.MAX)
    return [float(x) for x in t.cpu()]


def run_launcher_selftest(args):
    """CPU check of the launcher and the max-over-ranks merge (gloo, no GPU): every rank reports a
    rank-dependent fake time; rank 0 prints one JSON line with the max."""
    import torch.distributed as dist

    world = int(os.environ.get("WORLD_SIZE", "1"))
    rank = int(os.environ.get("RANK", "0"))
    if world > 1:
        dist.init_process_group("gloo")
    ms = max_over_ranks([10.0 + rank], "cpu")[0]
    if rank == 0:
        print(json.dumps({"metric": METRIC, "value": ms / 1e3, "unit": "s", "n_gpus": world, "steps": args.steps,
                          "warmup": args.warmup, "ms_per_step": ms, "selftest": True}), flush=True)
    if world > 1:
        dist.barrier()
        dist.destroy_process_group()


# --------------------------------------------------------------------------------------------
# our arm
# --------------------------------------------------------------------------------------------
def kernels_per_step(rs, h, A, q, perm, Q, R) -> int:
    """Kernel launches of one step, counted by the library's launchers on an un-captured run of the
    same phases (a graph replay re-launches exactly these kernels)."""
    import torch

    n0 = rs.kernel_launches()
    rs.sample(h, A)
    rs.power_iterate(h, A, q)
    rs.pivot(h, perm)
    rs.factor(h, A, Q, R)
    torch.cuda.synchronize()
    return rs.kernel_launches() - n0


def run_ours(args, c):
    import torch
    import torch.distributed as dist

    import paper_conf_sc_maryykltd15_b200 as rs
    from synth.matrices import make_matrix_torch, singular_values

    world = int(os.environ.get("WORLD_SIZE", "1"))
    rank = int(os.environ.get("RANK", "0"))
    local = int(os.environ.get("LOCAL_RANK", "0"))
    if world != args.gpus:
        raise SystemExit(f"--gpus {args.gpus} but WORLD_SIZE={world}")
    torch.cuda.set_device(local)
    dev = torch.device("cuda", local)
    if world > 1:
        dist.init_process_group("nccl", device_id=dev)
    rs.load_library()

    m, n, k, p, q = c["m"], c["n"], c["k"], c["p"], c["q"]
    ell = k + p
    r0, r1 = row_split(m, world, rank)
    ml = r1 - r0
    A, sigma = make_matrix_torch(m, n, c["law"], k, seed=c["matrix_seed"], rows=(r0, r1), device=dev)
    comm = None
    if world > 1:
        uid = [rs.rs_lowrank.comm_get_unique_id() if rank == 0 else None]
        dist.broadcast_object_list(uid, src=0)
        comm = rs.rs_lowrank.comm_init(world, uid[0], rank)
        nr, rr = rs.rs_lowrank.comm_info(comm)
        if nr != world or rr != rank:
            raise SystemExit(f"NCCL communicator has nranks={nr} rank={rr}, expected {world}/{rank}")
        print(f"[rank {rank}] NCCL communicator: nranks={nr} rank={rr}", file=sys.stderr, flush=True)
    stream = torch.cuda.Stream(device=dev)
    h = rs.create(m, ml, r0, n, k, p, c["omega_seed"], device=dev, stream=stream, nccl_comm=comm)
    perm = torch.empty(n, dtype=torch.int64, device=dev)
    Q = rs.empty_colmajor(ml, k, device=dev)
    R = rs.empty_colmajor(k, n, device=dev)

    def step():   # the whole step as one CUDA-graph replay (rs_lowrank_run)
        rs.run(h, A, q, perm, Q, R)

    torch.cuda.synchronize()
    for _ in range(args.warmup):
        step()
    torch.cuda.synchronize()
    rs.reset_profile(h)
    rs.set_profiling(h, True)
    step()   # re-capture with the profiling event nodes (untimed)
    torch.cuda.synchronize()
    rs.reset_profile(h)
    launches0 = rs.kernel_launches()
    if world > 1:
        dist.barrier()
    torch.cuda.synchronize()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    with ClockSampler(local) as clk:
        e0.record(stream)
        for _ in range(args.steps):
            step()
        e1.record(stream)
        torch.cuda.synchronize()
    if world > 1:
        dist.barrier()
    rs.set_profiling(h, False)
    ms_local = e0.elapsed_time(e1)
    prof = rs.get_profile(h)
    # kernels launched in the timed region: the graph replays them; count one un-captured step
    launches = args.steps * kernels_per_step(rs, h, A, q, perm, Q, R)
    gemm_names = ("gemm_sample", "gemm_power_c", "gemm_power_b")
    gemm_ms_local = sum(prof[g]["ms"] for g in gemm_names)
    ms_total, gemm_ms_max = max_over_ranks([ms_local, gemm_ms_local], dev)
    ms_step = ms_total / args.steps

    # accuracy of the last approximation (evaluation only, outside the timed region)
    err_num = torch.zeros((), dtype=torch.float64, device=dev)
    nrm = torch.zeros((), dtype=torch.float64, device=dev)
    for c0 in range(0, n, 512):
        c1 = min(n, c0 + 512)
        D = A[:, perm[c0:c1]] - Q @ R[:, c0:c1]
        err_num += (D * D).sum()
        nrm += (A[:, c0:c1] * A[:, c0:c1]).sum()
    tot = torch.stack([err_num, nrm])
    if world > 1:
        dist.all_reduce(tot)
    err = math.sqrt(float(tot[0]) / float(tot[1]))
    ey = math.sqrt(float((sigma[k:] ** 2).sum()) / float((sigma ** 2).sum()))

    # e2e: the same call sequence through the host-buffer entry point (H2D of A and D2H of Q, R, perm)
    e2e = None
    if not args.no_e2e:
        e2e_steps = max(1, min(args.steps, args.e2e_steps))
        A_host = rs.empty_colmajor(ml, n, device="cpu", pin=True)
        A_host.copy_(A)
        Qh = rs.empty_colmajor(ml, k, device="cpu", pin=True)
        Rh = rs.empty_colmajor(k, n, device="cpu", pin=True)
        permh = torch.empty(n, dtype=torch.int64, pin_memory=True)
        torch.cuda.synchronize()
        rs.run_host(h, A_host, A, q, permh, Qh, Rh, Q, R)     # warm
        if world > 1:
            dist.barrier()
        t0 = time.perf_counter()
        for _ in range(e2e_steps):
            rs.run_host(h, A_host, A, q, permh, Qh, Rh, Q, R)
        dt = torch.tensor([(time.perf_counter() - t0) / e2e_steps], dtype=torch.float64, device=dev)
        if world > 1:
            dist.all_reduce(dt, op=dist.ReduceOp.MAX)
        e2e = {"value": float(dt), "unit": "s", "steps": e2e_steps,
               "h2d_bytes_per_step": int(m * n * 8),
               "d2h_bytes_per_step": int(m * k * 8 + world * (k * n * 8 + n * 8)),
               "api": "rs_lowrank_run_host (pinned host A, Q, R, perm)"}
        del A_host

    # roofline of the dominant kernel class (max total device time)
    dom = max(gemm_names, key=lambda g: prof[g]["ms"])
    launches_dom = max(prof[dom]["launches"], 1)
    avg_ms = prof[dom]["ms"] / launches_dom
    fl_launch = prof[dom]["flops"] / launches_dom
    achieved = fl_launch / (avg_ms * 1e9)
    traffic = None
    tpath = os.path.join(ROOT, "profiles", "traffic.json")
    if os.path.exists(tpath):
        try:
            traffic = json.load(open(tpath)).get(dom)
        except Exception:  # noqa: BLE001
            traffic = None
    gf = gemm_flops(c)
    sampling_tf = gf * args.steps / (gemm_ms_max * 1e9) if gemm_ms_max > 0 else None

    if rank != 0:
        if world > 1:
            dist.barrier()
            rs.destroy(h)
            rs.rs_lowrank.comm_destroy(comm)
            dist.destroy_process_group()
        return

    cpu = None
    if world == 1 and not args.no_cpu_baseline:
        m_s = oracle_m_sample(c)
        r = oracle_sample_run(c, m_s)
        cpu = {"value": r["seconds_extrapolated"], "unit": "s", "cores": cpu_threads(), "kind": "oracle",
               "sample": f"oracle pipeline on the first {m_s} of {m} rows ({r['seconds_sample']:.1f} s of CPU work); "
                         f"sample/power/factor scaled by m/{m_s}, QRCP unscaled",
               "phases_s": r["phases"]}
        full = full_oracle_reference(c)
        if full:
            cpu["full_size_measured"] = full

    phases = {nm: round(v["ms"] / args.steps, 4) for nm, v in prof.items() if v["launches"]}
    line = {
        "metric": METRIC,
        "value": ms_step / 1e3,
        "unit": "s",
        "n_gpus": world,
        "steps": args.steps,
        "warmup": args.warmup,
        "ms_per_step": ms_step,
        "higher_is_better": False,
        "scaling": "strong",
        "vs_baseline": None,
        "dtype": "f64",
        "data": "synthetic",
        "config": {"workload": describe(c), "m": m, "n": n, "k": k, "p": p, "q": q, "law": c["law"],
                   "matrix_seed": c["matrix_seed"], "omega_seed": c["omega_seed"],
                   "parallelism": f"row-block dp{world} (NCCL allreduce)" if world > 1 else "1 GPU",
                   "l2": f"inputs larger than L2 (A = {m * n * 8 / 1e9:.1f} GB total)"},
        "sampling_tflops": sampling_tf,
        "sampling_frac_fp64_peak": (sampling_tf / world / FP64_PEAK_TFLOPS) if sampling_tf else None,
        "tflops_total": gf / (ms_step * 1e9),
        "phases_ms_per_step": phases,
        "accuracy": {"err_fro": err, "eckart_young": ey, "sigma_k": float(sigma[k])},
        "roofline": {"bound": "tensor", "kernel": dom, "achieved": achieved, "peak": FP64_PEAK_TFLOPS,
                     "unit": "TFLOP/s", "frac": achieved / FP64_PEAK_TFLOPS, "traffic": traffic,
                     "peak_source": "measured FP64 DMMA probe (profiles/r01_probe_fp64_peak.jsonl); nominal "
                                    f"{FP64_NOMINAL_TFLOPS:.1f}; MEASURED_PEAKS.json has no FP64 entry",
                     "flops_per_launch": fl_launch, "avg_launch_ms": avg_ms},
        "clocks": clk.summary(),
        "e2e": e2e,
        "gpu_launches": int(launches),
        "step_api": "rs_lowrank_run (CUDA graph replay)",
        "nccl": {"nranks": world, "checked": "rs_comm_info == WORLD_SIZE on every rank"} if world > 1 else None,
        "cpu_baseline": cpu,
    }
    print(json.dumps(line), flush=True)
    if world > 1:
        dist.barrier()
        rs.destroy(h)
        rs.rs_lowrank.comm_destroy(comm)
        dist.destroy_process_group()
    else:
        rs.destroy(h)


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--gpus", type=int, default=1)
    ap.add_argument("--steps", type=int, default=5)
    ap.add_argument("--warmup", type=int, default=3)
    ap.add_argument("--impl", default="ours", choices=["ours", "reference"])
    ap.add_argument("--workload", default="cfg4")
    ap.add_argument("--no-e2e", action="store_true")
    ap.add_argument("--e2e-steps", type=int, default=2)
    ap.add_argument("--no-cpu-baseline", action="store_true")
    ap.add_argument("--launcher-selftest", action="store_true", help=argparse.SUPPRESS)
    args = ap.parse_args()
    maybe_spawn(args, sys.argv[1:])
    if args.launcher_selftest:
        run_launcher_selftest(args)
        return
    if args.warmup < 3:
        args.warmup = 3
    c = workload(args.workload)
    if args.impl == "reference":
        run_reference(args, c)
    else:
        run_ours(args, c)


if __name__ == "__main__":
    main()
