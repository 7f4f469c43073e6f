#!/bin/bash
mkdir -p gpurun_out
SKIP_BENCH=1 TIMING_CFG="cfg4 cfg2" bash scripts/gpu_check.sh
timeout 600 python scripts/bench_qp3.py --ms 50000 --reps 5 > gpurun_out/fig7.jsonl 2> gpurun_out/fig7.err; echo "fig7 rc=$?"; cat gpurun_out/fig7.jsonl
