#!/bin/bash
mkdir -p gpurun_out
SKIP_TESTS=1 NCU=1 bash scripts/gpu_check.sh
RS_QRCP_TIMING=1 timeout 300 python scripts/gpu_timing.py --cfg cfg1 --reps 1 2>&1 | grep -i "qrcp\|rep"
timeout 600 python scripts/bench_qp3.py --ms 2500,10000,20000,50000 --reps 5 > gpurun_out/fig7.jsonl 2> gpurun_out/fig7.err; echo "fig7 rc=$?"; cat gpurun_out/fig7.jsonl
RS_QRCP_NO_CLUSTER=1 timeout 600 python scripts/bench_qp3.py --ms 50000 --qs 0 --reps 5 2>/dev/null | head -2
