#!/bin/bash
# QRCP per-phase cycle counts (RS_QRCP_TIMING) at cfg2's B (l = 110, n = 5000, k = 100)
mkdir -p gpurun_out
python __graft_entry__.py build > gpurun_out/build.log 2>&1 || { tail -20 gpurun_out/build.log; exit 1; }
RS_QRCP_TIMING=1 timeout 300 python scripts/gpu_timing.py --cfg cfg2 --reps 2 2>&1 | grep -i "QRCP\|rep"
RS_QRCP_TIMING=1 RS_QRCP_SMEM=1 timeout 300 python scripts/gpu_timing.py --cfg cfg2 --reps 2 2>&1 | grep -i "QRCP\|rep"
