#!/bin/bash
mkdir -p gpurun_out
SKIP_BENCH=1 TIMING_CFG="cfg2 cfg4" bash scripts/gpu_check.sh
RS_QRCP_TIMING=1 timeout 300 python scripts/gpu_timing.py --cfg cfg2 --reps 1 2>&1 | grep QRCP
RS_QRCP_TIMING=1 RS_QRCP_SMEM=1 timeout 300 python scripts/gpu_timing.py --cfg cfg2 --reps 1 2>&1 | grep QRCP
timeout 600 ncu --set full --clock-control none --import-source on -k regex:chol_tile -c 1 \
    -o gpurun_out/ncu_chol_tile_cfg2 -f python scripts/gpu_timing.py --cfg cfg2 --reps 0 > gpurun_out/ncu_chol.log 2>&1
echo "ncu chol rc=$?"
