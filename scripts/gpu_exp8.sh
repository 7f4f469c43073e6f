#!/bin/bash
mkdir -p gpurun_out
TIMING_CFG="cfg4 cfg2" NCU=1 bash scripts/gpu_check.sh
timeout 600 ncu --set full --clock-control none --import-source on -k regex:mc_persist -s 1 -c 1 \
    -o gpurun_out/ncu_mc_persist_factor_cfg4 -f python scripts/gpu_timing.py --cfg cfg4 --reps 0 > gpurun_out/ncu_mcp.log 2>&1
echo "ncu mcp rc=$?"
