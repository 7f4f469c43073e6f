#!/bin/bash
mkdir -p gpurun_out
nvcc -gencode arch=compute_100a,code=sm_100a -O3 -o /tmp/fp64_ops probes/fp64_ops.cu && /tmp/fp64_ops | tee gpurun_out/probe_fp64_ops.jsonl
SKIP_BENCH=1 TIMING_CFG="cfg4 cfg2" bash scripts/gpu_check.sh
RS_MC_WM=1 timeout 300 python scripts/gpu_timing.py --cfg cfg4 > gpurun_out/timing_cfg4_wm1.json 2>&1
grep -A1 '"gemm_power_c"' gpurun_out/timing_cfg4_wm1.json | tail -1; grep -A1 '"gemm_sample"' gpurun_out/timing_cfg4_wm1.json | tail -1
