#!/bin/bash
mkdir -p gpurun_out
SKIP_BENCH=1 TIMING_CFG="cfg2 cfg4" bash scripts/gpu_check.sh
for gm in 1 2; do
  RS_PHILOX_GENMODE=$gm timeout 300 python scripts/gpu_timing.py --cfg cfg4 > gpurun_out/timing_genmode$gm.json 2>&1
  echo "genmode $gm"; grep -A1 '"gemm_sample"' gpurun_out/timing_genmode$gm.json | tail -1
done
timeout 600 ncu --set full --clock-control none --import-source on -k regex:mc_gemm_kernel -s 2 -c 1 \
    -o gpurun_out/ncu_mc_gemm_kernel_cfg2 -f python scripts/gpu_timing.py --cfg cfg2 --reps 0 > gpurun_out/ncu_mc.log 2>&1
echo "ncu mc rc=$?"
timeout 600 ncu --set full --clock-control none --import-source on -k regex:chol_tile -c 1 \
    -o gpurun_out/ncu_chol_tile_cfg2 -f python scripts/gpu_timing.py --cfg cfg2 --reps 0 > gpurun_out/ncu_chol.log 2>&1
echo "ncu chol rc=$?"
