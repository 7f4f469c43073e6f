#!/bin/bash
mkdir -p gpurun_out
bash scripts/gpu_check.sh
for cs in 2 4; do
  RS_PHILOX_CLUSTER=$cs timeout 300 python scripts/gpu_timing.py --cfg cfg4 > gpurun_out/timing_cs$cs.json 2>&1
  echo "cs=$cs"; grep -A3 '"gemm_sample"' gpurun_out/timing_cs$cs.json | head -4
done
timeout 600 ncu --metrics gpu__time_duration.sum --clock-control none -c 200 --csv --log-file gpurun_out/launches_cfg4.csv python bench.py --steps 1 --warmup 1 --no-e2e --no-cpu-baseline > gpurun_out/ncu_bench.log 2>&1; echo "ncu rc=$?"
