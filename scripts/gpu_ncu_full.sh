#!/bin/bash
# ncu --set full captures of the GEMM kernels at cfg2 (one launch each) -> gpurun_out/ncu_*.ncu-rep
mkdir -p gpurun_out
python __graft_entry__.py build > gpurun_out/build.log 2>&1 || exit 1
CFG=${CFG:-cfg2}
for kn in ${KERNELS:-kc_philox_kernel mc_gemm_kernel kc_gemm_kernel syrk_kernel}; do
  timeout 600 ncu --set full --clock-control none --import-source on -k regex:$kn -c 1 \
    -o gpurun_out/ncu_${kn}_$CFG -f python scripts/gpu_timing.py --cfg $CFG --reps 0 > gpurun_out/ncu_${kn}.log 2>&1
  echo "$kn rc=$?"
done
ls -la gpurun_out/*.ncu-rep
