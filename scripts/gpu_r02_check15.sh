#!/bin/bash
# r02 check 15: ncu --set full of the KC and MC GEMMs, TSA and SYRK at cfg4 (CSV exported on the box)
mkdir -p gpurun_out
python __graft_entry__.py build > gpurun_out/build.log 2>&1 || exit 1
timeout 1500 ncu --set full --clock-control none --import-source on -k regex:"kc_gemm_pwg|mc_gemm_pwg|tsa_kernel|syrk_kernel" -c 4 -o /tmp/r02_k python scripts/gpu_timing.py --cfg cfg4 --reps 1 > gpurun_out/r02_ncu_k.log 2>&1; echo "ncu rc=$?"
ncu -i /tmp/r02_k.ncu-rep --page raw --csv > gpurun_out/r02_ncu_k_raw.csv 2>/dev/null
ncu -i /tmp/r02_k.ncu-rep --page source --csv --print-source sass > gpurun_out/r02_ncu_k_src.csv 2>/dev/null
ls -la gpurun_out/r02_ncu_k*
