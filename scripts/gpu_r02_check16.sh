#!/bin/bash
# r02 check 16: ncu --set full of the KC GEMM (B = C~A), the ring sample GEMM and TSA at cfg4
mkdir -p gpurun_out
python __graft_entry__.py build > gpurun_out/build.log 2>&1 || exit 1
for k in kc_gemm_pwg kc_sample_ring tsa_kernel; do
  timeout 900 ncu --set full --clock-control none --import-source on -k regex:$k -c 1 -o /tmp/r02_$k python scripts/gpu_timing.py --cfg cfg4 --reps 1 > gpurun_out/r02_ncu_$k.log 2>&1; echo "ncu $k rc=$?"
  ncu -i /tmp/r02_$k.ncu-rep --page raw --csv > gpurun_out/r02_ncu_${k}_raw.csv 2>/dev/null
  ncu -i /tmp/r02_$k.ncu-rep --page source --csv --print-source sass > gpurun_out/r02_ncu_${k}_src.csv 2>/dev/null
done
ls -la gpurun_out/r02_ncu_*_raw.csv
