#!/bin/bash
# r02 check 10: source-level ncu of the latency-bound small kernels at cfg4 (Cholesky, QRCP)
mkdir -p gpurun_out
python __graft_entry__.py build > gpurun_out/build.log 2>&1 || exit 1
timeout 900 ncu --set full --clock-control none --import-source on -k regex:"chol_tile|qrcp_flag" -c 2 -o /tmp/r02_small python scripts/gpu_timing.py --cfg cfg4 --m 125000 --reps 1 > gpurun_out/r02_ncu_small.log 2>&1; echo "ncu rc=$?"
ncu -i /tmp/r02_small.ncu-rep --page raw --csv > gpurun_out/r02_ncu_small_raw.csv 2>/dev/null
ncu -i /tmp/r02_small.ncu-rep --page source --csv --print-source sass > gpurun_out/r02_ncu_small_src.csv 2>/dev/null
ls -la gpurun_out/r02_ncu_small*
