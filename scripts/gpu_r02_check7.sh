#!/bin/bash
# r02 check 7: ring chunk size / depth sweep; ncu of the chosen variant exported to CSV on the box
mkdir -p gpurun_out
for flags in "-DRS_RG_CH=128 -DRS_RG_R=8" "-DRS_RG_CH=256 -DRS_RG_R=8" "-DRS_RG_CH=128 -DRS_RG_R=4"; do
  export RS_EXTRA_NVCC_FLAGS="$flags"
  python __graft_entry__.py build > gpurun_out/build.log 2>&1 || { tail -30 gpurun_out/build.log; exit 1; }
  for m in 1000000 125000; do
    timeout 300 python scripts/gpu_timing.py --cfg cfg4 --m $m 2>&1 | python -c "
import sys,json; t=sys.stdin.read(); j=json.loads(t[t.index('{'):]); print('[$flags] m=$m', {k: round(v['ms_per_rep'],3) for k,v in j.items() if isinstance(v,dict) and k.startswith('gemm')})"
  done
done
export RS_EXTRA_NVCC_FLAGS="-DRS_RG_CH=256"
python __graft_entry__.py build > gpurun_out/build.log 2>&1
timeout 900 ncu --set full --clock-control none --import-source on -k regex:kc_sample_ring -c 1 -o /tmp/r02_ncu_ring python scripts/gpu_timing.py --cfg cfg4 --m 125000 --reps 1 > gpurun_out/r02_ncu_ring.log 2>&1; echo "ncu rc=$?"
ncu -i /tmp/r02_ncu_ring.ncu-rep --page raw --csv > gpurun_out/r02_ncu_ring_m125k_raw.csv 2>/dev/null
ncu -i /tmp/r02_ncu_ring.ncu-rep --page source --csv --print-source sass > gpurun_out/r02_ncu_ring_m125k_src.csv 2>/dev/null
ls -la gpurun_out/*.csv
