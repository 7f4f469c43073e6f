#!/bin/bash
# r02 check 6: ring sample GEMM chunk size (RS_RG_CH) at cfg4 and at the N = 8 per-rank slice;
# ncu full capture of the ring kernel at cfg4
mkdir -p gpurun_out
for flags in "" "-DRS_RG_CH=256" "-DRS_RG_CH=1024 -DRS_RG_R=3"; do
  export RS_EXTRA_NVCC_FLAGS="$flags"
  python __graft_entry__.py build > gpurun_out/build.log 2>&1 || { tail -30 gpurun_out/build.log; exit 1; }
  for m in 1000000 125000; do
    timeout 300 python scripts/gpu_timing.py --cfg cfg4 --m $m 2>&1 | python -c "
import sys,json; t=sys.stdin.read(); j=json.loads(t[t.index('{'):]); print('[$flags] m=$m', {k: round(v['ms_per_rep'],3) for k,v in j.items() if isinstance(v,dict) and k.startswith('gemm')})"
  done
done
unset RS_EXTRA_NVCC_FLAGS
python __graft_entry__.py build > gpurun_out/build.log 2>&1
timeout 900 ncu --set full --clock-control none --import-source on -k regex:kc_sample_ring -c 1 -o gpurun_out/r02_ncu_ring_cfg4 python scripts/gpu_timing.py --cfg cfg4 --reps 1 > gpurun_out/r02_ncu_ring.log 2>&1; echo "ncu rc=$?"
timeout 900 ncu --set full --clock-control none --import-source on -k regex:kc_sample_ring -c 1 -o gpurun_out/r02_ncu_ring_m125k python scripts/gpu_timing.py --cfg cfg4 --m 125000 --reps 1 > gpurun_out/r02_ncu_ring2.log 2>&1; echo "ncu2 rc=$?"
