#!/bin/bash
# r02 check 9: ring L2 cache hints (A evict-first, Omega chunks evict-last) vs none: time + DRAM bytes;
# QRCP with cooperative_groups grid sync vs the counter barrier
mkdir -p gpurun_out
for flags in "" "-DRS_DEV_RING_NO_HINTS" "-DRS_DEV_QRCP_CGSYNC"; do
  export RS_EXTRA_NVCC_FLAGS="$flags"
  python __graft_entry__.py build > gpurun_out/build.log 2>&1 || { tail -30 gpurun_out/build.log; exit 1; }
  for m in 1000000 125000; do
    timeout 300 python scripts/gpu_timing.py --cfg cfg4 --m $m 2>&1 | python -c "
import sys,json; t=sys.stdin.read(); j=json.loads(t[t.index('{'):]); print('[$flags] m=$m', {k: round(v['ms_per_rep'],3) for k,v in j.items() if isinstance(v,dict) and k in ('gemm_sample','qrcp','reduce')})"
  done
  if [ "$flags" != "-DRS_DEV_QRCP_CGSYNC" ]; then
    timeout 600 ncu --metrics dram__bytes_read.sum,dram__bytes_write.sum,gpu__time_duration.sum --clock-control none -k regex:kc_sample_ring -c 1 --csv python scripts/gpu_timing.py --cfg cfg4 --reps 1 2>/dev/null | grep -E "dram__|gpu__time" | cut -d, -f12- | sed "s/^/[$flags] /"
  fi
done
