#!/bin/bash
# r02 experiment: split count of the tail-fold KC GEMM (B := C~ A): the time-model chooser against
# the old wave-score chooser (-DRS_DEV_KC_SPLITS_OLD), cfg4 / cfg2 / cfg3 and the cfg4 N = 8 slice
mkdir -p gpurun_out
for flags in "" "-DRS_DEV_KC_SPLITS_OLD" ""; do
  export RS_EXTRA_NVCC_FLAGS="$flags"
  python __graft_entry__.py build > gpurun_out/build.log 2>&1 || { tail -30 gpurun_out/build.log; exit 1; }
  for c in cfg4 cfg2 cfg3; do
    timeout 300 python scripts/gpu_timing.py --cfg $c --reps 3 2>&1 | python -c "
import sys,json; t=sys.stdin.read(); j=json.loads(t[t.index('{'):]); print('[$flags] $c', {k: round(v['ms_per_rep'],3) for k,v in j.items() if isinstance(v,dict) and k in ('gemm_power_b','reduce')})"
  done
  timeout 300 python scripts/rank_slice.py --cfg cfg4 --ranks 8 2>/dev/null | python -c "
import sys,json
for l in sys.stdin:
  if l.startswith('{'): j=json.loads(l); print('[$flags] slice8', round(j['ms_per_step'],3), round(j['phases_ms']['gemm_power_b'],3))"
done
