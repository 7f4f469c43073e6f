#!/bin/bash
# r02 experiment: split count of the tail-fold KC GEMM (B := C~ A), forced by -DRS_DEV_KC_S
mkdir -p gpurun_out
for flags in "" "-DRS_DEV_KC_S=34" "-DRS_DEV_KC_S=30" "-DRS_DEV_KC_S=53" ""; do
  export RS_EXTRA_NVCC_FLAGS="$flags"
  python __graft_entry__.py build > gpurun_out/build.log 2>&1 || { tail -30 gpurun_out/build.log; exit 1; }
  for c in cfg4 cfg2; do
    timeout 300 python scripts/gpu_timing.py --cfg $c --reps 3 2>&1 | python -c "
import sys,json; t=sys.stdin.read(); j=json.loads(t[t.index('{'):]); print('[$flags] $c', {k: round(v['ms_per_rep'],3) for k,v in j.items() if isinstance(v,dict) and k in ('gemm_power_b','reduce')})"
  done
done
