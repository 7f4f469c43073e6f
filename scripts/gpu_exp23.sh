#!/bin/bash
# A/B at cfg4 in one session: RS-BM32 reference vs production forms, and GEMM ring depths
# (compile-time -DRS_BM32_REF / -DRS_PHX_NS / RS_KC_NS / RS_MC_NS), each timed twice
mkdir -p gpurun_out
for flags in "" "-DRS_BM32_REF" "-DRS_PHX_NS=5 -DRS_KC_NS=6 -DRS_MC_NS=6" "-DRS_PHX_NS=6 -DRS_KC_NS=7 -DRS_MC_NS=5"; do
  RS_EXTRA_NVCC_FLAGS="$flags" python __graft_entry__.py build > gpurun_out/build.log 2>&1 || { tail -20 gpurun_out/build.log; exit 1; }
  for rep in 1 2; do
    RS_EXTRA_NVCC_FLAGS="$flags" timeout 300 python scripts/gpu_timing.py --cfg cfg4 2>&1 | python -c "
import sys,json; t=sys.stdin.read(); j=json.loads(t[t.index('{'):]); print('[$flags]', {k: round(v['ms_per_rep'],3) for k,v in j.items() if isinstance(v,dict) and k.startswith('gemm')})"
  done
done
