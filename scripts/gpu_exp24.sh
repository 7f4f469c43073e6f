#!/bin/bash
# Producer waits with a suspend-time hint (NANOSLEEP.SYNCS) vs spinning (-DRS_NO_WAIT_HINT), crossed
# with the RS-BM32 production vs reference forms (-DRS_BM32_REF), cfg4 (+ cfg2); GPU tests first
mkdir -p gpurun_out
python __graft_entry__.py build > gpurun_out/build.log 2>&1 || { tail -20 gpurun_out/build.log; exit 1; }
timeout 1200 python -m pytest tests -q -m gpu -x > gpurun_out/gpu_tests24.log 2>&1; echo "tests rc=$?"; tail -2 gpurun_out/gpu_tests24.log
for flags in "" "-DRS_BM32_REF" "-DRS_NO_WAIT_HINT" "-DRS_NO_WAIT_HINT -DRS_BM32_REF"; do
  RS_EXTRA_NVCC_FLAGS="$flags" python __graft_entry__.py build > gpurun_out/build.log 2>&1 || { tail -20 gpurun_out/build.log; exit 1; }
  for c in cfg4 cfg2; do
    RS_EXTRA_NVCC_FLAGS="$flags" timeout 300 python scripts/gpu_timing.py --cfg $c 2>&1 | python -c "
import sys,json; t=sys.stdin.read(); j=json.loads(t[t.index('{'):]); print('[$flags] $c', {k: round(v['ms_per_rep'],3) for k,v in j.items() if isinstance(v,dict)})"
  done
done
