#!/bin/bash
# r02 check 12: tile Cholesky with 1/sqrt(d_k) formed once by the publisher vs by every thread
mkdir -p gpurun_out
python __graft_entry__.py build > gpurun_out/build.log 2>&1 || { tail -30 gpurun_out/build.log; exit 1; }
timeout 1200 python -m pytest tests/test_gpu_parity.py tests/test_gpu_fallback.py -q -x -k "cfg1 or ragged or fallback or rank_deficient or exact" > gpurun_out/r02_gpu_tests12.log 2>&1; echo "tests rc=$?"; tail -2 gpurun_out/r02_gpu_tests12.log; grep -E "^E " gpurun_out/r02_gpu_tests12.log | head -5
for flags in "" "-DRS_DEV_CHOL_RSQRT_ALL"; do
  export RS_EXTRA_NVCC_FLAGS="$flags"
  python __graft_entry__.py build > gpurun_out/build.log 2>&1 || exit 1
  for c in cfg4 cfg3; do
  timeout 300 python scripts/gpu_timing.py --cfg $c 2>&1 | python -c "
import sys,json; t=sys.stdin.read(); j=json.loads(t[t.index('{'):]); print('[$flags] $c', {k: round(v['ms_per_rep'],3) for k,v in j.items() if isinstance(v,dict) and k in ('chol','qrcp','other','apply')})"
  done
done
