#!/bin/bash
# r02 check 14: fenced slot release in every ring kernel (TSA, SYRK, ring sample, KC) vs deferred
mkdir -p gpurun_out
for flags in "" "-DRS_RELEASE_FENCE_ALL -DRS_RELEASE_FENCE"; do
  export RS_EXTRA_NVCC_FLAGS="$flags"
  python __graft_entry__.py build > gpurun_out/build.log 2>&1 || { tail -30 gpurun_out/build.log; exit 1; }
  for m in 1000000 125000; do
    timeout 300 python scripts/gpu_timing.py --cfg cfg4 --m $m 2>&1 | python -c "
import sys,json; t=sys.stdin.read(); j=json.loads(t[t.index('{'):]); print('[$flags] m=$m', {k: round(v['ms_per_rep'],3) for k,v in j.items() if isinstance(v,dict) and k in ('gemm_sample','gemm_power_c','gemm_power_b','gram','apply','factor')})"
  done
done
export RS_EXTRA_NVCC_FLAGS="-DRS_RELEASE_FENCE_ALL -DRS_RELEASE_FENCE"
python __graft_entry__.py build > gpurun_out/build.log 2>&1
timeout 1200 python -m pytest tests/test_gpu_parity.py tests/test_gpu_multirank.py -q -x -k "not baseline_shapes and not cfg4_full" > gpurun_out/r02_gpu_tests14.log 2>&1; echo "tests(fence) rc=$?"; tail -2 gpurun_out/r02_gpu_tests14.log
