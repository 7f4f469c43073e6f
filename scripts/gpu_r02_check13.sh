#!/bin/bash
# r02 check 13: ring slot released at the end of its own stage behind a CTA fence (MEMBAR.CTA waits for
# the warp's outstanding LDS) instead of one stage later: timing, and the overlap stress on the
# MMA-warp-issuer KC kernel that exposed the race
mkdir -p gpurun_out
for flags in "" "-DRS_RELEASE_FENCE"; do
  export RS_EXTRA_NVCC_FLAGS="$flags"
  python __graft_entry__.py build > gpurun_out/build.log 2>&1 || { tail -30 gpurun_out/build.log; exit 1; }
  for m in 1000000 125000; do
    timeout 300 python scripts/gpu_timing.py --cfg cfg4 --m $m 2>&1 | python -c "
import sys,json; t=sys.stdin.read(); j=json.loads(t[t.index('{'):]); print('[$flags] m=$m', {k: round(v['ms_per_rep'],3) for k,v in j.items() if isinstance(v,dict) and k.startswith('gemm')})"
  done
done
export RS_EXTRA_NVCC_FLAGS="-DRS_RELEASE_FENCE -DRS_DEV_KC_NO_PWG"
python __graft_entry__.py build > gpurun_out/build.log 2>&1 || exit 1
bad=0; ok=0
for i in $(seq 1 30); do
  timeout 300 python -m pytest tests/test_gpu_multirank.py -q -x -k "test_multirank_pipeline_matches_oracle and 20000-1000" > gpurun_out/r02_fence_$i.log 2>&1
  if [ $? -eq 0 ]; then ok=$((ok+1)); else bad=$((bad+1)); fi
done
echo "[$RS_EXTRA_NVCC_FLAGS] overlapped multirank: ok=$ok bad=$bad"
