#!/bin/bash
# r02 check 8: blocked Cholesky (chol_b16_kernel) + ring polling back-off: GPU suite subset, timing
mkdir -p gpurun_out
python __graft_entry__.py build > gpurun_out/build.log 2>&1 || { tail -30 gpurun_out/build.log; exit 1; }
timeout 1800 python -m pytest tests -q -m gpu -x -k "not baseline_shapes and not cfg4_full and not racecheck" > gpurun_out/r02_gpu_tests8.log 2>&1; echo "tests rc=$?"; tail -2 gpurun_out/r02_gpu_tests8.log; grep -E "^E |^FAILED" gpurun_out/r02_gpu_tests8.log | head -8
for flags in "" "-DRS_DEV_CHOL_TILE"; do
  export RS_EXTRA_NVCC_FLAGS="$flags"
  python __graft_entry__.py build > gpurun_out/build.log 2>&1 || { tail -30 gpurun_out/build.log; exit 1; }
  for m in 1000000 125000; do
    timeout 300 python scripts/gpu_timing.py --cfg cfg4 --m $m 2>&1 | python -c "
import sys,json; t=sys.stdin.read(); j=json.loads(t[t.index('{'):]); print('[$flags] m=$m', {k: round(v['ms_per_rep'],3) for k,v in j.items() if isinstance(v,dict)})"
  done
done
