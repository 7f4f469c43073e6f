#!/bin/bash
# r02: KC tail fold on the producer warpgroup's idle warps -- parity, then A/B timing against
# -DRS_DEV_NO_TAIL on the same box (cfg4 / cfg2 / cfg3)
mkdir -p gpurun_out
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv,noheader
python __graft_entry__.py build > gpurun_out/build.log 2>&1 || { tail -30 gpurun_out/build.log; exit 1; }
timeout 1200 python -m pytest tests/test_gpu_parity.py -q -x -k "tail or ragged_and_multitile or baseline_shapes or cfg4_full or deterministic or graph" > gpurun_out/r02_tail_tests.log 2>&1; echo "tests rc=$?"; tail -3 gpurun_out/r02_tail_tests.log
for flags in "" "-DRS_DEV_NO_TAIL" ""; do
  export RS_EXTRA_NVCC_FLAGS="$flags"
  python __graft_entry__.py build > gpurun_out/build.log 2>&1 || { tail -30 gpurun_out/build.log; exit 1; }
  for c in cfg4 cfg2 cfg3; do
    timeout 300 python scripts/gpu_timing.py --cfg $c --reps 3 2>&1 | python -c "
import sys,json; t=sys.stdin.read(); j=json.loads(t[t.index('{'):]); print('[$flags] $c', {k: round(v['ms_per_rep'],3) for k,v in j.items() if isinstance(v,dict) and 'ms_per_rep' in v})"
  done
done
