#!/bin/bash
# r02 check 18: ring generators' slot wait with relaxed polls (no CCTL.IVALL per try) vs acquire polls
mkdir -p gpurun_out
for flags in "" "-DRS_DEV_RING_ACQ_POLL" ""; do
  export RS_EXTRA_NVCC_FLAGS="$flags"
  python __graft_entry__.py build > gpurun_out/build.log 2>&1 || { tail -30 gpurun_out/build.log; exit 1; }
  for m in 1000000 125000; do
    timeout 300 python scripts/gpu_timing.py --cfg cfg4 --m $m 2>&1 | python -c "
import sys,json; t=sys.stdin.read(); j=json.loads(t[t.index('{'):]); print('[$flags] m=$m', {k: round(v['ms_per_rep'],3) for k,v in j.items() if isinstance(v,dict) and k in ('gemm_sample','gemm_power_b')})"
  done
done
unset RS_EXTRA_NVCC_FLAGS
python __graft_entry__.py build > gpurun_out/build.log 2>&1
timeout 600 python -m pytest tests/test_gpu_parity.py -q -x -k "sample or cfg4_full or graph" > gpurun_out/r02_gpu_tests18.log 2>&1; echo "tests rc=$?"; tail -2 gpurun_out/r02_gpu_tests18.log
