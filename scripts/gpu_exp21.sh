#!/bin/bash
# QRCP grid variants: counter barrier + records + winner column (default), per-record polling, 4 lanes, old barrier kernel
mkdir -p gpurun_out
python __graft_entry__.py build > gpurun_out/build.log 2>&1 || { tail -20 gpurun_out/build.log; exit 1; }
timeout 900 python -m pytest tests/test_gpu_parity.py -q -x > gpurun_out/gpu_tests21.log 2>&1; echo "tests rc=$?"; tail -2 gpurun_out/gpu_tests21.log
for v in "X=1" "RS_QRCP_POLL=1" "RS_QRCP_LPC4=1" "RS_QRCP_BARRIER=1"; do
  env $v RS_QRCP_TIMING=1 timeout 300 python scripts/gpu_timing.py --cfg cfg2 --reps 2 2>&1 | grep "QRCP" | tail -1
  env $v timeout 300 python scripts/gpu_timing.py --cfg cfg2 2>&1 | python -c "
import sys,json; t=sys.stdin.read(); j=json.loads(t[t.index('{'):]); print('cfg2 $v qrcp', round(j['qrcp']['ms_per_rep'],3))"
done
