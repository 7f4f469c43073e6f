#!/bin/bash
# QRCP flag kernel: GPU tests + phase timing + A/B against the barrier kernel
mkdir -p gpurun_out
python __graft_entry__.py build > gpurun_out/build.log 2>&1 || { tail -20 gpurun_out/build.log; exit 1; }
timeout 900 python -m pytest tests -q -m gpu -x > gpurun_out/gpu_tests20.log 2>&1; echo "tests rc=$?"; tail -3 gpurun_out/gpu_tests20.log
RS_QRCP_TIMING=1 timeout 300 python scripts/gpu_timing.py --cfg cfg2 --reps 2 2>&1 | grep "QRCP" | tail -1
RS_QRCP_TIMING=1 RS_QRCP_BARRIER=1 timeout 300 python scripts/gpu_timing.py --cfg cfg2 --reps 2 2>&1 | grep "QRCP" | tail -1
for v in "" "RS_QRCP_BARRIER=1"; do
env $v timeout 300 python scripts/gpu_timing.py --cfg cfg2 2>&1 | python -c "
import sys,json; t=sys.stdin.read(); j=json.loads(t[t.index('{'):]); print('cfg2 $v', {k: round(v['ms_per_rep'],3) for k,v in j.items() if isinstance(v,dict)})"
done
