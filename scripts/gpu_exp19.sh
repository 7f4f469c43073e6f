#!/bin/bash
# QRCP v3 (REDUX top-2, batched flat staging, reciprocal reflector): GPU tests + phase timing
mkdir -p gpurun_out
python __graft_entry__.py build > gpurun_out/build.log 2>&1 || { tail -20 gpurun_out/build.log; exit 1; }
timeout 900 python -m pytest tests -q -m gpu -x > gpurun_out/gpu_tests19.log 2>&1; echo "tests rc=$?"; tail -3 gpurun_out/gpu_tests19.log
RS_QRCP_TIMING=1 timeout 300 python scripts/gpu_timing.py --cfg cfg2 --reps 2 2>&1 | grep "QRCP NB" | tail -1
RS_QRCP_TIMING=1 timeout 300 python scripts/gpu_timing.py --cfg cfg2 --m 50000 --n 2500 --k 54 --q 0 --reps 2 2>&1 | grep "QRCP NB" | tail -1
for c in cfg2; do
timeout 300 python scripts/gpu_timing.py --cfg $c 2>&1 | python -c "
import sys,json; t=sys.stdin.read(); j=json.loads(t[t.index('{'):]); print('$c', {k: round(v['ms_per_rep'],3) for k,v in j.items() if isinstance(v,dict)})"
done
timeout 300 python scripts/gpu_timing.py --cfg cfg2 --m 50000 --n 2500 --k 54 --q 0 2>&1 | python -c "
import sys,json; t=sys.stdin.read(); j=json.loads(t[t.index('{'):]); print('fig7', {k: round(v['ms_per_rep'],3) for k,v in j.items() if isinstance(v,dict)})"
