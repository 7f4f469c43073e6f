#!/bin/bash
# RS-BM32 fast forms: exhaustive self-test + Omega/sample parity + cfg4 timing
mkdir -p gpurun_out
python __graft_entry__.py build > gpurun_out/build.log 2>&1 || { tail -20 gpurun_out/build.log; exit 1; }
timeout 600 python -m pytest tests/test_gpu_parity.py -q -x > gpurun_out/parity17.log 2>&1; echo "parity rc=$?"; tail -3 gpurun_out/parity17.log
for c in cfg4 cfg2; do
timeout 300 python scripts/gpu_timing.py --cfg $c 2>&1 | python -c "
import sys,json; t=sys.stdin.read(); j=json.loads(t[t.index('{'):]); print('$c', {k: round(v['ms_per_rep'],3) for k,v in j.items() if isinstance(v,dict)})"
done
