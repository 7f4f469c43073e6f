#!/bin/bash
# r02 check 17: TSA with all loads of a k-step issued before its DMMAs and an incremental ring slot
mkdir -p gpurun_out
python __graft_entry__.py build > gpurun_out/build.log 2>&1 || { tail -30 gpurun_out/build.log; exit 1; }
for m in 1000000 125000; do
  timeout 300 python scripts/gpu_timing.py --cfg cfg4 --m $m 2>&1 | python -c "
import sys,json; t=sys.stdin.read(); j=json.loads(t[t.index('{'):]); print('m=$m', {k: round(v['ms_per_rep'],3) for k,v in j.items() if isinstance(v,dict)})"
done
timeout 900 python -m pytest tests/test_gpu_parity.py tests/test_gpu_adaptive.py -q -x -k "ragged or cfg1 or graph or adaptive or wide" > gpurun_out/r02_gpu_tests17.log 2>&1; echo "tests rc=$?"; tail -2 gpurun_out/r02_gpu_tests17.log
timeout 600 ncu --metrics gpu__time_duration.sum,sm__inst_executed_pipe_tensor_subpipe_dmma.avg.pct_of_peak_sustained_active --clock-control none -k regex:tsa_kernel -c 1 --csv python scripts/gpu_timing.py --cfg cfg4 --reps 1 2>/dev/null | grep -E "gpu__time|dmma" | cut -d, -f12-
