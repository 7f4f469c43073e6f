#!/bin/bash
mkdir -p gpurun_out
SKIP_BENCH=1 TIMING_CFG="cfg4 cfg2" bash scripts/gpu_check.sh
RS_QRCP_TIMING=1 timeout 300 python scripts/gpu_timing.py --cfg cfg2 --reps 1 2>&1 | grep QRCP
RS_MC_NO_PERSIST=1 timeout 300 python scripts/gpu_timing.py --cfg cfg4 2>&1 | python -c "
import sys,json; t=sys.stdin.read(); j=json.loads(t[t.index('{'):]); print('no-persist', {k: round(v['ms_per_rep'],3) for k,v in j.items() if isinstance(v,dict)})"
timeout 600 python scripts/bench_qp3.py --ms 50000 --reps 5 > gpurun_out/fig7.jsonl 2> gpurun_out/fig7.err; echo "fig7 rc=$?"; cat gpurun_out/fig7.jsonl
