#!/bin/bash
mkdir -p gpurun_out
SKIP_BENCH=1 TIMING_CFG="cfg4 cfg2" bash scripts/gpu_check.sh
RS_MC_NO_TMA3D=1 timeout 300 python scripts/gpu_timing.py --cfg cfg4 2>&1 | python -c "
import sys,json; t=sys.stdin.read(); j=json.loads(t[t.index('{'):]); print('no-3d', {k: round(v['ms_per_rep'],3) for k,v in j.items() if isinstance(v,dict)})"
