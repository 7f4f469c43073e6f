#!/bin/bash
# persistent MC warp-half mapping A/B (RS_MCP_WMAP) at cfg4 + parity of the interleaved mapping
mkdir -p gpurun_out
python __graft_entry__.py build > gpurun_out/build.log 2>&1 || { tail -20 gpurun_out/build.log; exit 1; }
RS_MCP_WMAP=1 timeout 900 python -m pytest tests/test_gpu_parity.py -q -x -k "multitile or wide" > gpurun_out/gpu_tests22.log 2>&1; echo "tests rc=$?"; tail -2 gpurun_out/gpu_tests22.log
for v in 0 1 0 1; do
RS_MCP_WMAP=$v timeout 300 python scripts/gpu_timing.py --cfg cfg4 2>&1 | python -c "
import sys,json; t=sys.stdin.read(); j=json.loads(t[t.index('{'):]); print('WMAP=$v', {k: round(v['ms_per_rep'],3) for k,v in j.items() if isinstance(v,dict)})"
done
