#!/bin/bash
# Philox-sample cluster size sweep at cfg4 (RS_PHILOX_CLUSTER = 1, 2, 4)
mkdir -p gpurun_out
python __graft_entry__.py build > gpurun_out/build.log 2>&1 || exit 1
for v in 1 2 4; do
  RS_PHILOX_CLUSTER=$v timeout 300 python scripts/gpu_timing.py --cfg cfg4 2>&1 | python -c "
import sys,json; t=sys.stdin.read(); j=json.loads(t[t.index('{'):]); print('CS=$v', {k: round(v['ms_per_rep'],3) for k,v in j.items() if isinstance(v,dict)})"
done
