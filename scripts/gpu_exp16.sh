#!/bin/bash
# Per-rank slices of cfg4 (m = 1e6 / N) for the 2/4/8-GPU projection + ncu of the persistent MC
mkdir -p gpurun_out
python __graft_entry__.py build > gpurun_out/build.log 2>&1 || exit 1
for mm in 500000 250000 125000; do
  timeout 300 python scripts/gpu_timing.py --cfg cfg4 --m $mm > gpurun_out/slice_$mm.json 2>&1
  grep "rep 3" gpurun_out/slice_$mm.json
  python -c "
import json; t=open('gpurun_out/slice_$mm.json').read(); j=json.loads(t[t.index('{'):]); print('m=$mm', {k: round(v['ms_per_rep'],3) for k,v in j.items() if isinstance(v,dict)})"
done
timeout 600 ncu --set full --clock-control none --import-source on -k regex:mc_persist -c 1 \
    -o gpurun_out/ncu_mc_persist_cfg4 -f python scripts/gpu_timing.py --cfg cfg4 --reps 0 > gpurun_out/ncu_mcp.log 2>&1
echo "ncu mcp rc=$?"
