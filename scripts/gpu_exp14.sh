#!/bin/bash
mkdir -p gpurun_out
python __graft_entry__.py build > gpurun_out/build.log 2>&1 || exit 1
timeout 600 python -m pytest tests -q -m gpu -x > gpurun_out/gpu_tests.log 2>&1; echo "tests rc=$?"; tail -2 gpurun_out/gpu_tests.log
timeout 600 ncu --set full --clock-control none --import-source on -k regex:qrcp_cluster -c 1 \
    -o gpurun_out/ncu_qrcp_cluster_fig7 -f python scripts/gpu_timing.py --cfg cfg2 --m 50000 --n 2500 --k 54 --q 0 --reps 0 > gpurun_out/ncu_qc.log 2>&1
echo "ncu qc rc=$?"
timeout 600 ncu --set full --clock-control none --import-source on -k regex:chol_tile -c 1 \
    -o gpurun_out/ncu_chol_tile2 -f python scripts/gpu_timing.py --cfg cfg2 --reps 0 > gpurun_out/ncu_ct.log 2>&1
echo "ncu ct rc=$?"
for v in "" "RS_KC_PWG=1" "RS_CHOL_TPT=2"; do
  env $v timeout 300 python scripts/gpu_timing.py --cfg cfg4 2>&1 | python -c "
import sys,json; t=sys.stdin.read(); j=json.loads(t[t.index('{'):]); print('$v', {k: round(v['ms_per_rep'],3) for k,v in j.items() if isinstance(v,dict)})"
done
