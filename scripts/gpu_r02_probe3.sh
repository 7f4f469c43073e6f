#!/bin/bash
# r02 probe 3: does the r01 overlap defect come back with the r01-default (non-producer-warpgroup)
# KC / MC GEMM kernels?  The r01 library (tree .r01 = commit 76c4c9a, runtime A/B switches), 30
# fresh processes per variant, RS_MR_OVERLAP=1 (the ranks' kernels overlap on the one GPU)
mkdir -p gpurun_out
cd .r01
python __graft_entry__.py build > ../gpurun_out/build_r01.log 2>&1 || { tail -20 ../gpurun_out/build_r01.log; exit 1; }
for v in "RS_KC_NO_PWG=1 RS_MC_NO_PWG=1" "RS_KC_NO_PWG=1" "RS_MC_NO_PWG=1"; do
  bad=0; ok=0; tag=$(echo $v | tr -d ' =_')
  for i in $(seq 1 30); do
    env $v RS_MR_OVERLAP=1 timeout 300 python -m pytest tests/test_gpu_multirank.py -q -x -k "test_multirank_pipeline_matches_oracle and 20000-1000" > ../gpurun_out/r02_ovl_${tag}_$i.log 2>&1
    if [ $? -eq 0 ]; then ok=$((ok+1)); else bad=$((bad+1)); fi
  done
  echo "[$v] overlap repro: ok=$ok bad=$bad"
done
