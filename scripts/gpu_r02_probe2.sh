#!/bin/bash
# r02 probe 2: the r01 overlapped repro (test hook, token off) in 30 fresh processes; racecheck
# analysis per kernel; full GPU suite against the new fixed-order oracle
mkdir -p gpurun_out
python __graft_entry__.py build > gpurun_out/build.log 2>&1 || { tail -20 gpurun_out/build.log; exit 1; }
bad=0; ok=0
for i in $(seq 1 30); do
  RS_MR_OVERLAP=1 timeout 300 python -m pytest tests/test_gpu_multirank.py -q -x -k "test_multirank_pipeline_matches_oracle and 20000-1000" > gpurun_out/r02_ovl_$i.log 2>&1
  if [ $? -eq 0 ]; then ok=$((ok+1)); else bad=$((bad+1)); fi
done
echo "overlap repro: ok=$ok bad=$bad"
timeout 1200 compute-sanitizer --tool racecheck --racecheck-report analysis --print-limit 200 python scripts/sanitize_run.py > gpurun_out/r02_racecheck_analysis.log 2>&1; echo "racecheck rc=$?"; tail -3 gpurun_out/r02_racecheck_analysis.log
timeout 1500 python -m pytest tests -q -m gpu -x > gpurun_out/r02_gpu_tests.log 2>&1; echo "tests rc=$?"; tail -3 gpurun_out/r02_gpu_tests.log
