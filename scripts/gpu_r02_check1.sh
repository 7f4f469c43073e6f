#!/bin/bash
# r02 check 1: the deferred ring-slot release: overlapped multi-rank repro with the
# default kernels and with the non-producer-warpgroup KC kernel that failed 6-8/30 before the fix;
# then the GPU suite, smoke and a cfg4 bench line
mkdir -p gpurun_out
for flags in "-DRS_DEV_KC_NO_PWG" ""; do
  export RS_EXTRA_NVCC_FLAGS="$flags"
  python __graft_entry__.py build > gpurun_out/build.log 2>&1 || { tail -30 gpurun_out/build.log; exit 1; }
  bad=0; ok=0; tag=$(echo "x$flags" | tr -d ' -=')
  for i in $(seq 1 30); do
    timeout 300 python -m pytest tests/test_gpu_multirank.py -q -x -k "test_multirank_pipeline_matches_oracle and 20000-1000" > gpurun_out/r02_fix_${tag}_$i.log 2>&1
    if [ $? -eq 0 ]; then ok=$((ok+1)); else bad=$((bad+1)); fi
  done
  echo "[$flags] overlapped multirank after the fix: ok=$ok bad=$bad"
done
unset RS_EXTRA_NVCC_FLAGS
python __graft_entry__.py build > gpurun_out/build.log 2>&1 || exit 1
RS_PARITY_LOG=gpurun_out/r02_parity_log.jsonl timeout 2400 python -m pytest tests -q -m gpu -x -rA > gpurun_out/r02_gpu_tests.log 2>&1; echo "tests rc=$?"; tail -5 gpurun_out/r02_gpu_tests.log
timeout 300 python __graft_entry__.py > gpurun_out/r02_smoke.log 2>&1; echo "smoke rc=$?"; tail -1 gpurun_out/r02_smoke.log
timeout 900 python bench.py --steps 10 --warmup 3 > gpurun_out/r02_bench.json 2> gpurun_out/r02_bench.err; echo "bench rc=$?"; cat gpurun_out/r02_bench.json | head -c 1500; tail -3 gpurun_out/r02_bench.err
