#!/bin/bash
# r02 check 3: graph on an internal stream; full GPU suite (incl. sanitizers); cfg4 bench line
mkdir -p gpurun_out
python __graft_entry__.py build > gpurun_out/build.log 2>&1 || { tail -30 gpurun_out/build.log; exit 1; }
RS_PARITY_LOG=gpurun_out/r02_parity_log3.jsonl timeout 2700 python -m pytest tests -q -m gpu -rA > gpurun_out/r02_gpu_tests3.log 2>&1; echo "tests rc=$?"; tail -3 gpurun_out/r02_gpu_tests3.log; grep -E "^FAILED|^ERROR" gpurun_out/r02_gpu_tests3.log | head -10
timeout 300 python __graft_entry__.py > gpurun_out/r02_smoke.log 2>&1; echo "smoke rc=$?"; tail -1 gpurun_out/r02_smoke.log
timeout 900 python bench.py --steps 10 --warmup 3 > gpurun_out/r02_bench3.json 2> gpurun_out/r02_bench3.err; echo "bench rc=$?"; head -c 1200 gpurun_out/r02_bench3.json; echo; tail -3 gpurun_out/r02_bench3.err
