#!/bin/bash
# r02 probe 1: overlapped multi-rank bisect (20 fresh processes) + racecheck/synccheck of one small pipeline
mkdir -p gpurun_out
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv
python __graft_entry__.py build > gpurun_out/build.log 2>&1 || { tail -20 gpurun_out/build.log; exit 1; }
timeout 1500 python scripts/mr_overlap_probe.py --procs 20 > gpurun_out/r02_mr_probe.log 2>&1; echo "probe rc=$?"
grep SUMMARY gpurun_out/r02_mr_probe.log
timeout 900 compute-sanitizer --tool racecheck --racecheck-report all python scripts/sanitize_run.py > gpurun_out/r02_racecheck.log 2>&1; echo "racecheck rc=$?"; tail -5 gpurun_out/r02_racecheck.log
timeout 600 compute-sanitizer --tool synccheck python scripts/sanitize_run.py > gpurun_out/r02_synccheck.log 2>&1; echo "synccheck rc=$?"; tail -5 gpurun_out/r02_synccheck.log
