#!/bin/bash
# r02 evidence: GPU suite, smoke, cfg4 bench line (+ cfg2/cfg3), ncu launch list of one step and a
# full capture of the dominant kernel (exported to CSV on the box), per-rank slices
mkdir -p gpurun_out
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv,noheader
python __graft_entry__.py build > gpurun_out/build.log 2>&1 || { tail -30 gpurun_out/build.log; exit 1; }
RS_PARITY_LOG=gpurun_out/r02_parity_final.jsonl timeout 2700 python -m pytest tests -q -m gpu -rA > gpurun_out/r02_gpu_tests_final.log 2>&1; echo "tests rc=$?"; tail -2 gpurun_out/r02_gpu_tests_final.log; grep -E "^FAILED|^ERROR" gpurun_out/r02_gpu_tests_final.log | head
timeout 300 python __graft_entry__.py > gpurun_out/r02_smoke_final.log 2>&1; echo "smoke rc=$?"; tail -1 gpurun_out/r02_smoke_final.log
timeout 900 python bench.py > gpurun_out/r02_bench_final.json 2> gpurun_out/r02_bench_final.err; echo "bench rc=$?"; head -c 600 gpurun_out/r02_bench_final.json; echo
for c in cfg2 cfg3; do timeout 600 python bench.py --workload $c --no-cpu-baseline > gpurun_out/r02_bench_$c.json 2>/dev/null; echo "bench $c rc=$?"; head -c 300 gpurun_out/r02_bench_$c.json; echo; done
timeout 600 python bench.py --impl reference --steps 1 --warmup 3 > gpurun_out/r02_bench_reference.json 2>/dev/null; echo "ref rc=$?"; head -c 300 gpurun_out/r02_bench_reference.json; echo
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none --kernel-name-base demangled --kernel-name regex:'rs::' --csv --log-file gpurun_out/r02_launches_cfg4.csv python bench.py --steps 1 --warmup 3 --no-e2e --no-cpu-baseline > gpurun_out/r02_ncu_bench.log 2>&1; echo "ncu launches rc=$?"
timeout 900 ncu --set full --clock-control none --import-source on -k regex:kc_sample_ring -c 1 -o /tmp/r02_ring python scripts/gpu_timing.py --cfg cfg4 --reps 1 > gpurun_out/r02_ncu_ring_cfg4.log 2>&1; echo "ncu full rc=$?"
ncu -i /tmp/r02_ring.ncu-rep --page raw --csv > gpurun_out/r02_ncu_ring_cfg4_raw.csv 2>/dev/null
timeout 600 python scripts/rank_slice.py --cfg cfg4 --ranks 1 2 4 8 > gpurun_out/r02_rank_slices_final.jsonl 2>/dev/null; echo "slices rc=$?"; cut -c1-200 gpurun_out/r02_rank_slices_final.jsonl
