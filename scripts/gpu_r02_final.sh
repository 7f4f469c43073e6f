#!/bin/bash
# r02 evidence: GPU suite, smoke, cfg4 bench line (+ cfg2/cfg3), the reference (oracle) arm, ncu
# launch list of one step, full ncu captures of the dominant kernel and of the tail-fold KC GEMM
# (exported to CSV on the box), per-rank slices.  Output names carry the tag $1 (default r02).
T=${1:-r02}
mkdir -p gpurun_out
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv,noheader
python __graft_entry__.py build > gpurun_out/build.log 2>&1 || { tail -30 gpurun_out/build.log; exit 1; }
RS_PARITY_LOG=gpurun_out/${T}_parity.jsonl timeout 2700 python -m pytest tests -q -m gpu -rA > gpurun_out/${T}_gpu_tests.log 2>&1; echo "tests rc=$?"; tail -2 gpurun_out/${T}_gpu_tests.log; grep -E "^FAILED|^ERROR" gpurun_out/${T}_gpu_tests.log | head
timeout 300 python __graft_entry__.py > gpurun_out/${T}_smoke.log 2>&1; echo "smoke rc=$?"; tail -1 gpurun_out/${T}_smoke.log
timeout 900 python bench.py > gpurun_out/${T}_bench_cfg4.json 2> gpurun_out/${T}_bench_cfg4.err; echo "bench rc=$?"; head -c 600 gpurun_out/${T}_bench_cfg4.json; echo
for c in cfg2 cfg3; do timeout 600 python bench.py --workload $c --no-cpu-baseline > gpurun_out/${T}_bench_$c.json 2>/dev/null; echo "bench $c rc=$?"; head -c 300 gpurun_out/${T}_bench_$c.json; echo; done
timeout 600 python bench.py --impl reference --steps 1 --warmup 3 > gpurun_out/${T}_bench_reference_cfg4.json 2>/dev/null; echo "ref rc=$?"; head -c 300 gpurun_out/${T}_bench_reference_cfg4.json; echo
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none --kernel-name-base demangled --kernel-name regex:'rs::' --csv --log-file gpurun_out/${T}_launches_cfg4.csv python bench.py --steps 1 --warmup 3 --no-e2e --no-cpu-baseline > gpurun_out/${T}_ncu_bench.log 2>&1; echo "ncu launches rc=$?"
timeout 900 ncu --set full --clock-control none --import-source on -k regex:kc_sample_ring -c 1 -o /tmp/${T}_ring python scripts/gpu_timing.py --cfg cfg4 --reps 1 > gpurun_out/${T}_ncu_ring.log 2>&1; echo "ncu ring rc=$?"
ncu -i /tmp/${T}_ring.ncu-rep --page raw --csv > gpurun_out/${T}_ncu_ring_cfg4_raw.csv 2>/dev/null
timeout 900 ncu --set full --clock-control none --import-source on -k regex:kc_gemm_pwg -c 1 -o /tmp/${T}_kc python scripts/gpu_timing.py --cfg cfg4 --reps 1 > gpurun_out/${T}_ncu_kc.log 2>&1; echo "ncu kc rc=$?"
ncu -i /tmp/${T}_kc.ncu-rep --page raw --csv > gpurun_out/${T}_ncu_kc_cfg4_raw.csv 2>/dev/null
timeout 600 python scripts/rank_slice.py --cfg cfg4 --ranks 1 2 4 8 > gpurun_out/${T}_rank_slices.jsonl 2> gpurun_out/${T}_rank_slices.err; echo "slices rc=$?"; cut -c1-200 gpurun_out/${T}_rank_slices.jsonl
