#!/bin/bash
# Round evidence: GPU tests, smoke, bench lines (cfg4 default, cfg2, cfg3), ncu launch list (cfg4),
# one ncu --set full capture of the dominant kernel (Philox-fused sample GEMM, cfg4).
mkdir -p gpurun_out
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv
python __graft_entry__.py build > gpurun_out/build.log 2>&1 || { tail -20 gpurun_out/build.log; exit 1; }
timeout 1500 python -m pytest tests -q -m gpu -x > gpurun_out/gpu_tests.log 2>&1; echo "tests rc=$?"; tail -2 gpurun_out/gpu_tests.log
timeout 300 python __graft_entry__.py > gpurun_out/smoke.log 2>&1; echo "smoke rc=$?"; tail -1 gpurun_out/smoke.log
timeout 900 python bench.py > gpurun_out/bench_cfg4.json 2> gpurun_out/bench_cfg4.err; echo "bench cfg4 rc=$?"; cut -c1-400 gpurun_out/bench_cfg4.json
timeout 600 python bench.py --workload cfg2 > gpurun_out/bench_cfg2.json 2> gpurun_out/bench_cfg2.err; echo "bench cfg2 rc=$?"; cut -c1-300 gpurun_out/bench_cfg2.json
timeout 600 python bench.py --workload cfg3 --no-cpu-baseline > gpurun_out/bench_cfg3.json 2> gpurun_out/bench_cfg3.err; echo "bench cfg3 rc=$?"; cut -c1-300 gpurun_out/bench_cfg3.json
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none --kernel-name-base demangled \
    --kernel-name regex:'rs::' --csv --log-file gpurun_out/launches_cfg4.csv \
    python bench.py --steps 1 --warmup 1 --no-e2e --no-cpu-baseline > gpurun_out/ncu_bench.log 2>&1
echo "ncu launches rc=$?"; python scripts/ncu_summary.py gpurun_out/launches_cfg4.csv | head -20
timeout 900 ncu --set full --clock-control none --import-source on -k regex:kc_philox -c 1 \
    -o gpurun_out/ncu_philox_cfg4 -f python scripts/gpu_timing.py --cfg cfg4 --reps 0 > gpurun_out/ncu_phx.log 2>&1
echo "ncu full rc=$?"
