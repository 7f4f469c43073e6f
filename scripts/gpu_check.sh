#!/bin/bash
# Round GPU check (run under gpurun from the repo root): build, GPU tests, smoke, bench.
# Outputs land in gpurun_out/ (merged back by gpurun).
mkdir -p gpurun_out
nvidia-smi --query-gpu=name,clocks.sm,clocks.max.sm --format=csv
python __graft_entry__.py build > gpurun_out/build.log 2>&1 || { tail -20 gpurun_out/build.log; exit 1; }
if [ "${SKIP_TESTS:-0}" != 1 ]; then
  timeout ${TEST_TIMEOUT:-1500} python -m pytest tests -q -m gpu -x ${PYTEST_ARGS:-} > gpurun_out/gpu_tests.log 2>&1
  echo "tests rc=$?"; tail -5 gpurun_out/gpu_tests.log
  timeout 300 python __graft_entry__.py > gpurun_out/smoke.log 2>&1; echo "smoke rc=$?"; tail -2 gpurun_out/smoke.log
fi
if [ "${SKIP_BENCH:-0}" != 1 ]; then
  timeout 900 python bench.py ${BENCH_ARGS:-} > gpurun_out/bench.json 2> gpurun_out/bench.err
  echo "bench rc=$?"; cat gpurun_out/bench.json; tail -3 gpurun_out/bench.err
fi
if [ -n "${TIMING_CFG:-}" ]; then
  for c in $TIMING_CFG; do
    timeout 300 python scripts/gpu_timing.py --cfg $c > gpurun_out/timing_$c.json 2>&1; echo "timing $c rc=$?"
    python - "$c" <<'PY'
import json, sys
t = open(f"gpurun_out/timing_{sys.argv[1]}.json").read()
j = json.loads(t[t.index("{"):])
print({k: round(v["ms_per_rep"], 3) for k, v in j.items() if isinstance(v, dict)}, "gemm_tflops", j.get("gemm_tflops"))
PY
  done
fi
if [ "${NCU:-0}" = 1 ]; then
  timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none --kernel-name-base demangled \
    --kernel-name regex:'rs::' --csv --log-file gpurun_out/launches_cfg4.csv \
    python bench.py --steps 1 --warmup 1 --no-e2e --no-cpu-baseline > gpurun_out/ncu_bench.log 2>&1
  echo "ncu rc=$?"; python scripts/ncu_summary.py gpurun_out/launches_cfg4.csv | head -30
fi
