#!/bin/bash
# r02 check 4: Omega written as st.async tx bytes (own ring too); racecheck; parity subset; cfg4
# timing A/B against the generic-store variant; ncu launch list + full capture of the sample GEMM;
# the CPU oracle on the full cfg4 (host cores)
mkdir -p gpurun_out
nproc; free -g | head -2
python __graft_entry__.py build > gpurun_out/build.log 2>&1 || { tail -30 gpurun_out/build.log; exit 1; }
timeout 1500 python -m pytest tests/test_gpu_parity.py tests/test_gpu_sanitizer.py tests/test_gpu_adaptive.py -q -x -k "not baseline_shapes and not cfg4_full" > gpurun_out/r02_gpu_tests4.log 2>&1; echo "tests rc=$?"; tail -2 gpurun_out/r02_gpu_tests4.log; grep -E "^FAILED" gpurun_out/r02_gpu_tests4.log | head
for flags in "" "-DRS_PHX_LOCAL_STS"; do
  RS_EXTRA_NVCC_FLAGS="$flags" python __graft_entry__.py build > gpurun_out/build.log 2>&1 || { tail -30 gpurun_out/build.log; exit 1; }
  RS_EXTRA_NVCC_FLAGS="$flags" timeout 300 python scripts/gpu_timing.py --cfg cfg4 2>&1 | python -c "
import sys,json; t=sys.stdin.read(); j=json.loads(t[t.index('{'):]); print('[$flags] cfg4', {k: round(v['ms_per_rep'],3) for k,v in j.items() if isinstance(v,dict)}, 'gemm_tflops', j.get('gemm_tflops'))"
done
python __graft_entry__.py build > gpurun_out/build.log 2>&1
timeout 900 ncu --metrics gpu__time_duration.sum --clock-control none --csv --log-file gpurun_out/r02_launches_cfg4.csv python bench.py --steps 1 --warmup 3 --no-e2e --no-cpu-baseline > gpurun_out/r02_ncu_bench.log 2>&1; echo "ncu launches rc=$?"
timeout 900 ncu --set full --clock-control none --import-source on -k regex:kc_philox -c 1 -o gpurun_out/r02_ncu_philox_cfg4 python scripts/gpu_timing.py --cfg cfg4 --reps 1 > gpurun_out/r02_ncu_phx.log 2>&1; echo "ncu full rc=$?"
timeout 1500 python scripts/oracle_full.py --cfg cfg4 > gpurun_out/r02_oracle_full_cfg4.json 2> gpurun_out/r02_oracle_full_cfg4.err; echo "oracle full rc=$?"; cat gpurun_out/r02_oracle_full_cfg4.json; tail -3 gpurun_out/r02_oracle_full_cfg4.err
