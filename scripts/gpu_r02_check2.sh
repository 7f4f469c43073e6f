#!/bin/bash
# r02 check 2: TSA kernel correctness (parity, multirank, sanitizers) and cfg4 phase timing; ring
# depth with the deferred slot release; per-rank slices (N = 1, 2, 4, 8)
mkdir -p gpurun_out
python __graft_entry__.py build > gpurun_out/build.log 2>&1 || { tail -30 gpurun_out/build.log; exit 1; }
timeout 1500 python -m pytest tests/test_gpu_parity.py tests/test_gpu_multirank.py tests/test_gpu_fallback.py tests/test_gpu_adaptive.py tests/test_gpu_sanitizer.py -q -x -rA -k "not baseline_shapes and not cfg4_full" > gpurun_out/r02_gpu_tests2.log 2>&1; echo "tests rc=$?"; tail -3 gpurun_out/r02_gpu_tests2.log; grep -E "FAILED|Error" gpurun_out/r02_gpu_tests2.log | head -5
for flags in "" "-DRS_KC_NS=5 -DRS_PHX_NS=5" "-DRS_KC_NS=6 -DRS_PHX_NS=6"; do
  RS_EXTRA_NVCC_FLAGS="$flags" python __graft_entry__.py build > gpurun_out/build.log 2>&1 || { tail -30 gpurun_out/build.log; exit 1; }
  RS_EXTRA_NVCC_FLAGS="$flags" timeout 300 python scripts/gpu_timing.py --cfg cfg4 2>&1 | python -c "
import sys,json; t=sys.stdin.read(); j=json.loads(t[t.index('{'):]); print('[$flags] cfg4', {k: round(v['ms_per_rep'],3) for k,v in j.items() if isinstance(v,dict)}, 'gemm_tflops', j.get('gemm_tflops'))"
done
python __graft_entry__.py build > gpurun_out/build.log 2>&1
timeout 600 python scripts/rank_slice.py --cfg cfg4 --ranks 1 2 4 8 > gpurun_out/r02_rank_slices.jsonl 2> gpurun_out/r02_rank_slices.err; echo "slices rc=$?"; cat gpurun_out/r02_rank_slices.jsonl | cut -c1-400
timeout 600 ncu --set full --clock-control none --import-source on -k regex:tsa_kernel -c 2 -o gpurun_out/r02_ncu_tsa python scripts/gpu_timing.py --cfg cfg4 --reps 1 > gpurun_out/r02_ncu_tsa.log 2>&1; echo "ncu rc=$?"
