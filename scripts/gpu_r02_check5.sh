#!/bin/bash
# r02 check 5: sample GEMM with the L2 ring of Omega chunks (kc_sample_ring_kernel): parity, timing
mkdir -p gpurun_out
python __graft_entry__.py build > gpurun_out/build.log 2>&1 || { tail -30 gpurun_out/build.log; exit 1; }
timeout 300 python scripts/gpu_timing.py --cfg cfg2 > gpurun_out/r02_t5_cfg2.txt 2>&1; echo "cfg2 rc=$?"; tail -3 gpurun_out/r02_t5_cfg2.txt | cut -c1-600
timeout 900 python -m pytest tests/test_gpu_parity.py -q -x -k "sample or baseline_shapes or cfg4_full or ragged" > gpurun_out/r02_gpu_tests5.log 2>&1; echo "tests rc=$?"; tail -3 gpurun_out/r02_gpu_tests5.log; grep -E "^E " gpurun_out/r02_gpu_tests5.log | head -5
timeout 300 python scripts/gpu_timing.py --cfg cfg4 2>&1 | python -c "
import sys,json; t=sys.stdin.read(); j=json.loads(t[t.index('{'):]); print('cfg4', {k: round(v['ms_per_rep'],3) for k,v in j.items() if isinstance(v,dict)}, 'gemm_tflops', j.get('gemm_tflops'))"
timeout 300 python scripts/gpu_timing.py --cfg cfg3 2>&1 | python -c "
import sys,json; t=sys.stdin.read(); j=json.loads(t[t.index('{'):]); print('cfg3', {k: round(v['ms_per_rep'],3) for k,v in j.items() if isinstance(v,dict)}, 'gemm_tflops', j.get('gemm_tflops'))"
timeout 600 python -m pytest tests/test_gpu_multirank.py tests/test_gpu_nccl.py -q -x > gpurun_out/r02_gpu_tests5b.log 2>&1; echo "tests2 rc=$?"; tail -2 gpurun_out/r02_gpu_tests5b.log
timeout 600 python scripts/rank_slice.py --cfg cfg4 --ranks 8 4 > gpurun_out/r02_rank_slices5.jsonl 2>/dev/null; echo "slices rc=$?"; cut -c1-300 gpurun_out/r02_rank_slices5.jsonl
