#!/bin/bash
# r02 check 11: Cholesky of 128 < n <= 256 as 2 x 2 blocks on the one-CTA tile kernel (cfg3's l = 220)
mkdir -p gpurun_out
python __graft_entry__.py build > gpurun_out/build.log 2>&1 || { tail -30 gpurun_out/build.log; exit 1; }
timeout 1500 python -m pytest tests/test_gpu_parity.py tests/test_gpu_fallback.py tests/test_gpu_adaptive.py -q -x -k "ragged or baseline_shapes or fallback or adaptive" > gpurun_out/r02_gpu_tests11.log 2>&1; echo "tests rc=$?"; tail -2 gpurun_out/r02_gpu_tests11.log; grep -E "^E " gpurun_out/r02_gpu_tests11.log | head -5
for flags in "" "-DRS_DEV_CHOL_CLUSTER_256"; do
  export RS_EXTRA_NVCC_FLAGS="$flags"
  python __graft_entry__.py build > gpurun_out/build.log 2>&1 || exit 1
  timeout 300 python scripts/gpu_timing.py --cfg cfg3 2>&1 | python -c "
import sys,json; t=sys.stdin.read(); j=json.loads(t[t.index('{'):]); print('[$flags] cfg3', {k: round(v['ms_per_rep'],3) for k,v in j.items() if isinstance(v,dict)})"
done
