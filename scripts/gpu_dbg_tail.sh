mkdir -p gpurun_out
python __graft_entry__.py build > gpurun_out/build.log 2>&1 || { tail -30 gpurun_out/build.log; exit 1; }
timeout 300 python scripts/debug_tail.py 2>&1 | tail -8
for c in cfg4 cfg2; do
timeout 300 python scripts/gpu_timing.py --cfg $c --reps 3 2>&1 | python -c "
import sys,json; t=sys.stdin.read(); j=json.loads(t[t.index('{'):]) if '{' in t else print(t[-600:]); print('$c', {k: round(v['ms_per_rep'],3) for k,v in j.items() if isinstance(v,dict) and k.startswith('gemm')})"
done
