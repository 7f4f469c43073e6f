#!/bin/bash
# r02 experiment: ring sample kernel time against its split count (rounds of the persistent grid),
# with the narrow 40th tile (default) and with it dropped (-DRS_DEV_RING_DROP_TAIL, a timing-only
# switch that skipped the tail columns; removed from the library after the experiment, see
# profiles/r02_ring_splits.jsonl)
mkdir -p gpurun_out
for flags in "" "-DRS_DEV_RING_S=11" "-DRS_DEV_RING_S=22" "-DRS_DEV_RING_S=7" "-DRS_DEV_RING_DROP_TAIL -DRS_DEV_RING_S=11" "-DRS_DEV_RING_DROP_TAIL -DRS_DEV_RING_S=15" "-DRS_DEV_RING_DROP_TAIL -DRS_DEV_RING_S=30" ""; do
  export RS_EXTRA_NVCC_FLAGS="$flags"
  python __graft_entry__.py build > gpurun_out/build.log 2>&1 || { tail -30 gpurun_out/build.log; exit 1; }
  for c in cfg4 cfg2; do
    timeout 300 python scripts/gpu_timing.py --cfg $c --reps 3 2>&1 | python -c "
import sys,json; t=sys.stdin.read(); j=json.loads(t[t.index('{'):]); print('[$flags] $c', {k: round(v['ms_per_rep'],3) for k,v in j.items() if isinstance(v,dict) and k.startswith('gemm_s')})"
  done
done
