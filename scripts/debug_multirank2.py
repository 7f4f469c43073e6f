"""Development aid: repeat the multi-rank test harness and localise any difference in B."""
import sys

sys.path.insert(0, '.')
import numpy as np  # noqa: E402

import paper_conf_sc_maryykltd15_b200 as rs  # noqa: E402
import tests.test_gpu_multirank as T  # noqa: E402
from oracle import pipeline as OPL  # noqa: E402
from synth.matrices import make_matrix  # noqa: E402
from tests.gpu_helpers import rel  # noqa: E402

rs.load_library()
m, n, k, p, q = 20000, 1000, 50, 10, 1
A, _ = make_matrix(m, n, "exp-k", k, seed=m + 14)
o = OPL.rs_lowrank(A, k, p, q, T.SEED)
for it in range(8):
    ranks, calls = T._run_ranks(A, 2, k, p, q)
    B = ranks[0]["B"]
    e = rel(B, o.B)
    d = np.abs(B - o.B)
    bad_rows = sorted(set(np.where(d > 1e-9 * np.abs(o.B).max())[0]))
    bad_cols = sorted(set(np.where(d > 1e-9 * np.abs(o.B).max())[1]))
    print(f"it {it}: rel {e:.3e} calls {calls} bad rows {bad_rows[:12]} ncols {len(bad_cols)} cols {bad_cols[:8]} "
          f"perm eq {list(ranks[0]['perm'][:k]) == list(o.perm[:k])}", flush=True)
