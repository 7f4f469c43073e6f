"""Development aid: first multi-rank pipeline call in a fresh process, B checked against the oracle."""
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
ranks, calls = T._run_ranks(A, 2, k, p, q)
o = OPL.rs_lowrank(A, k, p, q, T.SEED)
d = np.abs(ranks[0]["B"] - o.B)
bad = d > 1e-9 * np.abs(o.B).max()
print(f"rel B {rel(ranks[0]['B'], o.B):.3e} rel R {rel(ranks[0]['R'], o.R):.3e} bad rows {sorted(set(np.where(bad)[0]))[:12]} "
      f"bad cols {len(set(np.where(bad)[1]))} B1==B0 {np.array_equal(ranks[0]['B'], ranks[1]['B'])}", flush=True)
