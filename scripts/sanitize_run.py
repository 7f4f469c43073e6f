"""One small rank-k approximation through the C ABI (every kernel family of the fixed-rank path),
for compute-sanitizer runs:  compute-sanitizer --tool racecheck python scripts/sanitize_run.py"""
import argparse
import os
import sys

sys.path.insert(0, os.path.dirname(os.path.dirname(os.path.abspath(__file__))))

import numpy as np  # noqa: E402
import torch  # noqa: E402

import paper_conf_sc_maryykltd15_b200 as rs  # noqa: E402
from synth.matrices import make_matrix  # noqa: E402

ap = argparse.ArgumentParser()
ap.add_argument("--m", type=int, default=2000)
ap.add_argument("--n", type=int, default=1000)
ap.add_argument("--k", type=int, default=50)
ap.add_argument("--p", type=int, default=10)
ap.add_argument("--q", type=int, default=1)
a = ap.parse_args()
rs.load_library()
A, _ = make_matrix(a.m, a.n, "exp-k", a.k, seed=7)
Ad = rs.empty_colmajor(a.m, a.n)
Ad.copy_(torch.from_numpy(A))
perm, Q, R, h = rs.rs_lowrank.rs_lowrank(Ad, a.k, a.p, a.q, seed=0x5C15)   # the phases
rs.run(h, Ad, a.q, perm, Q, R)   # the whole step captured as a CUDA graph, then replayed
rs.run(h, Ad, a.q, perm, Q, R)
torch.cuda.synchronize()
rs.destroy(h)
print("ok", float(np.abs(Q.cpu().numpy().T @ Q.cpu().numpy() - np.eye(a.k)).max()))
