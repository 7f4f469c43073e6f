"""Development aid: where does B go wrong?  B captured (synchronously) after each stage."""
import sys
import threading

sys.path.insert(0, '.')
import numpy as np  # noqa: E402
import torch  # noqa: E402

import paper_conf_sc_maryykltd15_b200 as rs  # noqa: E402
import tests.test_gpu_multirank as T  # noqa: E402
from oracle import pipeline as OPL  # noqa: E402
from paper_conf_sc_maryykltd15_b200.partition import row_split  # noqa: E402
from synth.matrices import make_matrix  # noqa: E402
from tests.gpu_helpers import rel, to_dev, to_np  # noqa: E402

import os  # noqa: E402

SYNC = os.environ.get("MR_SYNC", "sample,power,pivot").split(",")
rs.load_library()
m, n, k, p, q = 20000, 1000, 50, 10, 1
A, _ = make_matrix(m, n, "exp-k", k, seed=m + 14)
WARM = os.environ.get("MR_WARM", "none")  # single-threaded warm-up (loads kernels) before the ranks
if WARM != "none":
    hw = rs.create(m, m, 0, n, k, p, T.SEED)
    Aw = to_dev(A)
    rs.sample(hw, Aw)
    if WARM in ("power", "all"):
        rs.power_iterate(hw, Aw, q)
    torch.cuda.synchronize()
    rs.destroy(hw)
    del Aw
nranks = 2
comm = T.InProcessAllreduce(nranks)
res = [dict() for _ in range(nranks)]


def work(r):
    torch.cuda.set_device(0)
    r0, r1 = row_split(m, nranks, r)
    st = torch.cuda.Stream()
    with torch.cuda.stream(st):
        Ad = to_dev(np.asfortranarray(A[r0:r1]))
        st.synchronize()
        h = rs.create(m, r1 - r0, r0, n, k, p, T.SEED, stream=st)
        rs.rs_lowrank.set_allreduce_hook(h, nranks, r, comm.hook(r, st))
        perm = torch.empty(n, dtype=torch.int64, device="cuda")
        Q = rs.empty_colmajor(r1 - r0, k)
        R = rs.empty_colmajor(k, n)
        rs.sample(h, Ad)
        if "sample" in SYNC or "sample" == "factor":
            res[r]["sample"] = to_np(rs.get_sample(h))
        rs.power_iterate(h, Ad, q)
        if "power" in SYNC or "power" == "factor":
            res[r]["power"] = to_np(rs.get_sample(h))
        rs.pivot(h, perm)
        if "pivot" in SYNC or "pivot" == "factor":
            res[r]["pivot"] = to_np(rs.get_sample(h))
        rs.factor(h, Ad, Q, R)
        if "factor" in SYNC or "factor" == "factor":
            res[r]["factor"] = to_np(rs.get_sample(h))
        rs.destroy(h)


ts = [threading.Thread(target=work, args=(r,)) for r in range(nranks)]
[t.start() for t in ts]
[t.join() for t in ts]
o = OPL.rs_lowrank(A, k, p, q, T.SEED)
print(SYNC, {st: f"{rel(res[0][st], o.B0 if st == 'sample' else o.B):.2e}" for st in res[0]}, flush=True)
