"""Development aid: two independent single-rank handles in two host threads on one GPU (first
calls in a fresh process), each checked against the oracle."""
import sys
import threading

sys.path.insert(0, '.')
import numpy as np  # noqa: E402
import torch  # noqa: E402

import paper_conf_sc_maryykltd15_b200 as rs  # noqa: E402
from oracle import pipeline as OPL  # noqa: E402
from synth.matrices import make_matrix  # noqa: E402
from tests.gpu_helpers import rel, to_dev, to_np  # noqa: E402

rs.load_library()
k, p, q = 50, 10, 1
mats = [make_matrix(10000, 1000, "exp-k", k, seed=s)[0] for s in (11, 12)]
want = [OPL.rs_lowrank(A, k, p, q, 0x5C15) for A in mats]
out = [None, None]


def work(i):
    torch.cuda.set_device(0)
    st = torch.cuda.Stream()
    with torch.cuda.stream(st):
        Ad = to_dev(mats[i])
        st.synchronize()
        perm, Q, R, h = rs.rs_lowrank.rs_lowrank(Ad, k, p, q, 0x5C15)
        out[i] = to_np(rs.get_sample(h))
        rs.destroy(h)


ts = [threading.Thread(target=work, args=(i,)) for i in range(2)]
[t.start() for t in ts]
[t.join() for t in ts]
print("concurrent handles: B rel", [f"{rel(out[i], want[i].B):.2e}" for i in range(2)], flush=True)
