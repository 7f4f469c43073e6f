"""Development aid: multi-rank (allreduce hook) pipeline on one GPU, B checked after every stage."""
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

rs.load_library()
m, n, k, p, q = 20000, 1000, 50, 10, 1
A, _ = make_matrix(m, n, "exp-k", k, seed=m + 14)
o = OPL.rs_lowrank(A, k, p, q, T.SEED)
for nranks in (1, 2):
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
            if nranks > 1:
                rs.rs_lowrank.set_allreduce_hook(h, nranks, r, comm.hook(r, st))
            perm = torch.empty(n, dtype=torch.int64, device="cuda")
            Q = rs.empty_colmajor(r1 - r0, k)
            R = rs.empty_colmajor(k, n)
            rs.sample(h, Ad)
            rs.power_iterate(h, Ad, q)
            res[r]["power"] = to_np(rs.get_sample(h))
            rs.pivot(h, perm)
            res[r]["pivot"] = to_np(rs.get_sample(h))
            res[r]["perm"] = perm.cpu().numpy()
            rs.factor(h, Ad, Q, R)
            res[r]["factor"] = to_np(rs.get_sample(h))
            res[r]["R"] = to_np(R)
            rs.destroy(h)

    ts = [threading.Thread(target=work, args=(r,)) for r in range(nranks)]
    [t.start() for t in ts]
    [t.join() for t in ts]
    r0 = res[0]
    print(f"nranks={nranks}: B rel after power {rel(r0['power'], o.B):.3e} pivot {rel(r0['pivot'], o.B):.3e} "
          f"factor {rel(r0['factor'], o.B):.3e}; perm eq {list(r0['perm'][:k]) == list(o.perm[:k])}; "
          f"R rel {rel(r0['R'], o.R):.3e}; calls {comm.calls}", flush=True)
    d = np.abs(r0['factor'] - o.B)
    i, j = np.unravel_index(np.argmax(d), d.shape)
    print("   max |dB| at", (i, j), d[i, j], "rows with dB > 1e-9:", sorted(set(np.where(d > 1e-9)[0]))[:10],
          "cols:", len(set(np.where(d > 1e-9)[1])), flush=True)
