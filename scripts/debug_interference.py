"""Development aid: is the single-rank pipeline bitwise stable while another stream keeps the GPU
busy (perturbed CTA scheduling)?  Runs the pipeline repeatedly next to a torch matmul loop."""
import sys
import threading

sys.path.insert(0, '.')
import numpy as np  # noqa: E402
import torch  # noqa: E402

import paper_conf_sc_maryykltd15_b200 as rs  # noqa: E402
from synth.matrices import make_matrix  # noqa: E402
from tests.gpu_helpers import to_dev, to_np  # noqa: E402

rs.load_library()
m, n, k, p, q = 10000, 1000, 50, 10, 1
A, _ = make_matrix(m, n, "exp-k", k, seed=20014)
Ad = to_dev(A)
stop = threading.Event()


def noise():
    torch.cuda.set_device(0)
    s = torch.cuda.Stream()
    with torch.cuda.stream(s):
        x = torch.randn(2048, 2048, device="cuda")
        while not stop.is_set():
            for _ in range(20):
                x = (x @ x).tanh_()
            s.synchronize()


def run():
    perm, Q, R, h = rs.rs_lowrank.rs_lowrank(Ad, k, p, q, 0x5C15)
    B = to_np(rs.get_sample(h))
    rs.destroy(h)
    return B, to_np(R), perm.cpu().numpy()


B0, R0, P0 = run()
t = threading.Thread(target=noise)
t.start()
bad = 0
for i in range(40):
    B, R, P = run()
    if not (np.array_equal(B, B0) and np.array_equal(R, R0) and np.array_equal(P, P0)):
        bad += 1
        print("run", i, "differs: B", float(np.abs(B - B0).max()), "R", float(np.abs(R - R0).max()), flush=True)
stop.set()
t.join()
print("interference runs differing:", bad, "of 40", flush=True)
