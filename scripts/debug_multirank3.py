"""Development aid: does the pipeline depend on a zeroed workspace?  Fill it with garbage first."""
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
_create = rs.create


def create_garbage(*a, **kw):
    h = _create(*a, **kw)
    with torch.cuda.stream(h.stream):
        h.workspace.view(torch.float64)[:] = float("nan") if GARBAGE == "nan" else 1.2345e3
        h.stream.synchronize()
    return h


rs.create = create_garbage
m, n, k, p, q = 20000, 1000, 50, 10, 1
A, _ = make_matrix(m, n, "exp-k", k, seed=m + 14)
o = OPL.rs_lowrank(A, k, p, q, T.SEED)
for GARBAGE in ("val", "nan"):
    for nranks in (1, 2):
        try:
            ranks, calls = T._run_ranks(A, nranks, k, p, q)
            B = ranks[0]["B"]
            print(f"{GARBAGE} nranks={nranks}: B rel {rel(B, o.B):.3e}  R rel {rel(ranks[0]['R'], o.R):.3e}", flush=True)
        except Exception as e:  # noqa: BLE001
            print(f"{GARBAGE} nranks={nranks}: error {e}", flush=True)
