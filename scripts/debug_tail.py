"""Development aid: B after one power pass (B := C~ A through the KC GEMM, tail fold when
n % 128 <= 16) against the oracle, main and tail columns separately."""
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)
import numpy as np  # noqa: E402
import torch  # noqa: E402

import paper_conf_sc_maryykltd15_b200 as rs  # noqa: E402
from oracle import pipeline as OPL  # noqa: E402

SEED = 0x5C15
for (m, n, k, p) in [(2000, 400, 120, 8), (3000, 1032, 100, 10), (6000, 900, 400, 10), (3000, 1036, 60, 4),
                     (3000, 1040, 40, 8)]:
    rng = np.random.default_rng(m + n)
    A = np.asfortranarray(rng.standard_normal((m, n)))
    h = rs.create(m, m, 0, n, k, p, SEED)
    try:
        Ad = torch.from_numpy(A.T.copy()).cuda().t()
        rs.sample(h, Ad)
        rs.power_iterate(h, Ad, 1)
        torch.cuda.synchronize()
        B = rs.get_sample(h).cpu().numpy()
        Bo = OPL.power_iterate(A, OPL.sample(A, k + p, SEED), 1)
        t0 = (n // 128) * 128
        e = lambda x, y: float(np.linalg.norm(x - y) / max(np.linalg.norm(y), 1e-300))
        print(f"m={m} n={n} l={k+p}: B main {e(B[:, :t0], Bo[:, :t0]):.2e} tail {e(B[:, t0:], Bo[:, t0:]):.2e}",
              flush=True)
    except Exception as ex:  # noqa: BLE001
        print(f"m={m} n={n} l={k+p}: ERROR {ex}", flush=True)
    finally:
        rs.destroy(h)
