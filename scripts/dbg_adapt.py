import numpy as np, torch, sys
sys.path.insert(0, '.')
import paper_conf_sc_maryykltd15_b200 as rs
from tests.gpu_helpers import to_dev, to_np, rel
from oracle import adaptive as AD, pipeline as OPL
from synth.matrices import make_matrix
m, n, lmax, inc, q = 3000, 500, 160, 8, 0
A, _ = make_matrix(m, n, "exp-paper", 50, seed=21)
o = AD.adaptive_sample(A, 1e-4, inc, q, 0x5C15, lmax)
Ad = to_dev(A)
h = rs.create(m, m, 0, n, lmax, 0, 0x5C15)
ell, est, hist = rs.sample_adaptive(h, Ad, 1e-4, inc, q)
print("ell", ell, o.ell)
B = to_np(rs.get_sample(h)); print("relB", rel(B, o.B))
perm = torch.empty(n, dtype=torch.int64, device="cuda")
rs.pivot(h, perm)
T, Rh, gaps = rs.get_pivot_data(h)
perm = perm.cpu().numpy()
po, Rho, To, go = OPL.pivot(o.B, ell)
print("perm eq", (perm[:ell] == po[:ell]).mean(), "min gap", min(go))
print("T shape", T.shape, To.shape, "relT", rel(to_np(T), To) if list(perm[:ell])==list(po[:ell]) else None)
print("Rhat rel", rel(np.abs(to_np(Rh)), np.abs(Rho)))
Q = rs.empty_colmajor(m, lmax); R = rs.empty_colmajor(lmax, n)
rs.factor(h, Ad, Q, R)
Qn, Rn = to_np(Q)[:, :ell], to_np(R)[:ell]
print("QtQ", np.abs(Qn.T@Qn-np.eye(ell)).max())
Qo, Rbo, Ro = OPL.factor(A, po, To, ell)
print("relR", rel(Rn, Ro), "relQ", rel(Qn, Qo))
print("e", OPL.approx_error(A, perm, Qn, Rn), OPL.approx_error(A, po, Qo, Ro))
# check columns first ell: A P1 = Q R[:, :ell]
print("first-k exact", np.linalg.norm(A[:, perm[:ell]] - Qn @ Rn[:, :ell]))
