"""Overlapped multi-rank probe.

N ranks' handles run the whole pipeline in N host threads on ONE GPU with their kernels
overlapping (no token), every reduction routed through rs_lowrank_set_allreduce_hook.  The hook
records each rank's PRE-reduction buffer at every reduction point.  The same pipeline is then run
again in the same process with the ranks serialised (known good), and the two recordings are
compared call by call: the first differing (call, rank) names the segment of the pipeline where the
overlapped run went wrong.

  python scripts/mr_overlap_probe.py --procs 30            # 30 fresh processes, summary line
  python scripts/mr_overlap_probe.py --child               # one process, one JSON line
"""
import argparse
import json
import os
import subprocess
import sys
import threading

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)


class _DevBuf:
    def __init__(self, ptr, count):
        self.__cuda_array_interface__ = {"shape": (count,), "typestr": "<f8", "data": (ptr, False),
                                         "version": 3, "strides": None}


def child(args):
    import numpy as np
    import torch

    import paper_conf_sc_maryykltd15_b200 as rs
    from paper_conf_sc_maryykltd15_b200.partition import row_split
    from synth.matrices import make_matrix

    rs.load_library()
    m, n, k, p, q, nr = args.m, args.n, args.k, args.p, args.q, args.nranks
    A, _ = make_matrix(m, n, "exp-k", k, seed=m + 7 * nr)

    def run(serial):
        rec = [[] for _ in range(nr)]
        out = [None] * nr
        errs = [None] * nr
        bar = threading.Barrier(nr, timeout=300)
        token = threading.Lock()
        bufs = [None] * nr

        def hook(r, stream):
            def fn(buf, count, sp):
                stream.synchronize()
                v = torch.as_tensor(_DevBuf(buf, count), device="cuda")
                rec[r].append(v.cpu().numpy().copy())
                bufs[r] = (buf, count)
                if serial:
                    token.release()
                bar.wait()
                if r == 0:
                    torch.cuda.synchronize()
                    views = [torch.as_tensor(_DevBuf(b, c), device="cuda") for b, c in bufs]
                    tot = views[0].cpu().numpy().copy()
                    for x in views[1:]:
                        tot += x.cpu().numpy()
                    src = torch.from_numpy(tot)
                    for x in views:
                        x.copy_(src)
                    torch.cuda.synchronize()
                bar.wait()
                if serial:
                    token.acquire()
            return fn

        def work(r):
            if serial:
                token.acquire()
            try:
                torch.cuda.set_device(0)
                r0, r1 = row_split(m, nr, r)
                st = torch.cuda.Stream()
                with torch.cuda.stream(st):
                    Ad = rs.empty_colmajor(r1 - r0, n)
                    Ad.copy_(torch.from_numpy(np.asfortranarray(A[r0:r1])))
                    st.synchronize()
                    h = rs.create(m, r1 - r0, r0, n, k, p, 0x5C15, stream=st)
                    try:
                        rs.rs_lowrank.set_allreduce_hook(h, nr, r, hook(r, st))
                        perm = torch.empty(n, dtype=torch.int64, device="cuda")
                        Q = rs.empty_colmajor(r1 - r0, k)
                        R = rs.empty_colmajor(k, n)
                        rs.sample(h, Ad)
                        rs.power_iterate(h, Ad, q)
                        rs.pivot(h, perm)
                        rs.factor(h, Ad, Q, R)
                        st.synchronize()
                        out[r] = dict(B=rs.get_sample(h).cpu().numpy(), R=R.cpu().numpy(), Q=Q.cpu().numpy())
                    finally:
                        rs.destroy(h)
            except BaseException as e:  # noqa: BLE001
                errs[r] = repr(e)
                bar.abort()
            finally:
                if serial:
                    token.release()

        ts = [threading.Thread(target=work, args=(r,)) for r in range(nr)]
        for t in ts:
            t.start()
        for t in ts:
            t.join()
        return rec, out, errs

    rec_o, out_o, err_o = run(serial=False)
    rec_s, out_s, err_s = run(serial=True)
    res = {"loading": os.environ.get("CUDA_MODULE_LOADING", "default"), "errs": [err_o, err_s],
           "ncalls": [len(rec_o[0]), len(rec_s[0])]}
    first = None
    for c in range(min(len(rec_o[0]), len(rec_s[0]))):
        for r in range(nr):
            a, b = rec_o[r][c], rec_s[r][c]
            if a.shape != b.shape or not np.array_equal(a, b):
                d = np.abs(a - b) if a.shape == b.shape else np.array([np.inf])
                nz = np.nonzero(d)[0]
                first = {"call": c, "rank": r, "count": int(a.size), "maxdiff": float(d.max()),
                         "nbad": int(nz.size), "bad_first": int(nz[0]) if nz.size else -1,
                         "bad_last": int(nz[-1]) if nz.size else -1,
                         "rel": float(np.linalg.norm(a - b) / max(np.linalg.norm(b), 1e-300))}
                break
        if first:
            break
    res["first_diff"] = first
    if out_o[0] is not None and out_s[0] is not None:
        B0, B1 = out_o[0]["B"], out_s[0]["B"]
        res["B_rel"] = float(np.linalg.norm(B0 - B1) / np.linalg.norm(B1))
        res["B_equal"] = bool(np.array_equal(B0, B1))
    # per-call layout of the partial that first differs (l_pad x n column-major for B partials)
    print(json.dumps(res), flush=True)


def parent(args):
    stats = {"ok": 0, "bad": 0, "error": 0, "first_calls": {}}
    for i in range(args.procs):
        env = dict(os.environ)
        cmd = [sys.executable, os.path.abspath(__file__), "--child"] + [
            f"--{k}={getattr(args, k)}" for k in ("m", "n", "k", "p", "q", "nranks")]
        r = subprocess.run(cmd, capture_output=True, text=True, env=env, timeout=600)
        line = [x for x in r.stdout.splitlines() if x.startswith("{")]
        if r.returncode != 0 or not line:
            stats["error"] += 1
            print(f"[{i}] rc={r.returncode} {r.stderr[-800:]}", flush=True)
            continue
        j = json.loads(line[-1])
        if j.get("first_diff") is None and j.get("B_equal", False):
            stats["ok"] += 1
        else:
            stats["bad"] += 1
            c = str((j.get("first_diff") or {}).get("call"))
            stats["first_calls"][c] = stats["first_calls"].get(c, 0) + 1
        print(f"[{i}] {line[-1]}", flush=True)
    print("SUMMARY " + json.dumps(stats), flush=True)


if __name__ == "__main__":
    ap = argparse.ArgumentParser()
    ap.add_argument("--child", action="store_true")
    ap.add_argument("--procs", type=int, default=20)
    ap.add_argument("--m", type=int, default=20000)
    ap.add_argument("--n", type=int, default=1000)
    ap.add_argument("--k", type=int, default=50)
    ap.add_argument("--p", type=int, default=10)
    ap.add_argument("--q", type=int, default=1)
    ap.add_argument("--nranks", type=int, default=2)
    a = ap.parse_args()
    child(a) if a.child else parent(a)
