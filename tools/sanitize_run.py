"""Small workload for compute-sanitizer (racecheck / synccheck / initcheck /
memcheck): the tiled SpMV at n = 1024 (tiles_x = 4, every vector scheme with
its paired element / rowptr schemes), the fused calc_p + SpMV, and a few CG
iterations, with single flips in cross-tile halo cells so the cold paths run.

    compute-sanitizer --tool racecheck python tools/sanitize_run.py [--n 1024]
"""
from __future__ import annotations

import argparse
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--n", type=int, default=1024)
    ap.add_argument("--schemes", default="0,1,2,3,4")
    a = ap.parse_args()
    import torch
    import gen
    from paper_conf_cluster_pawelczakmpm17_b200 import abft
    torch.cuda.set_device(0)
    n = a.n
    N = n * n
    ctx = abft.Context(0)
    v, c, r = gen.tealeaf_csr(n, device="cuda")
    for S in [int(t) for t in a.schemes.split(",")]:
        es = S if S != abft.SECDED128 else abft.SECDED64
        A = abft.Matrix(v, c.to(torch.int32), r.to(torch.int32), N, N, es, S, stencil_n=n)
        assert A.encode(ctx) == 0
        x = abft.Vector.from_values(ctx, torch.from_numpy(gen.uniform_pm1(N, 3)).cuda(), S)
        if S != abft.NONE:
            for i in (255, 256 + 7 * n, 511 + 8 * n, 768 + 15 * n):
                abft.inject_bitflip(ctx, x.data, 64 * i + 40)
            abft.inject_bitflip(ctx, A.val, 64 * (5 * (300 + 8 * n) + 1) + 3)
        y = abft.Vector.empty(N, S)
        cnt = abft.Counters()
        dot = torch.zeros(1, dtype=torch.float64, device="cuda")
        abft.spmv(ctx, A, x, y, cnt, dot=dot)
        if S in (abft.NONE, abft.SED, abft.SECDED64):
            r_ = abft.Vector.from_values(ctx, torch.from_numpy(gen.uniform_pm1(N, 4)).cuda(), S)
            p2 = abft.Vector.empty(N, S)
            abft.calc_p_spmv(ctx, A, x, r_, 0.5, p2, y, cnt, dot=dot)
        b = abft.Vector.from_values(ctx, gen.tealeaf_rhs(n).cuda(), S)
        xs = abft.Vector.from_values(ctx, gen.tealeaf_rhs(n).cuda(), S)
        rr, pp, ww = (abft.Vector.empty(N, S) for _ in range(3))
        res = abft.cg_solve(ctx, A, b, xs, rr, pp, ww, tol=1e-10, max_iters=6, due_policy=1, counts=cnt, poll_every=3)
        torch.cuda.synchronize()
        print(f"scheme {S}: cg iters {res.iters} counts {int(cnt.read().sum())}", flush=True)
        if S == abft.SECDED64:   # the bench's arrangement: PDL between the CG kernels (early window TMA)
            ctx.set_pdl(True)
            res = abft.cg_solve(ctx, A, b, xs, rr, pp, ww, tol=1e-10, max_iters=6, due_policy=1, counts=cnt,
                                poll_every=3)
            ctx.set_pdl(False)
            torch.cuda.synchronize()
            print(f"scheme {S} + PDL: cg iters {res.iters}", flush=True)
    # peer-memory halos between two loopback ranks (calc_p's stores into the
    # neighbour's ghost rows, arrival flags, the SpMV's wait)
    m, P = 256, 2
    S = abft.SECDED64
    rows = m // P
    ctxs, As, vecs = [], [], []
    for q in range(P):
        vq, cq, rq = gen.strip_csr(m, q * rows, (q + 1) * rows, ny=m, col_offset=m, device="cuda")
        cx = abft.Context(0)
        Aq = abft.Matrix(vq, cq.to(torch.int32), rq.to(torch.int32), rows * m, rows * m + 2 * m, S, S, row_base=m,
                         col_base=0, stencil_n=m)
        assert Aq.encode(cx) == 0
        bq = torch.zeros(rows * m + 2 * m, dtype=torch.float64, device="cuda")
        bq[m:m + rows * m] = gen.tealeaf_rhs(m, q * rows, (q + 1) * rows, ny=m).cuda()
        bv = abft.Vector.from_values(cx, bq, S)
        xv = abft.Vector.from_values(cx, bq.clone(), S)
        ctxs.append(cx)
        As.append(Aq)
        vecs.append([bv, xv] + [abft.Vector.empty(rows * m + 2 * m, S) for _ in range(3)])
    d = abft.Loopback(P, 0)
    d.set_peer_halo(True)
    res = d.cg_solve(ctxs, As, m, vecs, tol=1e-10, max_iters=8, due_policy=1, counts=[abft.Counters() for _ in range(P)],
                     poll_every=4)
    torch.cuda.synchronize()
    d.close()
    print(f"loopback peer halo: iters {[r.iters for r in res]}", flush=True)


if __name__ == "__main__":
    main()
