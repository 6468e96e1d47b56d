"""Per-scheme overhead sweep (BASELINE.json config 3; mirrors the paper's
Figs 4/5/9) on the G-TEA grid (default 8192^2, row-block chunks).

    python tools/sweep.py [--grid 8192] [--iters 200] [--out gpurun_out/sweep.json]

For every scheme s in none/SED/SECDED64/SECDED128/CRC32C: (i) all structures
protected with s, (ii) one structure at a time (CSR elements, row pointers,
dense vectors) with the others unprotected.  Each configuration runs a fixed
window of protected CG iterations (tol 0) after one warm-up solve; reported
per-iteration time and overhead vs the unprotected twin.  SECDED128 on CSR
elements maps to E-SECDED (reading R3).  SECDED128/CRC32C vectors (groups of
2/4 doubles) run the generic kernels (the tiled SpMV fast path is G = 1 only).

--intervals 1,2,4,...: additionally the check-interval sweep of the paper's
Figs 6-8: the whole CSR matrix (elements + row pointers) protected
with SED / SECDED64 / CRC32C, vectors unprotected, matrix checked (detection
only) every N-th access and range-checked otherwise.
"""
from __future__ import annotations

import argparse
import json
import os
import sys

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))
sys.path.insert(0, ROOT)


def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--grid", type=int, default=8192)
    ap.add_argument("--iters", type=int, default=200)
    ap.add_argument("--reps", type=int, default=2)
    ap.add_argument("--out", default=os.path.join(ROOT, "gpurun_out", "sweep.json"))
    ap.add_argument("--intervals", default="", help="comma-separated check intervals (matrix-only configs)")
    ap.add_argument("--no-schemes", action="store_true", help="skip the per-scheme sweep")
    ap.add_argument("--only", default="SED,SECDED64,CRC32C", help="schemes of the interval sweep")
    a = ap.parse_args()
    import torch
    import bench
    from paper_conf_cluster_pawelczakmpm17_b200 import abft
    torch.cuda.set_device(0)
    P = bench.build_problem(a.grid, a.grid, 0, 1, torch.device("cuda", 0))
    ctx = abft.Context(0)
    names = ["NONE", "SED", "SECDED64", "SECDED128", "CRC32C"]
    configs = [("all", "NONE", ("NONE", "NONE", "NONE"), 1)]
    if not a.no_schemes:
        for s in names[1:]:
            configs.append(("all", s, (s, s, s), 1))
        for s in names[1:]:
            configs.append(("elements", s, (s, "NONE", "NONE"), 1))
            configs.append(("rowptr", s, ("NONE", s, "NONE"), 1))
            configs.append(("vectors", s, ("NONE", "NONE", s), 1))
    for N in [int(t) for t in a.intervals.split(",") if t]:
        for s in a.only.split(","):
            configs.append(("matrix", s, (s, s, "NONE"), N))
    rows = []
    base = None
    for (what, s, (es, rs, vs), interval) in configs:
        sol = bench.Solver(abft, ctx, P, getattr(abft, es), getattr(abft, rs), getattr(abft, vs),
                           check_interval=interval)
        sol.step(0.0, 5)   # warm-up (graph capture, attributes)
        best = None
        for _ in range(a.reps):
            e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
            torch.cuda.synchronize()
            e0.record()
            it, st = sol.step(0.0, a.iters)
            e1.record()
            torch.cuda.synchronize()
            ms = e0.elapsed_time(e1) / max(it, 1)
            best = ms if best is None else min(best, ms)
        if what == "all" and s == "NONE":
            base = best
        # per-kernel-class breakdown: one extra profiled (non-graph) step
        abft.profile(ctx, 15)
        it2, _ = sol.step(0.0, a.iters)
        torch.cuda.synchronize()
        ms_cls, n_cls = abft.profile_read(ctx)
        abft.profile(ctx, 0)
        kms = {k: (ms_cls[i] / n_cls[i] if n_cls[i] else None) for i, k in enumerate(["spmv", "calc_ur", "calc_p", "reductions"])}
        row = {"structures": what, "scheme": s, "elem": es, "rowptr": rs, "vectors": vs, "check_interval": interval,
               "iter_ms": best,
               "overhead_pct": None if base is None else 100.0 * (best / base - 1.0),
               "cg_gbs": 152.0 * P["N"] / (best / 1000.0) / 1e9, "kernel_ms": kms}
        rows.append(row)
        print(json.dumps(row), flush=True)
        del sol
        torch.cuda.empty_cache()
    out = {"grid": a.grid, "chunks": len(P["chunks"]), "iters_per_config": a.iters, "rows": rows}
    os.makedirs(os.path.dirname(a.out), exist_ok=True)
    json.dump(out, open(a.out, "w"), indent=1)


if __name__ == "__main__":
    main()
