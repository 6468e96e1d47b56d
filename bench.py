"""bench.py — protected CG (BASELINE.json config 2) on B200, one JSON line.

    python bench.py [--gpus N --steps K --warmup W] [--impl reference] [--grid 4096]

A step is one pass of the whole hot path (rows a0-a7) over the
4096^2 G-TEA problem: re-encode the CSR matrix (a0) and the vectors b, x0 (a1),
then the protected CG solve to tol 1e-10 (a2-a6) with fault counters (a7).
`value` = CG iterations per second of the protected solve (inputs resident in
HBM); `e2e` = the same through the C ABI from pinned HOST buffers (H2D of the
raw matrix + b and D2H of x inside every step).  The unprotected twin (scheme
NONE everywhere, same kernels) is timed the same way for the overhead figure.
N > 1 (torchrun): weak scaling, each rank owns a 4096-row strip of a
4096 x 4096N grid, halos + dots over NCCL; value = it/s x N (4096^2-equivalent).
"""
from __future__ import annotations

import argparse
import json
import os
import statistics
import subprocess
import sys
import threading
import time

ROOT = os.path.dirname(os.path.abspath(__file__))
sys.path.insert(0, ROOT)

METRIC = "protected CG iters/sec and SpMV HBM GB/s vs peak; ECC overhead % vs unprotected"
SPMV_BYTES_PER_ROW = 80    # val 40 + col 20 + rowptr 4 + p 8 + w 8
CG_BYTES_PER_ROW = 152     # SpMV 80 + calc_ur 48 + calc_p 24
# fused calc_p: the SpMV reads p_{k-1} and r and writes p_k
FUSED_SPMV_BYTES_PER_ROW = 96   # val 40 + col 20 + rowptr 4 + p_{k-1} 8 + r 8 + p_k 8 + w 8
FUSED_CG_BYTES_PER_ROW = 144    # fused SpMV 96 + calc_ur 48


def _peaks():
    try:
        with open(os.path.join(ROOT, "MEASURED_PEAKS.json")) as f:
            p = json.load(f)
        return float(p["hbm_gbs"]), "measured (MEASURED_PEAKS.json hbm_gbs)"
    except Exception:
        return 6650.0, "fallback (B200_PROFILING.md 6.65 TB/s)"


class ClockSampler:
    """nvidia-smi clocks + throttle reasons DURING the timed region."""
    Q = ("clocks.sm,clocks.max.sm,clocks_event_reasons.hw_slowdown,clocks_event_reasons.hw_thermal_slowdown,"
         "clocks_event_reasons.sw_thermal_slowdown,clocks_event_reasons.sw_power_cap,power.draw")

    def __init__(self, index: int):
        self.index, self.rows, self.proc = index, [], None

    def __enter__(self):
        try:
            self.proc = subprocess.Popen(["nvidia-smi", "-i", str(self.index), "--query-gpu=" + self.Q,
                                          "--format=csv,noheader,nounits", "-lms", "200"],
                                         stdout=subprocess.PIPE, stderr=subprocess.DEVNULL, text=True)
            self.t = threading.Thread(target=self._read, daemon=True)
            self.t.start()
        except Exception:
            self.proc = None
        return self

    def _read(self):
        for line in self.proc.stdout:
            parts = [p.strip() for p in line.split(",")]
            if len(parts) >= 7:
                self.rows.append(parts)

    def __exit__(self, *a):
        if self.proc:
            self.proc.terminate()
            try:
                self.proc.wait(timeout=5)
            except Exception:
                self.proc.kill()

    def summary(self):
        if not self.rows:
            return {"sm_mhz": None, "sm_max_mhz": None, "reasons": ["unsampled"]}
        sm = [float(r[0]) for r in self.rows if r[0].replace(".", "").isdigit()]
        mx = [float(r[1]) for r in self.rows if r[1].replace(".", "").isdigit()]
        names = ["hw_slowdown", "hw_thermal_slowdown", "sw_thermal_slowdown", "sw_power_cap"]
        reasons = sorted({names[k] for r in self.rows for k in range(4) if r[2 + k].lower() == "active"})
        return {"sm_mhz": statistics.median(sm) if sm else None, "sm_max_mhz": max(mx) if mx else None,
                "reasons": reasons, "samples": len(self.rows)}


# ------------------------------------------------------------------ problem
def chunk_layout(n: int, ny: int, rank: int, world: int, chunk_rows=None):
    """This rank's row-block chunks (no arrays) of an n x ny grid split into
    `world` strips of ny/world grid rows: global grid rows, row_base / col_base
    in the rank's halo-extended vector, rows and column-window width (<= 2^24
    for the 24-bit element index, reading R7)."""
    import gen
    rows = ny // world
    y0r, y1r = rank * rows, (rank + 1) * rows
    halo = n if world > 1 else 0
    out = []
    for (c0, c1, cb) in gen.chunk_plan(n, y1r - y0r, chunk_rows=chunk_rows, halo=world > 1):
        # local grid rows [c0, c1) of this rank's strip; vector index = halo + local row index
        row_base = halo + c0 * n
        col_base = max(0, row_base - n) if world > 1 or c0 > 0 else 0
        ncols = min(halo + (y1r - y0r) * n + halo, row_base + (c1 - c0) * n + n) - col_base
        out.append(dict(gy0=y0r + c0, gy1=y0r + c1, row_base=row_base, col_base=col_base, nrows=(c1 - c0) * n,
                        ncols=ncols))
    return out


def build_problem(n: int, ny: int, rank: int, world: int, device, chunk_rows=None):
    """Raw (unencoded) device arrays of this rank's strip of the n x ny G-TEA
    grid, as row-block chunks whose column windows fit the 24-bit element index
    (reading R7)."""
    import torch
    import gen
    if ny % world:
        raise ValueError(f"{ny} grid rows do not split into {world} equal strips")
    rows = ny // world
    y0r, y1r = rank * rows, (rank + 1) * rows
    halo = n if world > 1 else 0
    chunks = []
    for L in chunk_layout(n, ny, rank, world, chunk_rows):
        val, col, rowptr = gen.strip_csr(n, L["gy0"], L["gy1"], ny=ny, device=device,
                                         col_offset=L["row_base"] - L["col_base"])
        chunks.append(dict(val=val.contiguous(), col=col.to(torch.int32).contiguous(),
                           rowptr=rowptr.to(torch.int32).contiguous(), row_base=L["row_base"],
                           col_base=L["col_base"], nrows=L["nrows"], ncols=L["ncols"]))
    b = gen.tealeaf_rhs(n, y0r, y1r, ny=ny, device=device)
    N = (y1r - y0r) * n
    return dict(chunks=chunks, b=b.contiguous(), N=N, n=n, halo=halo)


class Solver:
    """One configuration (protected or unprotected twin) of the solve."""

    def __init__(self, abft, ctx, P, es, rs, vs, dist=None, check_interval=1, sr=False, peer=False):
        import torch
        self.abft, self.ctx, self.P, self.dist = abft, ctx, P, dist
        self.peer = peer and dist is not None and not sr   # peer-memory halos
        self.check_interval = check_interval
        self.es, self.rs, self.vs = es, rs, vs
        N, halo = P["N"], P["halo"]
        dev = P["b"].device
        self.A, self.raw = [], []
        for ch in P["chunks"]:
            M = abft.Matrix(ch["val"], ch["col"].clone(), ch["rowptr"], ch["nrows"], ch["ncols"], es, rs,
                            row_base=ch["row_base"], col_base=ch["col_base"], stencil_n=P["n"])
            rp_raw = torch.zeros_like(M.rowptr)
            rp_raw[:ch["nrows"] + 1] = ch["rowptr"]
            self.A.append(M)
            self.raw.append((ch["col"], rp_raw))
        n_ext = N + 2 * halo
        self.sr = sr   # single-reduction CG: a sixth vector s
        self.vecs = [abft.Vector.empty(n_ext, vs, device=dev) for _ in range(6 if sr else 5)]  # b x r p w [s]
        self.counts = abft.Counters(device=dev)
        self.b_raw = P["b"]
        self.N, self.halo = N, halo

    def load_inputs(self, host=None):
        """(Re)place the raw inputs: from device copies, or from pinned host buffers (e2e)."""
        for i, (M, (col_raw, rp_raw)) in enumerate(zip(self.A, self.raw)):
            if host is None:
                M.col.copy_(col_raw)
                M.rowptr.copy_(rp_raw)
            else:
                hv, hc, hr = host["chunks"][i]
                M.val.copy_(hv, non_blocking=True)
                M.col.copy_(hc, non_blocking=True)
                M.rowptr[:M.nrows + 1].copy_(hr, non_blocking=True)
                M.rowptr[M.nrows + 1:].zero_()
        src_b = self.b_raw if host is None else host["b"]
        b, x = self.vecs[0], self.vecs[1]
        h = self.halo
        b.data[h:h + self.N].copy_(src_b, non_blocking=True)
        x.data[h:h + self.N].copy_(src_b, non_blocking=True)

    def step(self, tol, max_iters, host=None):
        """a0 + a1 + a2..a7: returns the iteration count."""
        self.load_inputs(host)
        for M in self.A:
            st = M.encode(self.ctx)
            if st != 0:
                raise RuntimeError(f"encode failed: {self.abft.last_error()}")
        self.vecs[0].encode(self.ctx)
        self.vecs[1].encode(self.ctx)
        if self.sr:
            if self.dist is not None:
                res = self.dist.cg_solve_sr(self.ctx, self.A, self.halo, *self.vecs, tol=tol, max_iters=max_iters,
                                            due_policy=1, counts=self.counts, poll_every=32)
            else:
                res = self.abft.cg_solve_sr(self.ctx, self.A, *self.vecs, tol=tol, max_iters=max_iters, due_policy=1,
                                            counts=self.counts, poll_every=32)
        elif self.dist is not None:
            # peer-memory halos name this solver's p: map the neighbours' p once
            # (collective), and never leave another solver's mapping enabled
            owner = getattr(self.dist, "_peer_owner", None)
            if owner is not (self if self.peer else None):
                self.dist.disable_peer_halo()
                self.dist._peer_owner = None
                if self.peer:
                    self.dist.enable_peer_halo(self.vecs[3])
                    self.dist._peer_owner = self
            res = self.dist.cg_solve(self.ctx, self.A, self.halo, *self.vecs, tol=tol, max_iters=max_iters,
                                     due_policy=1, counts=self.counts, poll_every=32,
                                     check_interval=self.check_interval)
        else:
            res = self.abft.cg_solve(self.ctx, self.A, *self.vecs, tol=tol, max_iters=max_iters, due_policy=1,
                                     counts=self.counts, poll_every=32, check_interval=self.check_interval)
        return res.iters, res.status


def host_inputs(P):
    """Pinned host copies of the raw inputs (the e2e leg's H2D source)."""
    chunks = [(c["val"].cpu().pin_memory(), c["col"].cpu().pin_memory(), c["rowptr"].cpu().pin_memory())
              for c in P["chunks"]]
    return {"chunks": chunks, "b": P["b"].cpu().pin_memory()}


def timed(solver, steps, warmup, tol, max_iters, dist_on, host=None, out_host=None, profile=0):
    import torch
    import torch.distributed as dist
    abft = solver.abft
    for _ in range(warmup):
        solver.step(tol, max_iters, host)
    torch.cuda.synchronize()
    if dist_on:
        dist.barrier()
    if profile:
        abft.profile(solver.ctx, profile)
    l0 = abft.launch_count()
    e0, e1 = torch.cuda.Event(enable_timing=True), torch.cuda.Event(enable_timing=True)
    iters = 0
    statuses = set()
    e0.record()
    for _ in range(steps):
        it, st = solver.step(tol, max_iters, host)
        if out_host is not None:
            x = solver.vecs[1]
            out_host.copy_(x.data[solver.halo:solver.halo + solver.N], non_blocking=True)
        iters += it
        statuses.add(st)
    e1.record()
    torch.cuda.synchronize()
    launches = abft.launch_count() - l0
    ms = e0.elapsed_time(e1)
    prof = abft.profile_read(solver.ctx) if profile else None
    if profile:
        abft.profile(solver.ctx, 0)
    if dist_on:
        t = torch.tensor([ms], dtype=torch.float64, device="cuda")
        dist.all_reduce(t, op=dist.ReduceOp.MAX)
        ms = float(t.item())
        dist.barrier()
    return dict(ms=ms, iters=iters, launches=launches, prof=prof, statuses=statuses)


def read_traffic():
    """dram bytes per SpMV launch from the committed ncu --set full summary (or None)."""
    p = os.path.join(ROOT, "profiles", "spmv_traffic.json")
    try:
        with open(p) as f:
            t = json.load(f)
    except Exception:
        return None
    b = t.get("bytes_per_launch")
    if not isinstance(b, (int, float)) or b != b:   # a failed capture leaves NaN: report null
        return None
    return t


def traffic_matches(t, grid, world, fused):
    """The stored capture is per SpMV launch of one workload (grid, ranks,
    calc_p arrangement); another workload's line reports traffic null."""
    return bool(t) and t.get("grid", 4096) == grid and t.get("n_gpus", 1) == world and t.get("fused", False) == fused


# ------------------------------------------------------------------ oracle legs
UNIT = "CG it/s (4096^2-equivalent)"


def cpu_info():
    model = None
    try:
        with open("/proc/cpuinfo") as f:
            for line in f:
                if line.startswith("model name"):
                    model = line.split(":", 1)[1].strip()
                    break
    except Exception:
        pass
    return {"model": model, "nproc": os.cpu_count()}


def oracle_sample(strip_rows=128, iters=3, grid=4096):
    """The CPU oracle (never tuned) on a bounded sample of the 4096^2 workload
    itself: the grid rows [grid/2, grid/2 + strip_rows) of the 4096^2 G-TEA
    matrix (config-2 schemes, read from their own input window), through `iters`
    CG iterations' worth of the oracle's hot-path calls (protected SpMV + p.w,
    calc_ur, calc_p), single-threaded and pinned to one host core; scaled to the
    whole 4096^2 iteration by rows.  Returns (it/s, cores, sample text)."""
    import numpy as np
    import gen
    import oracle as orc
    n = grid
    y0, y1 = n // 2, n // 2 + strip_rows
    w0, w1 = y0 - 1, y1 + 1
    rows = strip_rows * n
    v, c, r = gen.strip_csr(n, y0, y1, ny=n, col_offset=n)
    S = orc.SECDED64
    A = orc.Matrix(v.numpy(), c.numpy().astype(np.uint32), r.numpy().astype(np.uint32), rows, (w1 - w0) * n, S, S,
                   row_base=n, col_base=0)
    A.encode()
    W = (w1 - w0) * n
    p = orc.vec_encode(gen.uniform_pm1(W, 5), S)
    x = orc.vec_encode(gen.uniform_pm1(rows, 6), S)
    rv = orc.vec_encode(gen.uniform_pm1(rows, 7), S)
    out = np.zeros(W, dtype=np.uint64)
    old = os.sched_getaffinity(0)
    core = min(old)
    try:
        os.sched_setaffinity(0, {core})
        t0 = time.perf_counter()
        for _ in range(iters):
            orc.spmv(A, p, W, S, out, W, None, want_dot=True)
            w = out[n:n + rows].copy()
            pl = p[n:n + rows].copy()
            orc.calc_ur(x, pl, rv, w, rows, S, 1e-3, None)
            orc.calc_p(pl, rv, rows, S, 0.5, None)
        per_iter = (time.perf_counter() - t0) / iters
    finally:
        os.sched_setaffinity(0, old)
    its = 1.0 / (per_iter * (n * n) / rows)
    ci = cpu_info()
    sample = (f"{iters} CG iterations of the oracle's hot-path calls (protected SpMV + p.w, calc_ur, calc_p; "
              f"E-SECDED + R-SECDED64 + V-SECDED64) on grid rows [{y0}, {y1}) of the {n}^2 G-TEA matrix "
              f"({rows} of {n * n} rows), {per_iter:.3f} s per sampled iteration, scaled by rows to the whole "
              f"{n}^2 iteration; pinned to host core {core} ({ci['model']}, nproc {ci['nproc']})")
    return its, 1, sample


def run_reference(args):
    rank = int(os.environ.get("RANK", "0"))
    if rank != 0:
        return
    vals = []
    sample = ""
    for _ in range(args.warmup):
        oracle_sample(32, 1)
    t0 = time.perf_counter()
    for _ in range(args.steps):
        v, cores, sample = oracle_sample(args.oracle_rows, 1)
        vals.append(v)
    wall = time.perf_counter() - t0
    val = statistics.median(vals)
    line = {"impl": "reference", "metric": METRIC, "value": val, "unit": UNIT,
            "n_gpus": args.gpus, "steps": args.steps, "warmup": args.warmup,
            "ms_per_step": 1000.0 * wall / max(args.steps, 1), "higher_is_better": True, "scaling": "weak",
            "vs_baseline": None, "dtype": "f64", "data": "synthetic",
            "config": {"workload": "tealeaf-4096x4096-cg-full-ecc", "grid": 4096, "sample_strip_rows": args.oracle_rows},
            "cpu_baseline": {"value": val, "unit": UNIT, "cores": cores, "kind": "oracle", "sample": sample,
                             "cpu": cpu_info()},
            "e2e": {"value": val, "unit": UNIT, "h2d_bytes_per_step": 0, "d2h_bytes_per_step": 0}}
    print(json.dumps(line), flush=True)


# ------------------------------------------------------------------ main
def main():
    ap = argparse.ArgumentParser()
    ap.add_argument("--gpus", type=int, default=1)
    ap.add_argument("--steps", type=int, default=3)
    ap.add_argument("--warmup", type=int, default=3)
    ap.add_argument("--impl", default="ours", choices=["ours", "reference"])
    ap.add_argument("--grid", type=int, default=None, help="grid side (default 4096; 16384 with --mode strong)")
    ap.add_argument("--tol", type=float, default=1e-10)
    ap.add_argument("--max-iters", type=int, default=20000)
    ap.add_argument("--oracle-rows", type=int, default=64, help="grid rows of the 4096^2 strip the oracle legs time")
    ap.add_argument("--mode", default="weak", choices=["weak", "strong"],
                    help="N > 1: weak = a grid x grid strip per GPU (config 2 per GPU); strong = config 4, one "
                         "fixed grid x grid problem (default grid 16384) split into N strips")
    ap.add_argument("--chunk-rows", type=int, default=None, help="grid rows per row-block chunk (default: fit 2^24 cols)")
    ap.add_argument("--no-cpu-baseline", action="store_true")
    ap.add_argument("--no-e2e", action="store_true")
    ap.add_argument("--fuse", action="store_true", help="main line on the fused calc_p path (DESIGN.md §6.1)")
    ap.add_argument("--no-pdl", action="store_true", help="plain launches in the CG loop (DESIGN.md §6.2)")
    ap.add_argument("--no-fused-extra", action="store_true", help="skip the fused-calc_p side measurement")
    ap.add_argument("--peer-halo", action="store_true",
                    help="N > 1: p's halo stored by the neighbours' calc_p over NVLink peer memory (DESIGN.md §8)")
    ap.add_argument("--no-sr-extra", action="store_true",
                    help="skip the single-reduction CG side measurement (DESIGN.md §4.1)")
    args = ap.parse_args()
    if args.impl == "reference":
        return run_reference(args)
    if args.grid is None:
        args.grid = 16384 if args.mode == "strong" else 4096

    import torch
    import torch.distributed as dist
    world = int(os.environ.get("WORLD_SIZE", "1"))
    rank = int(os.environ.get("RANK", "0"))
    local = int(os.environ.get("LOCAL_RANK", "0"))
    torch.cuda.set_device(local)
    dist_on = world > 1
    if dist_on:
        dist.init_process_group("nccl", device_id=torch.device("cuda", local))
    from paper_conf_cluster_pawelczakmpm17_b200 import abft

    ny = args.grid * world if args.mode == "weak" else args.grid
    P = build_problem(args.grid, ny, rank, world, torch.device("cuda", local), args.chunk_rows)
    ctx = abft.Context(local)
    # fused calc_p (opt-in) runs on the single-GPU tiled path (the dist path exchanges p halos unfused)
    fused = args.fuse and not dist_on
    ctx.set_fused_cg(fused)
    ctx.set_pdl(not args.no_pdl)
    spmv_bpr = FUSED_SPMV_BYTES_PER_ROW if fused else SPMV_BYTES_PER_ROW
    cg_bpr = FUSED_CG_BYTES_PER_ROW if fused else CG_BYTES_PER_ROW
    dobj = abft.Dist(rank, world, local) if dist_on else None
    prot = Solver(abft, ctx, P, abft.SECDED64, abft.SECDED64, abft.SECDED64, dobj, peer=args.peer_halo)
    with ClockSampler(local) as clk:
        r_p = timed(prot, args.steps, args.warmup, args.tol, args.max_iters, dist_on)
        # roofline pass: same workload, every SpMV launch bracketed by CUDA events on
        # the launch stream (event-timed solves launch kernels directly, no graph)
        r_ps = timed(prot, args.steps, 0, args.tol, args.max_iters, dist_on, profile=1)
    clocks = clk.summary()
    # per-kernel breakdown: one extra, untimed, fully profiled step
    r_pk = timed(prot, 1, 0, args.tol, args.max_iters, dist_on, profile=15)
    del prot
    twin = Solver(abft, ctx, P, abft.NONE, abft.NONE, abft.NONE, dobj, peer=args.peer_halo)
    r_u = timed(twin, args.steps, max(1, args.warmup // 2), args.tol, args.max_iters, dist_on)
    r_uk = timed(twin, 1, 0, args.tol, args.max_iters, dist_on, profile=15)
    del twin

    # side measurement: the other calc_p arrangement (fused <-> unfused), protected and unprotected
    alt = None
    if not dist_on and not args.no_fused_extra:
        ctx.set_fused_cg(not fused)
        a_p = Solver(abft, ctx, P, abft.SECDED64, abft.SECDED64, abft.SECDED64, dobj)
        r_ap = timed(a_p, args.steps, 1, args.tol, args.max_iters, dist_on)
        r_apk = timed(a_p, 1, 0, args.tol, args.max_iters, dist_on, profile=15)
        del a_p
        a_u = Solver(abft, ctx, P, abft.NONE, abft.NONE, abft.NONE, dobj)
        r_au = timed(a_u, args.steps, 1, args.tol, args.max_iters, dist_on)
        del a_u
        ctx.set_fused_cg(fused)
        eq_ = P["N"] / float(4096 * 4096)
        ip, iu = r_ap["ms"] / max(r_ap["iters"], 1), r_au["ms"] / max(r_au["iters"], 1)
        ms_a, n_a = r_apk["prof"]
        alt = {"fused_calc_p": not fused,
               "value": r_ap["iters"] / (r_ap["ms"] / 1000.0) * eq_,
               "unprotected_value": r_au["iters"] / (r_au["ms"] / 1000.0) * eq_,
               "overhead_pct_per_iter": 100.0 * (ip / iu - 1.0),
               "bytes_per_row_per_iter": CG_BYTES_PER_ROW if fused else FUSED_CG_BYTES_PER_ROW,
               "kernel_ms": {"spmv": ms_a[0] / max(n_a[0], 1), "calc_ur": ms_a[1] / max(n_a[1], 1),
                             "calc_p": ms_a[2] / max(n_a[2], 1), "reductions": ms_a[3] / max(n_a[3], 1)}}

    # side measurement: the single-reduction CG (one reduction per iteration), protected and unprotected
    alt_sr = None
    if not args.no_sr_extra:
        s_p = Solver(abft, ctx, P, abft.SECDED64, abft.SECDED64, abft.SECDED64, dobj, sr=True)
        r_sp = timed(s_p, args.steps, 1, args.tol, args.max_iters, dist_on)
        del s_p
        s_u = Solver(abft, ctx, P, abft.NONE, abft.NONE, abft.NONE, dobj, sr=True)
        r_su = timed(s_u, args.steps, 1, args.tol, args.max_iters, dist_on)
        del s_u
        eq_ = P["N"] / float(4096 * 4096)
        ip, iu = r_sp["ms"] / max(r_sp["iters"], 1), r_su["ms"] / max(r_su["iters"], 1)
        alt_sr = {"value": world * r_sp["iters"] / (r_sp["ms"] / 1000.0) * eq_,
                  "unprotected_value": world * r_su["iters"] / (r_su["ms"] / 1000.0) * eq_,
                  "iters_per_step": r_sp["iters"] / args.steps,
                  "overhead_pct_per_iter": 100.0 * (ip / iu - 1.0), "bytes_per_row_per_iter": CG_BYTES_PER_ROW,
                  "statuses": sorted(r_sp["statuses"])}

    e2e = None
    if not args.no_e2e:
        prot = Solver(abft, ctx, P, abft.SECDED64, abft.SECDED64, abft.SECDED64, dobj)
        host = host_inputs(P)
        out_host = torch.empty(P["N"], dtype=torch.float64).pin_memory()
        r_e = timed(prot, args.steps, 1, args.tol, args.max_iters, dist_on, host=host, out_host=out_host)
        h2d = sum(t.numel() * t.element_size() for c in host["chunks"] for t in c) + host["b"].numel() * 8
        e2e = {"value": world * r_e["iters"] / (r_e["ms"] / 1000.0) * P["N"] / float(4096 * 4096),
               "unit": UNIT,
               "h2d_bytes_per_step": h2d, "d2h_bytes_per_step": P["N"] * 8}
        del prot

    if rank != 0:
        if dist_on:
            dist.destroy_process_group()
        return

    N = P["N"]
    eq = N / float(4096 * 4096)   # 4096^2-equivalent: scale by rows per GPU
    its = r_p["iters"] / (r_p["ms"] / 1000.0) * eq
    its_u = r_u["iters"] / (r_u["ms"] / 1000.0) * eq
    peak, peak_src = _peaks()
    ms_t, n_t = r_ps["prof"]         # roofline pass: SpMV launches only
    spmv_ms = ms_t[0] / max(n_t[0], 1)
    spmv_gbs = spmv_bpr * N / (spmv_ms / 1000.0) / 1e9 if spmv_ms > 0 else None
    ms_cls, n_cls = r_pk["prof"]     # separate profiled step: all kernel classes
    ms_u, n_u = r_uk["prof"]
    traffic = read_traffic()
    iter_ms_p = r_p["ms"] / max(r_p["iters"], 1)
    iter_ms_u = r_u["ms"] / max(r_u["iters"], 1)
    line = {
        "metric": METRIC,
        "value": world * its,
        "unit": UNIT,
        "n_gpus": world,
        "steps": args.steps,
        "warmup": args.warmup,
        "ms_per_step": r_p["ms"] / args.steps,
        "higher_is_better": True,
        "scaling": args.mode if world > 1 else "weak",
        "vs_baseline": None,
        "dtype": "f64",
        "data": "synthetic",
        "config": {"workload": f"tealeaf-{args.grid}x{ny}-cg-full-ecc", "grid": args.grid, "grid_rows": ny,
                   "rows_per_gpu": N,
                   "chunks": len(P["chunks"]),
                   "schemes": {"elements": "E-SECDED", "rowptr": "R-SECDED64", "vectors": "V-SECDED64"},
                   "tol": args.tol, "iters_per_step": r_p["iters"] / args.steps,
                   "l2": f"inputs larger than L2 ({cg_bpr * N / 1e9:.2f} GB moved per CG iteration vs 126 MB L2)",
                   "parallelism": f"row-block strips x{world}" if world > 1 else "single GPU",
                   "fused_calc_p": fused, "pdl": not args.no_pdl and not dist_on, "bytes_per_row_per_iter": cg_bpr,
                   "halo": ("peer-memory" if args.peer_halo else "nccl send/recv") if world > 1 else None},
        "roofline": {"bound": "hbm",
                     "kernel": "k_spmv_tile (fused calc_p + protected SpMV + p.w)" if fused
                     else "k_spmv_tile (protected SpMV + p.w)",
                     "achieved": spmv_gbs, "peak": peak, "unit": "GB/s",
                     "frac": (spmv_gbs / peak) if spmv_gbs else None,
                     "traffic": traffic.get("bytes_per_launch") if traffic_matches(traffic, args.grid, world, fused) else None,
                     "bytes_per_launch_algorithmic": spmv_bpr * N, "peak_source": peak_src,
                     "avg_launch_ms": spmv_ms},
        "cg_bandwidth": {"achieved_gbs": cg_bpr * N / (iter_ms_p / 1000.0) / 1e9,
                         "frac_of_measured": cg_bpr * N / (iter_ms_p / 1000.0) / 1e9 / peak,
                         "frac_of_8tbs": cg_bpr * N / (iter_ms_p / 1000.0) / 1e9 / 8000.0,
                         "bytes_per_row_per_iter": cg_bpr},
        "kernel_ms": {"spmv": ms_cls[0] / max(n_cls[0], 1), "calc_ur": ms_cls[1] / max(n_cls[1], 1),
                      "calc_p": ms_cls[2] / max(n_cls[2], 1), "reductions": ms_cls[3] / max(n_cls[3], 1),
                      "note": "one extra untimed step with every kernel class bracketed by events"},
        "unprotected": {"value": world * its_u, "iter_ms": iter_ms_u, "iters_per_step": r_u["iters"] / args.steps,
                        "spmv_ms": ms_u[0] / max(n_u[0], 1), "calc_ur_ms": ms_u[1] / max(n_u[1], 1),
                        "calc_p_ms": ms_u[2] / max(n_u[2], 1), "reductions_ms": ms_u[3] / max(n_u[3], 1)},
        "overhead_pct_per_iter": 100.0 * (iter_ms_p / iter_ms_u - 1.0),
        "alt_calc_p_arrangement": alt,
        "alt_single_reduction_cg": alt_sr,
        "clocks": clocks,
        "gpu_launches": r_p["launches"],
        "e2e": e2e,
    }
    if world == 1 and not args.no_cpu_baseline:
        v, cores, sample = oracle_sample(2 * args.oracle_rows, 3)
        line["cpu_baseline"] = {"value": v, "unit": UNIT, "cores": cores, "kind": "oracle", "sample": sample,
                                "cpu": cpu_info()}
    print(json.dumps(line), flush=True)
    if dist_on:
        dist.destroy_process_group()


if __name__ == "__main__":
    main()
