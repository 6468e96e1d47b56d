"""Multi-rank host logic on CPU (torch.distributed gloo, world size 2 and 4).

Each rank owns a strip of grid rows of the G-TEA problem with one ghost grid
row above/below its local vectors.  Per CG iteration the ranks
exchange the encoded boundary rows of p (ECC travels with the data), run the
oracle SpMV / calc_ur / calc_p on their strip, and all-gather one RED-1
subtree root per dot product, combining them with the top of the tree.  This is
the algorithm `abft_cg_solve_dist` runs over NCCL; here it is checked against
the single-process oracle CG: identical iteration count, bit-identical x and r,
and fault counters that sum to the single-process counts (owner rule).
"""
import os

import numpy as np
import pytest
import torch
import torch.distributed as dist
import torch.multiprocessing as mp

import gen
import oracle as orc

N_GRID = 32


def _single(scheme, flips):
    n = N_GRID
    N = n * n
    v, c, r = gen.tealeaf_csr(n)
    es = rs = orc.SECDED64
    A = orc.Matrix(v.numpy(), c.numpy().astype(np.uint32), r.numpy().astype(np.uint32), N, N, es, rs)
    A.encode()
    b = gen.tealeaf_rhs(n).numpy()
    B = orc.vec_encode(b, scheme)
    X = B.copy()
    for (i, bit) in flips:
        X[i] ^= np.uint64(1 << bit)
    R, P, W = (np.zeros_like(B) for _ in range(3))
    cnt = orc.new_counts()
    st, res = orc.cg_solve(A, B, X, R, P, W, scheme, 1e-10, 500, 1, cnt)
    return res.iters, X[:N], R[:N], cnt


def _worker(rank, world, port, scheme, flips, q):
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        n = N_GRID
        rows = n // world
        y0, y1 = rank * rows, (rank + 1) * rows
        N = rows * n
        h = n
        v, c, r = gen.strip_csr(n, y0, y1, ny=n, col_offset=h)
        es = rs = orc.SECDED64
        A = orc.Matrix(v.numpy(), c.numpy().astype(np.uint32), r.numpy().astype(np.uint32), N, N + 2 * h, es, rs,
                       row_base=h, col_base=0)
        A.encode()
        b = gen.tealeaf_rhs(n, y0, y1, ny=n).numpy()
        ext = N + 2 * h

        def vec(vals=None):
            out = np.zeros(ext, dtype=np.uint64)
            if vals is not None:
                out[h:h + N] = orc.vec_encode(vals, scheme)[:N]
            return out

        B, X = vec(b), vec(b)
        for (i, bit) in flips:  # global index -> owner rank's local slot
            if y0 * n <= i < y1 * n:
                X[h + i - y0 * n] ^= np.uint64(1 << bit)
        R, Pv, W = vec(), vec(), vec()
        cnt = orc.new_counts()

        def halo(a):
            t = torch.from_numpy(a.view(np.int64))
            reqs = []
            if rank > 0:
                reqs.append(dist.isend(t[h:2 * h].clone(), rank - 1))
                top = torch.empty(h, dtype=torch.int64)
                reqs.append(dist.irecv(top, rank - 1))
            if rank < world - 1:
                reqs.append(dist.isend(t[N:N + h].clone(), rank + 1))
                bot = torch.empty(h, dtype=torch.int64)
                reqs.append(dist.irecv(bot, rank + 1))
            for rq in reqs:
                rq.wait()
            if rank > 0:
                a[0:h] = top.numpy().view(np.uint64)
            if rank < world - 1:
                a[h + N:] = bot.numpy().view(np.uint64)

        def combine(root):
            g = [torch.zeros(1, dtype=torch.float64) for _ in range(world)]
            dist.all_gather(g, torch.tensor([root], dtype=torch.float64))
            return orc.tree_sum(np.array([x.item() for x in g]))

        loc = slice(h, h + N)
        halo(X)
        orc.spmv(A, X, ext, scheme, W, ext, cnt)
        _, rr0_loc = orc.cg_init_r(B[loc], W[loc], R[loc], Pv[loc], N, scheme, cnt)
        rr0 = rro = combine(rr0_loc)
        iters = 0
        for k in range(1, 501):
            halo(Pv)
            _, pw_loc = orc.spmv(A, Pv, ext, scheme, W, ext, cnt, want_dot=True)
            pw = combine(pw_loc)
            alpha = rro / pw
            xl, pl, rl, wl = X[loc].copy(), Pv[loc].copy(), R[loc].copy(), W[loc].copy()
            _, rrn_loc = orc.calc_ur(xl, pl, rl, wl, N, scheme, alpha, cnt)
            X[loc], Pv[loc], R[loc], W[loc] = xl, pl, rl, wl
            rrn = combine(rrn_loc)
            iters = k
            if np.sqrt(rrn) <= 1e-10 * np.sqrt(rr0):
                break
            beta = rrn / rro
            pl, rl = Pv[loc].copy(), R[loc].copy()
            orc.calc_p(pl, rl, N, scheme, beta, cnt)
            Pv[loc], R[loc] = pl, rl
            rro = rrn
        q.put((rank, iters, X[loc].copy(), R[loc].copy(), cnt))
    finally:
        dist.destroy_process_group()


@pytest.mark.parametrize("world", [2, 4])
@pytest.mark.parametrize("scheme_name", ["SECDED64", "SED"])
def test_distributed_cg_matches_single_process(world, scheme_name):
    scheme = getattr(orc, scheme_name)
    orc.build()
    flips = [(5, 7), (300, 40), (700, 63), (1000, 2)]   # single flips in x0 on several ranks
    it1, x1, r1, cnt1 = _single(scheme, flips)
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = 29500 + world * 7 + scheme
    procs = [ctx.Process(target=_worker, args=(rk, world, port, scheme, flips, q)) for rk in range(world)]
    for p in procs:
        p.start()
    out = [q.get(timeout=300) for _ in range(world)]
    for p in procs:
        p.join(timeout=60)
        assert p.exitcode == 0
    out.sort(key=lambda t: t[0])
    assert all(o[1] == it1 for o in out), ([o[1] for o in out], it1)
    xg = np.concatenate([o[2] for o in out])
    rg = np.concatenate([o[3] for o in out])
    assert np.array_equal(xg, x1)
    assert np.array_equal(rg, r1)
    cnt = sum(o[4] for o in out)
    assert np.array_equal(cnt, cnt1), (cnt, cnt1)


@pytest.mark.parametrize("world", [1, 2, 4, 8])
@pytest.mark.parametrize("grid", [4096, 8192, 16384])
@pytest.mark.parametrize("mode", ["weak", "strong"])
def test_bench_chunk_layout_fits_element_index(world, grid, mode):
    """bench.py's per-rank chunks (weak scaling: a grid x grid strip per rank of
    a grid x grid*world grid; strong scaling, config 4: grid/world rows of a
    fixed grid x grid grid) cover the strip and keep every column window within
    E-SECDED's 24-bit index and R-SECDED's 28-bit nnz (reading R7), at the
    sizes the driver runs (no arrays are built)."""
    import bench
    ny = grid * world if mode == "weak" else grid
    rows = ny // world
    for rank in {0, world // 2, world - 1}:
        L = bench.chunk_layout(grid, ny, rank, world)
        halo = grid if world > 1 else 0
        assert L[0]["row_base"] == halo and L[0]["gy0"] == rank * rows and L[-1]["gy1"] == (rank + 1) * rows
        for a, b in zip(L[:-1], L[1:]):
            assert a["gy1"] == b["gy0"] and b["row_base"] == a["row_base"] + a["nrows"]
        for c in L:
            assert c["ncols"] <= 1 << 24 and 5 * c["nrows"] <= (1 << 28) - 1
            assert c["nrows"] % 256 == 0 and (c["row_base"] - halo) % 256 == 0
            # the window covers the chunk's rows and one grid row either side (ghost rows for world > 1)
            assert c["col_base"] <= max(0, c["row_base"] - grid)
            assert c["col_base"] + c["ncols"] >= min(c["row_base"] + c["nrows"] + grid, halo + grid * rows + halo)


def test_bench_traffic_null_for_failed_capture(tmp_path, monkeypatch):
    """bench.py's roofline `traffic` comes from profiles/spmv_traffic.json; a
    failed ncu capture leaves NaN there, which must be reported as null (a NaN
    would make the JSON line invalid)."""
    import json
    import bench
    (tmp_path / "profiles").mkdir()
    f = tmp_path / "profiles" / "spmv_traffic.json"
    monkeypatch.setattr(bench, "ROOT", str(tmp_path))
    f.write_text('{"bytes_per_launch": NaN}')
    assert bench.read_traffic() is None
    f.write_text(json.dumps({"bytes_per_launch": 1336580796.0}))
    assert bench.read_traffic()["bytes_per_launch"] == 1336580796.0
    f.unlink()
    assert bench.read_traffic() is None


def test_bench_traffic_only_for_the_captured_workload():
    """The stored DRAM bytes are per launch of one workload: other grids, rank
    counts or the fused arrangement report traffic null."""
    import bench
    t = {"bytes_per_launch": 1.0, "grid": 4096, "n_gpus": 1, "fused": False}
    assert bench.traffic_matches(t, 4096, 1, False)
    assert not bench.traffic_matches(t, 16384, 1, False)
    assert not bench.traffic_matches(t, 4096, 2, False)
    assert not bench.traffic_matches(t, 4096, 1, True)
    assert not bench.traffic_matches(None, 4096, 1, False)


# ---------------------------------------------------------------- peer-memory halo handshake
def _peer_worker(rank, world, port, q):
    """Dist.enable_peer_halo's host logic over gloo with the CUDA IPC calls
    faked: every rank publishes (handle, offset) of its p and of its flag
    words, maps its neighbours' and hands abft_dist_set_peer_halo rank-1's p
    and flags[1], rank+1's p and flags[0]."""
    os.environ["MASTER_ADDR"] = "127.0.0.1"
    os.environ["MASTER_PORT"] = str(port)
    dist.init_process_group("gloo", rank=rank, world_size=world)
    try:
        import ctypes as C
        from paper_conf_cluster_pawelczakmpm17_b200 import abft
        P_BASE, F_BASE = 0x10000000, 0x20000000   # fake device addresses of rank r: base + r * 0x1000

        class FakeLib:
            def abft_dist_flags(self, h, out):
                out._obj.value = F_BASE + rank * 0x1000
                return 0

            def abft_ipc_get_handle(self, ptr, hb, off):   # handle = allocation base, 8 bytes LE
                o = 8 if ptr.value >= F_BASE else 16
                base = ptr.value - o
                buf = (C.c_uint8 * 64).from_address(hb.value)
                for i in range(8):
                    buf[i] = base >> (8 * i) & 0xFF
                off._obj.value = o
                return 0

            def abft_ipc_open_handle(self, hb, off, out):
                buf = (C.c_uint8 * 64).from_address(hb.value)
                out._obj.value = sum(buf[i] << (8 * i) for i in range(8)) + off
                return 0

            def abft_ipc_close_handle(self, ptr, off):
                return 0

            def abft_dist_set_peer_halo(self, h, enable, pp, pf):
                if enable:
                    pa = (C.c_void_p * 2).from_address(pp.value)
                    fa = (C.c_void_p * 2).from_address(pf.value)
                    self.got = ([pa[0], pa[1]], [fa[0], fa[1]])
                return 0

        fake = FakeLib()
        real = abft._lib
        abft._lib = fake
        try:
            d = abft.Dist.__new__(abft.Dist)
            d.h, d.rank, d.nranks = C.c_void_p(1), rank, world

            class FakeVec:
                class data:
                    @staticmethod
                    def data_ptr():
                        return P_BASE + rank * 0x1000

            d.enable_peer_halo(FakeVec())
            q.put((rank, fake.got))
        finally:
            abft._lib = real
    finally:
        dist.destroy_process_group()


@pytest.mark.parametrize("world", [2, 3])
def test_peer_halo_handshake_gloo(world):
    ctx = mp.get_context("spawn")
    q = ctx.Queue()
    port = 29650 + world
    procs = [ctx.Process(target=_peer_worker, args=(r, world, port, q)) for r in range(world)]
    for p in procs:
        p.start()
    got = dict(q.get(timeout=240) for _ in range(world))
    for p in procs:
        p.join(timeout=60)
        assert p.exitcode == 0
    P_BASE, F_BASE = 0x10000000, 0x20000000
    for r in range(world):
        pp, pf = got[r]
        up, dn = r > 0, r < world - 1
        # rank-1's and rank+1's p, mapped at their own addresses (handle + offset)
        assert pp[0] == (P_BASE + (r - 1) * 0x1000 if up else None)
        assert pp[1] == (P_BASE + (r + 1) * 0x1000 if dn else None)
        # rank-1 is signalled in its flags[1] (+4 bytes), rank+1 in its flags[0]
        assert pf[0] == (F_BASE + (r - 1) * 0x1000 + 4 if up else None)
        assert pf[1] == (F_BASE + (r + 1) * 0x1000 if dn else None)
