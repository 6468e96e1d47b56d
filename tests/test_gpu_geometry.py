"""GPU parity at the PRODUCTION geometry (S§8(c) A4 and
PIN-15, SURVEY.md:564, :605).

Every earlier tiled-path test used n = 256, where tiles_x = 1 and every tile
is both a left and a right grid edge.  Here:

* n = 1024 (tiles_x = 4): the tiled SpMV (every vector scheme, one chunk and
  two chunks) and the fused calc_p + SpMV, with single and same-word double
  flips in the cross-tile halo cells x = 255/256, 511/512, 767/768 at the
  tile-row edges y = 7/8, 15/16, the middle rows and the grid's first / last
  row, in the elements of those rows and in their row pointers — bit-exact
  words, counters, scrubbed storage and dot;
* 4096^2 (config 2, N = 2^24): one full SpMV + calc_ur + calc_p bit-exact
  against the oracle, including the element with col = 2^24 - 1 (the E-SECDED
  capacity edge, reading R4) with a flipped index bit, and the encoded matrix;
* 8192^2 (config 3) in its 5 row-block chunks (reading R7): the whole SpMV on
  the GPU, compared with the oracle on sampled strips around every chunk
  boundary and the grid's edges (the oracle computes those rows one by one from
  their own input window), with flips inside the strips;
* tiled CG to convergence at 512^2 (tiles_x = 2): equal iterations, bit-exact
  x / r / p / w and counters.

The 4096^2 test runs the (single-threaded) oracle's independent calls in
parallel worker processes; each call is the unmodified oracle."""
import multiprocessing as mp
import os
import tempfile

import numpy as np
import pytest
import torch

import gen
import oracle as orc
from gpu_helpers import col_words, gpu_matrix, gpu_vec_from_words, oracle_matrix, rowptr_words, val_words, words_of

pytestmark = pytest.mark.gpu

TILE_TY = 8


@pytest.fixture(scope="module")
def abft():
    from paper_conf_cluster_pawelczakmpm17_b200 import build
    build.build()
    from paper_conf_cluster_pawelczakmpm17_b200 import abft as A
    return A


@pytest.fixture(scope="module")
def ctx(abft):
    return abft.Context(0)


def _schemes(S):
    if S == orc.NONE:
        return orc.NONE, orc.NONE
    if S == orc.CRC32C:
        return orc.CRC32C, orc.CRC32C
    return orc.SECDED64, (orc.SECDED128 if S == orc.SECDED128 else orc.SECDED64)


def halo_cells(n):
    """Cells on both sides of every 256-wide tile column edge, on both sides of
    tile-row edges, and on the grid's edges."""
    xs = sorted({0, n - 1} | {x for t in range(256, n, 256) for x in (t - 1, t)})
    ys = sorted({0, TILE_TY - 1, TILE_TY, 2 * TILE_TY - 1, 2 * TILE_TY, n // 2 - 1, n // 2, n - 1})
    return [x + y * n for y in ys for x in xs]


def periodic_encoded(N, S, seed, period=1 << 20):
    """Oracle-encoded words of a random vector repeating with `period` (a
    multiple of every group size): the oracle encodes `period` values, the
    words are tiled (each codeword depends only on its own group)."""
    base = orc.vec_encode(gen.uniform_pm1(period, seed), S)[:period]
    reps = -(-N // period)
    out = np.tile(base, reps)[:orc.vec_padded_len(N, S)]
    if len(out) < orc.vec_padded_len(N, S):
        out = np.concatenate([out, np.zeros(orc.vec_padded_len(N, S) - len(out), dtype=np.uint64)])
    return out.copy()


def _flip_words(abft, ctx, wo, g, idx, rng, double=False, nbits=64, tensor=None):
    for i in idx:
        for b in rng.choice(nbits, 2 if double else 1, replace=False):
            wo[i] ^= type(wo[i])(1 << int(b))
            abft.inject_bitflip(ctx, tensor if tensor is not None else g.data, nbits * int(i) + int(b))


def _flip_elems(abft, ctx, Ao, Ag, elems, rng):
    for e in elems:
        b = int(rng.integers(96))
        if b < 64:
            Ao.val[e] ^= np.uint64(1 << b)
            abft.inject_bitflip(ctx, Ag.val, 64 * int(e) + b)
        else:
            Ao.col[e] ^= np.uint32(1 << (b - 64))
            abft.inject_bitflip(ctx, Ag.col, 32 * int(e) + b - 64)


# ------------------------------------------------------------------ n = 1024
@pytest.mark.parametrize("vs", ["NONE", "SED", "SECDED64", "SECDED128", "CRC32C"])
@pytest.mark.parametrize("splits", [(), (513,)])
def test_tiled_spmv_1024_cross_tile(abft, ctx, vs, splits):
    n = 1024
    N = n * n
    S = getattr(orc, vs)
    es, rs = _schemes(S)
    if splits and S not in (orc.SECDED64, orc.NONE):
        pytest.skip("chunked geometry: config-2 schemes")
    rng = np.random.default_rng(1024 + S + len(splits))
    xo = orc.vec_encode(gen.uniform_pm1(N, 41), S)
    xg = gpu_vec_from_words(abft, xo, N, S)
    cells = halo_cells(n)
    ys = [0] + list(splits) + [n]
    Aos, Ags = [], []
    for y0, y1 in zip(ys[:-1], ys[1:]):
        v, c, r = gen.strip_csr(n, y0, y1, ny=n, col_offset=y0 * n)
        v, c, r = v.numpy(), c.numpy().astype(np.uint32), r.numpy().astype(np.uint32)
        rows = (y1 - y0) * n
        Ao, st_o = oracle_matrix(v, c, r, rows, N, es, rs, row_base=y0 * n)
        Ag, st_g = gpu_matrix(abft, ctx, v, c, r, rows, N, es, rs, row_base=y0 * n, stencil_n=n)
        assert st_o == st_g == 0
        assert np.array_equal(col_words(Ag), Ao.col) and np.array_equal(rowptr_words(Ag), Ao.rowptr)
        if S != orc.NONE:
            own = [i - y0 * n for i in cells if y0 * n <= i < y1 * n]
            _flip_elems(abft, ctx, Ao, Ag, [5 * i + int(rng.integers(5)) for i in own[::3]], rng)
            rp = sorted(set(own[1::7]))
            _flip_words(abft, ctx, Ao.rowptr, None, rp, rng, nbits=32, tensor=Ag.rowptr)
        Aos.append(Ao)
        Ags.append(Ag)
    if S != orc.NONE:
        _flip_words(abft, ctx, xo, xg, cells[::2], rng)                   # single flips in halo cells
        _flip_words(abft, ctx, xo, xg, [cells[5], cells[-4]], rng, True)  # + two same-word doubles (DUE)
    out_o = np.zeros(N, dtype=np.uint64)
    cnt_o = orc.new_counts()
    for Ao in Aos:
        orc.spmv(Ao, xo, N, S, out_o, N, cnt_o, want_dot=True)
    dot_o = orc.dot_red1(orc.vec_masked(xo, N, S), orc.vec_masked(out_o, N, S))
    yg = abft.Vector.empty(N, S)
    cnt_g = abft.Counters()
    dot_g = torch.zeros(1, dtype=torch.float64, device="cuda")
    abft.spmv(ctx, Ags, xg, yg, cnt_g, dot=dot_g)
    torch.cuda.synchronize()
    assert np.array_equal(cnt_g.read(), cnt_o), (cnt_g.read(), cnt_o)
    assert np.array_equal(words_of(yg)[:N], out_o[:N])
    assert np.array_equal(words_of(xg)[:N], xo[:N])
    for Ao, Ag in zip(Aos, Ags):
        assert np.array_equal(val_words(Ag), Ao.val) and np.array_equal(col_words(Ag), Ao.col)
        assert np.array_equal(rowptr_words(Ag), Ao.rowptr)
    assert dot_g.item() == dot_o


@pytest.mark.parametrize("vs", ["SED", "SECDED64"])
@pytest.mark.parametrize("double", [False, True])
def test_fused_calc_p_spmv_1024_cross_tile(abft, ctx, vs, double):
    n = 1024
    N = n * n
    S = getattr(orc, vs)
    rng = np.random.default_rng(77 + S + 10 * double)
    po = orc.vec_encode(gen.uniform_pm1(N, 51) * 2.0, S)
    ro = orc.vec_encode(gen.uniform_pm1(N, 52) * 2.0, S)
    pg, rg = gpu_vec_from_words(abft, po, N, S), gpu_vec_from_words(abft, ro, N, S)
    v, c, r = gen.tealeaf_csr(n)
    v, c, r = v.numpy(), c.numpy().astype(np.uint32), r.numpy().astype(np.uint32)
    Ao, _ = oracle_matrix(v, c, r, N, N, orc.SECDED64, orc.SECDED64)
    Ag, _ = gpu_matrix(abft, ctx, v, c, r, N, N, orc.SECDED64, orc.SECDED64, stencil_n=n)
    cells = halo_cells(n)
    _flip_words(abft, ctx, po, pg, cells[::2], rng, double)
    _flip_words(abft, ctx, ro, rg, cells[1::3], rng, double)
    _flip_elems(abft, ctx, Ao, Ag, [5 * i + 1 for i in cells[::5]], rng)
    beta = -0.61
    pn_o, rn_o = po.copy(), ro.copy()
    cnt_o = orc.new_counts()
    orc.calc_p(pn_o, rn_o, N, S, beta, cnt_o)
    out_o = np.zeros(N, dtype=np.uint64)
    orc.spmv(Ao, pn_o, N, S, out_o, N, cnt_o)
    dot_o = orc.dot_red1(orc.vec_masked(pn_o, N, S), orc.vec_masked(out_o, N, S))
    pp_o = po.copy()
    orc.vec_check(pp_o, N, S, counts=None, scrub=True)
    pout, yg = abft.Vector.empty(N, S), abft.Vector.empty(N, S)
    cnt_g = abft.Counters()
    dot_g = torch.zeros(1, dtype=torch.float64, device="cuda")
    abft.calc_p_spmv(ctx, Ag, pg, rg, beta, pout, yg, cnt_g, dot=dot_g)
    torch.cuda.synchronize()
    assert np.array_equal(cnt_g.read(), cnt_o), (cnt_g.read(), cnt_o)
    keep = np.uint64(~np.uint64((1 << (1 if S == orc.SED else 8)) - 1))
    def same(a, b):
        va, vb = (a & keep).view(np.float64), (b & keep).view(np.float64)
        return bool(np.all((a == b) | (np.isnan(va) & np.isnan(vb))))
    assert same(words_of(pout)[:N], pn_o[:N]) and same(words_of(yg)[:N], out_o[:N])
    assert np.array_equal(words_of(rg)[:N], rn_o[:N]) and np.array_equal(words_of(pg)[:N], pp_o[:N])
    assert np.array_equal(val_words(Ag), Ao.val) and np.array_equal(col_words(Ag), Ao.col)
    d = dot_g.item()
    assert d == dot_o or (np.isnan(d) and np.isnan(dot_o))


# ------------------------------------------------------------------ 4096^2 (config 2)
_SHARED = {}


def _job_spmv(tmp):
    """Oracle: encode the 4096^2 matrix, apply the element / rowptr flips, SpMV (+ dot)."""
    d = _SHARED
    N = d["N"]
    A = orc.Matrix(d["v"], d["c"], d["rp"], N, N, orc.SECDED64, orc.SECDED64)
    st = A.encode()
    np.save(os.path.join(tmp, "col_enc.npy"), A.col)
    np.save(os.path.join(tmp, "rp_enc.npy"), A.rowptr)
    for (e, b) in d["eflips"]:
        if b < 64:
            A.val[e] ^= np.uint64(1 << b)
        else:
            A.col[e] ^= np.uint32(1 << (b - 64))
    for (i, b) in d["rflips"]:
        A.rowptr[i] ^= np.uint32(1 << b)
    p = d["p"].copy()
    out = np.zeros(N, dtype=np.uint64)
    cnt = orc.new_counts()
    _, dot = orc.spmv(A, p, N, orc.SECDED64, out, N, cnt, want_dot=True)
    for name, a in (("spmv_out", out), ("spmv_cnt", cnt), ("spmv_p", p), ("spmv_val", A.val), ("spmv_col", A.col),
                    ("spmv_rp", A.rowptr)):
        np.save(os.path.join(tmp, name + ".npy"), a)
    return st, dot


def _job_ur(tmp):
    d = _SHARED
    x, p, r, w = (d[k].copy() for k in ("x", "p", "rv", "w"))
    cnt = orc.new_counts()
    _, rrn = orc.calc_ur(x, p, r, w, d["N"], orc.SECDED64, d["alpha"], cnt)
    for name, a in (("ur_x", x), ("ur_p", p), ("ur_r", r), ("ur_w", w), ("ur_cnt", cnt)):
        np.save(os.path.join(tmp, name + ".npy"), a)
    return rrn


def _job_p(tmp):
    d = _SHARED
    p, r = d["p"].copy(), d["rv"].copy()
    cnt = orc.new_counts()
    orc.calc_p(p, r, d["N"], orc.SECDED64, d["beta"], cnt)
    for name, a in (("p_p", p), ("p_r", r), ("p_cnt", cnt)):
        np.save(os.path.join(tmp, name + ".npy"), a)
    return 0


@pytest.mark.slow
def test_full_4096_spmv_ur_p(abft, ctx):
    n = 4096
    N = n * n
    S = orc.SECDED64
    rng = np.random.default_rng(4096)
    v, c, r = gen.tealeaf_csr(n)
    v, c, r = v.numpy(), c.numpy().astype(np.uint32), r.numpy().astype(np.uint32)
    assert int(c.max()) == (1 << 24) - 1   # the E-SECDED capacity edge (reading R4)
    cells = halo_cells(n)
    x, p, rr, w = (periodic_encoded(N, S, 60 + k) for k in range(4))
    for k, arr in enumerate((x, p, rr, w)):
        for i in sorted(set(cells[k::4])):
            arr[i] ^= np.uint64(1 << int(rng.integers(64)))
    last = N - 1
    # flips: col index bits of the element with col = 2^24-1 (row N-1's diagonal,
    # and its out-of-grid east / north neighbours, stored with col = i), plus
    # elements and row pointers in cross-tile halo rows
    eflips = [(5 * last + 2, 64 + 23), (5 * last + 4, 64 + 5), (5 * last + 3, 7)]
    eflips += [(5 * i + int(rng.integers(5)), int(rng.integers(96))) for i in cells[::6]]
    rflips = [(i, int(rng.integers(32))) for i in sorted(set(cells[2::9]))] + [(N, 3)]
    _SHARED.update(dict(N=N, v=v, c=c, rp=r, p=p, x=x, rv=rr, w=w, eflips=eflips, rflips=rflips, alpha=0.731,
                        beta=-0.25))
    with tempfile.TemporaryDirectory() as tmp:
        # the workers fork here and see _SHARED as it is now
        with mp.get_context("fork").Pool(3) as pool:
            j_ur = pool.apply_async(_job_ur, (tmp,))
            j_p = pool.apply_async(_job_p, (tmp,))
            j_sp = pool.apply_async(_job_spmv, (tmp,))
            # ---- GPU side (same inputs) while the oracle runs
            Ag = abft.Matrix(torch.from_numpy(v).cuda(), torch.from_numpy(c.view(np.int32)).cuda(),
                             torch.from_numpy(r.view(np.int32)).cuda(), N, N, S, S, stencil_n=n)
            assert Ag.encode(ctx) == 0
            col_enc_g, rp_enc_g = col_words(Ag).copy(), rowptr_words(Ag).copy()
            for (e, b) in eflips:
                if b < 64:
                    abft.inject_bitflip(ctx, Ag.val, 64 * e + b)
                else:
                    abft.inject_bitflip(ctx, Ag.col, 32 * e + b - 64)
            for (i, b) in rflips:
                abft.inject_bitflip(ctx, Ag.rowptr, 32 * i + b)
            pg = gpu_vec_from_words(abft, p, N, S)
            yg = abft.Vector.empty(N, S)
            cnt_sp = abft.Counters()
            dot_g = torch.zeros(1, dtype=torch.float64, device="cuda")
            abft.spmv(ctx, Ag, pg, yg, cnt_sp, dot=dot_g)
            torch.cuda.synchronize()
            out_g, p_after = words_of(yg)[:N].copy(), words_of(pg)[:N].copy()
            val_g, col_g, rp_g = val_words(Ag).copy(), col_words(Ag).copy(), rowptr_words(Ag).copy()
            cnt_sp_g = cnt_sp.read()
            del Ag, yg
            # calc_ur
            xg, pg2, rg, wg = (gpu_vec_from_words(abft, a, N, S) for a in (x, p, rr, w))
            cnt_ur = abft.Counters()
            rrn_g = torch.zeros(1, dtype=torch.float64, device="cuda")
            abft.calc_ur(ctx, xg, pg2, rg, wg, 0.731, rrn=rrn_g, counts=cnt_ur)
            torch.cuda.synchronize()
            ur_g = [words_of(t)[:N].copy() for t in (xg, pg2, rg, wg)]
            cnt_ur_g = cnt_ur.read()
            del xg, pg2, rg, wg
            # calc_p
            pg3, rg3 = gpu_vec_from_words(abft, p, N, S), gpu_vec_from_words(abft, rr, N, S)
            cnt_p = abft.Counters()
            abft.calc_p(ctx, pg3, rg3, -0.25, counts=cnt_p)
            torch.cuda.synchronize()
            p_g = [words_of(t)[:N].copy() for t in (pg3, rg3)]
            cnt_p_g = cnt_p.read()
            st_o, dot_o = j_sp.get(timeout=1800)
            rrn_o = j_ur.get(timeout=1800)
            j_p.get(timeout=1800)
        _SHARED.clear()
        L = lambda k: np.load(os.path.join(tmp, k + ".npy"))  # noqa: E731
        assert st_o == 0
        # a0 at the capacity edge: encoded col / rowptr words
        assert np.array_equal(col_enc_g, L("col_enc")) and np.array_equal(rp_enc_g, L("rp_enc"))
        # a3: words, dot, counters, scrubbed storage
        assert np.array_equal(cnt_sp_g, L("spmv_cnt")), (cnt_sp_g, L("spmv_cnt"))
        assert np.array_equal(out_g, L("spmv_out")[:N])
        assert dot_g.item() == dot_o
        assert np.array_equal(p_after, L("spmv_p")[:N])
        assert np.array_equal(val_g, L("spmv_val")) and np.array_equal(col_g, L("spmv_col"))
        assert np.array_equal(rp_g, L("spmv_rp"))
        assert cnt_sp_g[orc.ELEM, S, orc.COR] > 0 and cnt_sp_g[orc.ELEM, S, orc.DET] == cnt_sp_g[orc.ELEM, S, orc.COR]
        # a4
        assert np.array_equal(cnt_ur_g, L("ur_cnt"))
        for got, k in zip(ur_g, ("ur_x", "ur_p", "ur_r", "ur_w")):
            assert np.array_equal(got, L(k)[:N]), k
        assert rrn_g.item() == rrn_o
        # a5
        assert np.array_equal(cnt_p_g, L("p_cnt"))
        assert np.array_equal(p_g[0], L("p_p")[:N]) and np.array_equal(p_g[1], L("p_r")[:N])


# ------------------------------------------------------------------ 8192^2 (config 3), 5 chunks
@pytest.mark.slow
def test_8192_five_chunk_spmv_sampled(abft, ctx):
    n = 8192
    N = n * n
    S = orc.SECDED64
    plan = gen.chunk_plan(n)
    assert len(plan) == 5
    rng = np.random.default_rng(8192)
    xo = periodic_encoded(N, S, 81)
    # sampled strips: 3 grid rows each side of every chunk boundary, the first and last rows
    # (each strip lies inside one chunk: the rows on both sides of a boundary are two strips)
    strips = [(0, 3), (n - 3, n)] + [s for (y0, _, _) in plan[1:] for s in ((y0 - 3, y0), (y0, y0 + 3))]
    cells = []
    for (y0, y1) in strips:
        for y in range(y0, y1):
            cells += [x + y * n for x in (0, 255, 256, 4095, 4096, n - 1)]
    vflip = [(i, int(rng.integers(64))) for i in cells[::3]]
    for (i, b) in vflip:
        xo[i] ^= np.uint64(1 << b)
    xg = gpu_vec_from_words(abft, xo, N, S)
    eflips, rflips = [], []
    for i in cells[1::4]:
        eflips.append((5 * i + int(rng.integers(5)), int(rng.integers(96))))
    for i in cells[2::11]:
        rflips.append((i, int(rng.integers(32))))
    Ags = []
    dev = torch.device("cuda")
    for (y0, y1, cb) in plan:
        val, col, rowptr = gen.chunk_csr(n, y0, y1, cb, ny=n, device=dev)
        rows = (y1 - y0) * n
        ncols = min(n, y1 + 1) * n - cb
        M = abft.Matrix(val, col.to(torch.int32), rowptr.to(torch.int32), rows, ncols, S, S, row_base=y0 * n,
                        col_base=cb, stencil_n=n)
        assert M.encode(ctx) == 0
        for (e, b) in eflips:
            le = e - 5 * y0 * n
            if 0 <= le < 5 * rows:
                if b < 64:
                    abft.inject_bitflip(ctx, M.val, 64 * le + b)
                else:
                    abft.inject_bitflip(ctx, M.col, 32 * le + b - 64)
        for (i, b) in rflips:
            li = i - y0 * n
            if 0 <= li < rows:
                abft.inject_bitflip(ctx, M.rowptr, 32 * li + b)
        Ags.append((M, y0, y1, cb))
    yg = abft.Vector.empty(N, S)
    cnt_g = abft.Counters()
    abft.spmv(ctx, [m for (m, _, _, _) in Ags], xg, yg, cnt_g)
    torch.cuda.synchronize()
    out_g = words_of(yg)
    cnt_tot = orc.new_counts()
    for (s0, s1) in strips:
        # the GPU chunk holding the strip, and the strip's encoded col words in that chunk's indexing
        (M, y0, y1, cb) = next(t for t in Ags if t[1] <= s0 and s1 <= t[2])
        v1, c1, r1 = gen.chunk_csr(n, s0, s1, cb, ny=n)
        rows = (s1 - s0) * n
        A1, st1 = oracle_matrix(v1.numpy(), c1.numpy().astype(np.uint32), r1.numpy().astype(np.uint32), rows,
                                min(n, y1 + 1) * n - cb, S, S)
        assert st1 == 0
        le0 = 5 * (s0 - y0) * n
        colw = M.col[le0:le0 + 5 * rows].cpu().numpy().view(np.uint32)
        # after the SpMV scrubbed every flipped element these are the clean encoded words
        assert np.array_equal(colw, A1.col)
        # the oracle SpMV of the strip from its own input window [w0, w1) grid rows
        w0, w1 = max(0, s0 - 1), min(n, s1 + 1)
        v2, c2, r2 = gen.strip_csr(n, s0, s1, ny=n, col_offset=(s0 - w0) * n)
        A2 = orc.Matrix(v2.numpy(), c2.numpy().astype(np.uint32), r2.numpy().astype(np.uint32), rows,
                        (w1 - w0) * n, S, S, row_base=(s0 - w0) * n, col_base=0)
        assert A2.encode() == 0
        for (e, b) in eflips:
            le = e - 5 * s0 * n
            if 0 <= le < 5 * rows:
                if b < 64:
                    A2.val[le] ^= np.uint64(1 << b)
                else:
                    A2.col[le] ^= np.uint32(1 << (b - 64))
        for (i, b) in rflips:
            li = i - s0 * n
            if 0 <= li < rows:
                A2.rowptr[li] ^= np.uint32(1 << b)
        win = xo[w0 * n:w1 * n].copy()
        out = np.zeros(len(win), dtype=np.uint64)
        orc.spmv(A2, win, len(win), S, out, len(win), cnt_tot)
        assert np.array_equal(out_g[s0 * n:s1 * n], out[(s0 - w0) * n:(s1 - w0) * n]), (s0, s1)
        assert np.array_equal(words_of(xg)[s0 * n:s1 * n], win[(s0 - w0) * n:(s1 - w0) * n])
        assert np.array_equal(M.val[le0:le0 + 5 * rows].view(torch.int64).cpu().numpy().view(np.uint64), A2.val)
    # every flip sits in a sampled strip: the whole-matrix counters equal the strips' sum
    assert np.array_equal(cnt_g.read(), cnt_tot), (cnt_g.read(), cnt_tot)
    assert cnt_tot[orc.VEC, S, orc.COR] == len(vflip)


# ------------------------------------------------------------------ tiled CG to convergence, 512^2
@pytest.mark.slow
def test_tiled_cg_512_converged(abft, ctx):
    n = 512
    N = n * n
    S = orc.SECDED64
    v, c, r = gen.tealeaf_csr(n)
    v, c, r = v.numpy(), c.numpy().astype(np.uint32), r.numpy().astype(np.uint32)
    Ao, _ = oracle_matrix(v, c, r, N, N, S, S)
    Ag, _ = gpu_matrix(abft, ctx, v, c, r, N, N, S, S, stencil_n=n)
    rng = np.random.default_rng(512)
    cells = halo_cells(n)
    _flip_elems(abft, ctx, Ao, Ag, [5 * i + 2 for i in cells[::4]], rng)
    bo = orc.vec_encode(gen.tealeaf_rhs(n).numpy(), S)
    xo = bo.copy()
    bg = gpu_vec_from_words(abft, bo, N, S)
    xg = gpu_vec_from_words(abft, xo, N, S)
    _flip_words(abft, ctx, xo, xg, cells[1::4], rng)
    ro, po, wo = (np.zeros_like(bo) for _ in range(3))
    cnt_o = orc.new_counts()
    st, res_o = orc.cg_solve(Ao, bo, xo, ro, po, wo, S, 1e-10, 5000, 0, cnt_o)
    rg, pg, wg = (abft.Vector.empty(N, S) for _ in range(3))
    cnt_g = abft.Counters()
    res_g = abft.cg_solve(ctx, Ag, bg, xg, rg, pg, wg, tol=1e-10, max_iters=5000, due_policy=0, counts=cnt_g)
    torch.cuda.synchronize()
    assert st == 0 and res_g.status == 0
    assert res_g.iters == res_o.iters and res_o.iters > 250
    assert res_g.rr0 == res_o.rr0 and res_g.rrn == res_o.rrn
    for g, o in ((xg, xo), (rg, ro), (pg, po), (wg, wo)):
        assert np.array_equal(words_of(g)[:N], o[:N])
    assert np.array_equal(cnt_g.read(), cnt_o)
