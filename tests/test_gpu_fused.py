"""GPU parity of the fused calc_p + SpMV path (S§8(f) row f3):
calc_p of iteration k (p = enc(fma(beta, p, r))) computed inside
the tiled SpMV of iteration k+1.  Checked against the oracle's UNFUSED
sequence (or_calc_p then or_spmv; or_cg_solve): new p, w, p.w, counters and
scrubbed operands bit-exact, with single / same-word double flips in p, r
(tile halo rows and chunk edges included) and in the matrix; and whole CG
solves (converged, max_iters odd / even, DUE abort, chunked) bit-exact in
iterations, rr0, rrn, x, r, p, w and counters, fused and unfused alike."""
import numpy as np
import pytest
import torch

import gen
import oracle as orc
from gpu_helpers import gpu_matrix, gpu_vec_from_words, oracle_matrix, words_of

pytestmark = pytest.mark.gpu

N_GRID = 256
KEEP_BITS = {0: 0, 1: 1, 2: 8}


@pytest.fixture(scope="module")
def abft():
    from paper_conf_cluster_pawelczakmpm17_b200 import build
    build.build()
    from paper_conf_cluster_pawelczakmpm17_b200 import abft as A
    return A


@pytest.fixture(scope="module")
def ctx(abft):
    return abft.Context(0)


def _same(a, b, S):
    """Bit-exact except where both values are NaN (reading R25)."""
    keep = np.uint64(~np.uint64((1 << KEEP_BITS[S]) - 1))
    va, vb = (a & keep).view(np.float64), (b & keep).view(np.float64)
    return bool(np.all((a == b) | (np.isnan(va) & np.isnan(vb))))


def _matrices(abft, ctx, n, splits, es, rs):
    ys = [0] + list(splits) + [n]
    Aos, Ags = [], []
    for y0, y1 in zip(ys[:-1], ys[1:]):
        v, c, r = gen.strip_csr(n, y0, y1, ny=n, col_offset=y0 * n)
        v, c, r = v.numpy(), c.numpy().astype(np.uint32), r.numpy().astype(np.uint32)
        rows = (y1 - y0) * n
        Ao, _ = oracle_matrix(v, c, r, rows, n * n, es, rs, row_base=y0 * n, col_base=0)
        Ag, _ = gpu_matrix(abft, ctx, v, c, r, rows, n * n, es, rs, row_base=y0 * n, col_base=0, stencil_n=n)
        Aos.append(Ao)
        Ags.append(Ag)
    return Aos, Ags


def _flip_vec(abft, ctx, wo, g, idx, rng, double):
    for i in idx:
        bits = rng.choice(64, 2 if double else 1, replace=False)
        for b in bits:
            wo[i] ^= np.uint64(1 << int(b))
            abft.inject_bitflip(ctx, g.data, 64 * int(i) + int(b))


@pytest.mark.parametrize("vs", ["NONE", "SED", "SECDED64"])
@pytest.mark.parametrize("splits", [(), (40,)])
@pytest.mark.parametrize("faults", ["none", "single", "double"])
def test_calc_p_spmv_parity(abft, ctx, vs, splits, faults):
    n = N_GRID
    N = n * n
    S = getattr(orc, vs)
    if S == orc.NONE and faults != "none":
        pytest.skip("no code to check")
    es, rs = (orc.NONE, orc.NONE) if S == orc.NONE else (orc.SECDED64, orc.SECDED64)
    rng = np.random.default_rng(3 + len(splits) + 7 * ["none", "single", "double"].index(faults))
    po = orc.vec_encode(gen.uniform_pm1(N, 21) * 2.0, S)
    ro = orc.vec_encode(gen.uniform_pm1(N, 22) * 2.0, S)
    pg = gpu_vec_from_words(abft, po, N, S)
    rg = gpu_vec_from_words(abft, ro, N, S)
    Aos, Ags = _matrices(abft, ctx, n, splits, es, rs)
    if faults != "none":
        # p / r flips: random, tile halo rows (grid rows 7/8, 15/16), chunk edges, domain corners
        edge = [7 * n + 3, 8 * n + 255, 15 * n, 16 * n - 1, 40 * n, 40 * n - 1, 0, N - 1]
        _flip_vec(abft, ctx, po, pg, sorted(set(list(rng.choice(N, 24, replace=False)) + edge)), rng,
                  faults == "double")
        _flip_vec(abft, ctx, ro, rg, sorted(set(int(i) for i in rng.choice(N, 24, replace=False))), rng,
                  faults == "double")
        for Ao, Ag in zip(Aos, Ags):   # single matrix flips (corrected)
            for e in rng.choice(Ao.nnz, 4, replace=False):
                b = int(rng.integers(64))
                Ao.val[e] ^= np.uint64(1 << b)
                abft.inject_bitflip(ctx, Ag.val, 64 * int(e) + b)
    beta = 0.37
    # oracle, unfused: calc_p in place on a copy of p, then the SpMV of the new p
    pn_o, rn_o = po.copy(), ro.copy()
    cnt_o = orc.new_counts()
    orc.calc_p(pn_o, rn_o, N, S, beta, cnt_o)
    out_o = np.zeros(N, dtype=np.uint64)
    for Ao in Aos:
        orc.spmv(Ao, pn_o, N, S, out_o, N, cnt_o, want_dot=True)
    dot_o = orc.dot_red1(orc.vec_masked(pn_o, N, S), orc.vec_masked(out_o, N, S))
    # what the fused kernel leaves in p_prev: single flips scrubbed, DUE words as stored
    pp_o = po.copy()
    orc.vec_check(pp_o, N, S, counts=None, scrub=True)

    pout = abft.Vector.empty(N, S)
    yg = abft.Vector.empty(N, S)
    cnt_g = abft.Counters()
    dot_g = torch.zeros(1, dtype=torch.float64, device="cuda")
    abft.calc_p_spmv(ctx, Ags, pg, rg, beta, pout, yg, cnt_g, dot=dot_g)
    torch.cuda.synchronize()
    assert np.array_equal(cnt_g.read(), cnt_o), (cnt_g.read(), cnt_o)
    assert _same(words_of(pout)[:N], pn_o[:N], S)
    assert _same(words_of(yg)[:N], out_o, S)
    assert np.array_equal(words_of(rg)[:N], rn_o[:N])
    assert np.array_equal(words_of(pg)[:N], pp_o[:N])
    d = dot_g.item()
    assert d == dot_o or (np.isnan(d) and np.isnan(dot_o))


def test_calc_p_spmv_rejects_group_schemes(abft, ctx):
    n = N_GRID
    N = n * n
    S = orc.SECDED128
    _, Ags = _matrices(abft, ctx, n, (), orc.SECDED64, orc.SECDED128)
    v = [gpu_vec_from_words(abft, orc.vec_encode(gen.uniform_pm1(N, 5 + j), S), N, S) for j in range(4)]
    with pytest.raises(abft.AbftError):
        abft.calc_p_spmv(ctx, Ags, v[0], v[1], 0.5, v[2], v[3])


def _cg(abft, ctx, vs, max_iters, policy=1, splits=(), fused=True, poll=16, inject=None):
    n = N_GRID
    N = n * n
    S = getattr(orc, vs)
    es, rs = (orc.NONE, orc.NONE) if S == orc.NONE else (orc.SECDED64, orc.SECDED64)
    Aos, Ags = _matrices(abft, ctx, n, splits, es, rs)
    bo = orc.vec_encode(gen.tealeaf_rhs(n).numpy(), S)
    xo = bo.copy()
    bg = gpu_vec_from_words(abft, bo, N, S)
    xg = gpu_vec_from_words(abft, xo, N, S)
    if inject:
        inject(Aos, Ags, bo, bg, xo, xg)
    ro, po, wo = (np.zeros_like(bo) for _ in range(3))
    cnt_o = orc.new_counts()
    Ao = Aos[0] if len(Aos) == 1 else _whole(abft, ctx, n, es, rs, Aos)
    st_o, res_o = orc.cg_solve(Ao, bo, xo, ro, po, wo, S, 1e-10, max_iters, policy, cnt_o)
    rg, pg, wg = (abft.Vector.empty(N, S) for _ in range(3))
    cnt_g = abft.Counters()
    ctx.set_fused_cg(fused)
    try:
        res_g = abft.cg_solve(ctx, Ags if len(Ags) > 1 else Ags[0], bg, xg, rg, pg, wg, tol=1e-10,
                              max_iters=max_iters, due_policy=policy, counts=cnt_g, poll_every=poll)
    finally:
        ctx.set_fused_cg(False)
    return dict(st_o=st_o, res_o=res_o, res_g=res_g, cnt_o=cnt_o, cnt_g=cnt_g.read(), S=S, N=N,
                pairs=[(xo, words_of(xg)), (ro, words_of(rg)), (po, words_of(pg)), (wo, words_of(wg))])


def _whole(abft, ctx, n, es, rs, Aos):
    """The oracle solves the unchunked matrix (the same rows; the chunks only
    change how the GPU launches), with the chunks' injected flips applied."""
    v, c, r = gen.tealeaf_csr(n)
    v, c, r = v.numpy(), c.numpy().astype(np.uint32), r.numpy().astype(np.uint32)
    A, _ = oracle_matrix(v, c, r, n * n, n * n, es, rs)
    off = 0
    for Ao in Aos:
        A.val[off:off + Ao.nnz] = Ao.val
        A.col[off:off + Ao.nnz] = Ao.col
        off += Ao.nnz
    return A


def _assert_same(R):
    assert R["res_g"].status == R["st_o"], (R["res_g"].status, R["st_o"])
    assert R["res_g"].iters == R["res_o"].iters
    assert R["res_g"].rr0 == R["res_o"].rr0 and R["res_g"].rrn == R["res_o"].rrn
    for o, g in R["pairs"]:
        assert _same(g[:R["N"]], o[:R["N"]], R["S"])
    assert np.array_equal(R["cnt_g"], R["cnt_o"]), (R["cnt_g"], R["cnt_o"])


@pytest.mark.parametrize("vs", ["NONE", "SED", "SECDED64"])
@pytest.mark.parametrize("max_iters", [5000, 41, 40])
@pytest.mark.parametrize("fused", [True, False])
def test_fused_cg_parity(abft, ctx, vs, max_iters, fused):
    R = _cg(abft, ctx, vs, max_iters, fused=fused, poll=7)
    _assert_same(R)
    if max_iters == 5000:
        assert R["st_o"] == orc.OK
    else:
        assert R["st_o"] == orc.E_NOT_CONVERGED and R["res_o"].iters == max_iters


@pytest.mark.parametrize("policy", [0, 1])
def test_fused_cg_faults(abft, ctx, policy):
    """Single flips in the matrix, b and x0 (corrected, counted once) and one
    same-word double flip in an element (DUE: abort stops at init, continue
    runs on with the masked stored bits), chunked matrix."""
    def inject(Aos, Ags, bo, bg, xo, xg):
        rng = np.random.default_rng(11)
        for Ao, Ag in zip(Aos, Ags):
            for e in rng.choice(Ao.nnz, 6, replace=False):
                b = int(rng.integers(96))
                if b < 64:
                    Ao.val[e] ^= np.uint64(1 << b)
                    abft.inject_bitflip(ctx, Ag.val, 64 * int(e) + b)
                else:
                    Ao.col[e] ^= np.uint32(1 << (b - 64))
                    abft.inject_bitflip(ctx, Ag.col, 32 * int(e) + b - 64)
        Ao, Ag = Aos[-1], Ags[-1]
        Ao.val[33] ^= np.uint64(0b1001 << 20)
        abft.inject_bitflip(ctx, Ag.val, 64 * 33 + 20)
        abft.inject_bitflip(ctx, Ag.val, 64 * 33 + 23)
        for wo, g in ((bo, bg), (xo, xg)):
            for i in rng.choice(len(wo), 5, replace=False):
                b = int(rng.integers(64))
                wo[i] ^= np.uint64(1 << b)
                abft.inject_bitflip(ctx, g.data, 64 * int(i) + b)
    R = _cg(abft, ctx, "SECDED64", 300, policy=policy, splits=(40, 200), inject=inject)
    _assert_same(R)
    assert R["st_o"] == (orc.E_DUE if policy == 0 else orc.OK)


def test_fused_cg_matches_unfused_poll_variants(abft, ctx):
    """Graph replays (poll even / odd -> rounded up) and direct issue give the same solve."""
    ref = _cg(abft, ctx, "SECDED64", 77, fused=False, poll=5)
    for poll in (1, 2, 16):
        R = _cg(abft, ctx, "SECDED64", 77, fused=True, poll=poll)
        assert R["res_g"].iters == ref["res_g"].iters == 77
        for (_, g), (_, gr) in zip(R["pairs"], ref["pairs"]):
            assert np.array_equal(g, gr)
        assert np.array_equal(R["cnt_g"], ref["cnt_g"])
