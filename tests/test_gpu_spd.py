"""GPU parity on general (non-stencil) sparse SPD matrices, G-SPD (S§8(f) f4,
gen/spd.py): variable row lengths (5..~16 entries), unsorted-by-stencil
columns, through the generic gather SpMV.  Protected SpMV and CG vs the
oracle for every scheme, with single / same-word double flips in elements,
row pointers and the input vector: outputs, iterations, counters and
scrubbed storage bit-exact."""
import numpy as np
import pytest
import torch

import gen
import oracle as orc
from gpu_helpers import col_words, gpu_matrix, gpu_vec_from_words, oracle_matrix, rowptr_words, val_words, words_of

pytestmark = pytest.mark.gpu
SCHEMES = ["NONE", "SED", "SECDED64", "SECDED128", "CRC32C"]
KEEP = {0: 0, 1: 1, 2: 8, 3: 5, 4: 8}


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
    keep = np.uint64(~np.uint64((1 << KEEP[S]) - 1))
    va, vb = (a & keep).view(np.float64), (b & keep).view(np.float64)
    return bool(np.all((a == b) | (np.isnan(va) & np.isnan(vb))))


def _schemes(S):
    return (orc.NONE, orc.NONE) if S == orc.NONE else ((orc.CRC32C, orc.CRC32C) if S == orc.CRC32C else
                                                        (orc.SECDED64 if S != orc.SED else orc.SED, S))


def _inject(abft, ctx, Ao, Ag, xo, xg, rng, double, N):
    for e in rng.choice(Ao.nnz, 30, replace=False):
        bits = rng.choice(96, 2 if double else 1, replace=False)
        for b in bits:
            b = int(b)
            if b < 64:
                Ao.val[e] ^= np.uint64(1 << b)
                abft.inject_bitflip(ctx, Ag.val, 64 * int(e) + b)
            else:
                Ao.col[e] ^= np.uint32(1 << (b - 64))
                abft.inject_bitflip(ctx, Ag.col, 32 * int(e) + b - 64)
    for g in rng.choice(len(Ao.rowptr), 6, replace=False):
        b = int(rng.integers(32))
        Ao.rowptr[g] ^= np.uint32(1 << b)
        abft.inject_bitflip(ctx, Ag.rowptr, 32 * int(g) + b)
    if xo is not None:
        for i in rng.choice(N, 20, replace=False):
            for b in rng.choice(64, 2 if double else 1, replace=False):
                xo[i] ^= np.uint64(1 << int(b))
                abft.inject_bitflip(ctx, xg.data, 64 * int(i) + int(b))


@pytest.mark.parametrize("vs", SCHEMES)
@pytest.mark.parametrize("faults", ["none", "single", "double"])
def test_spd_spmv_parity(abft, ctx, vs, faults):
    N = 3000
    S = getattr(orc, vs)
    if S == orc.NONE and faults != "none":
        pytest.skip("no code")
    es, rs = _schemes(S)
    v, c, r = gen.random_spd_csr(N, 4, 17)
    Ao, st = oracle_matrix(v, c, r, N, N, es, rs)
    assert st == 0
    Ag, st = gpu_matrix(abft, ctx, v, c, r, N, N, es, rs)
    assert st == 0
    assert np.array_equal(col_words(Ag), Ao.col) and np.array_equal(rowptr_words(Ag), Ao.rowptr)
    xo = orc.vec_encode(gen.uniform_pm1(N, 18) * 2.0, S)
    xg = gpu_vec_from_words(abft, xo, N, S)
    if faults != "none":
        _inject(abft, ctx, Ao, Ag, xo, xg, np.random.default_rng(19), faults == "double", N)
    yo = np.zeros_like(xo)
    cnt_o = orc.new_counts()
    _, dot_o = orc.spmv(Ao, xo, N, S, yo, N, cnt_o, want_dot=True)
    yg = abft.Vector.empty(N, S)
    cnt_g = abft.Counters()
    dot_g = torch.zeros(1, dtype=torch.float64, device="cuda")
    abft.spmv(ctx, Ag, xg, yg, cnt_g, dot=dot_g)
    torch.cuda.synchronize()
    assert np.array_equal(cnt_g.read(), cnt_o), (cnt_g.read()[:, S], cnt_o[:, S])
    assert _same(words_of(yg)[:N], yo[:N], S)
    d = dot_g.item()
    assert d == dot_o or (np.isnan(d) and np.isnan(dot_o))
    assert np.array_equal(val_words(Ag), Ao.val) and np.array_equal(col_words(Ag), Ao.col)
    assert np.array_equal(rowptr_words(Ag), Ao.rowptr)
    assert np.array_equal(words_of(xg)[:N], xo[:N])


@pytest.mark.parametrize("vs", SCHEMES)
@pytest.mark.parametrize("faults", [False, True])
def test_spd_cg_parity(abft, ctx, vs, faults):
    N = 2000
    S = getattr(orc, vs)
    es, rs = _schemes(S)
    v, c, r = gen.random_spd_csr(N, 5, 23)
    Ao, _ = oracle_matrix(v, c, r, N, N, es, rs)
    Ag, _ = gpu_matrix(abft, ctx, v, c, r, N, N, es, rs)
    bo = orc.vec_encode(gen.uniform_pm1(N, 24), S)
    xo = bo.copy()
    bg = gpu_vec_from_words(abft, bo, N, S)
    xg = gpu_vec_from_words(abft, xo, N, S)
    if faults and S != orc.NONE:
        _inject(abft, ctx, Ao, Ag, xo, xg, np.random.default_rng(25), False, N)
    ro, po, wo = (np.zeros_like(bo) for _ in range(3))
    cnt_o = orc.new_counts()
    st_o, res_o = orc.cg_solve(Ao, bo, xo, ro, po, wo, S, 1e-10, 3000, 1, cnt_o)
    rg, pg, wg = (abft.Vector.empty(N, S) for _ in range(3))
    cnt_g = abft.Counters()
    res_g = abft.cg_solve(ctx, Ag, bg, xg, rg, pg, wg, tol=1e-10, max_iters=3000, due_policy=1, counts=cnt_g,
                          poll_every=9)
    assert res_g.status == st_o and res_g.iters == res_o.iters
    assert res_g.rr0 == res_o.rr0 and res_g.rrn == res_o.rrn
    for o, g in ((xo, xg), (ro, rg), (po, pg), (wo, wg)):
        assert _same(words_of(g)[:N], o[:N], S)
    assert np.array_equal(cnt_g.read(), cnt_o)
    if faults and S in (orc.SECDED64, orc.SECDED128):   # single flips in distinct codewords: all corrected
        assert cnt_o[:, S, orc.UNC].sum() == 0 and cnt_o[:, S, orc.COR].sum() > 0
