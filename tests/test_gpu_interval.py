"""GPU parity of interval checking: the SpMV's
matrix check modes (detection only / range only) on the generic and the tiled
kernel, and the CG with check interval N (device-side access counter, final
integrity check), bit-exact vs the oracle: outputs, counts, stored words,
iterations and solutions."""
import numpy as np
import pytest
import torch

import gen
import oracle as orc
from gpu_helpers import col_words, gpu_matrix, gpu_vec_from_words, oracle_matrix, rowptr_words, val_words, words_of

pytestmark = pytest.mark.gpu


@pytest.fixture(scope="module")
def abft():
    from paper_conf_cluster_pawelczakmpm17_b200 import build
    build.build()
    from paper_conf_cluster_pawelczakmpm17_b200 import abft as A
    return A


@pytest.fixture(scope="module")
def ctx(abft):
    return abft.Context(0)


def _flip_matrix(abft, ctx, Ao, Ag, rng, n_el, n_rp, double=False):
    for e in rng.choice(Ao.nnz, n_el, replace=False):
        for b in rng.choice(96, 2 if double else 1, replace=False):
            b = int(b)
            if b < 64:
                Ao.val[e] ^= np.uint64(1 << b)
                abft.inject_bitflip(ctx, Ag.val, 64 * int(e) + b)
            else:
                Ao.col[e] ^= np.uint32(1 << (b - 64))
                abft.inject_bitflip(ctx, Ag.col, 32 * int(e) + b - 64)
    for g in rng.choice(len(Ao.rowptr), n_rp, replace=False):
        b = int(rng.integers(28, 32)) if not double else int(rng.integers(32))   # check bits: rows stay valid
        Ao.rowptr[g] ^= np.uint32(1 << b)
        abft.inject_bitflip(ctx, Ag.rowptr, 32 * int(g) + b)


@pytest.mark.parametrize("mode", ["DETECT", "RANGE"])
@pytest.mark.parametrize("n,stencil", [(48, False), (256, True)])
@pytest.mark.parametrize("double", [False, True])
def test_spmv_mode_parity(abft, ctx, mode, n, stencil, double):
    N = n * n
    S = orc.SECDED64
    v, c, r = gen.tealeaf_csr(n)
    v, c, r = v.numpy(), c.numpy().astype(np.uint32), r.numpy().astype(np.uint32)
    Ao, _ = oracle_matrix(v, c, r, N, N, S, S)
    Ag, _ = gpu_matrix(abft, ctx, v, c, r, N, N, S, S, stencil_n=n if stencil else 0)
    rng = np.random.default_rng(7 + n + double)
    _flip_matrix(abft, ctx, Ao, Ag, rng, 30, 10, double)
    x = gen.uniform_pm1(N, 11)
    xo = orc.vec_encode(x, S)
    xg = gpu_vec_from_words(abft, xo, N, S)
    out_o = np.zeros(N, dtype=np.uint64)
    cnt_o = orc.new_counts()
    _, dot_o = orc.spmv(Ao, xo, N, S, out_o, N, cnt_o, want_dot=True, mode=getattr(orc, "MODE_" + mode))
    yg = abft.Vector.empty(N, S)
    cnt_g = abft.Counters()
    dot_g = torch.zeros(1, dtype=torch.float64, device="cuda")
    abft.spmv(ctx, Ag, xg, yg, cnt_g, dot=dot_g, mode=getattr(abft, "CHECK_" + mode))
    torch.cuda.synchronize()
    assert np.array_equal(cnt_g.read(), cnt_o), (cnt_g.read()[:2], cnt_o[:2])
    assert np.array_equal(words_of(yg)[:N], out_o)
    assert dot_g.item() == dot_o
    # nothing scrubbed in either mode
    assert np.array_equal(val_words(Ag), Ao.val) and np.array_equal(col_words(Ag), Ao.col)
    assert np.array_equal(rowptr_words(Ag), Ao.rowptr)
    if mode == "RANGE":
        assert cnt_o[:, :, :3].sum() == 0
    elif not double:
        assert cnt_o[orc.ELEM, S, orc.COR] == 0 and cnt_o[orc.ELEM, S, orc.UNC] > 0


def test_check_all_detect_only_parity(abft, ctx):
    n = 40
    N = n * n
    S = orc.SECDED64
    v, c, r = gen.tealeaf_csr(n)
    v, c, r = v.numpy(), c.numpy().astype(np.uint32), r.numpy().astype(np.uint32)
    Ao, _ = oracle_matrix(v, c, r, N, N, S, S)
    Ag, _ = gpu_matrix(abft, ctx, v, c, r, N, N, S, S)
    _flip_matrix(abft, ctx, Ao, Ag, np.random.default_rng(5), 20, 8)
    xo = orc.vec_encode(gen.uniform_pm1(N, 2), S)
    xg = gpu_vec_from_words(abft, xo, N, S)
    for i in (3, 77, 1500):
        xo[i] ^= np.uint64(1 << 40)
        abft.inject_bitflip(ctx, xg.data, 64 * i + 40)
    cnt_o = orc.new_counts()
    Ao.check(cnt_o, scrub=2)
    orc.vec_check(xo, N, S, cnt_o, scrub=2)
    cnt_g = abft.Counters()
    abft.check_all(ctx, Ag, [xg], cnt_g, scrub=2)
    assert np.array_equal(cnt_g.read(), cnt_o)
    assert cnt_o[:, :, orc.COR].sum() == 0 and cnt_o[:, :, orc.UNC].sum() == 31
    assert np.array_equal(val_words(Ag), Ao.val) and np.array_equal(words_of(xg)[:N], xo)


def _cg_interval(abft, ctx, n, N_int, stencil, policy, nflip, max_iters=5000, seed=1):
    Nn = n * n
    S = orc.SECDED64
    v, c, r = gen.tealeaf_csr(n)
    v, c, r = v.numpy(), c.numpy().astype(np.uint32), r.numpy().astype(np.uint32)
    Ao, _ = oracle_matrix(v, c, r, Nn, Nn, S, S)
    Ag, _ = gpu_matrix(abft, ctx, v, c, r, Nn, Nn, S, S, stencil_n=n if stencil else 0)
    rng = np.random.default_rng(seed)
    for e in rng.choice(Ao.nnz, nflip, replace=False):   # persistent low-mantissa flips (solve still converges)
        b = int(rng.integers(0, 8))
        Ao.val[e] ^= np.uint64(1 << b)
        abft.inject_bitflip(ctx, Ag.val, 64 * int(e) + b)
    b = gen.tealeaf_rhs(n).numpy()
    bo = orc.vec_encode(b, S)
    xo = bo.copy()
    bg, xg = gpu_vec_from_words(abft, bo, Nn, S), gpu_vec_from_words(abft, xo, Nn, S)
    ro, po, wo = (np.zeros_like(bo) for _ in range(3))
    cnt_o = orc.new_counts()
    st_o, res_o = orc.cg_solve(Ao, bo, xo, ro, po, wo, S, 1e-10, max_iters, policy, cnt_o, check_interval=N_int)
    rg, pg, wg = (abft.Vector.empty(Nn, S) for _ in range(3))
    cnt_g = abft.Counters()
    res_g = abft.cg_solve(ctx, Ag, bg, xg, rg, pg, wg, tol=1e-10, max_iters=max_iters, due_policy=policy,
                          counts=cnt_g, poll_every=8, check_interval=N_int)
    return st_o, res_o, res_g, xo, words_of(xg)[:Nn], cnt_o, cnt_g.read(), Ao, Ag


@pytest.mark.parametrize("N_int", [2, 5, 64])
@pytest.mark.parametrize("n,stencil", [(32, False), (256, True)])
def test_cg_interval_parity(abft, ctx, N_int, n, stencil):
    st_o, res_o, res_g, xo, xg, cnt_o, cnt_g, Ao, Ag = _cg_interval(abft, ctx, n, N_int, stencil, 1, 4,
                                                                   max_iters=60 if n == 256 else 5000)
    assert res_g.status == st_o and res_g.iters == res_o.iters
    assert res_g.rrn == res_o.rrn
    assert np.array_equal(xg, xo)
    assert np.array_equal(cnt_g, cnt_o), (cnt_g[0], cnt_o[0])
    K = res_o.iters
    expect = 4 * (K // N_int + 1 + (1 if K % N_int else 0))
    assert cnt_o[orc.ELEM, orc.SECDED64].tolist() == [expect, 0, expect, 0]
    assert np.array_equal(val_words(Ag), Ao.val)        # never scrubbed


def test_cg_interval_abort(abft, ctx):
    st_o, res_o, res_g, xo, xg, cnt_o, cnt_g, *_ = _cg_interval(abft, ctx, 32, 3, False, 0, 1)
    assert st_o == orc.E_DUE and res_g.status == orc.E_DUE and res_g.iters == res_o.iters == 0
    assert np.array_equal(cnt_g, cnt_o) and np.array_equal(xg, xo)
    # clean solve, interval larger than the iteration count: no counts, same answer as N = 1
    st_o, res_o, res_g, xo, xg, cnt_o, cnt_g, *_ = _cg_interval(abft, ctx, 32, 1000, False, 0, 0)
    assert st_o == orc.OK and res_g.status == 0 and cnt_g.sum() == 0
    st1, r1, rg1, xo1, xg1, *_ = _cg_interval(abft, ctx, 32, 1, False, 0, 0)
    assert np.array_equal(xg, xg1) and rg1.iters == res_g.iters
