"""GPU parity of the protected Chebyshev iteration and TeaLeaf's spectrum
estimate (S§8(f) f4; abft_cheby_solve / abft_cg_spectrum)
against the oracle (or_cheby_solve, or_cg_solve_log + numpy eigvalsh of the
Lanczos tridiagonal): iterations, status, rr0 / rrn, every stored word of u, r,
p, w and every counter bit-exact with the same bounds; the GPU's Sturm-bisection
bounds equal the oracle's eigvalsh bounds to 1e-12 relative."""
import numpy as np
import pytest
import torch

import gen
import oracle as orc
from gpu_helpers import gpu_vec_from_words, words_of

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


def _schemes(S):
    if S == orc.NONE:
        return orc.NONE, orc.NONE
    if S == orc.CRC32C:
        return orc.CRC32C, orc.CRC32C
    return orc.SECDED64, (orc.SECDED128 if S == orc.SECDED128 else orc.SECDED64)


def gershgorin_max(n):
    """Upper spectrum bound of the G-TEA matrix: the largest absolute row sum."""
    v, c, r = gen.tealeaf_csr(n)
    return float(np.abs(v.numpy()).reshape(-1, 5).sum(axis=1).max())


def _setup(abft, ctx, n, S, stencil):
    N = n * n
    es, rs = _schemes(S)
    v, c, r = gen.tealeaf_csr(n)
    v, c, r = v.numpy(), c.numpy().astype(np.uint32), r.numpy().astype(np.uint32)
    Ao = orc.Matrix(v, c, r, N, N, es, rs)
    assert Ao.encode() == 0
    Ag = abft.Matrix(torch.from_numpy(v).cuda(), torch.from_numpy(c.view(np.int32)).cuda(),
                     torch.from_numpy(r.view(np.int32)).cuda(), N, N, es, rs, stencil_n=stencil)
    assert Ag.encode(ctx) == 0
    return Ao, Ag


@pytest.mark.parametrize("vs", ["NONE", "SED", "SECDED64", "SECDED128", "CRC32C"])
@pytest.mark.parametrize("n,stencil,max_iters", [(32, 0, 2000), (256, 256, 60)])
def test_cheby_parity(abft, ctx, vs, n, stencil, max_iters):
    S = getattr(orc, vs)
    N = n * n
    Ao, Ag = _setup(abft, ctx, n, S, stencil)
    lo, hi = 0.95, gershgorin_max(n)   # lambda_min = 1 (A 1 = 1, PIN-8) with a margin; Gershgorin above
    bo = orc.vec_encode(gen.tealeaf_rhs(n).numpy(), S)
    vo = [bo.copy(), bo.copy()] + [np.zeros_like(bo) for _ in range(3)]   # b u r p w
    cnt_o = orc.new_counts()
    st, ro = orc.cheby_solve(Ao, *vo, S, lo, hi, 1e-10, max_iters, 1, cnt_o)
    vg = [gpu_vec_from_words(abft, bo, N, S), gpu_vec_from_words(abft, bo, N, S)] + \
         [abft.Vector.empty(N, S) for _ in range(3)]
    cnt_g = abft.Counters()
    rg = abft.cheby_solve(ctx, Ag, *vg, lo, hi, tol=1e-10, max_iters=max_iters, due_policy=1, counts=cnt_g,
                          poll_every=8)
    torch.cuda.synchronize()
    assert rg.status == st and rg.iters == ro.iters and rg.rr0 == ro.rr0 and rg.rrn == ro.rrn
    for name, g, o in zip("burpw", vg, vo):
        a, b = words_of(g)[:N], o[:N]
        assert np.array_equal(a, b), name
    assert np.array_equal(cnt_g.read(), cnt_o)
    if n == 32:
        assert st == 0


@pytest.mark.parametrize("n,stencil", [(32, 0), (256, 256)])
def test_spectrum_estimate(abft, ctx, n, stencil):
    S = orc.SECDED64
    N = n * n
    Ao, Ag = _setup(abft, ctx, n, S, stencil)
    bo = orc.vec_encode(gen.tealeaf_rhs(n).numpy(), S)
    vo = [bo.copy(), bo.copy()] + [np.zeros_like(bo) for _ in range(3)]
    st, ro, al, bl = orc.cg_solve_log(Ao, *vo, S, 0.0, 20, 1, None)
    lo_o, hi_o = orc.lanczos_bounds(al, bl)
    vg = [gpu_vec_from_words(abft, bo, N, S), gpu_vec_from_words(abft, bo, N, S)] + \
         [abft.Vector.empty(N, S) for _ in range(3)]
    lo, hi, rg = abft.cg_spectrum(ctx, Ag, *vg, steps=20)
    assert rg.iters == ro.iters == 20
    assert np.array_equal(words_of(vg[1])[:N], vo[1][:N])   # the CG steps themselves are bit-exact
    assert abs(lo - lo_o) <= 1e-12 * lo_o and abs(hi - hi_o) <= 1e-12 * hi_o


def test_cheby_single_flips_and_due(abft, ctx):
    """Flips before the solve: singles corrected (bit-identical solve); a
    same-word double flip in u0 under policy abort stops after init."""
    n, S = 256, orc.SECDED64
    N = n * n
    lo, hi = 0.95, gershgorin_max(n)
    for double in (False, True):
        Ao, Ag = _setup(abft, ctx, n, S, n)
        bo = orc.vec_encode(gen.tealeaf_rhs(n).numpy(), S)
        uo = bo.copy()
        ug = gpu_vec_from_words(abft, bo, N, S)
        rng = np.random.default_rng(5 + double)
        for i in rng.choice(N, 6, replace=False):
            bits = rng.choice(64, 2 if double else 1, replace=False)
            for b in bits:
                uo[i] ^= np.uint64(1 << int(b))
                abft.inject_bitflip(ctx, ug.data, 64 * int(i) + int(b))
        vo = [bo.copy(), uo] + [np.zeros_like(bo) for _ in range(3)]
        cnt_o = orc.new_counts()
        st, ro = orc.cheby_solve(Ao, *vo, S, lo, hi, 1e-10, 40, 0, cnt_o)
        vg = [gpu_vec_from_words(abft, bo, N, S), ug] + [abft.Vector.empty(N, S) for _ in range(3)]
        cnt_g = abft.Counters()
        rg = abft.cheby_solve(ctx, Ag, *vg, lo, hi, tol=1e-10, max_iters=40, due_policy=0, counts=cnt_g)
        torch.cuda.synchronize()
        assert rg.status == st and rg.iters == ro.iters
        assert np.array_equal(words_of(vg[1])[:N], vo[1][:N]) and np.array_equal(cnt_g.read(), cnt_o)
        if double:
            assert st == orc.E_DUE and ro.iters == 0
