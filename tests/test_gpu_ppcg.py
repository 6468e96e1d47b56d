"""GPU parity of the protected PPCG (S§8(f) f4, reading R34;
abft_ppcg_solve) against the oracle's or_ppcg_solve: iterations, status,
rr0 / rrn, every stored word of x, r, p, w, z and every counter bit-exact —
every vector scheme, generic and tiled SpMV, converged and max_iters stops,
single flips (corrected) and a DUE under policy abort."""
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


def _run(abft, ctx, n, S, inner, max_iters, stencil, flips=0, double=False, policy=1):
    N = n * n
    es, rs = _schemes(S)
    v, c, r = gen.tealeaf_csr(n)
    v, c, r = v.numpy(), c.numpy().astype(np.uint32), r.numpy().astype(np.uint32)
    lo, hi = 0.95, float(np.abs(v).reshape(-1, 5).sum(axis=1).max())
    Ao = orc.Matrix(v, c, r, N, N, es, rs)
    assert Ao.encode() == 0
    Ag = abft.Matrix(torch.from_numpy(v).cuda(), torch.from_numpy(c.view(np.int32)).cuda(),
                     torch.from_numpy(r.view(np.int32)).cuda(), N, N, es, rs, stencil_n=stencil)
    assert Ag.encode(ctx) == 0
    bo = orc.vec_encode(gen.tealeaf_rhs(n).numpy(), S)
    xo = bo.copy()
    xg = gpu_vec_from_words(abft, bo, N, S)
    rng = np.random.default_rng(17 + n + flips)
    for i in rng.choice(N, flips, replace=False):
        for b in rng.choice(64, 2 if double else 1, replace=False):
            xo[i] ^= np.uint64(1 << int(b))
            abft.inject_bitflip(ctx, xg.data, 64 * int(i) + int(b))
    vo = [bo.copy(), xo] + [np.zeros_like(bo) for _ in range(6)]    # b x r p w z rin pin
    cnt_o = orc.new_counts()
    st, ro = orc.ppcg_solve(Ao, *vo, S, lo, hi, inner, 1e-10, max_iters, policy, cnt_o)
    vg = [gpu_vec_from_words(abft, bo, N, S), xg] + [abft.Vector.empty(N, S) for _ in range(6)]
    cnt_g = abft.Counters()
    rg = abft.ppcg_solve(ctx, Ag, *vg, lo, hi, inner=inner, tol=1e-10, max_iters=max_iters, due_policy=policy,
                         counts=cnt_g, poll_every=4)
    torch.cuda.synchronize()
    return st, ro, rg, vo, [words_of(t) for t in vg], cnt_o, cnt_g.read(), N


@pytest.mark.parametrize("vs", ["NONE", "SED", "SECDED64", "SECDED128", "CRC32C"])
@pytest.mark.parametrize("n,stencil,max_iters,inner", [(32, 0, 500, 4), (256, 256, 12, 3)])
def test_ppcg_parity(abft, ctx, vs, n, stencil, max_iters, inner):
    S = getattr(orc, vs)
    st, ro, rg, vo, vg, co, cg, N = _run(abft, ctx, n, S, inner, max_iters, stencil)
    assert rg.status == st and rg.iters == ro.iters and rg.rr0 == ro.rr0 and rg.rrn == ro.rrn
    for name, a, b in zip(["b", "x", "r", "p", "w", "z", "rin", "pin"], vg, vo):
        assert np.array_equal(a[:N], b[:N]), name
    assert np.array_equal(cg, co)
    if n == 32:
        assert st == 0


@pytest.mark.parametrize("double", [False, True])
def test_ppcg_flips(abft, ctx, double):
    S = orc.SECDED64
    st, ro, rg, vo, vg, co, cg, N = _run(abft, ctx, 256, S, 4, 10, 256, flips=6, double=double, policy=0)
    assert rg.status == st and rg.iters == ro.iters
    assert np.array_equal(vg[1][:N], vo[1][:N]) and np.array_equal(cg, co)
    if double:
        assert st == orc.E_DUE and ro.iters == 0
    else:
        assert cg[orc.VEC, S, orc.COR] == 6
