"""GPU parity of the single-reduction protected CG (S§8(f) f3; DESIGN.md
§4.1, reading R28; abft_cg_solve_sr) against the oracle's or_cg_solve_sr:
iterations, status, rr0 / rrn, every stored word of x, r, p, w, s and every
counter bit-exact — every vector scheme, generic and tiled SpMV, converged
and max_iters stops, scheduled single flips (corrected) and a DUE under policy
abort."""
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


def _same(a, b, S):
    k = {orc.NONE: 0, orc.SED: 1, orc.SECDED64: 8, orc.SECDED128: 5, orc.CRC32C: 8}[S]
    keep = np.uint64(~np.uint64((1 << k) - 1)) if k else np.uint64(0xFFFFFFFFFFFFFFFF)
    va, vb = (a & keep).view(np.float64), (b & keep).view(np.float64)
    return bool(np.all((a == b) | (np.isnan(va) & np.isnan(vb))))


def _both(abft, ctx, n, S, max_iters, stencil=0, faults=(), policy=1, poll=8):
    N = n * n
    es, rs = _schemes(S)
    v, c, r = gen.tealeaf_csr(n)
    v, c, r = v.numpy(), c.numpy().astype(np.uint32), r.numpy().astype(np.uint32)
    Ao = orc.Matrix(v, c, r, N, N, es, rs)
    assert Ao.encode() == 0
    bo = orc.vec_encode(gen.tealeaf_rhs(n).numpy(), S)
    vo = [bo.copy(), bo.copy()] + [np.zeros_like(bo) for _ in range(4)]   # b x r p w s
    cnt_o = orc.new_counts()
    st, res_o = orc.cg_solve_sr(Ao, *vo, S, 1e-10, max_iters, policy, cnt_o,
                                faults=orc.fault_schedule(list(faults)) if faults else None)
    Ag = abft.Matrix(torch.from_numpy(v).cuda(), torch.from_numpy(c.view(np.int32)).cuda(),
                     torch.from_numpy(r.view(np.int32)).cuda(), N, N, es, rs, stencil_n=stencil)
    assert Ag.encode(ctx) == 0
    vg = [gpu_vec_from_words(abft, bo, N, S), gpu_vec_from_words(abft, bo, N, S)] + \
         [abft.Vector.empty(N, S) for _ in range(4)]
    if faults:
        ctx.set_faults(list(faults), Ag, vg[:5])
    cnt_g = abft.Counters()
    try:
        res_g = abft.cg_solve_sr(ctx, Ag, *vg, tol=1e-10, max_iters=max_iters, due_policy=policy, counts=cnt_g,
                                 poll_every=poll)
    finally:
        if faults:
            ctx.set_faults([])
    torch.cuda.synchronize()
    return st, res_o, res_g, vo, [words_of(t) for t in vg], cnt_o, cnt_g.read()


@pytest.mark.parametrize("vs", ["NONE", "SED", "SECDED64", "SECDED128", "CRC32C"])
@pytest.mark.parametrize("n,stencil,max_iters", [(32, 0, 400), (256, 256, 45)])
def test_sr_parity(abft, ctx, vs, n, stencil, max_iters):
    S = getattr(orc, vs)
    st, ro, rg, vo, vg, co, cg = _both(abft, ctx, n, S, max_iters, stencil)
    assert rg.status == st and rg.iters == ro.iters
    assert rg.rr0 == ro.rr0 and (rg.rrn == ro.rrn or (np.isnan(rg.rrn) and np.isnan(ro.rrn)))
    N = n * n
    for name, a, b in zip("bxrpws", vg, vo):
        assert _same(a[:N], b[:N], S), name
    assert np.array_equal(cg, co)
    if n == 32:
        assert st == 0


@pytest.mark.parametrize("stencil", [0, 256])
def test_sr_scheduled_single_flips(abft, ctx, stencil):
    n, S = 256, orc.SECDED64
    N = n * n
    rng = np.random.default_rng(9 + stencil)
    faults, used = [], set()
    while len(faults) < 60:
        t = int(rng.choice([orc.F_VAL, orc.F_COL, orc.F_X, orc.F_R, orc.F_P, orc.F_W]))
        k = int(rng.integers(1, 30))
        w = int(rng.integers(5 * N if t in (orc.F_VAL, orc.F_COL) else N))
        key = ("el", w) if t in (orc.F_VAL, orc.F_COL) else (t, w)
        if key in used:
            continue
        used.add(key)
        faults.append((k, t, w, int(rng.integers(32 if t == orc.F_COL else 64))))
    st, ro, rg, vo, vg, co, cg = _both(abft, ctx, n, S, 40, stencil, faults)
    assert rg.status == st == orc.E_NOT_CONVERGED and rg.iters == ro.iters == 40
    assert np.array_equal(vg[1][:N], vo[1][:N]) and np.array_equal(cg, co)
    assert cg[:, :, orc.COR].sum() == 60 and cg[:, :, orc.UNC].sum() == 0


@pytest.mark.parametrize("t", [orc.F_P, orc.F_X, orc.F_W])
def test_sr_due_abort(abft, ctx, t):
    n, S = 256, orc.SECDED64
    st, ro, rg, vo, vg, co, cg = _both(abft, ctx, n, S, 40, n, [(7, t, 1234, 3), (7, t, 1234, 50)], policy=0)
    assert st == rg.status == orc.E_DUE and rg.iters == ro.iters == 7
    assert np.array_equal(cg, co) and np.array_equal(vg[1][:n * n], vo[1][:n * n])
