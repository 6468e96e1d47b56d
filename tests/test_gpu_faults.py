"""GPU parity of the scheduled fault harness (S§8(c) O10; BASELINE config 1's
mid-solve variant): faults (iteration k, target, word, bit) applied by a
device-side kernel before init (k = 0) or before iteration k's SpMV, inside
the CUDA-graph replays of the solve (abft_ctx_set_faults).  Compared with the
oracle's or_cg_solve_sched on the same schedule: iterations, status, rrn, x
and every fault counter bit-exact."""
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


def _same(a, b, S):
    k = {orc.SED: 1, orc.SECDED64: 8}.get(S, 0)
    keep = np.uint64(~np.uint64((1 << k) - 1))
    va, vb = (a & keep).view(np.float64), (b & keep).view(np.float64)
    return bool(np.all((a == b) | (np.isnan(va) & np.isnan(vb))))


def _both(abft, ctx, n, es, rs, vs, faults, policy, max_iters, stencil=0, poll=8):
    N = n * n
    v, c, r = gen.tealeaf_csr(n)
    v, c, r = v.numpy(), c.numpy().astype(np.uint32), r.numpy().astype(np.uint32)
    Ao = orc.Matrix(v, c, r, N, N, es, rs)
    assert Ao.encode() == 0
    bo = orc.vec_encode(gen.tealeaf_rhs(n).numpy(), vs)
    xo = bo.copy()
    ro, po, wo = (np.zeros_like(bo) for _ in range(3))
    cnt_o = orc.new_counts()
    st, res_o = orc.cg_solve_sched(Ao, bo.copy(), xo, ro, po, wo, vs, 1e-10, max_iters, policy, cnt_o,
                                   faults=orc.fault_schedule(faults))
    Ag = abft.Matrix(torch.from_numpy(v).cuda(), torch.from_numpy(c.view(np.int32)).cuda(),
                     torch.from_numpy(r.view(np.int32)).cuda(), N, N, es, rs, stencil_n=stencil)
    assert Ag.encode(ctx) == 0
    bg, xg = gpu_vec_from_words(abft, bo, N, vs), gpu_vec_from_words(abft, bo, N, vs)
    rg, pg, wg = (abft.Vector.empty(N, vs) for _ in range(3))
    ctx.set_faults(faults, Ag, (bg, xg, rg, pg, wg))
    cnt_g = abft.Counters()
    try:
        res_g = abft.cg_solve(ctx, Ag, bg, xg, rg, pg, wg, tol=1e-10, max_iters=max_iters, due_policy=policy,
                              counts=cnt_g, poll_every=poll)
    finally:
        ctx.set_faults([])
    torch.cuda.synchronize()
    return dict(st=st, res_o=res_o, res_g=res_g, xo=xo[:N], xg=words_of(xg)[:N], cnt_o=cnt_o, cnt_g=cnt_g.read())


def _schedule(rng, n, nnz, rp_len, count, targets, kmax):
    N = n * n
    out, used = [], set()
    while len(out) < count:
        t = int(rng.choice(targets))
        k = 0 if t in (orc.F_B,) else int(rng.integers(0 if t in (orc.F_VAL, orc.F_COL, orc.F_ROWPTR, orc.F_X) else 1,
                                                        kmax + 1))
        if t in (orc.F_VAL, orc.F_COL):
            w = int(rng.integers(nnz))
            key, bit = ("el", w), int(rng.integers(64 if t == orc.F_VAL else 32))
        elif t == orc.F_ROWPTR:
            w = int(rng.integers(rp_len))
            key, bit = ("rp", w // 2), int(rng.integers(32))
        else:
            w = int(rng.integers(N))
            key, bit = (t, w), int(rng.integers(64))
        if key in used:
            continue
        used.add(key)
        out.append((k, t, w, bit))
    return out


@pytest.mark.parametrize("seed", [1, 2, 3])
def test_config1_mid_solve(abft, ctx, seed):
    """Config 1 (32^2, E-SECDED / R-SED / V-SED, policy continue): 100 single
    flips before init over val / col / rowptr / b / x0, plus 30 mid-solve flips
    on r / p / w / x at random iterations."""
    n = 32
    rng = np.random.default_rng(seed)
    pre = _schedule(rng, n, 5 * n * n, n * n + 1, 100, [orc.F_VAL, orc.F_COL, orc.F_ROWPTR, orc.F_B, orc.F_X], 0)
    pre = [(0,) + f[1:] for f in pre]
    mid = _schedule(rng, n, 5 * n * n, n * n + 1, 30, [orc.F_R, orc.F_P, orc.F_W, orc.F_X], 15)
    mid = [f if f[0] > 0 else (1,) + f[1:] for f in mid]
    R = _both(abft, ctx, n, orc.SECDED64, orc.SED, orc.SED, pre + mid, 1, 400)
    assert np.array_equal(R["cnt_g"], R["cnt_o"]), (R["cnt_g"], R["cnt_o"])
    assert R["res_g"].iters == R["res_o"].iters and R["res_g"].status == R["st"]
    assert _same(R["xg"], R["xo"], orc.SED)
    assert R["cnt_g"][orc.ELEM, orc.SECDED64, orc.UNC] == 0 and R["cnt_g"][orc.ELEM, orc.SECDED64, orc.COR] > 0


@pytest.mark.parametrize("stencil", [0, 256])
def test_config2_schemes_mid_solve_singles(abft, ctx, stencil):
    """Config-2 schemes on the 256^2 grid (tiled and generic SpMV): single
    flips into every target at random iterations are corrected before use —
    iterations and x bit-identical to the oracle's scheduled solve."""
    n = 256
    rng = np.random.default_rng(40 + stencil)
    S = orc.SECDED64
    f = _schedule(rng, n, 5 * n * n, n * n + 2, 120, list(range(8)), 60)
    R = _both(abft, ctx, n, S, S, S, f, 1, 80, stencil=stencil)
    assert R["st"] == R["res_g"].status == orc.E_NOT_CONVERGED
    assert R["res_g"].iters == R["res_o"].iters and R["res_g"].rrn == R["res_o"].rrn
    assert np.array_equal(R["xg"], R["xo"])
    assert np.array_equal(R["cnt_g"], R["cnt_o"])
    assert R["cnt_g"][:, :, orc.UNC].sum() == 0


@pytest.mark.parametrize("t,k", [(orc.F_P, 13), (orc.F_X, 9), (orc.F_VAL, 21), (orc.F_W, 13)])
def test_due_abort_mid_solve_in_graph(abft, ctx, t, k):
    """A same-word double flip at iteration k (inside a CUDA-graph replay,
    poll 8): abort after exactly iteration k where it is read, nothing where it
    is overwritten (w)."""
    n = 256
    S = orc.SECDED64
    word = 3000 if t != orc.F_VAL else 5 * 3000 + 1
    R = _both(abft, ctx, n, S, S, S, [(k, t, word, 7), (k, t, word, 44)], 0, 40, stencil=n)
    assert R["res_g"].status == R["st"] and R["res_g"].iters == R["res_o"].iters
    if t != orc.F_W:
        assert R["st"] == orc.E_DUE and R["res_o"].iters == k
    else:
        assert R["st"] == orc.E_NOT_CONVERGED and not R["cnt_o"].any()
    assert np.array_equal(R["cnt_g"], R["cnt_o"])
    assert np.array_equal(R["xg"], R["xo"])
