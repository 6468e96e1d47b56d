"""GPU parity of the CG vector kernels (S§8(a) rows a4 calc_ur and a5 calc_p)
through the C ABI vs the oracle, for every vector scheme: full reduction
blocks (the lane-split group codecs of V-SECDED128 / V-CRC) and ragged tails,
with single and same-word double flips in every operand: stored words, r.r,
counts and scrubbing bit-exact."""
import math

import numpy as np
import pytest
import torch

import gen
import oracle as orc
from gpu_helpers import gpu_vec_from_words, words_of

pytestmark = pytest.mark.gpu

SCHEMES = ["NONE", "SED", "SECDED64", "SECDED128", "CRC32C"]


@pytest.fixture(scope="module")
def abft():
    from paper_conf_cluster_pawelczakmpm17_b200 import build
    build.build()
    from paper_conf_cluster_pawelczakmpm17_b200 import abft as A
    return A


@pytest.fixture(scope="module")
def ctx(abft):
    return abft.Context(0)


def _vecs(abft, n, S, k, rng, nflip, double):
    host, dev = [], []
    for j in range(k):
        w = orc.vec_encode(gen.uniform_pm1(n, 30 + j) * 3.0, S)
        g = gpu_vec_from_words(abft, w, n, S)
        if S != orc.NONE:
            for i in rng.choice(n, nflip, replace=False):
                for b in rng.choice(64, 2 if double else 1, replace=False):
                    w[int(i)] ^= np.uint64(1 << int(b))
                    abft.inject_bitflip(ctx_of[0], g.data, 64 * int(i) + int(b))
        host.append(w)
        dev.append(g)
    return host, dev


ctx_of = [None]


def _same(a, b, S):
    keep = np.uint64(~np.uint64((1 << {0: 0, 1: 1, 2: 8, 3: 5, 4: 8}[S]) - 1))
    va, vb = (a & keep).view(np.float64), (b & keep).view(np.float64)
    return bool(np.all((a == b) | (np.isnan(va) & np.isnan(vb))))


@pytest.mark.parametrize("vs", SCHEMES)
@pytest.mark.parametrize("n", [4096, 1000])
@pytest.mark.parametrize("double", [False, True])
def test_calc_ur_parity(abft, ctx, vs, n, double):
    ctx_of[0] = ctx
    S = getattr(orc, vs)
    rng = np.random.default_rng(n + 3 * double + 11 * S)
    (xo, po, ro, wo), (xg, pg, rg, wg) = _vecs(abft, n, S, 4, rng, 7, double)
    alpha = 0.37
    cnt_o = orc.new_counts()
    _, rrn_o = orc.calc_ur(xo, po, ro, wo, n, S, alpha, cnt_o)
    cnt_g = abft.Counters()
    rrn_g = torch.zeros(1, dtype=torch.float64, device="cuda")
    abft.calc_ur(ctx, xg, pg, rg, wg, alpha, rrn=rrn_g, counts=cnt_g)
    torch.cuda.synchronize()
    assert np.array_equal(cnt_g.read(), cnt_o), (cnt_g.read()[2], cnt_o[2])
    for ho, gv in ((xo, xg), (po, pg), (ro, rg), (wo, wg)):
        assert _same(words_of(gv)[:len(ho)], ho, S)
    assert rrn_g.item() == rrn_o or (math.isnan(rrn_g.item()) and math.isnan(rrn_o))
    if S == orc.SECDED64 and not double:
        assert cnt_o[orc.VEC, S].tolist() == [28, 28, 0, 0]


@pytest.mark.parametrize("vs", SCHEMES)
@pytest.mark.parametrize("n", [4096, 1000])
@pytest.mark.parametrize("double", [False, True])
def test_calc_p_parity(abft, ctx, vs, n, double):
    ctx_of[0] = ctx
    S = getattr(orc, vs)
    rng = np.random.default_rng(7 * n + double + 5 * S)
    (po, ro), (pg, rg) = _vecs(abft, n, S, 2, rng, 9, double)
    beta = -0.81
    cnt_o = orc.new_counts()
    orc.calc_p(po, ro, n, S, beta, cnt_o)
    cnt_g = abft.Counters()
    abft.calc_p(ctx, pg, rg, beta, counts=cnt_g)
    torch.cuda.synchronize()
    assert np.array_equal(cnt_g.read(), cnt_o)
    assert _same(words_of(pg)[:len(po)], po, S) and _same(words_of(rg)[:len(ro)], ro, S)
