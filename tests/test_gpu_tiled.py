"""GPU parity of the tiled stencil SpMV fast path (stencil_n hint set,
n % 256 == 0) and of row-block chunks (reading R7): bit-exact outputs, dots,
counts and scrubbed storage vs the oracle, including flips in tile halos and
across chunk boundaries, and a ragged last tile (rows not a multiple of 16)."""
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


def _chunks(n, splits):
    """Row-block chunks of the n x n G-TEA matrix at grid-row boundaries `splits`."""
    out = []
    ys = [0] + list(splits) + [n]
    for y0, y1 in zip(ys[:-1], ys[1:]):
        v, c, r = gen.strip_csr(n, y0, y1, ny=n, col_offset=y0 * n)
        out.append((v.numpy(), c.numpy().astype(np.uint32), r.numpy().astype(np.uint32), y0 * n, (y1 - y0) * n))
    return out


def _flip(abft, ctx, Ao, Ag, xo, xg, rng, n_el, n_rp, xs):
    for e in rng.choice(Ao.nnz, n_el, replace=False):
        b = int(rng.integers(96))
        if b < 64:
            Ao.val[e] ^= np.uint64(1 << b)
            abft.inject_bitflip(ctx, Ag.val, 64 * int(e) + b)
        else:
            Ao.col[e] ^= np.uint32(1 << (b - 64))
            abft.inject_bitflip(ctx, Ag.col, 32 * int(e) + b - 64)
    for g in rng.choice(len(Ao.rowptr), n_rp, replace=False):
        b = int(rng.integers(32))
        Ao.rowptr[g] ^= np.uint32(1 << b)
        abft.inject_bitflip(ctx, Ag.rowptr, 32 * int(g) + b)


def _schemes(S):
    """Element / rowptr schemes paired with vector scheme S in the tiled tests:
    CRC32C everywhere for CRC32C (table-driven E-CRC / R-CRC / V-CRC), R-SECDED128
    with V-SECDED128, E-SECDED + R-SECDED64 otherwise."""
    if S == orc.NONE:
        return orc.NONE, orc.NONE
    if S == orc.CRC32C:
        return orc.CRC32C, orc.CRC32C
    return orc.SECDED64, (orc.SECDED128 if S == orc.SECDED128 else orc.SECDED64)


@pytest.mark.parametrize("vs", ["NONE", "SED", "SECDED64", "SECDED128", "CRC32C"])
@pytest.mark.parametrize("splits", [(), (40,), (16, 100)])
@pytest.mark.parametrize("faults", [False, True])
def test_tiled_spmv_parity(abft, ctx, vs, splits, faults):
    n = 256
    N = n * n
    S = getattr(orc, vs)
    es, rs = _schemes(S)
    rng = np.random.default_rng(7 + len(splits) + 10 * faults)
    x = gen.uniform_pm1(N, 11)
    xo = orc.vec_encode(x, S)
    xg = gpu_vec_from_words(abft, xo, N, S)
    if faults and S != orc.NONE:
        # vector flips, including tile halo rows (grid rows 15/16, 31/32) and chunk edges
        idx = list(rng.choice(N, 20, replace=False)) + [15 * n + 3, 16 * n + 255, 40 * n, 40 * n - 1, 100 * n + 7]
        for i in set(int(i) for i in idx):
            b = int(rng.integers(64))
            xo[i] ^= np.uint64(1 << b)
            abft.inject_bitflip(ctx, xg.data, 64 * i + b)
    Aos, Ags = [], []
    for (v, c, r, base, rows) in _chunks(n, splits):
        Ao, _ = oracle_matrix(v, c, r, rows, N, es, rs, row_base=base, col_base=0)
        Ag, _ = gpu_matrix(abft, ctx, v, c, r, rows, N, es, rs, row_base=base, col_base=0, stencil_n=n)
        if faults and S != orc.NONE:
            _flip(abft, ctx, Ao, Ag, xo, xg, rng, 8, 3, [])
        Aos.append(Ao)
        Ags.append(Ag)
    out_o = np.zeros(N, dtype=np.uint64)
    cnt_o = orc.new_counts()
    dots = []
    for Ao in Aos:
        d, dot = orc.spmv(Ao, xo, N, S, out_o, N, cnt_o, want_dot=True)
        dots.append(dot)
    yg = abft.Vector.empty(N, S)
    cnt_g = abft.Counters()
    dot_g = torch.zeros(1, dtype=torch.float64, device="cuda")
    abft.spmv(ctx, Ags, xg, yg, cnt_g, dot=dot_g)
    torch.cuda.synchronize()
    assert np.array_equal(cnt_g.read(), cnt_o), (cnt_g.read(), cnt_o)
    assert np.array_equal(words_of(yg)[:N], out_o)
    for Ao, Ag in zip(Aos, Ags):
        assert np.array_equal(val_words(Ag), Ao.val) and np.array_equal(col_words(Ag), Ao.col)
        assert np.array_equal(rowptr_words(Ag), Ao.rowptr)
    assert np.array_equal(words_of(xg)[:N], xo)
    if not splits:
        assert dot_g.item() == dots[0]
    else:
        # chunk dots combine through the RED-1 tree over the whole vector
        masked_x = orc.vec_masked(xo, N, S)
        masked_y = orc.vec_masked(out_o, N, S)
        assert dot_g.item() == orc.dot_red1(masked_x, masked_y)


@pytest.mark.parametrize("vs", ["SECDED64", "SECDED128", "CRC32C"])
def test_tiled_cg_parity(abft, ctx, vs):
    n = 256
    N = n * n
    S = getattr(orc, vs)
    es, rs = _schemes(S)
    v, c, r = gen.tealeaf_csr(n)
    v, c, r = v.numpy(), c.numpy().astype(np.uint32), r.numpy().astype(np.uint32)
    Ao, _ = oracle_matrix(v, c, r, N, N, es, rs)
    Ag, _ = gpu_matrix(abft, ctx, v, c, r, N, N, es, rs, stencil_n=n)
    b = gen.tealeaf_rhs(n).numpy()
    bo = orc.vec_encode(b, S)
    xo = bo.copy()
    bg = gpu_vec_from_words(abft, bo, N, S)
    xg = gpu_vec_from_words(abft, xo, N, S)
    ro, po, wo = (np.zeros_like(bo) for _ in range(3))
    cnt_o = orc.new_counts()
    st, res_o = orc.cg_solve(Ao, bo, xo, ro, po, wo, S, 1e-10, 40, 1, cnt_o)
    rg, pg, wg = (abft.Vector.empty(N, S) for _ in range(3))
    cnt_g = abft.Counters()
    res_g = abft.cg_solve(ctx, Ag, bg, xg, rg, pg, wg, tol=1e-10, max_iters=40, due_policy=1, counts=cnt_g)
    assert res_g.iters == res_o.iters == 40
    assert res_g.rrn == res_o.rrn
    assert np.array_equal(words_of(xg)[:N], xo)
    assert np.array_equal(cnt_g.read(), cnt_o)


@pytest.mark.parametrize("seed", [1, 2, 3])
def test_tiled_spmv_rowptr_due_parity(abft, ctx, seed):
    """Same-word double flips in rowptr entries (DUE, used as masked stored bits
    under policy continue): rows may point anywhere in [0, nnz] or outside it;
    the tiled kernel must fall back to global reads and match the oracle."""
    n = 256
    N = n * n
    S = orc.SECDED64
    rng = np.random.default_rng(100 + seed)
    v, c, r = gen.tealeaf_csr(n)
    v, c, r = v.numpy(), c.numpy().astype(np.uint32), r.numpy().astype(np.uint32)
    Ao, _ = oracle_matrix(v, c, r, N, N, S, S)
    Ag, _ = gpu_matrix(abft, ctx, v, c, r, N, N, S, S, stencil_n=n)
    for g in rng.choice(N // 2, 6, replace=False):
        i = 2 * int(g) + int(rng.integers(2))
        for b in rng.choice(28, 2, replace=False):   # value bits: the decoded entry really moves
            Ao.rowptr[i] ^= np.uint32(1 << int(b))
            abft.inject_bitflip(ctx, Ag.rowptr, 32 * i + int(b))
    x = gen.uniform_pm1(N, 5)
    xo = orc.vec_encode(x, S)
    xg = gpu_vec_from_words(abft, xo, N, S)
    out_o = np.zeros(N, dtype=np.uint64)
    cnt_o = orc.new_counts()
    orc.spmv(Ao, xo, N, S, out_o, N, cnt_o)
    yg = abft.Vector.empty(N, S)
    cnt_g = abft.Counters()
    abft.spmv(ctx, Ag, xg, yg, cnt_g)
    torch.cuda.synchronize()
    assert np.array_equal(cnt_g.read(), cnt_o)
    assert np.array_equal(words_of(yg)[:N], out_o)
