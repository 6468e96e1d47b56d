"""GPU parity of CRC32C single-bit correction (1EC4ED, DESIGN.md
§3.5 reading R9) vs the oracle: every stored bit position of an E-CRC row
flipped in some row (tiled and generic SpMV, interval detect-only access),
R-CRC octets and V-CRC quads in the SpMV input, check_all count-only / scrub /
detect-only, and multi-bit flips (DUE, never miscorrected).  Counters, outputs
and scrubbed storage bit-exact."""
import numpy as np
import pytest
import torch

import gen
import oracle as orc
from gpu_helpers import col_words, gpu_matrix, gpu_vec_from_words, oracle_matrix, rowptr_words, val_words, words_of

pytestmark = pytest.mark.gpu
S = orc.CRC32C


@pytest.fixture(scope="module")
def abft():
    from paper_conf_cluster_pawelczakmpm17_b200 import build
    build.build()
    from paper_conf_cluster_pawelczakmpm17_b200 import abft as A
    return A


@pytest.fixture(scope="module")
def ctx(abft):
    return abft.Context(0)


def _both(abft, ctx, n, stencil):
    v, c, r = gen.tealeaf_csr(n)
    v, c, r = v.numpy(), c.numpy().astype(np.uint32), r.numpy().astype(np.uint32)
    N = n * n
    Ao, _ = oracle_matrix(v, c, r, N, N, S, S)
    Ag, _ = gpu_matrix(abft, ctx, v, c, r, N, N, S, S, stencil_n=n if stencil else 0)
    return Ao, Ag, N


def _flip_el(abft, ctx, Ao, Ag, e, b):
    if b < 64:
        Ao.val[e] ^= np.uint64(1 << b)
        abft.inject_bitflip(ctx, Ag.val, 64 * e + b)
    else:
        Ao.col[e] ^= np.uint32(1 << (b - 64))
        abft.inject_bitflip(ctx, Ag.col, 32 * e + b - 64)


@pytest.mark.parametrize("stencil", [True, False])
@pytest.mark.parametrize("nbits", [1, 2, 4])
@pytest.mark.parametrize("mode", [0, 1])
def test_crc_spmv_fix_parity(abft, ctx, stencil, nbits, mode):
    n = 256 if stencil else 48
    Ao, Ag, N = _both(abft, ctx, n, stencil)
    rng = np.random.default_rng(100 * nbits + stencil + 7 * mode)
    # E-CRC: row 3 r + 1 gets row bit r (all 480 positions with nbits = 1)
    rows = range(480) if nbits == 1 else range(0, 480, 5)
    for r in rows:
        row = (3 * r + 1) % N
        bits = [r] if nbits == 1 else list(rng.choice(480, nbits, replace=False))
        for b in bits:
            _flip_el(abft, ctx, Ao, Ag, 5 * row + int(b) // 96, int(b) % 96)
    # R-CRC octets and V-CRC quads of the input
    for g in rng.choice(len(Ao.rowptr) // 8 - 1, 40, replace=False):
        for b in rng.choice(256, nbits, replace=False):
            Ao.rowptr[8 * g + b // 32] ^= np.uint32(1 << int(b % 32))
            abft.inject_bitflip(ctx, Ag.rowptr, 256 * int(g) + int(b))
    xo = orc.vec_encode(gen.uniform_pm1(N, 3) * 2.0, S)
    xg = gpu_vec_from_words(abft, xo, N, S)
    for q in rng.choice(N // 4, 60, replace=False):
        for b in rng.choice(256, nbits, replace=False):
            xo[4 * q + b // 64] ^= np.uint64(1 << int(b % 64))
            abft.inject_bitflip(ctx, xg.data, 256 * int(q) + int(b))
    yo = np.zeros_like(xo)
    cnt_o = orc.new_counts()
    orc.spmv(Ao, xo, N, S, yo, N, cnt_o, mode=mode)
    yg = abft.Vector.empty(N, S)
    cnt_g = abft.Counters()
    abft.spmv(ctx, Ag, xg, yg, cnt_g, mode=mode)
    torch.cuda.synchronize()
    cg = cnt_g.read()
    assert np.array_equal(cg, cnt_o), (cg, cnt_o)
    if nbits == 1 and mode == 0:
        assert cg[orc.ELEM, S, orc.COR] == 480 and cg[orc.ELEM, S, orc.UNC] == 0
        assert cg[orc.ROWPTR, S, orc.UNC] == 0 and cg[orc.VEC, S, orc.UNC] == 0
    if nbits > 1:
        assert cg[:, S, orc.COR].sum() == 0
    keep = np.uint64(~np.uint64(0xFF))
    both_nan = np.isnan((words_of(yg)[:N] & keep).view(np.float64)) & np.isnan((yo[:N] & keep).view(np.float64))
    assert np.all((words_of(yg)[:N] == yo[:N]) | both_nan)
    assert np.array_equal(val_words(Ag), Ao.val) and np.array_equal(col_words(Ag), Ao.col)
    assert np.array_equal(rowptr_words(Ag), Ao.rowptr)
    assert np.array_equal(words_of(xg)[:N], xo[:N])


@pytest.mark.parametrize("scrub", [0, 1, 2])
def test_crc_check_all_parity(abft, ctx, scrub):
    Ao, Ag, N = _both(abft, ctx, 40, False)
    rng = np.random.default_rng(5 + scrub)
    for e in rng.choice(Ao.nnz, 30, replace=False):
        _flip_el(abft, ctx, Ao, Ag, int(e), int(rng.integers(96)))
    for g in rng.choice(len(Ao.rowptr), 10, replace=False):
        b = int(rng.integers(32))
        Ao.rowptr[g] ^= np.uint32(1 << b)
        abft.inject_bitflip(ctx, Ag.rowptr, 32 * int(g) + b)
    xo = orc.vec_encode(gen.uniform_pm1(N, 9), S)
    xg = gpu_vec_from_words(abft, xo, N, S)
    for i in rng.choice(N, 12, replace=False):
        b = int(rng.integers(64))
        xo[i] ^= np.uint64(1 << b)
        abft.inject_bitflip(ctx, xg.data, 64 * int(i) + b)
    cnt_o = orc.new_counts()
    Ao.check(cnt_o, scrub=scrub)
    orc.vec_check(xo, N, S, cnt_o, scrub=(scrub == 1))
    cnt_g = abft.Counters()
    abft.check_all(ctx, Ag, [xg] if scrub != 2 else [], cnt_g, scrub=scrub)
    cg = cnt_g.read()
    if scrub == 2:   # detection-only sweep covers the matrix; vectors are not part of it here
        cnt_o[orc.VEC] = 0
    assert np.array_equal(cg, cnt_o), (cg[:, S].tolist(), cnt_o[:, S].tolist())
    assert np.array_equal(col_words(Ag), Ao.col) and np.array_equal(val_words(Ag), Ao.val)
    assert np.array_equal(rowptr_words(Ag), Ao.rowptr)


# ------------------------------------------------ 2EC3ED (reading R9b)
@pytest.fixture
def two_ec(abft, ctx):
    orc.set_crc_correct(2)
    ctx.set_crc_correction(2)
    yield
    orc.set_crc_correct(1)
    ctx.set_crc_correction(1)


@pytest.mark.parametrize("stencil", [True, False])
@pytest.mark.parametrize("nbits", [2, 3])
def test_crc_2ec_spmv_parity(abft, ctx, two_ec, stencil, nbits):
    """Pair correction enabled: double flips in E-CRC rows, R-CRC octets and
    V-CRC quads of the SpMV input are corrected (both words scrubbed, counted
    once); triple flips stay DUEs — bit-exact against the oracle's 2EC3ED."""
    n = 256 if stencil else 48
    Ao, Ag, N = _both(abft, ctx, n, stencil)
    rng = np.random.default_rng(300 + 10 * nbits + stencil)
    for r in range(16):
        row = (37 * r + 5) % N
        for b in rng.choice(480, nbits, replace=False):
            _flip_el(abft, ctx, Ao, Ag, 5 * row + int(b) // 96, int(b) % 96)
    for g in rng.choice(len(Ao.rowptr) // 8 - 1, 16, replace=False):
        for b in rng.choice(256, nbits, replace=False):
            Ao.rowptr[8 * g + b // 32] ^= np.uint32(1 << int(b % 32))
            abft.inject_bitflip(ctx, Ag.rowptr, 256 * int(g) + int(b))
    xo = orc.vec_encode(gen.uniform_pm1(N, 4) * 2.0, S)
    xg = gpu_vec_from_words(abft, xo, N, S)
    for q in rng.choice(N // 4, 16, replace=False):
        for b in rng.choice(256, nbits, replace=False):
            xo[4 * q + b // 64] ^= np.uint64(1 << int(b % 64))
            abft.inject_bitflip(ctx, xg.data, 256 * int(q) + int(b))
    yo = np.zeros_like(xo)
    cnt_o = orc.new_counts()
    orc.spmv(Ao, xo, N, S, yo, N, cnt_o)
    yg = abft.Vector.empty(N, S)
    cnt_g = abft.Counters()
    abft.spmv(ctx, Ag, xg, yg, cnt_g)
    torch.cuda.synchronize()
    cg = cnt_g.read()
    assert np.array_equal(cg, cnt_o), (cg[:, S].tolist(), cnt_o[:, S].tolist())
    if nbits == 2:
        assert cg[orc.ELEM, S, orc.COR] == 16 and cg[orc.ROWPTR, S, orc.COR] == 16 and cg[orc.VEC, S, orc.COR] == 16
        assert cg[:, S, orc.UNC].sum() == 0
    else:
        assert cg[:, S, orc.COR].sum() == 0
    keep = np.uint64(~np.uint64(0xFF))
    both_nan = np.isnan((words_of(yg)[:N] & keep).view(np.float64)) & np.isnan((yo[:N] & keep).view(np.float64))
    assert np.all((words_of(yg)[:N] == yo[:N]) | both_nan)
    assert np.array_equal(val_words(Ag), Ao.val) and np.array_equal(col_words(Ag), Ao.col)
    assert np.array_equal(rowptr_words(Ag), Ao.rowptr)
    assert np.array_equal(words_of(xg)[:N], xo[:N])


@pytest.mark.parametrize("scrub", [0, 1, 2])
def test_crc_2ec_check_all_parity(abft, ctx, two_ec, scrub):
    Ao, Ag, N = _both(abft, ctx, 40, False)
    rng = np.random.default_rng(50 + scrub)
    for row in rng.choice(N, 8, replace=False):
        for b in rng.choice(480, 2, replace=False):
            _flip_el(abft, ctx, Ao, Ag, 5 * int(row) + int(b) // 96, int(b) % 96)
    for g in rng.choice(len(Ao.rowptr) // 8 - 1, 6, replace=False):
        for b in rng.choice(256, 2, replace=False):
            Ao.rowptr[8 * g + b // 32] ^= np.uint32(1 << int(b % 32))
            abft.inject_bitflip(ctx, Ag.rowptr, 256 * int(g) + int(b))
    xo = orc.vec_encode(gen.uniform_pm1(N, 10), S)
    xg = gpu_vec_from_words(abft, xo, N, S)
    for q in rng.choice(N // 4, 6, replace=False):
        for b in rng.choice(256, 2, replace=False):
            xo[4 * q + b // 64] ^= np.uint64(1 << int(b % 64))
            abft.inject_bitflip(ctx, xg.data, 256 * int(q) + int(b))
    cnt_o = orc.new_counts()
    Ao.check(cnt_o, scrub=scrub)
    orc.vec_check(xo, N, S, cnt_o, scrub=(scrub == 1))
    cnt_g = abft.Counters()
    abft.check_all(ctx, Ag, [xg] if scrub != 2 else [], cnt_g, scrub=scrub)
    cg = cnt_g.read()
    if scrub == 2:
        cnt_o[orc.VEC] = 0
    assert np.array_equal(cg, cnt_o), (cg[:, S].tolist(), cnt_o[:, S].tolist())
    assert np.array_equal(col_words(Ag), Ao.col) and np.array_equal(val_words(Ag), Ao.val)
    assert np.array_equal(rowptr_words(Ag), Ao.rowptr)
    if scrub != 2:
        assert np.array_equal(words_of(xg)[:N], xo[:N])
