"""Pins of the oracle's CRC32C single-bit correction (1EC4ED, P:260-278,
DESIGN.md §3.5 reading R9) against what the mathematics fixes, not against the
oracle itself:

* every single flip of every stored bit of a V-CRC quad / R-CRC octet / E-CRC
  row is corrected back to the exact original words and counted once;
* CRC32C has Hamming distance >= 6 at these codeword lengths (the
  HD test in test_oracle_codes.py re-proves it on the CRC itself), so 2, 3 and
  4 flips are never within distance 1 of a codeword: all DUE, nothing written;
* above the HD-6 length bound (message + 32 > 5243 bits) no correction is
  attempted: a single flip is a DUE.
"""
import numpy as np
import pytest

import gen
import oracle as orc

DET, COR, UNC = 0, 1, 2


def _vcrc_words(n_quads, seed):
    return orc.vec_encode(gen.uniform_pm1(4 * n_quads, seed) * 7.0, orc.CRC32C)


def test_vcrc_every_single_flip_corrected():
    base = _vcrc_words(1, 3)
    w = np.tile(base, 256)
    for b in range(256):                       # copy b gets stored bit b flipped
        w[4 * b + b // 64] ^= np.uint64(1 << (b % 64))
    cnt = orc.new_counts()
    orc.vec_check(w, len(w), orc.CRC32C, cnt, scrub=True)
    assert cnt[orc.VEC, orc.CRC32C, COR] == 256 and cnt[orc.VEC, orc.CRC32C, UNC] == 0
    assert np.array_equal(w, np.tile(base, 256))


@pytest.mark.parametrize("k", [2, 3, 4])
def test_vcrc_2_to_4_flips_all_due(k):
    rng = np.random.default_rng(10 + k)
    trials = 600
    base = _vcrc_words(1, 5)
    w = np.tile(base, trials)
    for t in range(trials):
        for b in rng.choice(256, k, replace=False):
            w[4 * t + b // 64] ^= np.uint64(1 << int(b % 64))
    before = w.copy()
    cnt = orc.new_counts()
    orc.vec_check(w, len(w), orc.CRC32C, cnt, scrub=True)
    assert cnt[orc.VEC, orc.CRC32C, UNC] == trials and cnt[orc.VEC, orc.CRC32C, COR] == 0
    assert np.array_equal(w, before)


def _rcrc_matrix(nrows):
    """A matrix with nrows empty rows and R-CRC row pointers (octets of equal
    entries are valid; use distinct values so flips are not symmetric)."""
    rp = np.arange(nrows + 1, dtype=np.uint32) * 3
    val = np.ones(int(rp[-1]))
    col = np.zeros(int(rp[-1]), dtype=np.uint32)
    A = orc.Matrix(val, col, rp, nrows, 1, orc.NONE, orc.CRC32C)
    assert A.encode() == 0
    return A


def test_rcrc_every_single_flip_corrected():
    A = _rcrc_matrix(256 * 8 - 1)              # 256 octets
    ref = A.rowptr.copy()
    for g in range(256):                       # octet g gets stored bit g flipped
        A.rowptr[8 * g + g // 32] ^= np.uint32(1 << (g % 32))
    cnt = orc.new_counts()
    A.check(cnt, scrub=True)
    assert cnt[orc.ROWPTR, orc.CRC32C, COR] == 256 and cnt[orc.ROWPTR, orc.CRC32C, UNC] == 0
    assert np.array_equal(A.rowptr, ref)


@pytest.mark.parametrize("k", [2, 4])
def test_rcrc_multi_flips_due(k):
    rng = np.random.default_rng(20 + k)
    A = _rcrc_matrix(300 * 8 - 1)
    for g in range(300):
        for b in rng.choice(256, k, replace=False):
            A.rowptr[8 * g + b // 32] ^= np.uint32(1 << int(b % 32))
    before = A.rowptr.copy()
    cnt = orc.new_counts()
    A.check(cnt, scrub=True)
    assert cnt[orc.ROWPTR, orc.CRC32C, UNC] == 300 and cnt[orc.ROWPTR, orc.CRC32C, COR] == 0
    assert np.array_equal(A.rowptr, before)


def _ecrc_rows(nrows, L, seed):
    rng = np.random.default_rng(seed)
    rp = np.arange(nrows + 1, dtype=np.uint32) * L
    one = gen.uniform_pm1(L, seed) * 3.0
    cols = rng.choice(1000, L, replace=False).astype(np.uint32)
    A = orc.Matrix(np.tile(one, nrows), np.tile(cols, nrows), rp, nrows, 1000, orc.CRC32C, orc.NONE)
    assert A.encode() == 0
    return A


def _flip_elem_bit(A, e, b):
    if b < 64:
        A.val[e] ^= np.uint64(1 << b)
    else:
        A.col[e] ^= np.uint32(1 << (b - 64))


def test_ecrc_every_single_flip_corrected():
    L = 5                                      # the TeaLeaf row: 480 stored bits
    A = _ecrc_rows(96 * L, L, 7)
    rv, rc = A.val.copy(), A.col.copy()
    for r in range(96 * L):                    # row r gets stored bit r of the row flipped
        _flip_elem_bit(A, L * r + r // 96, r % 96)
    cnt = orc.new_counts()
    A.check(cnt, scrub=True)
    assert cnt[orc.ELEM, orc.CRC32C, COR] == 96 * L and cnt[orc.ELEM, orc.CRC32C, UNC] == 0
    assert np.array_equal(A.val, rv) and np.array_equal(A.col, rc)


@pytest.mark.parametrize("k", [2, 3, 4])
def test_ecrc_multi_flips_due(k):
    L = 5
    rng = np.random.default_rng(30 + k)
    A = _ecrc_rows(200, L, 9)
    for r in range(200):
        for b in rng.choice(96 * L, k, replace=False):
            _flip_elem_bit(A, L * r + int(b) // 96, int(b) % 96)
    bv, bc = A.val.copy(), A.col.copy()
    cnt = orc.new_counts()
    A.check(cnt, scrub=True)
    assert cnt[orc.ELEM, orc.CRC32C, UNC] == 200 and cnt[orc.ELEM, orc.CRC32C, COR] == 0
    assert np.array_equal(A.val, bv) and np.array_equal(A.col, bc)


def test_ecrc_no_correction_beyond_hd6_length():
    # 55 entries: 96 * 55 + 32 = 5312 > 5243 bits -> detect only
    L = 55
    A = _ecrc_rows(3, L, 11)
    for r in range(3):
        _flip_elem_bit(A, L * r + 7, 40 + r)
    cnt = orc.new_counts()
    A.check(cnt, scrub=True)
    assert cnt[orc.ELEM, orc.CRC32C, UNC] == 3 and cnt[orc.ELEM, orc.CRC32C, COR] == 0
    # 54 entries: 5216 bits, still corrected
    B = _ecrc_rows(2, 54, 12)
    ref = B.val.copy()
    _flip_elem_bit(B, 3, 17)
    cnt = orc.new_counts()
    B.check(cnt, scrub=True)
    assert cnt[orc.ELEM, orc.CRC32C, COR] == 1 and np.array_equal(B.val, ref)


def test_spmv_uses_the_corrected_row():
    """A corrected E-CRC row multiplies with its corrected values (SpMV of the
    flipped matrix == SpMV of the clean one) and the row is scrubbed."""
    n = 16
    v, c, r = gen.tealeaf_csr(n)
    v, c, r = v.numpy(), c.numpy().astype(np.uint32), r.numpy().astype(np.uint32)
    N = n * n
    A = orc.Matrix(v, c, r, N, N, orc.CRC32C, orc.CRC32C)
    B = orc.Matrix(v, c, r, N, N, orc.CRC32C, orc.CRC32C)
    assert A.encode() == 0 and B.encode() == 0
    x = orc.vec_encode(gen.uniform_pm1(N, 4), orc.CRC32C)
    for e, b in [(13, 52), (400, 70), (777, 90), (1000, 3)]:
        _flip_elem_bit(A, e, b)
    A.rowptr[40] ^= np.uint32(1 << 9)
    ya, yb = np.zeros_like(x), np.zeros_like(x)
    cnt = orc.new_counts()
    orc.spmv(A, x.copy(), N, orc.CRC32C, ya, N, cnt)
    orc.spmv(B, x.copy(), N, orc.CRC32C, yb, N, None)
    assert np.array_equal(ya, yb)
    assert cnt[orc.ELEM, orc.CRC32C, COR] == 4 and cnt[orc.ROWPTR, orc.CRC32C, COR] == 1
    assert np.array_equal(A.val, B.val) and np.array_equal(A.col, B.col) and np.array_equal(A.rowptr, B.rowptr)


# ---------------------------------------------------------------- 2EC3ED (reading R9b)
@pytest.fixture
def two_ec():
    orc.set_crc_correct(2)
    yield
    orc.set_crc_correct(1)


def test_2ec_vcrc_double_flips_corrected_triples_due(two_ec):
    """With HD 6, every double flip is the unique weight-2 explanation: corrected
    back exactly; a triple flip is never within distance 2 of another codeword:
    DUE, nothing written; singles stay corrected."""
    rng = np.random.default_rng(41)
    base = _vcrc_words(1, 8)
    for k, trials in ((1, 20), (2, 60), (3, 30)):
        w = np.tile(base, trials)
        for t in range(trials):
            for b in rng.choice(256, k, replace=False):
                w[4 * t + b // 64] ^= np.uint64(1 << int(b % 64))
        before = w.copy()
        cnt = orc.new_counts()
        orc.vec_check(w, len(w), orc.CRC32C, cnt, scrub=True)
        if k <= 2:
            assert cnt[orc.VEC, orc.CRC32C, COR] == trials and cnt[orc.VEC, orc.CRC32C, UNC] == 0
            assert np.array_equal(w, np.tile(base, trials))
        else:
            assert cnt[orc.VEC, orc.CRC32C, UNC] == trials and cnt[orc.VEC, orc.CRC32C, COR] == 0
            assert np.array_equal(w, before)


def test_2ec_rcrc_and_ecrc_double_flips_corrected(two_ec):
    rng = np.random.default_rng(42)
    A = _rcrc_matrix(40 * 8 - 1)
    ref = A.rowptr.copy()
    for g in range(40):
        for b in rng.choice(256, 2, replace=False):
            A.rowptr[8 * g + b // 32] ^= np.uint32(1 << int(b % 32))
    cnt = orc.new_counts()
    A.check(cnt, scrub=True)
    assert cnt[orc.ROWPTR, orc.CRC32C, COR] == 40 and cnt[orc.ROWPTR, orc.CRC32C, UNC] == 0
    assert np.array_equal(A.rowptr, ref)
    L = 5
    E = _ecrc_rows(12, L, 13)
    rv, rc = E.val.copy(), E.col.copy()
    for r in range(12):
        for b in rng.choice(96 * L, 2, replace=False):
            _flip_elem_bit(E, L * r + int(b) // 96, int(b) % 96)
    cnt = orc.new_counts()
    E.check(cnt, scrub=True)
    assert cnt[orc.ELEM, orc.CRC32C, COR] == 12 and cnt[orc.ELEM, orc.CRC32C, UNC] == 0
    assert np.array_equal(E.val, rv) and np.array_equal(E.col, rc)
