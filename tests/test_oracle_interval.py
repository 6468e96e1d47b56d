"""Pins of the oracle's interval checking ("less frequent correctness
checking", DESIGN.md §3.9 / reading R27): unchecked accesses only
range-check the matrix and use its stored bits (checked here against a dense
numpy matmul of the corrupted matrix), checked accesses detect without
correcting, and a CG with interval N reports a persistent matrix flip exactly
at accesses 0, N, 2N, ... plus the end-of-solve check (closed form)."""
import numpy as np
import pytest

import gen


def _mat(orc, n, es=None, rs=None):
    es = orc.SECDED64 if es is None else es
    rs = orc.SECDED64 if rs is None else rs
    v, c, r = gen.tealeaf_csr(n)
    A = orc.Matrix(v.numpy(), c.numpy().astype(np.uint32), r.numpy().astype(np.uint32), n * n, n * n, es, rs)
    assert A.encode() == orc.OK
    return A


def _dense_stored(orc, A):
    """Dense matrix of the STORED (possibly corrupted) values with masked columns."""
    N = A.nrows
    cm = 0x00FFFFFF if A.es in (orc.SECDED64, orc.SECDED128, orc.CRC32C) else (0x7FFFFFFF if A.es == orc.SED else ~0)
    D = np.zeros((N, N))
    rp = A.rowptr & np.uint32(0x0FFFFFFF if A.rs in (orc.SECDED64, orc.SECDED128, orc.CRC32C) else 0x7FFFFFFF)
    vals = A.val.view(np.float64)
    for i in range(N):
        for j in range(int(rp[i]), int(rp[i + 1])):
            c = int(A.col[j]) & cm
            if c < A.ncols:
                D[i, c] += vals[j]
    return D


def _run(orc, A, x, mode):
    N = A.nrows
    X = orc.vec_encode(x, orc.NONE)
    out = np.zeros(N, dtype=np.uint64)
    cnt = orc.new_counts()
    d = orc.spmv(A, X, N, orc.NONE, out, N, cnt, mode=mode)
    return out.view(np.float64).copy(), cnt, d


def _close(y, D, x):
    bound = 6 * np.finfo(float).eps * (np.abs(D) @ np.abs(x)) + 1e-300
    return np.all(np.abs(y - D @ x) <= bound)


@pytest.mark.parametrize("bit", [3, 52, 58])
def test_range_mode_uses_stored_bits(orc, bit):
    """without the integrity check a flipped value is used as stored;
    nothing is counted and nothing is scrubbed."""
    n = 8
    A = _mat(orc, n)
    e = 5 * 27 + 2                       # a diagonal element
    A.val[e] ^= np.uint64(1 << bit)
    stored = A.val.copy(), A.col.copy()
    x = gen.uniform_pm1(n * n, seed=4)
    y, cnt, d = _run(orc, A, x, orc.MODE_RANGE)
    assert d == 0 and cnt.sum() == 0
    assert np.array_equal(A.val, stored[0]) and np.array_equal(A.col, stored[1])
    assert _close(y, _dense_stored(orc, A), x)
    # the corrected access (N = 1) gives the clean product instead
    y1, cnt1, _ = _run(orc, A, x, orc.MODE_CORRECT)
    assert cnt1[orc.ELEM, orc.SECDED64].tolist() == [1, 1, 0, 0]
    assert _close(y1, _dense_stored(orc, A), x)          # A is scrubbed now
    assert not np.array_equal(y, y1)


def test_detect_mode_counts_singles_as_due(orc):
    """a checked access of interval mode detects but does not
    correct (the flip may already have been used): DUE, stored bits, no scrub."""
    n = 8
    A = _mat(orc, n)
    A.val[40] ^= np.uint64(1 << 60)
    A.col[77] ^= np.uint32(1 << 30)      # a flip in the column's ECC byte
    g = 9
    A.rowptr[2 * g] ^= np.uint32(1 << 29)   # a rowptr check bit (value unchanged)
    stored = A.val.copy(), A.col.copy(), A.rowptr.copy()
    x = gen.uniform_pm1(n * n, seed=5)
    y, cnt, d = _run(orc, A, x, orc.MODE_DETECT)
    assert cnt[orc.ELEM, orc.SECDED64].tolist() == [2, 0, 2, 0]
    assert cnt[orc.ROWPTR, orc.SECDED64].tolist() == [1, 0, 1, 0]
    assert d == 3
    assert all(np.array_equal(a, b) for a, b in zip((A.val, A.col, A.rowptr), stored))
    assert _close(y, _dense_stored(orc, A), x)
    # the detection-only check_all counts the same codewords, also without scrubbing
    cnt2 = orc.new_counts()
    assert A.check(cnt2, scrub=2) == 3
    assert cnt2[orc.ELEM, orc.SECDED64].tolist() == [2, 0, 2, 0]
    assert cnt2[orc.ROWPTR, orc.SECDED64].tolist() == [1, 0, 1, 0]
    assert all(np.array_equal(a, b) for a, b in zip((A.val, A.col, A.rowptr), stored))


@pytest.mark.parametrize("mode", ["MODE_RANGE", "MODE_DETECT"])
def test_unchecked_index_is_range_checked(orc, mode):
    """an index beyond ncols is skipped (contributes 0) and counted."""
    n = 4
    A = _mat(orc, n)
    A.col[22] = (A.col[22] & np.uint32(0xFF000000)) | np.uint32(0x00FFF000)   # 3 flips in the index: > ncols
    x = np.ones(n * n)
    y, cnt, d = _run(orc, A, x, getattr(orc, mode))
    assert cnt[orc.ELEM, orc.SECDED64, orc.RANGE] == 1
    D = _dense_stored(orc, A)
    assert _close(y, D, x)


def _cg(orc, A, n, N, policy=1, max_iters=5000):
    b = gen.tealeaf_rhs(n).numpy()
    B = orc.vec_encode(b, orc.SECDED64)
    X = B.copy()
    R, P, W = (np.zeros_like(B) for _ in range(3))
    cnt = orc.new_counts()
    st, res = orc.cg_solve(A, B, X, R, P, W, orc.SECDED64, 1e-10, max_iters, policy, cnt, check_interval=N)
    return st, res, X, cnt


@pytest.mark.parametrize("N", [2, 3, 7, 64])
def test_interval_cg_clean_is_unchanged(orc, N):
    """Interval checking changes when the matrix is checked, not the arithmetic:
    a clean solve is bit-identical to the every-access solve."""
    n = 16
    st1, r1, X1, c1 = _cg(orc, _mat(orc, n), n, 1)
    stN, rN, XN, cN = _cg(orc, _mat(orc, n), n, N)
    assert st1 == stN == orc.OK and r1.iters == rN.iters
    assert np.array_equal(X1, XN) and cN.sum() == 0 and c1.sum() == 0


@pytest.mark.parametrize("N", [2, 3, 7, 64])
def test_interval_cg_persistent_flip_counts(orc, N):
    """A matrix flip present from the start (policy continue) is reported as a
    DUE at every checked access a = 0, N, 2N, ... <= K and once more by the
    end-of-solve check when N does not divide K."""
    n = 16
    A = _mat(orc, n)
    A.val[5 * 100 + 2] ^= np.uint64(1)          # mantissa LSB of a diagonal value
    st, res, X, cnt = _cg(orc, A, n, N)
    K = res.iters
    assert st == orc.OK and K > 0
    expect = K // N + 1 + (1 if K % N else 0)
    assert cnt[orc.ELEM, orc.SECDED64].tolist() == [expect, 0, expect, 0]
    assert (A.val[5 * 100 + 2] & np.uint64(1)) != 0        # never scrubbed
    # every-access checking corrects it at access 0 instead
    A1 = _mat(orc, n)
    A1.val[5 * 100 + 2] ^= np.uint64(1)
    st1, r1, X1, c1 = _cg(orc, A1, n, 1)
    assert c1[orc.ELEM, orc.SECDED64].tolist() == [1, 1, 0, 0]


def test_interval_abort_and_final_check(orc):
    n = 16
    # abort policy: the DUE at access 0 stops the solve after init
    A = _mat(orc, n)
    A.val[3] ^= np.uint64(1 << 40)
    st, res, X, cnt = _cg(orc, A, n, 4, policy=0)
    assert st == orc.E_DUE and res.iters == 0
    assert cnt[orc.ELEM, orc.SECDED64].tolist() == [1, 0, 1, 0]
    # N larger than the iteration count: access 0 + the final check only
    A = _mat(orc, n)
    A.val[3] ^= np.uint64(1)
    st, res, X, cnt = _cg(orc, A, n, 100000)
    assert st == orc.OK
    assert cnt[orc.ELEM, orc.SECDED64].tolist() == [2, 0, 2, 0]
    # a flip that appears only at the final check turns OK into E_DUE under abort:
    # simulated by max_iters so that K % N != 0 and the flip is in a row pointer
    A = _mat(orc, n)
    st, res, X, cnt = _cg(orc, A, n, 5, policy=0, max_iters=7)
    assert st == orc.E_NOT_CONVERGED and cnt.sum() == 0
