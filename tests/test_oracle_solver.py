"""Pins of the oracle's SpMV / RED-1 / CG against closed
forms, library routines and the paper's invariants (S§8(c) PIN-8..PIN-14)."""
import math

import numpy as np
import pytest

import gen


def _mat(orc, n, es, rs, kind="tea", k=1.0):
    if kind == "tea":
        v, c, r = gen.tealeaf_csr(n)
    else:
        v, c, r = gen.const_k_csr(n, k)
    A = orc.Matrix(v.numpy(), c.numpy().astype(np.uint32), r.numpy().astype(np.uint32), n * n, n * n, es, rs)
    assert A.encode() == orc.OK
    return A, v.numpy(), c.numpy(), r.numpy()


def _dense(v, c, N):
    D = np.zeros((N, N))
    for i in range(N):
        for k in range(5):
            D[i, c[5 * i + k]] += v[5 * i + k]
    return D


def _spmv(orc, A, x, scheme):
    N = A.nrows
    xin = orc.vec_encode(x, scheme)
    out = np.zeros(orc.vec_padded_len(N, scheme), dtype=np.uint64)
    cnt = orc.new_counts()
    orc.spmv(A, xin, N, scheme, out, N, cnt)
    return orc.vec_masked(out, N, scheme), cnt


@pytest.mark.parametrize("scheme", ["NONE", "SED", "SECDED64", "SECDED128", "CRC32C"])
def test_pin8_row_sums_are_one(orc, scheme):
    s = getattr(orc, scheme)
    A, *_ = _mat(orc, 32, orc.SECDED64 if s != orc.CRC32C else orc.CRC32C, s if s != orc.NONE else orc.NONE)
    y, cnt = _spmv(orc, A, np.ones(32 * 32), s)
    assert np.max(np.abs(y - 1.0)) < 1e-12
    assert cnt.sum() == 0


def test_pin9_const_k_eigenpairs(orc):
    """A = I + K L_Neumann: v_kl(i,j) = cos(pi k (i+1/2)/n) cos(pi l (j+1/2)/n),
    lambda = 1 + K(4 sin^2(pi k/2n) + 4 sin^2(pi l/2n))."""
    n, K = 16, 0.7
    A, *_ = _mat(orc, n, orc.SECDED64, orc.SECDED64, kind="const", k=K)
    ii = np.arange(n)
    for (kx, ly) in [(0, 0), (1, 0), (3, 5), (15, 15)]:
        v = np.outer(np.cos(np.pi * ly * (ii + 0.5) / n), np.cos(np.pi * kx * (ii + 0.5) / n)).ravel()
        lam = 1 + K * (4 * math.sin(math.pi * kx / (2 * n)) ** 2 + 4 * math.sin(math.pi * ly / (2 * n)) ** 2)
        y, _ = _spmv(orc, A, v, orc.NONE)
        assert np.max(np.abs(y - lam * v)) < 1e-12


def test_pin12_symmetry_and_spmv_vs_dense(orc):
    n = 12
    A, v, c, r = _mat(orc, n, orc.SECDED64, orc.SECDED64)
    D = _dense(v, c, n * n)
    assert np.array_equal(D, D.T)
    rng = np.random.default_rng(0)
    a = gen.uniform_pm1(n * n, seed=1)
    b = gen.uniform_pm1(n * n, seed=2)
    Aa, _ = _spmv(orc, A, a, orc.NONE)
    Ab, _ = _spmv(orc, A, b, orc.NONE)
    assert abs(a @ Ab - b @ Aa) < 1e-13 * n * n
    # vs dense matmul: |err_i| <= 5 eps sum_k |a_ik x_k| (fma chain of 5 terms)
    ref = D @ a
    bound = 6 * np.finfo(float).eps * (np.abs(D) @ np.abs(a))
    assert np.all(np.abs(Aa - ref) <= bound + 1e-300)
    del rng


def test_red1_properties(orc):
    """RED-1 is a fixed-order sum: within the recursive-summation error bound of
    the exact sum; a single nonzero term is returned exactly; subtree roots
    combined by the tree equal the global value (P-invariance)."""
    for n in [1, 31, 256, 257, 1000, 5000]:
        a = gen.uniform_pm1(n, seed=n)
        b = gen.uniform_pm1(n, seed=n + 1)
        d = orc.dot_red1(a, b)
        exact = math.fsum((a[i] * b[i] for i in range(n)))  # products exact enough vs bound
        bound = (n + 20) * np.finfo(float).eps * float(np.sum(np.abs(a * b)))
        assert abs(d - exact) <= bound
    z = np.zeros(777)
    z[500] = 3.0
    assert orc.dot_red1(z, z) == 9.0
    n = 256 * 16
    a = gen.uniform_pm1(n, seed=9)
    blocks = orc.red1_blocks(a, a)
    for P in [1, 2, 4, 8]:
        roots = [orc.tree_sum(blocks[r * 16 // P:(r + 1) * 16 // P]) for r in range(P)]
        assert orc.tree_sum(np.array(roots)) == orc.dot_red1(a, a)


def _solve(orc, n, scheme, tol=1e-10, max_iters=5000, es=None, rs=None, b=None, x0=None, policy=1):
    es = orc.SECDED64 if es is None else es
    rs = orc.SECDED64 if rs is None else rs
    if scheme == orc.CRC32C:
        es, rs = orc.CRC32C, orc.CRC32C
    if scheme == orc.NONE:
        es, rs = orc.NONE, orc.NONE
    A, v, c, r = _mat(orc, n, es, rs)
    N = n * n
    b = gen.tealeaf_rhs(n).numpy() if b is None else b
    x0 = b if x0 is None else x0
    B = orc.vec_encode(b, scheme)
    X = orc.vec_encode(x0, scheme)
    R = np.zeros_like(B)
    Pv = np.zeros_like(B)
    W = np.zeros_like(B)
    cnt = orc.new_counts()
    st, res = orc.cg_solve(A, B, X, R, Pv, W, scheme, tol, max_iters, policy, cnt)
    return st, res, orc.vec_masked(X, N, scheme), (v, c, r), cnt


def _numpy_cg(D, b, x0, tol):
    """Plain textbook CG in numpy (library matmul; independent of the oracle)."""
    x = x0.copy()
    r = b - D @ x
    p = r.copy()
    rr0 = rro = r @ r
    for k in range(1, 10000):
        w = D @ p
        a = rro / (p @ w)
        x = x + a * p
        r = r - a * w
        rrn = r @ r
        if math.sqrt(rrn) <= tol * math.sqrt(rr0):
            return x, k
        p = r + (rrn / rro) * p
        rro = rrn
    return x, -1


@pytest.mark.parametrize("n", [2, 4, 8])
def test_pin11_tiny_grids_vs_dense_solve(orc, n):
    for scheme in [orc.NONE, orc.SED, orc.SECDED64, orc.SECDED128, orc.CRC32C]:
        st, res, x, (v, c, r), _ = _solve(orc, n, scheme, tol=1e-13)
        D = _dense(v, c, n * n)
        b = gen.tealeaf_rhs(n).numpy()
        xs = np.linalg.solve(D, b)
        cond = np.linalg.cond(D)
        k = {orc.NONE: 0, orc.SED: 1, orc.SECDED64: 8, orc.SECDED128: 5, orc.CRC32C: 8}[scheme]
        tol = max(1e-13 * cond, 4 * 2.0 ** (k - 52))
        assert st == orc.OK
        assert np.linalg.norm(x - xs) <= tol * np.linalg.norm(xs) * 10


def test_iteration_counts_match_numpy_cg(orc):
    """Unprotected oracle CG and a numpy CG agree on the iteration count (+-1,
    rounding order differs) and the solution (S§8(d): 32^2 -> 20 iterations)."""
    n = 32
    st, res, x, (v, c, r), _ = _solve(orc, n, orc.NONE)
    D = _dense(v, c, n * n)
    b = gen.tealeaf_rhs(n).numpy()
    xn, kn = _numpy_cg(D, b, b.copy(), 1e-10)
    assert abs(res.iters - kn) <= 1
    assert np.linalg.norm(x - xn) <= 1e-9 * np.linalg.norm(xn)


def test_pin10_krylov_iteration_counts(orc):
    """b = one eigenvector -> 1 iteration; m distinct eigencomponents -> m."""
    n, K = 16, 0.7
    ii = np.arange(n)
    vecs = []
    for (kx, ly) in [(1, 0), (3, 5), (7, 2)]:
        vecs.append(np.outer(np.cos(np.pi * ly * (ii + 0.5) / n), np.cos(np.pi * kx * (ii + 0.5) / n)).ravel())
    v, c, r = gen.const_k_csr(n, K)
    for m in [1, 2, 3]:
        b = sum(vecs[:m])
        A = orc.Matrix(v.numpy(), c.numpy().astype(np.uint32), r.numpy().astype(np.uint32), n * n, n * n,
                       orc.NONE, orc.NONE)
        A.encode()
        B = orc.vec_encode(b, orc.NONE)
        X = orc.vec_encode(np.zeros(n * n), orc.NONE)
        R, P, W = (np.zeros_like(B) for _ in range(3))
        st, res = orc.cg_solve(A, B, X, R, P, W, orc.NONE, 1e-10, 50, 1, None)
        assert st == orc.OK and res.iters == m


def test_pin13_masked_vs_unmasked(orc):
    """with ECC bits in the mantissa LSBs the solution norm stays within
    2.0e-11 % of the unprotected answer and iterations grow by < 1%."""
    n = 64
    st0, r0, x0, *_ = _solve(orc, n, orc.NONE)
    for scheme in [orc.SECDED64, orc.SECDED128, orc.CRC32C]:
        st, r1, x1, *_ = _solve(orc, n, scheme)
        assert st == orc.OK
        dev = abs(np.linalg.norm(x1) - np.linalg.norm(x0)) / np.linalg.norm(x0)
        assert dev <= 2.0e-13
        assert r1.iters <= math.floor(r0.iters * 1.01) + 0  # < 1% more


def test_pin14_injection_accounting(orc):
    """k single flips in distinct SECDED codewords of read-before-write targets
    are all corrected exactly once."""
    n = 16
    N = n * n
    A, *_ = _mat(orc, n, orc.SECDED64, orc.SECDED64)
    rng = np.random.default_rng(42)
    clean = A.val.copy(), A.col.copy(), A.rowptr.copy()
    elems = rng.choice(A.nnz, 20, replace=False)
    for e in elems:
        bit = int(rng.integers(0, 96))
        if bit < 64:
            A.val[e] ^= np.uint64(1 << bit)
        else:
            A.col[e] ^= np.uint32(1 << (bit - 64))
    groups = rng.choice(len(A.rowptr) // 2, 10, replace=False)
    for g in groups:
        bit = int(rng.integers(0, 64))
        A.rowptr[2 * g + bit // 32] ^= np.uint32(1 << (bit % 32))
    x = orc.vec_encode(gen.uniform_pm1(N, seed=3), orc.SECDED64)
    xs = rng.choice(N, 15, replace=False)
    for i in xs:
        x[i] ^= np.uint64(1 << int(rng.integers(0, 64)))
    out = np.zeros(N, dtype=np.uint64)
    cnt = orc.new_counts()
    d = orc.spmv(A, x, N, orc.SECDED64, out, N, cnt)
    assert d == 0
    assert cnt[orc.ELEM, orc.SECDED64].tolist() == [20, 20, 0, 0]
    assert cnt[orc.ROWPTR, orc.SECDED64].tolist() == [10, 10, 0, 0]
    assert cnt[orc.VEC, orc.SECDED64].tolist() == [15, 15, 0, 0]
    # scrubbed: the stored matrix is back to the clean encoding, a second pass counts nothing
    assert np.array_equal(A.val, clean[0]) and np.array_equal(A.col, clean[1]) and np.array_equal(A.rowptr, clean[2])
    cnt2 = orc.new_counts()
    orc.spmv(A, x, N, orc.SECDED64, out, N, cnt2)
    assert cnt2.sum() == 0


def test_double_flip_is_due_and_abort_policy(orc):
    n = 8
    N = n * n
    A, *_ = _mat(orc, n, orc.SECDED64, orc.SECDED64)
    A.val[17] ^= np.uint64(0b11)
    b = gen.tealeaf_rhs(n).numpy()
    B = orc.vec_encode(b, orc.SECDED64)
    X = B.copy()
    R, P, W = (np.zeros_like(B) for _ in range(3))
    cnt = orc.new_counts()
    st, res = orc.cg_solve(A, B, X, R, P, W, orc.SECDED64, 1e-10, 100, 0, cnt)
    assert st == orc.E_DUE and res.iters == 0
    assert cnt[orc.ELEM, orc.SECDED64, orc.UNC] == 1


def test_range_violation_skips_row(orc):
    """A rowptr corrupted past ECC (scheme NONE on elements, SED on rowptr with
    an even flip count) is caught by the range check."""
    n = 4
    A, *_ = _mat(orc, n, orc.NONE, orc.SED)
    A.rowptr[3] ^= np.uint32(0b11 << 20)          # 2 flips: parity still even, value > nnz
    x = orc.vec_encode(np.ones(n * n), orc.NONE)
    out = np.zeros(n * n, dtype=np.uint64)
    cnt = orc.new_counts()
    d = orc.spmv(A, x, n * n, orc.NONE, out, n * n, cnt)
    assert d == 2 and cnt[orc.ROWPTR, orc.SED, orc.RANGE] == 2   # rows 2 and 3 use entry 3
    y = out.view(np.float64)
    assert y[2] == 0.0 and y[3] == 0.0
    assert abs(y[4] - 1.0) < 1e-12
