"""Pins of the oracle's protected PPCG (polynomially preconditioned CG, S§8(f)
f4, reading R34) — fixed by:

* dense direct solves (numpy.linalg.solve);
* a plain numpy transcription of preconditioned CG whose preconditioner is the
  same m-step Chebyshev polynomial (library matmul): equal iteration counts
  (+-1) and solutions within tolerance;
* preconditioning theory: with a good polynomial the outer iteration count
  drops well below plain CG's;
* SECDED semantics: single flips in b, x0 and the matrix are corrected before
  use, so the solve is bit-identical to the fault-free one."""
import math

import numpy as np
import pytest

import gen
import oracle as orc


def _dense(v, c, N):
    D = np.zeros((N, N))
    for i in range(N):
        for k in range(5):
            D[i, c[5 * i + k]] += v[5 * i + k]
    return D


def _bounds(n):
    v, c, r = gen.tealeaf_csr(n)
    return 0.95, float(np.abs(v.numpy()).reshape(-1, 5).sum(axis=1).max())   # lambda_min = 1 (PIN-8), Gershgorin


def ppcg(n, S, inner, tol=1e-10, max_iters=2000, flips=None):
    v, c, r = gen.tealeaf_csr(n)
    N = n * n
    es = orc.NONE if S == orc.NONE else orc.SECDED64
    A = orc.Matrix(v.numpy(), c.numpy().astype(np.uint32), r.numpy().astype(np.uint32), N, N, es, es)
    assert A.encode() == 0
    b = gen.tealeaf_rhs(n).numpy()
    B, X = orc.vec_encode(b, S), orc.vec_encode(b, S)
    if flips:
        flips(A, B, X)
    R, P, W, Z, RI, PI = (np.zeros_like(B) for _ in range(6))
    lo, hi = _bounds(n)
    cnt = orc.new_counts()
    st, res = orc.ppcg_solve(A, B, X, R, P, W, Z, RI, PI, S, lo, hi, inner, tol, max_iters, 1, cnt)
    return st, res, X, orc.vec_masked(X, N, S), cnt, (v.numpy(), c.numpy(), b)


def numpy_ppcg(D, b, x0, lo, hi, m, tol):
    theta, delta = (hi + lo) / 2, (hi - lo) / 2
    sigma = theta / delta

    def prec(r):
        rho = 1 / sigma
        rin = r.copy()
        pin = rin / theta
        z = pin.copy()
        for _ in range(1, m):
            rn = 1 / (2 * sigma - rho)
            a, bb = rn * rho, 2 * rn / delta
            rho = rn
            rin = r - D @ z
            pin = a * pin + bb * rin
            z = z + pin
        return z

    x = x0.copy()
    r = b - D @ x
    rr0 = r @ r
    z = prec(r)
    rz = r @ z
    p = z.copy()
    for k in range(1, 10000):
        w = D @ p
        a = rz / (p @ w)
        x = x + a * p
        r = r - a * w
        if math.sqrt(r @ r) <= tol * math.sqrt(rr0):
            return x, k
        z = prec(r)
        rzn = r @ z
        p = z + (rzn / rz) * p
        rz = rzn
    return x, -1


@pytest.mark.parametrize("inner", [2, 5])
def test_ppcg_matches_numpy_and_dense_solve(inner):
    n = 32
    st, res, _, x, _, (v, c, b) = ppcg(n, orc.NONE, inner)
    D = _dense(v, c, n * n)
    lo, hi = _bounds(n)
    xn, kn = numpy_ppcg(D, b, b.copy(), lo, hi, inner, 1e-10)
    assert st == orc.OK and abs(res.iters - kn) <= 1
    xs = np.linalg.solve(D, b)
    assert np.linalg.norm(x - xs) <= 1e-8 * np.linalg.norm(xs)
    assert np.linalg.norm(x - xn) <= 1e-9 * np.linalg.norm(xn)


def test_ppcg_fewer_outer_iterations_than_cg():
    n = 64
    st, res, *_ = ppcg(n, orc.SECDED64, 6)
    v, c, r = gen.tealeaf_csr(n)
    N = n * n
    A = orc.Matrix(v.numpy(), c.numpy().astype(np.uint32), r.numpy().astype(np.uint32), N, N, orc.SECDED64,
                   orc.SECDED64)
    A.encode()
    B = orc.vec_encode(gen.tealeaf_rhs(n).numpy(), orc.SECDED64)
    X = B.copy()
    R, P, W = (np.zeros_like(B) for _ in range(3))
    st2, res2 = orc.cg_solve(A, B, X, R, P, W, orc.SECDED64, 1e-10, 5000, 1, None)
    assert st == st2 == orc.OK
    assert res.iters * 2 <= res2.iters


def test_ppcg_single_flips_bit_identical():
    n = 32
    N = n * n
    st0, res0, X0, *_ = ppcg(n, orc.SECDED64, 4)
    rng = np.random.default_rng(6)

    def flips(A, B, X):
        for i in rng.choice(N, 4, replace=False):
            B[i] ^= np.uint64(1 << int(rng.integers(64)))
        for i in rng.choice(N, 4, replace=False):
            X[i] ^= np.uint64(1 << int(rng.integers(64)))
        for e in rng.choice(5 * N, 5, replace=False):
            A.val[e] ^= np.uint64(1 << int(rng.integers(64)))

    st, res, X, _, cnt, _ = ppcg(n, orc.SECDED64, 4, flips=flips)
    assert st == st0 and res.iters == res0.iters and np.array_equal(X, X0)
    assert cnt[:, :, orc.COR].sum() == 13 and cnt[:, :, orc.UNC].sum() == 0
