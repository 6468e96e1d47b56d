"""Pins of the oracle's protected Chebyshev iteration and TeaLeaf's spectrum
estimate (S§8(f) f4, readings R32/R33) — fixed by:

* closed forms: the constant-K matrix A = I + K L_Neumann has the spectrum
  [1, 1 + 8K sin^2(pi (n-1) / 2n)] (PIN-9); with exactly those bounds the
  Chebyshev residual after k steps stays under the textbook bound
  2 c^k / (1 + c^2k) (c = (sqrt(kappa)-1)/(sqrt(kappa)+1)) and the converged
  answer equals numpy.linalg.solve;
* the Lanczos interval from CG's step coefficients lies inside the true
  spectrum (numpy.linalg.eigvalsh of the dense matrix) and its upper end is
  within 5 % of lambda_max after 30 CG steps;
* SECDED semantics: single flips in b, u0 and the matrix are corrected before
  use, so the solve is bit-identical to the fault-free one."""
import math

import numpy as np
import pytest

import gen
import oracle as orc


def _mat(n, kind="tea", K=1.0, S=orc.SECDED64):
    v, c, r = gen.tealeaf_csr(n) if kind == "tea" else gen.const_k_csr(n, K)
    es = orc.NONE if S == orc.NONE else orc.SECDED64
    A = orc.Matrix(v.numpy(), c.numpy().astype(np.uint32), r.numpy().astype(np.uint32), n * n, n * n, es, es)
    assert A.encode() == orc.OK
    return A, v.numpy(), c.numpy()


def _dense(v, c, N):
    D = np.zeros((N, N))
    for i in range(N):
        for k in range(5):
            D[i, c[5 * i + k]] += v[5 * i + k]
    return D


def cheby(n, S, lo, hi, b, u0, tol=1e-10, max_iters=5000, kind="tea", K=1.0, flips=None):
    A, v, c = _mat(n, kind, K, S)
    B, U = orc.vec_encode(b, S), orc.vec_encode(u0, S)
    if flips:
        flips(A, B, U)
    R, P, W = (np.zeros_like(B) for _ in range(3))
    cnt = orc.new_counts()
    st, res = orc.cheby_solve(A, B, U, R, P, W, S, lo, hi, tol, max_iters, 1, cnt)
    return st, res, U, orc.vec_masked(U, n * n, S), cnt, (v, c)


def test_cheby_exact_bounds_rate_and_solution():
    n, K = 16, 0.7
    N = n * n
    lmin, lmax = 1.0, 1.0 + 8 * K * math.sin(math.pi * (n - 1) / (2 * n)) ** 2
    kappa = lmax / lmin
    cfac = (math.sqrt(kappa) - 1) / (math.sqrt(kappa) + 1)
    b = gen.uniform_pm1(N, 3)
    u0 = np.zeros(N)
    rr0 = None
    for k in (5, 10, 20):
        st, res, _, _, _, _ = cheby(n, orc.NONE, lmin, lmax, b, u0, tol=0.0, max_iters=k, kind="const", K=K)
        rr0 = res.rr0
        # residual of u_{k-1} (the residual is computed before the update of step k)
        bound = 2 * cfac ** (k - 1) / (1 + cfac ** (2 * (k - 1)))
        assert math.sqrt(res.rrn) <= 1.0001 * bound * math.sqrt(rr0)
    st, res, _, u, _, (v, c) = cheby(n, orc.NONE, lmin, lmax, b, u0, tol=1e-12, kind="const", K=K)
    assert st == orc.OK
    xs = np.linalg.solve(_dense(v, c, N), b)
    assert np.linalg.norm(u - xs) <= 1e-10 * np.linalg.norm(xs)


def test_lanczos_bounds_inside_the_spectrum():
    n = 32
    N = n * n
    A, v, c = _mat(n, S=orc.NONE)
    ev = np.linalg.eigvalsh(_dense(v, c, N))
    b = gen.tealeaf_rhs(n).numpy()
    B = orc.vec_encode(b, orc.NONE)
    X = B.copy()
    R, P, W = (np.zeros_like(B) for _ in range(3))
    st, res, al, bl = orc.cg_solve_log(A, B, X, R, P, W, orc.NONE, 0.0, 30, 1, None)
    assert res.iters == 30 and len(al) == 30 and len(bl) == 29
    lo, hi = orc.lanczos_bounds(al, bl)
    assert ev[0] * (1 - 1e-12) <= lo and hi <= ev[-1] * (1 + 1e-12)
    assert hi >= 0.95 * ev[-1]   # (hence TeaLeaf's safety margin on eigmax)


@pytest.mark.parametrize("S", [orc.NONE, orc.SECDED64, orc.SED])
def test_tealeaf_cheby_with_lanczos_bound_matches_dense_solve(S):
    """TeaLeaf-style bounds: lambda_max from 30 CG steps' Lanczos data with a
    5 % margin, lambda_min = 1 (A = I + weighted graph Laplacian, A 1 = 1, PIN-8)
    with a 5 % margin; from u0 = b the iteration converges to the dense solve."""
    n = 32
    N = n * n
    A, v, c = _mat(n, S=S)
    b = gen.tealeaf_rhs(n).numpy()
    B = orc.vec_encode(b, S)
    X = B.copy()
    R, P, W = (np.zeros_like(B) for _ in range(3))
    st, res, al, bl = orc.cg_solve_log(A, B, X, R, P, W, S, 0.0, 30, 1, None)
    lo, hi = orc.lanczos_bounds(al, bl)
    st, res, _, u, _, (v, c) = cheby(n, S, 0.95, 1.05 * hi, b, b, tol=1e-10)
    assert st == orc.OK and res.iters > 0
    xs = np.linalg.solve(_dense(v, c, N), b)
    assert np.linalg.norm(u - xs) <= 1e-8 * np.linalg.norm(xs)


def test_cheby_single_flips_bit_identical():
    n = 32
    N = n * n
    b = gen.tealeaf_rhs(n).numpy()
    st0, res0, U0, *_ = cheby(n, orc.SECDED64, 0.9, 3.0, b, b)
    rng = np.random.default_rng(4)

    def flips(A, B, U):
        for i in rng.choice(N, 5, replace=False):
            B[i] ^= np.uint64(1 << int(rng.integers(64)))
        for i in rng.choice(N, 5, replace=False):
            U[i] ^= np.uint64(1 << int(rng.integers(64)))
        for e in rng.choice(5 * N, 6, replace=False):
            A.val[e] ^= np.uint64(1 << int(rng.integers(64)))

    st, res, U, _, cnt, _ = cheby(n, orc.SECDED64, 0.9, 3.0, b, b, flips=flips)
    assert st == st0 and res.iters == res0.iters and np.array_equal(U, U0)
    assert cnt[:, :, orc.COR].sum() == 16 and cnt[:, :, orc.UNC].sum() == 0
