"""Pins of the oracle's single-reduction CG (Chronopoulos-Gear, S§8(f) f3;
DESIGN.md §4.1, reading R28) — fixed by things other than the oracle itself:

* dense direct solves (numpy.linalg.solve) on 2^2 .. 8^2 grids, every scheme;
* Krylov theory: b with m distinct eigencomponents of a constant-K matrix
  converges in exactly m iterations (closed-form eigenvectors, PIN-9/10);
* a plain numpy transcription of the textbook Chronopoulos-Gear recurrence
  (library matmul) reaches the same iteration count and solution on G-TEA;
* in exact arithmetic single-reduction CG generates the same iterates as
  standard CG: equal iteration counts (+-1) and solutions within tolerance;
* O9/O10 accounting: single flips are corrected before use (the solve is
  bit-identical to the fault-free one), a DUE in p or s aborts exactly at the
  iteration that reads it."""
import math

import numpy as np
import pytest

import gen
import oracle as orc


def _problem(n, scheme, kind="tea", K=1.0):
    if kind == "tea":
        v, c, r = gen.tealeaf_csr(n)
    else:
        v, c, r = gen.const_k_csr(n, K)
    es = orc.NONE if scheme == orc.NONE else (orc.CRC32C if scheme == orc.CRC32C else orc.SECDED64)
    rs = es
    A = orc.Matrix(v.numpy(), c.numpy().astype(np.uint32), r.numpy().astype(np.uint32), n * n, n * n, es, rs)
    assert A.encode() == orc.OK
    return A, v.numpy(), c.numpy()


def _dense(v, c, N):
    D = np.zeros((N, N))
    for i in range(N):
        for k in range(5):
            D[i, c[5 * i + k]] += v[5 * i + k]
    return D


def sr_solve(n, scheme, b=None, x0=None, tol=1e-10, max_iters=5000, kind="tea", K=1.0, faults=None, policy=1):
    A, v, c = _problem(n, scheme, kind, K)
    N = n * n
    b = gen.tealeaf_rhs(n).numpy() if b is None else b
    x0 = b if x0 is None else x0
    B, X = orc.vec_encode(b, scheme), orc.vec_encode(x0, scheme)
    R, P, W, S = (np.zeros_like(B) for _ in range(4))
    cnt = orc.new_counts()
    st, res = orc.cg_solve_sr(A, B, X, R, P, W, S, scheme, tol, max_iters, policy, cnt,
                              faults=orc.fault_schedule(faults) if faults else None)
    return st, res, X, orc.vec_masked(X, N, scheme), cnt, (v, c)


def std_solve(n, scheme, tol=1e-10):
    A, v, c = _problem(n, scheme)
    b = gen.tealeaf_rhs(n).numpy()
    B = orc.vec_encode(b, scheme)
    X = B.copy()
    R, P, W = (np.zeros_like(B) for _ in range(3))
    st, res = orc.cg_solve(A, B, X, R, P, W, scheme, tol, 5000, 1, None)
    return st, res, orc.vec_masked(X, n * n, scheme)


def numpy_cg_cg(D, b, x0, tol):
    """Textbook Chronopoulos-Gear CG (numpy matmul)."""
    x = x0.copy()
    r = b - D @ x
    w = D @ r
    g, d = r @ r, w @ r
    rr0 = g
    a, beta = g / d, 0.0
    p = np.zeros_like(b)
    s = np.zeros_like(b)
    for k in range(1, 10000):
        p = r + beta * p
        s = w + beta * s
        x = x + a * p
        r = r - a * s
        w = D @ r
        gn, d = r @ r, w @ r
        if math.sqrt(gn) <= tol * math.sqrt(rr0):
            return x, k
        beta = gn / g
        a = gn / (d - beta * gn / a)
        g = gn
    return x, -1


@pytest.mark.parametrize("n", [2, 4, 8])
def test_sr_tiny_grids_vs_dense_solve(n):
    for scheme in [orc.NONE, orc.SED, orc.SECDED64, orc.SECDED128, orc.CRC32C]:
        st, res, _, x, _, (v, c) = sr_solve(n, scheme, tol=1e-13)
        D = _dense(v, c, n * n)
        b = gen.tealeaf_rhs(n).numpy()
        xs = np.linalg.solve(D, b)
        k = {orc.NONE: 0, orc.SED: 1, orc.SECDED64: 8, orc.SECDED128: 5, orc.CRC32C: 8}[scheme]
        tol = max(1e-13 * np.linalg.cond(D), 4 * 2.0 ** (k - 52))
        assert st == orc.OK
        assert np.linalg.norm(x - xs) <= tol * np.linalg.norm(xs) * 10


def test_sr_krylov_iteration_counts():
    n, K = 16, 0.7
    ii = np.arange(n)
    vecs = [np.outer(np.cos(np.pi * ly * (ii + 0.5) / n), np.cos(np.pi * kx * (ii + 0.5) / n)).ravel()
            for (kx, ly) in [(1, 0), (3, 5), (7, 2)]]
    for m in [1, 2, 3]:
        st, res, *_ = sr_solve(n, orc.NONE, b=sum(vecs[:m]), x0=np.zeros(n * n), kind="const", K=K, max_iters=50)
        assert st == orc.OK and res.iters == m


@pytest.mark.parametrize("n", [32, 64])
def test_sr_matches_numpy_recurrence_and_standard_cg(n):
    st, res, _, x, _, (v, c) = sr_solve(n, orc.NONE)
    D = _dense(v, c, n * n)
    b = gen.tealeaf_rhs(n).numpy()
    xn, kn = numpy_cg_cg(D, b, b.copy(), 1e-10)
    assert st == orc.OK and abs(res.iters - kn) <= 1
    assert np.linalg.norm(x - xn) <= 1e-9 * np.linalg.norm(xn)
    st2, res2, x2 = std_solve(n, orc.NONE)
    assert abs(res.iters - res2.iters) <= 1
    assert np.linalg.norm(x - x2) <= 1e-9 * np.linalg.norm(x2)
    # protected (config-2 schemes): the masked-vs-unmasked invariant of P:452-457
    st3, res3, _, x3, _, _ = sr_solve(n, orc.SECDED64)
    assert st3 == orc.OK and res3.iters <= math.floor(res.iters * 1.01) + 1
    assert abs(np.linalg.norm(x3) - np.linalg.norm(x)) / np.linalg.norm(x) <= 2.0e-13


def test_sr_single_flips_leave_the_solve_bit_identical():
    n = 32
    N = n * n
    st0, res0, X0, *_ = sr_solve(n, orc.SECDED64)
    rng = np.random.default_rng(3)
    faults, used = [], set()
    expect = 0
    for t in [orc.F_VAL, orc.F_COL, orc.F_X, orc.F_P, orc.F_R, orc.F_W, orc.F_S]:
        for _ in range(4):
            k = int(rng.integers(1, 10))
            w = int(rng.integers(5 * N if t in (orc.F_VAL, orc.F_COL) else N))
            key = ("el", w) if t in (orc.F_VAL, orc.F_COL) else (t, w)
            if key in used:
                continue
            used.add(key)
            faults.append((k, t, w, int(rng.integers(32 if t == orc.F_COL else 64))))
            expect += 1   # at the start of iteration k every target is read before it is rewritten
    st, res, X, _, cnt, _ = sr_solve(n, orc.SECDED64, faults=faults)
    assert st == orc.OK and res.iters == res0.iters and np.array_equal(X, X0)
    assert cnt[:, :, orc.COR].sum() == expect and cnt[:, :, orc.UNC].sum() == 0


@pytest.mark.parametrize("t", [orc.F_P, orc.F_S, orc.F_X, orc.F_R, orc.F_W])
def test_sr_due_aborts_at_its_iteration(t):
    """A same-word double flip (DUE) at the start of iteration 6: calc_sr reads
    x, p, s, r, w once each and rewrites p, s, x, r; the iteration's SpMV reads
    the NEW r and overwrites w, so the DUE is counted exactly once (O9), and
    policy abort stops after iteration 6 with ABFT_E_DUE."""
    n = 32
    st, res, _, _, cnt, _ = sr_solve(n, orc.SECDED64, faults=[(6, t, 77, 9), (6, t, 77, 40)], policy=0)
    assert st == orc.E_DUE and res.iters == 6
    assert cnt[:, :, orc.UNC].sum() == 1
