"""Oracle on general (non-stencil) sparse SPD matrices, G-SPD (S§8(f) f4;
gen/spd.py): pinned against a dense direct solve (numpy.linalg.solve) and a
dense matrix-vector product, i.e. against library routines, not the oracle."""
import numpy as np
import pytest

import gen
import oracle as orc


def _dense(v, c, r, n):
    A = np.zeros((n, n))
    for i in range(n):
        for j in range(r[i], r[i + 1]):
            A[i, c[j]] += v[j]
    return A


@pytest.mark.parametrize("scheme", [orc.NONE, orc.SED, orc.SECDED64, orc.CRC32C])
def test_spd_spmv_matches_dense(scheme):
    n = 400
    v, c, r = gen.random_spd_csr(n, 4, 5)
    A = orc.Matrix(v, c, r, n, n, scheme if scheme != orc.SED else orc.SED, scheme)
    assert A.encode() == 0
    x = orc.vec_encode(gen.uniform_pm1(n, 6), scheme)
    y = np.zeros_like(x)
    orc.spmv(A, x, n, scheme, y, n)
    xm = orc.vec_masked(x, n, scheme)
    ym = orc.vec_masked(y, n, scheme)
    ref = _dense(v, c, r, n) @ xm
    k = {orc.NONE: 0, orc.SED: 1, orc.SECDED64: 8, orc.CRC32C: 8}[scheme]
    # one rounding of the result to 2^k ulps plus the reordering of <= 17 terms
    tol = (2.0 ** (k - 52) + 40 * 2.0 ** -53) * (np.abs(_dense(v, c, r, n)) @ np.abs(xm)) + 1e-300
    assert np.all(np.abs(ym - ref) <= tol)


@pytest.mark.parametrize("scheme", [orc.NONE, orc.SECDED64])
def test_spd_cg_matches_dense_solve(scheme):
    n = 300
    v, c, r = gen.random_spd_csr(n, 5, 9)
    A = orc.Matrix(v, c, r, n, n, scheme, scheme)
    assert A.encode() == 0
    b = gen.uniform_pm1(n, 10)
    B = orc.vec_encode(b, scheme)
    X = B.copy()
    R, P, W = (np.zeros_like(B) for _ in range(3))
    st, res = orc.cg_solve(A, B, X, R, P, W, scheme, 1e-12, 2000, 1, None)
    assert st == orc.OK and res.iters > 5
    D = _dense(v, c, r, n)
    xs = np.linalg.solve(D, orc.vec_masked(B, n, scheme))
    xm = orc.vec_masked(X, n, scheme)
    cond = np.linalg.cond(D)
    assert np.linalg.norm(xm - xs) <= 1e-12 * cond * np.linalg.norm(xs) * 50 + 2.0 ** -44 * np.linalg.norm(xs)
