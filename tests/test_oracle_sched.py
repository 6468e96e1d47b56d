"""Pins for the oracle's O10 fault schedule (S§8(c) O10; PAPER.md P:82-97,
P:230-238): fault (k, target, word, bit) XOR-ed into the stored bits before
init (k = 0) or before iteration k's SpMV.

What fixes the expected values independently of the oracle's code:
* the unfused CG sequence's read-before-write structure (O8 / O9): which
  targets are read after a fault at iteration k and which are overwritten
  first (w always; p and r at k = 0) or never read again (b at k >= 1);
* SECDED corrects every single flip before the value is used, so a
  schedule of single flips leaves every iterate bit-identical to the
  fault-free solve;
* a same-word double flip is a DUE: under policy abort the solve
  stops with ABFT_E_DUE after exactly the iteration that first reads it."""
import numpy as np
import pytest

import gen
import oracle as orc

N_GRID = 32


def _problem(S=orc.SECDED64, n=N_GRID):
    N = n * n
    v, c, r = gen.tealeaf_csr(n)
    A = orc.Matrix(v.numpy(), c.numpy().astype(np.uint32), r.numpy().astype(np.uint32), N, N, orc.SECDED64,
                   orc.SECDED64)
    assert A.encode() == 0
    b = orc.vec_encode(gen.tealeaf_rhs(n).numpy(), S)
    return A, b, N


def _solve(S, faults, policy=1, max_iters=200):
    A, b, N = _problem(S)
    x = b.copy()
    r, p, w = (np.zeros_like(b) for _ in range(3))
    cnt = orc.new_counts()
    st, res = orc.cg_solve_sched(A, b, x, r, p, w, S, 1e-10, max_iters, policy, cnt,
                                 faults=orc.fault_schedule(faults) if faults else None)
    return st, res, x[:N], cnt


def _read_before_write(k, t):
    """Is a fault injected before iteration k (0 = before init) into target t
    read by the unfused sequence before the target is overwritten?"""
    if t in (orc.F_VAL, orc.F_COL, orc.F_ROWPTR):
        return True                       # every SpMV reads the matrix
    if t == orc.F_B:
        return k == 0                     # b is read only by init
    if t == orc.F_X:
        return True                       # init SpMV (k = 0) / calc_ur of iteration k
    if t in (orc.F_R, orc.F_P):
        return k >= 1                     # init writes r and p before reading them
    return False                          # w: every SpMV overwrites it before calc_ur reads it


def test_single_flips_leave_the_solve_bit_identical():
    S = orc.SECDED64
    st0, res0, x0, c0 = _solve(S, [])
    assert st0 == 0 and not c0.any()
    N = N_GRID * N_GRID
    rng = np.random.default_rng(10)
    faults, expect = [], 0
    used = set()
    for t in range(8):
        for _ in range(6):
            k = int(rng.integers(0, 12))
            if t == orc.F_ROWPTR:
                g = int(rng.integers(0, N // 2))
                key, word, bit = (t, g), 2 * g + int(rng.integers(2)), int(rng.integers(32))
            elif t in (orc.F_VAL, orc.F_COL):
                e = int(rng.integers(0, 5 * N))
                key, word, bit = ("el", e), e, int(rng.integers(64 if t == orc.F_VAL else 32))
            else:
                i = int(rng.integers(0, N))
                key, word, bit = (t, i), i, int(rng.integers(64))
            if key in used:
                continue
            used.add(key)
            faults.append((k, t, word, bit))
            expect += _read_before_write(k, t)
    st, res, x, cnt = _solve(S, faults)
    assert st == 0 and res.iters == res0.iters and res.rrn == res0.rrn
    assert np.array_equal(x, x0)
    total = cnt[:, :, orc.COR].sum()
    assert total == expect and cnt[:, :, orc.UNC].sum() == 0 and cnt[:, :, orc.DET].sum() == expect


# logical reads of the DUE word in iteration k before it is overwritten (O9: a
# DUE is counted at every logical read, never scrubbed): p is read by the SpMV,
# calc_ur and calc_p (which rewrites it); x and r by calc_ur (which rewrites
# them); a matrix element once by the SpMV
@pytest.mark.parametrize("t,k,dues", [(orc.F_P, 5, 3), (orc.F_X, 4, 1), (orc.F_R, 7, 1),
                                      (orc.F_VAL, 3, 1), (orc.F_W, 5, 0), (orc.F_B, 3, 0),
                                      (orc.F_P, 0, 0), (orc.F_R, 0, 0)])
def test_double_flip_abort_exactly_at_its_first_read(t, k, dues):
    S = orc.SECDED64
    _, res0, x0, _ = _solve(S, [], policy=0)
    word = 37 if t != orc.F_VAL else 5 * 37 + 2
    faults = [(k, t, word, 11), (k, t, word, 50)]
    st, res, x, cnt = _solve(S, faults, policy=0)
    if dues:
        assert st == orc.E_DUE and res.iters == k
        assert cnt[:, :, orc.UNC].sum() == dues and cnt[:, :, orc.COR].sum() == 0
    else:   # overwritten before any read (w; p / r before init) or never read again (b after init)
        assert st == 0 and res.iters == res0.iters and np.array_equal(x, x0)
        assert not cnt.any()


def test_faults_after_the_last_iteration_are_never_applied():
    S = orc.SECDED64
    st0, res0, x0, _ = _solve(S, [])
    faults = [(res0.iters + 1, orc.F_P, 3, 5), (res0.iters + 7, orc.F_VAL, 10, 60)]
    st, res, x, cnt = _solve(S, faults)
    assert st == 0 and res.iters == res0.iters and np.array_equal(x, x0) and not cnt.any()


def test_sed_vector_flip_mid_solve_is_a_detected_due():
    """V-SED: a single flip is detected but not correctable."""
    S = orc.SED
    faults = [(6, orc.F_X, 100, 40)]
    st, res, x, cnt = _solve(S, faults, policy=1)
    assert cnt[orc.VEC, S, orc.DET] == 1 and cnt[orc.VEC, S, orc.UNC] == 1
    st, res, x, cnt = _solve(S, faults, policy=0)
    assert st == orc.E_DUE and res.iters == 6
