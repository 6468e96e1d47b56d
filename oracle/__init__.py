"""ctypes wrapper of the CPU oracle (oracle/oracle.c).

TEST INFRASTRUCTURE ONLY: imported by tests/, __graft_entry__.smoke() and the
cpu_baseline / --impl reference legs of bench.py, never by the product package.
Arrays are numpy; f64 vectors are passed as their uint64 bit patterns so the
ECC bits in the mantissa survive the round trip.
"""
from __future__ import annotations

import ctypes as C
import os
import subprocess

import numpy as np

_HERE = os.path.dirname(os.path.abspath(__file__))
_SO = os.path.join(_HERE, "liboracle.so")
_SRC = os.path.join(_HERE, "oracle.c")

NONE, SED, SECDED64, SECDED128, CRC32C = range(5)
ELEM, ROWPTR, VEC = range(3)
DET, COR, UNC, RANGE = range(4)
CLEAN, CORRECTED, DUE = range(3)
I_E_SECDED, I_V_SECDED64, I_R_SECDED64, I_R_SECDED128, I_V_SECDED128 = range(5)
OK, E_INVALID, E_RANGE, E_SHAPE, E_DUE, E_NOT_CONVERGED = 0, -1, -2, -3, -4, -5


def build(force: bool = False) -> str:
    """Compile liboracle.so with gcc (plain C, no SIMD/OpenMP, no FP contraction)."""
    if force or not os.path.exists(_SO) or os.path.getmtime(_SO) < os.path.getmtime(_SRC):
        subprocess.check_call(["gcc", "-O2", "-std=c11", "-ffp-contract=off", "-shared", "-fPIC",
                               "-o", _SO, _SRC, "-lm"])
    return _SO


_lib = None


def lib():
    global _lib
    if _lib is None:
        _lib = C.CDLL(build())
        L = _lib
        u64p, u32p, dp = C.POINTER(C.c_uint64), C.POINTER(C.c_uint32), C.POINTER(C.c_double)
        L.or_crc32c.restype = C.c_uint32
        L.or_crc32c.argtypes = [C.c_char_p, C.c_size_t]
        L.or_inst_nbits.argtypes = [C.c_int]
        L.or_inst_column.argtypes = [C.c_int, C.c_int]
        L.or_inst_reserved.argtypes = [C.c_int, C.c_int]
        L.or_secded_check.argtypes = [C.c_int, u32p, C.POINTER(C.c_int)]
        L.or_secded_encode.argtypes = [C.c_int, u32p]
        L.or_secded_syndrome.argtypes = [C.c_int, u32p, C.POINTER(C.c_int), C.POINTER(C.c_int)]
        L.or_vec_padded_len.restype = C.c_int64
        L.or_vec_padded_len.argtypes = [C.c_int64, C.c_int]
        L.or_rowptr_padded_len.restype = C.c_int64
        L.or_rowptr_padded_len.argtypes = [C.c_int64, C.c_int]
        L.or_vec_encode.argtypes = [u64p, C.c_int64, C.c_int]
        L.or_vec_check.restype = C.c_int64
        L.or_vec_check.argtypes = [u64p, C.c_int64, C.c_int, dp, C.c_void_p, C.c_int]
        L.or_csr_encode.argtypes = [u64p, u32p, u32p, C.c_int64, C.c_int64, C.c_int64, C.c_int, C.c_int]
        L.or_dot_red1.restype = C.c_double
        L.or_dot_red1.argtypes = [dp, dp, C.c_int64]
        L.or_red1_blocks.argtypes = [dp, dp, C.c_int64, dp]
        L.or_tree_sum.restype = C.c_double
        L.or_tree_sum.argtypes = [dp, C.c_int64]
        L.or_spmv.restype = C.c_int64
        L.or_spmv.argtypes = [C.c_void_p, u64p, C.c_int64, C.c_int, u64p, C.c_int64, C.c_void_p, dp]
        L.or_spmv_mode.restype = C.c_int64
        L.or_spmv_mode.argtypes = [C.c_void_p, u64p, C.c_int64, C.c_int, u64p, C.c_int64, C.c_void_p, dp, C.c_int]
        L.or_check_csr.restype = C.c_int64
        L.or_check_csr.argtypes = [C.c_void_p, C.c_void_p, C.c_int]
        L.or_calc_ur.restype = C.c_int64
        L.or_calc_ur.argtypes = [u64p, u64p, u64p, u64p, C.c_int64, C.c_int, C.c_double, C.c_void_p, dp]
        L.or_calc_p.restype = C.c_int64
        L.or_calc_p.argtypes = [u64p, u64p, C.c_int64, C.c_int, C.c_double, C.c_void_p]
        L.or_cg_init_r.restype = C.c_int64
        L.or_cg_init_r.argtypes = [u64p, u64p, u64p, u64p, C.c_int64, C.c_int, C.c_void_p, dp]
        L.or_cg_solve.argtypes = [C.c_void_p, u64p, u64p, u64p, u64p, u64p, C.c_int, C.c_double, C.c_int,
                                  C.c_int, C.c_void_p, C.c_void_p]
        L.or_cg_solve_ex.argtypes = [C.c_void_p, u64p, u64p, u64p, u64p, u64p, C.c_int, C.c_double, C.c_int,
                                     C.c_int, C.c_void_p, C.c_void_p, C.c_int]
        L.or_cg_solve_sched.argtypes = [C.c_void_p, u64p, u64p, u64p, u64p, u64p, C.c_int, C.c_double, C.c_int,
                                        C.c_int, C.c_void_p, C.c_void_p, C.c_int, C.c_void_p, C.c_int]
        L.or_calc_sr.restype = C.c_int64
        L.or_calc_sr.argtypes = [u64p, u64p, u64p, u64p, u64p, C.c_int64, C.c_int, C.c_double, C.c_double,
                                 C.c_void_p]
        L.or_cg_solve_sr.argtypes = [C.c_void_p, u64p, u64p, u64p, u64p, u64p, u64p, C.c_int, C.c_double, C.c_int,
                                     C.c_int, C.c_void_p, C.c_void_p, C.c_void_p, C.c_int]
        L.or_cg_solve_log.argtypes = [C.c_void_p, u64p, u64p, u64p, u64p, u64p, C.c_int, C.c_double, C.c_int,
                                      C.c_int, C.c_void_p, C.c_void_p, dp, dp]
        L.or_cheby_solve.argtypes = [C.c_void_p, u64p, u64p, u64p, u64p, u64p, C.c_int, C.c_double, C.c_double,
                                     C.c_double, C.c_int, C.c_int, C.c_void_p, C.c_void_p]
        L.or_set_crc_correct.argtypes = [C.c_int]
        L.or_ppcg_solve.argtypes = [C.c_void_p, u64p, u64p, u64p, u64p, u64p, u64p, u64p, u64p, C.c_int,
                                    C.c_double, C.c_double, C.c_int, C.c_double, C.c_int, C.c_int, C.c_void_p,
                                    C.c_void_p]
        L.or_vec_masked.argtypes = [u64p, C.c_int64, C.c_int, dp]
        L.or_round_k.restype = C.c_uint64
        L.or_round_k.argtypes = [C.c_uint64, C.c_int]
    return _lib


def _p(a, t):
    assert a.flags["C_CONTIGUOUS"]
    return a.ctypes.data_as(C.POINTER(t))


class CSR(C.Structure):
    _fields_ = [("nrows", C.c_int64), ("ncols", C.c_int64), ("nnz", C.c_int64), ("row_base", C.c_int64),
                ("col_base", C.c_int64), ("val", C.POINTER(C.c_uint64)), ("col", C.POINTER(C.c_uint32)),
                ("rowptr", C.POINTER(C.c_uint32)), ("es", C.c_int), ("rs", C.c_int)]


class CGResult(C.Structure):
    _fields_ = [("iters", C.c_int32), ("status", C.c_int32), ("rr0", C.c_double), ("rrn", C.c_double)]


def new_counts() -> np.ndarray:
    """uint64 [target][scheme][det, cor, unc, range]"""
    return np.zeros((3, 5, 4), dtype=np.uint64)


# ---------------------------------------------------------------- codec hooks
def crc32c(data: bytes) -> int:
    return lib().or_crc32c(data, len(data))


def inst_nbits(inst: int) -> int:
    return lib().or_inst_nbits(inst)


def inst_columns(inst: int) -> list[int]:
    return [lib().or_inst_column(inst, b) for b in range(inst_nbits(inst))]


def inst_reserved(inst: int) -> list[int]:
    out = []
    k = 0
    while (b := lib().or_inst_reserved(inst, k)) >= 0 and k < 16:
        out.append(b)
        k += 1
    return out


def secded_check(inst: int, words: np.ndarray) -> tuple[int, int]:
    """Check/correct a container (uint32 words, in place). Returns (outcome, bit)."""
    words = np.ascontiguousarray(words, dtype=np.uint32)
    bit = C.c_int(-1)
    o = lib().or_secded_check(inst, _p(words, C.c_uint32), C.byref(bit))
    return o, bit.value


def secded_encode(inst: int, words: np.ndarray) -> np.ndarray:
    w = np.array(words, dtype=np.uint32, copy=True)
    lib().or_secded_encode(inst, _p(w, C.c_uint32))
    return w


def secded_syndrome(inst: int, words: np.ndarray) -> tuple[int, int]:
    w = np.ascontiguousarray(words, dtype=np.uint32)
    s, q = C.c_int(), C.c_int()
    lib().or_secded_syndrome(inst, _p(w, C.c_uint32), C.byref(s), C.byref(q))
    return s.value, q.value


# ---------------------------------------------------------------- vectors
def vec_padded_len(n: int, scheme: int) -> int:
    return lib().or_vec_padded_len(n, scheme)


def rowptr_padded_len(nrows: int, scheme: int) -> int:
    return lib().or_rowptr_padded_len(nrows, scheme)


def vec_encode(values: np.ndarray, scheme: int) -> np.ndarray:
    """f64 values -> padded encoded uint64 words."""
    n = len(values)
    out = np.zeros(vec_padded_len(n, scheme), dtype=np.uint64)
    out[:n] = np.ascontiguousarray(values, dtype=np.float64).view(np.uint64)
    lib().or_vec_encode(_p(out, C.c_uint64), n, scheme)
    return out


def vec_check(words: np.ndarray, n: int, scheme: int, counts=None, scrub=True):
    """Check all codewords (in place if scrub); returns (masked f64 values, dues)."""
    out = np.zeros(max(n, 1), dtype=np.float64)
    cp = counts.ctypes.data if counts is not None else None
    d = lib().or_vec_check(_p(words, C.c_uint64), n, scheme, _p(out, C.c_double), cp, int(scrub))
    return out[:n], d


def vec_masked(words: np.ndarray, n: int, scheme: int) -> np.ndarray:
    out = np.zeros(max(n, 1), dtype=np.float64)
    lib().or_vec_masked(_p(words, C.c_uint64), n, scheme, _p(out, C.c_double))
    return out[:n]


def round_k(u: int, k: int) -> int:
    return lib().or_round_k(u, k)


def dot_red1(a: np.ndarray, b: np.ndarray) -> float:
    a = np.ascontiguousarray(a, dtype=np.float64)
    b = np.ascontiguousarray(b, dtype=np.float64)
    return lib().or_dot_red1(_p(a, C.c_double), _p(b, C.c_double), len(a))


def red1_blocks(a: np.ndarray, b: np.ndarray) -> np.ndarray:
    a = np.ascontiguousarray(a, dtype=np.float64)
    b = np.ascontiguousarray(b, dtype=np.float64)
    out = np.zeros((len(a) + 255) // 256, dtype=np.float64)
    lib().or_red1_blocks(_p(a, C.c_double), _p(b, C.c_double), len(a), _p(out, C.c_double))
    return out


def tree_sum(v: np.ndarray) -> float:
    m = 1
    while m < len(v):
        m *= 2
    buf = np.zeros(m, dtype=np.float64)
    buf[:len(v)] = v
    return lib().or_tree_sum(_p(buf, C.c_double), m)


# ---------------------------------------------------------------- matrices
class Matrix:
    """An oracle-side CSR (chunk).  Holds numpy arrays: val as uint64 bits,
    col uint32, rowptr uint32 (padded for the rowptr scheme)."""

    def __init__(self, val, col, rowptr, nrows, ncols, es, rs, row_base=0, col_base=0):
        self.nrows, self.ncols, self.es, self.rs = int(nrows), int(ncols), es, rs
        self.nnz = int(rowptr[nrows])
        self.val = np.ascontiguousarray(np.asarray(val, dtype=np.float64).view(np.uint64)).copy()
        self.col = np.array(col, dtype=np.uint32, copy=True)
        rp = np.zeros(rowptr_padded_len(nrows, rs), dtype=np.uint32)
        rp[:nrows + 1] = rowptr[:nrows + 1]
        self.rowptr = rp
        self.row_base, self.col_base = int(row_base), int(col_base)

    def encode(self) -> int:
        return lib().or_csr_encode(_p(self.val, C.c_uint64), _p(self.col, C.c_uint32), _p(self.rowptr, C.c_uint32),
                                   self.nrows, self.ncols, self.nnz, self.es, self.rs)

    def cstruct(self) -> CSR:
        return CSR(self.nrows, self.ncols, self.nnz, self.row_base, self.col_base, _p(self.val, C.c_uint64),
                   _p(self.col, C.c_uint32), _p(self.rowptr, C.c_uint32), self.es, self.rs)

    def check(self, counts=None, scrub=True) -> int:
        """scrub: False count only, True count + scrub, 2 detection only."""
        s = self.cstruct()
        return lib().or_check_csr(C.byref(s), counts.ctypes.data if counts is not None else None, int(scrub))


# matrix check modes of one SpMV access
MODE_CORRECT, MODE_DETECT, MODE_RANGE = 0, 1, 2


def spmv(A: Matrix, x: np.ndarray, n_in: int, scheme: int, out: np.ndarray, n_out: int, counts=None,
         want_dot=False, mode=MODE_CORRECT):
    s = A.cstruct()
    dot = C.c_double(0.0)
    d = lib().or_spmv_mode(C.byref(s), _p(x, C.c_uint64), n_in, scheme, _p(out, C.c_uint64), n_out,
                           counts.ctypes.data if counts is not None else None, C.byref(dot) if want_dot else None,
                           int(mode))
    return (d, dot.value) if want_dot else d


def calc_ur(x, p, r, w, n, scheme, alpha, counts=None):
    rrn = C.c_double()
    d = lib().or_calc_ur(_p(x, C.c_uint64), _p(p, C.c_uint64), _p(r, C.c_uint64), _p(w, C.c_uint64), n, scheme,
                         alpha, counts.ctypes.data if counts is not None else None, C.byref(rrn))
    return d, rrn.value


def calc_p(p, r, n, scheme, beta, counts=None):
    return lib().or_calc_p(_p(p, C.c_uint64), _p(r, C.c_uint64), n, scheme, beta,
                           counts.ctypes.data if counts is not None else None)


def cg_init_r(b, w, r, p, n, scheme, counts=None):
    rr0 = C.c_double()
    d = lib().or_cg_init_r(_p(b, C.c_uint64), _p(w, C.c_uint64), _p(r, C.c_uint64), _p(p, C.c_uint64), n, scheme,
                           counts.ctypes.data if counts is not None else None, C.byref(rr0))
    return d, rr0.value


def cg_solve(A: Matrix, b, x, r, p, w, scheme, tol=1e-10, max_iters=10000, due_policy=1, counts=None,
             check_interval=1):
    """Protected CG on encoded uint64 vectors (x: in x0, out x).
    check_interval N > 1: the matrix is checked (detection only) on every N-th
    access and range-checked otherwise, plus a final check."""
    s = A.cstruct()
    res = CGResult()
    st = lib().or_cg_solve_ex(C.byref(s), _p(b, C.c_uint64), _p(x, C.c_uint64), _p(r, C.c_uint64),
                              _p(p, C.c_uint64), _p(w, C.c_uint64), scheme, tol, max_iters, due_policy, C.byref(res),
                              counts.ctypes.data if counts is not None else None, int(check_interval))
    return st, res


# O10 fault targets (S§8(c) O10): storage words of val (64-bit), col, rowptr
# (32-bit) and the CG vectors b, x, r, p, w (64-bit)
F_VAL, F_COL, F_ROWPTR, F_B, F_X, F_R, F_P, F_W = range(8)
FAULT_DTYPE = np.dtype([("iter", "<i4"), ("target", "<i4"), ("word", "<i8"), ("bit", "<i4"), ("pad", "<i4")])


def fault_schedule(entries) -> np.ndarray:
    """[(iteration k, target, storage-word index, bit), ...] -> packed schedule."""
    out = np.zeros(len(entries), dtype=FAULT_DTYPE)
    for i, (k, t, w, b) in enumerate(entries):
        out[i] = (k, t, w, b, 0)
    return out


def cg_solve_sched(A: Matrix, b, x, r, p, w, scheme, tol=1e-10, max_iters=10000, due_policy=1, counts=None,
                   check_interval=1, faults=None):
    """Protected CG with an O10 fault schedule: fault (k, target, word, bit) is
    XOR-ed into the stored bits before init (k = 0) or before iteration k's
    SpMV (S§8(c) O10)."""
    s = A.cstruct()
    res = CGResult()
    f = faults if faults is not None else np.zeros(0, dtype=FAULT_DTYPE)
    st = lib().or_cg_solve_sched(C.byref(s), _p(b, C.c_uint64), _p(x, C.c_uint64), _p(r, C.c_uint64),
                                 _p(p, C.c_uint64), _p(w, C.c_uint64), scheme, tol, max_iters, due_policy,
                                 C.byref(res), counts.ctypes.data if counts is not None else None,
                                 int(check_interval), f.ctypes.data if len(f) else None, len(f))
    return st, res

F_S = 8   # the single-reduction CG's extra vector s (or_cg_solve_sr)


def calc_sr(x, p, s, r, w, n, scheme, alpha, beta, counts=None):
    """Single-reduction CG update: p, s, x, r in place."""
    return lib().or_calc_sr(_p(x, C.c_uint64), _p(p, C.c_uint64), _p(s, C.c_uint64), _p(r, C.c_uint64),
                            _p(w, C.c_uint64), n, scheme, alpha, beta,
                            counts.ctypes.data if counts is not None else None)


def cg_solve_sr(A: Matrix, b, x, r, p, w, s, scheme, tol=1e-10, max_iters=10000, due_policy=1, counts=None,
                faults=None):
    """Protected single-reduction CG (Chronopoulos-Gear; S§8(f) f3)."""
    st = A.cstruct()
    res = CGResult()
    f = faults if faults is not None else np.zeros(0, dtype=FAULT_DTYPE)
    code = lib().or_cg_solve_sr(C.byref(st), _p(b, C.c_uint64), _p(x, C.c_uint64), _p(r, C.c_uint64),
                                _p(p, C.c_uint64), _p(w, C.c_uint64), _p(s, C.c_uint64), scheme, tol, max_iters,
                                due_policy, C.byref(res), counts.ctypes.data if counts is not None else None,
                                f.ctypes.data if len(f) else None, len(f))
    return code, res


def cg_solve_log(A: Matrix, b, x, r, p, w, scheme, tol=1e-10, max_iters=30, due_policy=1, counts=None):
    """Protected CG that also returns its step coefficients alpha_k, beta_k
    (the Lanczos data of TeaLeaf's spectrum estimate)."""
    s = A.cstruct()
    res = CGResult()
    al = np.zeros(max(max_iters, 1))
    bl = np.zeros(max(max_iters, 1))
    st = lib().or_cg_solve_log(C.byref(s), _p(b, C.c_uint64), _p(x, C.c_uint64), _p(r, C.c_uint64),
                               _p(p, C.c_uint64), _p(w, C.c_uint64), scheme, tol, max_iters, due_policy, C.byref(res),
                               counts.ctypes.data if counts is not None else None, _p(al, C.c_double),
                               _p(bl, C.c_double))
    return st, res, al[:res.iters], bl[:max(res.iters - 1, 0)] if res.iters else bl[:0]


def lanczos_bounds(alphas, betas):
    """Extreme eigenvalues of the Lanczos tridiagonal built from CG's step
    coefficients (T_jj = 1/a_j + b_{j-1}/a_{j-1}, T_{j,j+1} = sqrt(b_j)/a_j),
    by numpy.linalg.eigvalsh (library routine) — TeaLeaf's eigenvalue estimate."""
    k = len(alphas)
    T = np.zeros((k, k))
    for j in range(k):
        T[j, j] = 1.0 / alphas[j] + (betas[j - 1] / alphas[j - 1] if j > 0 else 0.0)
        if j + 1 < k:
            T[j, j + 1] = T[j + 1, j] = np.sqrt(betas[j]) / alphas[j]
    ev = np.linalg.eigvalsh(T)
    return float(ev[0]), float(ev[-1])


def cheby_solve(A: Matrix, b, u, r, p, w, scheme, eigmin, eigmax, tol=1e-10, max_iters=10000, due_policy=1,
                counts=None):
    """Protected Chebyshev iteration (TeaLeaf) with spectrum bounds [eigmin, eigmax]."""
    s = A.cstruct()
    res = CGResult()
    st = lib().or_cheby_solve(C.byref(s), _p(b, C.c_uint64), _p(u, C.c_uint64), _p(r, C.c_uint64),
                              _p(p, C.c_uint64), _p(w, C.c_uint64), scheme, float(eigmin), float(eigmax), tol,
                              max_iters, due_policy, C.byref(res), counts.ctypes.data if counts is not None else None)
    return st, res


def set_crc_correct(t: int):
    """CRC32C correction capability: 1 = 1EC4ED (default), 2 = 2EC3ED."""
    lib().or_set_crc_correct(int(t))


def ppcg_solve(A: Matrix, b, x, r, p, w, z, rin, pin, scheme, eigmin, eigmax, inner=10, tol=1e-10, max_iters=10000,
               due_policy=1, counts=None):
    """Protected polynomially preconditioned CG (TeaLeaf PPCG):
    the preconditioner is `inner` Chebyshev steps on [eigmin, eigmax] from z = 0."""
    s = A.cstruct()
    res = CGResult()
    st = lib().or_ppcg_solve(C.byref(s), *[_p(v, C.c_uint64) for v in (b, x, r, p, w, z, rin, pin)], scheme,
                             float(eigmin), float(eigmax), int(inner), tol, max_iters, due_policy, C.byref(res),
                             counts.ctypes.data if counts is not None else None)
    return st, res
