"""ctypes binding of libabft.so (include/abft.h) — argument marshalling only.

Every step of the hot path runs in the library's CUDA kernels; torch is used
for device memory, streams and process groups.  Importing this module fails
loudly if the compiled library is missing: there is no CPU fallback.
"""
from __future__ import annotations

import ctypes as C
import os

import torch

from . import build as _build

NONE, SED, SECDED64, SECDED128, CRC32C = range(5)
SCHEMES = {"none": NONE, "sed": SED, "secded64": SECDED64, "secded128": SECDED128, "crc32c": CRC32C}
ELEM, ROWPTR, VEC = range(3)
OK, E_INVALID, E_RANGE, E_SHAPE, E_DUE, E_NOT_CONVERGED, E_CUDA, E_NCCL = 0, -1, -2, -3, -4, -5, -6, -7

_SO = os.environ.get("ABFT_SO", _build.SO)   # override: kernel-variant timing tools only
if not os.path.exists(_SO):
    raise ImportError(f"libabft.so not built ({_SO}); run __graft_entry__.build() "
                      "or python -m paper_conf_cluster_pawelczakmpm17_b200.build")


class CSR(C.Structure):
    _fields_ = [("nrows", C.c_int64), ("ncols", C.c_int64), ("nnz", C.c_int64), ("row_base", C.c_int64),
                ("col_base", C.c_int64), ("val", C.c_void_p), ("col", C.c_void_p), ("rowptr", C.c_void_p),
                ("elem_scheme", C.c_int32), ("rowptr_scheme", C.c_int32), ("stencil_n", C.c_int64)]


class Vec(C.Structure):
    _fields_ = [("n", C.c_int64), ("data", C.c_void_p), ("scheme", C.c_int32)]


class CGOpts(C.Structure):
    _fields_ = [("tol", C.c_double), ("max_iters", C.c_int32), ("due_policy", C.c_int32), ("poll_every", C.c_int32),
                ("check_interval", C.c_int32)]


class Fault(C.Structure):
    _fields_ = [("iter", C.c_int32), ("target", C.c_int32), ("word", C.c_int64), ("bit", C.c_int32),
                ("chunk", C.c_int32)]


# abft_fault_target (S§8(c) O10)
F_VAL, F_COL, F_ROWPTR, F_B, F_X, F_R, F_P, F_W = range(8)


class CGResult(C.Structure):
    _fields_ = [("iters", C.c_int32), ("status", C.c_int32), ("rr0", C.c_double), ("rrn", C.c_double)]


_lib = C.CDLL(_SO)
_P = C.c_void_p
_sig = {
    "abft_ctx_create": (C.c_int, [C.c_int, C.POINTER(C.c_void_p)]),
    "abft_ctx_destroy": (C.c_int, [_P]),
    "abft_ctx_set_fused_cg": (C.c_int, [_P, C.c_int]),
    "abft_ctx_set_pdl": (C.c_int, [_P, C.c_int]),
    "abft_ctx_set_crc_correction": (C.c_int, [_P, C.c_int]),
    "abft_rowptr_padded_len": (C.c_int64, [C.c_int64, C.c_int32]),
    "abft_vec_padded_len": (C.c_int64, [C.c_int64, C.c_int32]),
    "abft_csr_encode": (C.c_int, [_P, C.POINTER(CSR), _P]),
    "abft_vec_encode": (C.c_int, [_P, C.POINTER(Vec), _P]),
    "abft_vec_decode": (C.c_int, [_P, C.POINTER(Vec), _P, _P, _P]),
    "abft_spmv": (C.c_int, [_P, C.POINTER(CSR), C.c_int, C.POINTER(Vec), C.POINTER(Vec), _P, _P, _P]),
    "abft_spmv_ex": (C.c_int, [_P, C.POINTER(CSR), C.c_int, C.POINTER(Vec), C.POINTER(Vec), _P, _P, C.c_int32, _P]),
    "abft_spmv_partials": (C.c_int, [_P, C.POINTER(CSR), C.c_int, C.POINTER(Vec), C.POINTER(Vec), _P, _P]),
    "abft_cg_solve": (C.c_int, [_P, C.POINTER(CSR), C.c_int, C.POINTER(Vec), C.POINTER(Vec), C.POINTER(Vec),
                                C.POINTER(Vec), C.POINTER(Vec), C.POINTER(CGOpts), C.POINTER(CGResult), _P, _P]),
    "abft_cg_solve_sr": (C.c_int, [_P, C.POINTER(CSR), C.c_int, C.POINTER(Vec), C.POINTER(Vec), C.POINTER(Vec),
                                   C.POINTER(Vec), C.POINTER(Vec), C.POINTER(Vec), C.POINTER(CGOpts),
                                   C.POINTER(CGResult), _P, _P]),
    "abft_cheby_solve": (C.c_int, [_P, C.POINTER(CSR), C.c_int, C.POINTER(Vec), C.POINTER(Vec), C.POINTER(Vec),
                                   C.POINTER(Vec), C.POINTER(Vec), C.c_double, C.c_double, C.POINTER(CGOpts),
                                   C.POINTER(CGResult), _P, _P]),
    "abft_ppcg_solve": (C.c_int, [_P, C.POINTER(CSR), C.c_int] + [C.POINTER(Vec)] * 8 +
                        [C.c_double, C.c_double, C.c_int, C.POINTER(CGOpts), C.POINTER(CGResult), _P, _P]),
    "abft_cg_spectrum": (C.c_int, [_P, C.POINTER(CSR), C.c_int, C.POINTER(Vec), C.POINTER(Vec), C.POINTER(Vec),
                                   C.POINTER(Vec), C.POINTER(Vec), C.c_int, C.POINTER(CGOpts),
                                   C.POINTER(C.c_double), C.POINTER(C.c_double), C.POINTER(CGResult), _P, _P]),
    "abft_check_all": (C.c_int, [_P, C.POINTER(CSR), C.c_int, C.POINTER(Vec), C.c_int, C.c_int, _P, _P]),
    "abft_calc_ur": (C.c_int, [_P, C.POINTER(Vec), C.POINTER(Vec), C.POINTER(Vec), C.POINTER(Vec), C.c_double, _P, _P,
                               _P]),
    "abft_calc_p": (C.c_int, [_P, C.POINTER(Vec), C.POINTER(Vec), C.c_double, _P, _P]),
    "abft_calc_p_spmv": (C.c_int, [_P, C.POINTER(CSR), C.c_int, C.POINTER(Vec), C.POINTER(Vec), C.c_double,
                                   C.POINTER(Vec), C.POINTER(Vec), _P, _P, _P]),
    "abft_inject_bitflip": (C.c_int, [_P, _P, C.c_uint64, _P]),
    "abft_ctx_set_faults": (C.c_int, [_P, _P, C.c_int, C.POINTER(CSR), C.c_int, _P]),
    "abft_counts_read": (C.c_int, [_P, _P, _P]),
    "abft_counts_reset": (C.c_int, [_P, _P]),
    "abft_launch_count": (C.c_uint64, []),
    "abft_profile": (C.c_int, [_P, C.c_int]),
    "abft_profile_read": (C.c_int, [_P, _P, _P]),
    "abft_last_error": (C.c_char_p, []),
    "abft_dist_init": (C.c_int, [C.POINTER(C.c_void_p), _P, C.c_int, C.c_int, C.c_int]),
    "abft_dist_get_unique_id": (C.c_int, [_P]),
    "abft_dist_destroy": (C.c_int, [_P]),
    "abft_cg_solve_dist": (C.c_int, [_P, _P, C.POINTER(CSR), C.c_int, C.c_int64, C.POINTER(Vec), C.POINTER(Vec),
                                     C.POINTER(Vec), C.POINTER(Vec), C.POINTER(Vec), C.POINTER(CGOpts),
                                     C.POINTER(CGResult), _P, _P]),
    "abft_dist_init_loopback": (C.c_int, [C.POINTER(C.c_void_p), C.c_int, C.c_int]),
    "abft_dist_set_peer_halo": (C.c_int, [_P, C.c_int, _P, _P]),
    "abft_dist_flags": (C.c_int, [_P, C.POINTER(C.c_void_p)]),
    "abft_ipc_get_handle": (C.c_int, [_P, _P, C.POINTER(C.c_int64)]),
    "abft_ipc_open_handle": (C.c_int, [_P, C.c_int64, C.POINTER(C.c_void_p)]),
    "abft_ipc_close_handle": (C.c_int, [_P, C.c_int64]),
    "abft_cg_solve_sr_dist": (C.c_int, [_P, _P, C.POINTER(CSR), C.c_int, C.c_int64, C.POINTER(Vec), C.POINTER(Vec),
                                        C.POINTER(Vec), C.POINTER(Vec), C.POINTER(Vec), C.POINTER(Vec),
                                        C.POINTER(CGOpts), C.POINTER(CGResult), _P, _P]),
    "abft_cg_solve_loopback_sr": (C.c_int, [_P, _P, _P, _P, C.c_int64, _P, C.POINTER(CGOpts), _P, _P, _P]),
    "abft_cg_solve_loopback": (C.c_int, [_P, _P, _P, _P, C.c_int64, _P, C.POINTER(CGOpts), _P, _P, _P]),
    "abft_codec_host_check": (C.c_int, [C.c_int, _P]),
    "abft_codec_host_encode": (None, [C.c_int, _P]),
}
for _name, (_res, _args) in _sig.items():
    _f = getattr(_lib, _name)
    _f.restype = _res
    _f.argtypes = _args

HEADER_SYMBOLS = sorted(_sig)


class AbftError(RuntimeError):
    def __init__(self, code: int, what: str):
        super().__init__(f"{what}: status {code}: {last_error()}")
        self.code = code


def last_error() -> str:
    return (_lib.abft_last_error() or b"").decode()


def _check(code: int, what: str, allow=()) -> int:
    if code != OK and code not in allow:
        raise AbftError(code, what)
    return code


def _stream(stream) -> int | None:
    if stream is None:
        return torch.cuda.current_stream().cuda_stream
    return stream.cuda_stream if hasattr(stream, "cuda_stream") else int(stream)


def launch_count() -> int:
    return int(_lib.abft_launch_count())


def rowptr_padded_len(nrows: int, scheme: int) -> int:
    return int(_lib.abft_rowptr_padded_len(nrows, scheme))


def vec_padded_len(n: int, scheme: int) -> int:
    return int(_lib.abft_vec_padded_len(n, scheme))


def codec_host_check(inst: int, words) -> int:
    buf = (C.c_uint32 * len(words))(*[int(w) for w in words])
    o = _lib.abft_codec_host_check(inst, C.cast(buf, C.c_void_p))
    words[:] = list(buf)
    return o


def codec_host_encode(inst: int, words) -> list:
    buf = (C.c_uint32 * len(words))(*[int(w) for w in words])
    _lib.abft_codec_host_encode(inst, C.cast(buf, C.c_void_p))
    return list(buf)


# ------------------------------------------------------------------ objects
class Context:
    """abft_ctx: owns reduction scratch and the device CG scalars."""

    def __init__(self, device: int | None = None):
        if not torch.cuda.is_available():
            raise RuntimeError("the ABFT CUDA path needs a GPU (no CPU fallback)")
        self.device = torch.cuda.current_device() if device is None else int(device)
        h = C.c_void_p()
        _check(_lib.abft_ctx_create(self.device, C.byref(h)), "abft_ctx_create")
        self.h = h

    def set_fused_cg(self, enable: bool):
        """Fused calc_p in the CG's SpMV (abft_ctx_set_fused_cg; default off)."""
        _check(_lib.abft_ctx_set_fused_cg(self.h, 1 if enable else 0), "abft_ctx_set_fused_cg")

    def set_crc_correction(self, bits: int):
        """CRC32C correction: 1 = 1EC4ED (default), 2 = 2EC3ED (abft_ctx_set_crc_correction)."""
        _check(_lib.abft_ctx_set_crc_correction(self.h, int(bits)), "abft_ctx_set_crc_correction")

    def set_pdl(self, enable: bool):
        """Programmatic dependent launch in the CG loop (abft_ctx_set_pdl; library default off)."""
        _check(_lib.abft_ctx_set_pdl(self.h, 1 if enable else 0), "abft_ctx_set_pdl")

    def set_faults(self, faults, A=None, vecs=None):
        """O10 fault schedule for the next CG solves on this context:
        faults = [(iter, target, word, bit[, chunk]), ...] (targets F_VAL ..
        F_W), A = the matrix / chunk list and vecs = (b, x, r, p, w) that the
        solve will be given.  An empty list clears it (abft_ctx_set_faults)."""
        fl = list(faults or [])
        arr = (Fault * max(len(fl), 1))()
        for i, f in enumerate(fl):
            k, t, w, b = f[:4]
            arr[i] = Fault(int(k), int(t), int(w), int(b), int(f[4]) if len(f) > 4 else 0)
        if fl:
            carr, nch = _chunks(A)
            vstructs = [v.cstruct() for v in vecs]
            vptr = (C.c_void_p * 5)(*[C.cast(C.pointer(v), C.c_void_p) for v in vstructs])
        else:
            carr, nch, vptr = None, 0, None
        _check(_lib.abft_ctx_set_faults(self.h, C.cast(arr, C.c_void_p), len(fl), carr, nch, vptr),
               "abft_ctx_set_faults")

    def close(self):
        if self.h:
            _lib.abft_ctx_destroy(self.h)
            self.h = None

    def __del__(self):
        try:
            self.close()
        except Exception:
            pass


class Vector:
    """A protected fp64 vector: `data` is a float64 device tensor of padded length
    whose bit patterns carry the ECC (never touch it with torch arithmetic)."""

    def __init__(self, data: torch.Tensor, n: int, scheme: int):
        assert data.dtype == torch.float64 and data.is_cuda and data.is_contiguous()
        assert data.numel() >= vec_padded_len(n, scheme)
        self.data, self.n, self.scheme = data, int(n), int(scheme)

    @classmethod
    def empty(cls, n: int, scheme: int, device="cuda"):
        return cls(torch.zeros(vec_padded_len(n, scheme), dtype=torch.float64, device=device), n, scheme)

    @classmethod
    def from_values(cls, ctx: Context, values: torch.Tensor, scheme: int, stream=None):
        v = cls.empty(values.numel(), scheme, device=values.device if values.is_cuda else "cuda")
        v.data[:values.numel()].copy_(values.reshape(-1))
        v.encode(ctx, stream)
        return v

    @classmethod
    def from_words(cls, words: torch.Tensor, n: int, scheme: int):
        """Wrap already-encoded 64-bit words (e.g. copied from the oracle)."""
        return cls(words.view(torch.float64), n, scheme)

    def cstruct(self) -> Vec:
        return Vec(self.n, self.data.data_ptr(), self.scheme)

    def encode(self, ctx: Context, stream=None):
        v = self.cstruct()
        _check(_lib.abft_vec_encode(ctx.h, C.byref(v), _stream(stream)), "abft_vec_encode")

    def decode(self, ctx: Context, counts: "Counters | None" = None, stream=None) -> torch.Tensor:
        out = torch.empty(max(self.n, 1), dtype=torch.float64, device=self.data.device)
        v = self.cstruct()
        _check(_lib.abft_vec_decode(ctx.h, C.byref(v), out.data_ptr(), counts.ptr if counts else None,
                                    _stream(stream)), "abft_vec_decode")
        return out[:self.n]

    def words(self) -> torch.Tensor:
        return self.data.view(torch.int64)


class Matrix:
    """A protected CSR matrix (one chunk): val float64 [nnz], col int32 [nnz]
    (ECC in its top bits after encode), rowptr int32 [padded]."""

    def __init__(self, val: torch.Tensor, col: torch.Tensor, rowptr: torch.Tensor, nrows: int, ncols: int,
                 elem_scheme: int, rowptr_scheme: int, row_base: int = 0, col_base: int = 0, stencil_n: int = 0):
        dev = val.device
        self.nrows, self.ncols = int(nrows), int(ncols)
        self.nnz = int(rowptr[nrows].item()) if rowptr.numel() > nrows else int(col.numel())
        self.es, self.rs = int(elem_scheme), int(rowptr_scheme)
        self.row_base, self.col_base, self.stencil_n = int(row_base), int(col_base), int(stencil_n)
        self.val = val.to(dtype=torch.float64).contiguous()
        self.col = col.to(dtype=torch.int32).contiguous()
        rp = torch.zeros(rowptr_padded_len(self.nrows, self.rs), dtype=torch.int32, device=dev)
        rp[:self.nrows + 1] = rowptr[:self.nrows + 1].to(device=dev, dtype=torch.int32)
        self.rowptr = rp

    def cstruct(self) -> CSR:
        return CSR(self.nrows, self.ncols, self.nnz, self.row_base, self.col_base, self.val.data_ptr(),
                   self.col.data_ptr(), self.rowptr.data_ptr(), self.es, self.rs, self.stencil_n)

    def encode(self, ctx: Context, stream=None) -> int:
        m = self.cstruct()
        return _lib.abft_csr_encode(ctx.h, C.byref(m), _stream(stream))


def _chunks(A) -> tuple:
    mats = A if isinstance(A, (list, tuple)) else [A]
    arr = (CSR * len(mats))(*[m.cstruct() for m in mats])
    return arr, len(mats)


class Counters:
    """Device abft_counts[3][5] (uint64 x4 each)."""

    def __init__(self, device="cuda"):
        self.t = torch.zeros(3 * 5 * 4, dtype=torch.int64, device=device)

    @property
    def ptr(self) -> int:
        return self.t.data_ptr()

    def reset(self, stream=None):
        _check(_lib.abft_counts_reset(self.ptr, _stream(stream)), "abft_counts_reset")

    def read(self, stream=None):
        import numpy as np
        host = (C.c_uint64 * 60)()
        _check(_lib.abft_counts_read(self.ptr, C.cast(host, C.c_void_p), _stream(stream)), "abft_counts_read")
        return np.array(list(host), dtype=np.uint64).reshape(3, 5, 4)


# matrix check modes of one SpMV access (abft_check_mode)
CHECK_CORRECT, CHECK_DETECT, CHECK_RANGE = 0, 1, 2


def spmv(ctx: Context, A, x: Vector, y: Vector, counts: Counters | None = None, dot: torch.Tensor | None = None,
         stream=None, mode: int = CHECK_CORRECT):
    arr, n = _chunks(A)
    vx, vy = x.cstruct(), y.cstruct()
    _check(_lib.abft_spmv_ex(ctx.h, arr, n, C.byref(vx), C.byref(vy), dot.data_ptr() if dot is not None else None,
                             counts.ptr if counts else None, int(mode), _stream(stream)), "abft_spmv_ex")


def spmv_partials(ctx: Context, A, x: Vector, y: Vector, counts: Counters | None = None, stream=None):
    """abft_spmv_partials: the CG SpMV kernel alone (p.w partials in ctx scratch, no reduction) — for timing."""
    arr, n = _chunks(A)
    vx, vy = x.cstruct(), y.cstruct()
    _check(_lib.abft_spmv_partials(ctx.h, arr, n, C.byref(vx), C.byref(vy), counts.ptr if counts else None,
                                   _stream(stream)), "abft_spmv_partials")


def cg_solve(ctx: Context, A, b: Vector, x: Vector, r: Vector, p: Vector, w: Vector, tol=1e-10, max_iters=10000,
             due_policy=0, counts: Counters | None = None, poll_every=16, stream=None,
             check_interval=1) -> CGResult:
    arr, n = _chunks(A)
    opts = CGOpts(tol, max_iters, due_policy, poll_every, check_interval)
    res = CGResult()
    vs = [v.cstruct() for v in (b, x, r, p, w)]
    code = _lib.abft_cg_solve(ctx.h, arr, n, *[C.byref(v) for v in vs], C.byref(opts), C.byref(res),
                              counts.ptr if counts else None, _stream(stream))
    _check(code, "abft_cg_solve", allow=(E_DUE, E_NOT_CONVERGED))
    return res


def cg_solve_sr(ctx: Context, A, b: Vector, x: Vector, r: Vector, p: Vector, w: Vector, s: Vector, tol=1e-10,
                max_iters=10000, due_policy=0, counts: Counters | None = None, poll_every=16, stream=None) -> CGResult:
    """Single-reduction protected CG (Chronopoulos-Gear; abft_cg_solve_sr)."""
    arr, n = _chunks(A)
    opts = CGOpts(tol, max_iters, due_policy, poll_every, 1)
    res = CGResult()
    vs = [v.cstruct() for v in (b, x, r, p, w, s)]
    code = _lib.abft_cg_solve_sr(ctx.h, arr, n, *[C.byref(v) for v in vs], C.byref(opts), C.byref(res),
                                 counts.ptr if counts else None, _stream(stream))
    _check(code, "abft_cg_solve_sr", allow=(E_DUE, E_NOT_CONVERGED))
    return res


def cheby_solve(ctx: Context, A, b: Vector, u: Vector, r: Vector, p: Vector, w: Vector, eigmin: float, eigmax: float,
                tol=1e-10, max_iters=10000, due_policy=0, counts: Counters | None = None, poll_every=16,
                stream=None) -> CGResult:
    """Protected Chebyshev iteration with spectrum bounds (abft_cheby_solve)."""
    arr, n = _chunks(A)
    opts = CGOpts(tol, max_iters, due_policy, poll_every, 1)
    res = CGResult()
    vs = [v.cstruct() for v in (b, u, r, p, w)]
    code = _lib.abft_cheby_solve(ctx.h, arr, n, *[C.byref(v) for v in vs], float(eigmin), float(eigmax),
                                 C.byref(opts), C.byref(res), counts.ptr if counts else None, _stream(stream))
    _check(code, "abft_cheby_solve", allow=(E_DUE, E_NOT_CONVERGED))
    return res


def ppcg_solve(ctx: Context, A, b: Vector, x: Vector, r: Vector, p: Vector, w: Vector, z: Vector, rin: Vector,
               pin: Vector, eigmin: float, eigmax: float, inner=10, tol=1e-10, max_iters=10000, due_policy=0,
               counts: Counters | None = None, poll_every=16, stream=None) -> CGResult:
    """Protected PPCG: CG with an `inner`-step Chebyshev preconditioner (abft_ppcg_solve)."""
    arr, n = _chunks(A)
    opts = CGOpts(tol, max_iters, due_policy, poll_every, 1)
    res = CGResult()
    vs = [v.cstruct() for v in (b, x, r, p, w, z, rin, pin)]
    code = _lib.abft_ppcg_solve(ctx.h, arr, n, *[C.byref(v) for v in vs], float(eigmin), float(eigmax), int(inner),
                                C.byref(opts), C.byref(res), counts.ptr if counts else None, _stream(stream))
    _check(code, "abft_ppcg_solve", allow=(E_DUE, E_NOT_CONVERGED))
    return res


def cg_spectrum(ctx: Context, A, b: Vector, x: Vector, r: Vector, p: Vector, w: Vector, steps=30, due_policy=1,
                counts: Counters | None = None, poll_every=16, stream=None):
    """TeaLeaf's Lanczos spectrum estimate from `steps` protected CG steps
    (abft_cg_spectrum): returns (eigmin, eigmax, CGResult)."""
    arr, n = _chunks(A)
    opts = CGOpts(0.0, steps, due_policy, poll_every, 1)
    res = CGResult()
    lo, hi = C.c_double(), C.c_double()
    vs = [v.cstruct() for v in (b, x, r, p, w)]
    _check(_lib.abft_cg_spectrum(ctx.h, arr, n, *[C.byref(v) for v in vs], int(steps), C.byref(opts), C.byref(lo),
                                 C.byref(hi), C.byref(res), counts.ptr if counts else None, _stream(stream)),
           "abft_cg_spectrum")
    return lo.value, hi.value, res


def calc_ur(ctx: Context, x: Vector, p: Vector, r: Vector, w: Vector, alpha: float,
            rrn: torch.Tensor | None = None, counts: Counters | None = None, stream=None):
    """a4: x = enc(fma(alpha, p, x)); r = enc(fma(-alpha, w, r)); rrn[0] = r.r (RED-1)."""
    vs = [v.cstruct() for v in (x, p, r, w)]
    _check(_lib.abft_calc_ur(ctx.h, *[C.byref(v) for v in vs], float(alpha),
                             rrn.data_ptr() if rrn is not None else None, counts.ptr if counts else None,
                             _stream(stream)), "abft_calc_ur")


def calc_p(ctx: Context, p: Vector, r: Vector, beta: float, counts: Counters | None = None, stream=None):
    """a5: p = enc(fma(beta, p, r))."""
    vp, vr = p.cstruct(), r.cstruct()
    _check(_lib.abft_calc_p(ctx.h, C.byref(vp), C.byref(vr), float(beta), counts.ptr if counts else None,
                            _stream(stream)), "abft_calc_p")


def calc_p_spmv(ctx: Context, A, p_prev: Vector, r: Vector, beta: float, p_out: Vector, y: Vector,
                counts: Counters | None = None, dot: torch.Tensor | None = None, stream=None):
    """a5 + a3 in one kernel: p_out = enc(fma(beta, p_prev, r)); y = A p_out (+ dot = p_out.y)."""
    arr, n = _chunks(A)
    vs = [v.cstruct() for v in (p_prev, r, p_out, y)]
    _check(_lib.abft_calc_p_spmv(ctx.h, arr, n, C.byref(vs[0]), C.byref(vs[1]), float(beta), C.byref(vs[2]),
                                 C.byref(vs[3]), dot.data_ptr() if dot is not None else None,
                                 counts.ptr if counts else None, _stream(stream)), "abft_calc_p_spmv")


def check_all(ctx: Context, A, vecs, counts: Counters | None = None, scrub=True, stream=None):
    if A is not None:
        arr, n = _chunks(A)
    else:
        arr, n = None, 0
    varr = (Vec * max(len(vecs), 1))(*[v.cstruct() for v in vecs])
    _check(_lib.abft_check_all(ctx.h, arr, n, varr, len(vecs), int(scrub), counts.ptr if counts else None,
                               _stream(stream)), "abft_check_all")


def inject_bitflip(ctx: Context, tensor: torch.Tensor, bit_offset: int, stream=None):
    """XOR one stored bit of a device tensor (bit offset within its storage)."""
    nbits = tensor.numel() * tensor.element_size() * 8
    if not 0 <= bit_offset < nbits:
        raise ValueError("bit offset out of range")
    _check(_lib.abft_inject_bitflip(ctx.h, tensor.data_ptr(), int(bit_offset), _stream(stream)), "abft_inject_bitflip")


def profile(ctx: Context, enable: bool):
    _check(_lib.abft_profile(ctx.h, int(enable)), "abft_profile")


def profile_read(ctx: Context):
    ms = (C.c_double * 4)()
    n = (C.c_int64 * 4)()
    _check(_lib.abft_profile_read(ctx.h, C.cast(ms, C.c_void_p), C.cast(n, C.c_void_p)), "abft_profile_read")
    return list(ms), list(n)


# ------------------------------------------------------------------ multi-GPU
class Dist:
    """abft_dist: an NCCL communicator for the row-block strips (one per rank)."""

    def __init__(self, rank: int, nranks: int, device: int, group=None):
        import torch.distributed as dist
        uid = torch.zeros(128, dtype=torch.uint8)
        if rank == 0:
            buf = (C.c_uint8 * 128)()
            _check(_lib.abft_dist_get_unique_id(C.cast(buf, C.c_void_p)), "abft_dist_get_unique_id")
            uid = torch.tensor(list(buf), dtype=torch.uint8)
        if nranks > 1:
            obj = [uid.tolist()]
            dist.broadcast_object_list(obj, src=0, group=group)
            uid = torch.tensor(obj[0], dtype=torch.uint8)
        raw = (C.c_uint8 * 128)(*uid.tolist())
        h = C.c_void_p()
        _check(_lib.abft_dist_init(C.byref(h), C.cast(raw, C.c_void_p), rank, nranks, device), "abft_dist_init")
        self.h, self.rank, self.nranks = h, rank, nranks

    def close(self):
        if self.h:
            self.disable_peer_halo()
            _lib.abft_dist_destroy(self.h)
            self.h = None

    def enable_peer_halo(self, p: "Vector", group=None):
        """Peer-memory halos (abft_dist_set_peer_halo) for solves whose p is the
        halo-extended vector `p`: every rank shares the CUDA IPC handles of its p
        and of its arrival flags (abft_ipc_get_handle, all-gathered over
        torch.distributed), maps its neighbours' (abft_ipc_open_handle) and hands
        the pointers to the transport.  Collective over the ranks."""
        import torch.distributed as dist
        flags = C.c_void_p()
        _check(_lib.abft_dist_flags(self.h, C.byref(flags)), "abft_dist_flags")
        mine = []
        for ptr in (p.data.data_ptr(), flags.value):
            hb = (C.c_uint8 * 64)()
            off = C.c_int64()
            _check(_lib.abft_ipc_get_handle(C.c_void_p(ptr), C.cast(hb, C.c_void_p), C.byref(off)),
                   "abft_ipc_get_handle")
            mine.append((bytes(hb), off.value))
        allh = [None] * self.nranks
        dist.all_gather_object(allh, mine, group=group)
        self._mapped = []
        peer_p = (C.c_void_p * 2)()
        peer_f = (C.c_void_p * 2)()
        for k, nb in enumerate((self.rank - 1, self.rank + 1)):
            if not 0 <= nb < self.nranks:
                continue
            ptrs = []
            for (hbytes, off) in allh[nb]:
                raw = (C.c_uint8 * 64)(*hbytes)
                out = C.c_void_p()
                _check(_lib.abft_ipc_open_handle(C.cast(raw, C.c_void_p), off, C.byref(out)), "abft_ipc_open_handle")
                self._mapped.append((out.value, off))
                ptrs.append(out.value)
            peer_p[k] = ptrs[0]
            # rank-1 is signalled through its flags[1], rank+1 through its flags[0]
            peer_f[k] = ptrs[1] + (4 if k == 0 else 0)
        _check(_lib.abft_dist_set_peer_halo(self.h, 1, C.cast(peer_p, C.c_void_p), C.cast(peer_f, C.c_void_p)),
               "abft_dist_set_peer_halo")

    def disable_peer_halo(self):
        if self.h:
            _lib.abft_dist_set_peer_halo(self.h, 0, None, None)
        for (ptr, off) in getattr(self, "_mapped", []):
            _lib.abft_ipc_close_handle(C.c_void_p(ptr), off)
        self._mapped = []

    def cg_solve(self, ctx: Context, A, n_halo: int, b, x, r, p, w, tol=1e-10, max_iters=10000, due_policy=0,
                 counts: Counters | None = None, poll_every=16, stream=None, check_interval=1) -> CGResult:
        arr, n = _chunks(A)
        opts = CGOpts(tol, max_iters, due_policy, poll_every, check_interval)
        res = CGResult()
        vs = [v.cstruct() for v in (b, x, r, p, w)]
        code = _lib.abft_cg_solve_dist(self.h, ctx.h, arr, n, int(n_halo), *[C.byref(v) for v in vs], C.byref(opts),
                                       C.byref(res), counts.ptr if counts else None, _stream(stream))
        _check(code, "abft_cg_solve_dist", allow=(E_DUE, E_NOT_CONVERGED))
        return res

    def cg_solve_sr(self, ctx: Context, A, n_halo: int, b, x, r, p, w, s, tol=1e-10, max_iters=10000, due_policy=0,
                    counts: Counters | None = None, poll_every=16, stream=None) -> CGResult:
        """Single-reduction CG on this rank's strip (abft_cg_solve_sr_dist)."""
        arr, n = _chunks(A)
        opts = CGOpts(tol, max_iters, due_policy, poll_every, 1)
        res = CGResult()
        vs = [v.cstruct() for v in (b, x, r, p, w, s)]
        code = _lib.abft_cg_solve_sr_dist(self.h, ctx.h, arr, n, int(n_halo), *[C.byref(v) for v in vs],
                                          C.byref(opts), C.byref(res), counts.ptr if counts else None, _stream(stream))
        _check(code, "abft_cg_solve_sr_dist", allow=(E_DUE, E_NOT_CONVERGED))
        return res


class Loopback:
    """abft_dist over the in-process loopback transport: `nranks` virtual ranks
    on one device, each with its own Context, chunks and halo-extended vectors
    (abft_dist_init_loopback / abft_cg_solve_loopback)."""

    def __init__(self, nranks: int, device: int = 0):
        h = C.c_void_p()
        _check(_lib.abft_dist_init_loopback(C.byref(h), int(nranks), int(device)), "abft_dist_init_loopback")
        self.h, self.nranks = h, int(nranks)

    def close(self):
        if self.h:
            _lib.abft_dist_destroy(self.h)
            self.h = None

    def set_peer_halo(self, enable: bool):
        """Peer-memory halos between the loopback ranks (abft_dist_set_peer_halo)."""
        _check(_lib.abft_dist_set_peer_halo(self.h, 1 if enable else 0, None, None), "abft_dist_set_peer_halo")

    def __del__(self):
        try:
            self.close()
        except Exception:
            pass

    def cg_solve(self, ctxs, As, n_halo: int, vecs, tol=1e-10, max_iters=10000, due_policy=0, counts=None,
                 poll_every=16, stream=None, check_interval=1):
        """ctxs[q], As[q] (matrix or chunk list), vecs[q] = (b, x, r, p, w), counts[q]
        for every rank q; returns the per-rank CGResult list."""
        return self._solve(_lib.abft_cg_solve_loopback, 5, ctxs, As, n_halo, vecs, tol, max_iters, due_policy,
                           counts, poll_every, stream, check_interval)

    def cg_solve_sr(self, ctxs, As, n_halo: int, vecs, tol=1e-10, max_iters=10000, due_policy=0, counts=None,
                    poll_every=16, stream=None):
        """Single-reduction CG on the loopback strips: vecs[q] = (b, x, r, p, w, s)."""
        return self._solve(_lib.abft_cg_solve_loopback_sr, 6, ctxs, As, n_halo, vecs, tol, max_iters, due_policy,
                           counts, poll_every, stream, 1)

    def _solve(self, fn, nv, ctxs, As, n_halo, vecs, tol, max_iters, due_policy, counts, poll_every, stream,
               check_interval):
        P = self.nranks
        assert len(ctxs) == len(As) == len(vecs) == P
        keep = []
        arrs = []
        nch = (C.c_int * P)()
        for q in range(P):
            arr, n = _chunks(As[q])
            keep.append(arr)
            arrs.append(C.cast(arr, C.c_void_p))
            nch[q] = n
        aptr = (C.c_void_p * P)(*arrs)
        cptr = (C.c_void_p * P)(*[c.h for c in ctxs])
        assert all(len(vecs[q]) == nv for q in range(P))
        vstructs = [v.cstruct() for q in range(P) for v in vecs[q]]
        vptr = (C.c_void_p * (nv * P))(*[C.cast(C.pointer(v), C.c_void_p) for v in vstructs])
        cnts = counts if counts is not None else [None] * P
        nptr = (C.c_void_p * P)(*[c.ptr if c is not None else None for c in cnts])
        opts = CGOpts(tol, max_iters, due_policy, poll_every, check_interval)
        res = (CGResult * P)()
        code = fn(self.h, cptr, aptr, nch, int(n_halo), vptr, C.byref(opts), C.cast(res, C.c_void_p), nptr,
                  _stream(stream))
        _check(code, fn.__name__, allow=(E_DUE, E_NOT_CONVERGED))
        return list(res)
