"""G-TEA: TeaLeaf-shaped 5-point CSR matrices.

Layout (reading R16): every row stores exactly 5 entries in stencil order
[i-n, i-1, i, i+1, i+n]; an out-of-grid neighbour is value +0.0
with col = i.  nnz = 5N, rowptr[i] = 5i.  Row index = x + y*n (x fastest).

Physics (reading R17, from TeaLeaf's public benchmark deck, NOT in PAPER.md):
domain [0,10]^2, background density 100 / energy 1e-4, four density-0.1
"pipe" states, dt = 0.004, face coefficient K = rx*(d1+d2)/(2*d1*d2) on interior
faces (0 on domain faces), diag = 1 + sum K, off-diagonal -K; b = x0 =
energy*density.

All functions take a torch device so large grids can be generated directly in
HBM; the same elementwise IEEE ops run on CPU and GPU, so the arrays are
bit-identical on either device.
"""
from __future__ import annotations

import numpy as np
import torch

# (x0, x1, y0, y1, density, energy): applied in order, later states win.
PIPE_STATES = [
    (0.0, 1.0, 1.0, 2.0, 0.1, 25.0),
    (1.0, 6.0, 1.0, 2.0, 0.1, 0.1),
    (5.0, 6.0, 1.0, 8.0, 0.1, 0.1),
    (5.0, 10.0, 7.0, 8.0, 0.1, 0.1),
]
DT = 0.004
EXTENT = 10.0


def _fields(n: int, y0: int, y1: int, device, kind: str, ny: int | None = None):
    """density, energy for grid rows [y0, y1) (+1 halo row each side, clamped later)."""
    ny = n if ny is None else ny
    dx = EXTENT / n
    dy = EXTENT / ny
    xs = (torch.arange(n, dtype=torch.float64, device=device) + 0.5) * dx
    ys = (torch.arange(y0, y1, dtype=torch.float64, device=device) + 0.5) * dy
    X = xs.unsqueeze(0).expand(y1 - y0, n)
    Y = ys.unsqueeze(1).expand(y1 - y0, n)
    dens = torch.full((y1 - y0, n), 100.0, dtype=torch.float64, device=device)
    ener = torch.full((y1 - y0, n), 1e-4, dtype=torch.float64, device=device)
    if kind == "tea":
        for (a, b, c, d, de, en) in PIPE_STATES:
            m = (X >= a) & (X < b) & (Y >= c) & (Y < d)
            dens = torch.where(m, torch.full_like(dens, de), dens)
            ener = torch.where(m, torch.full_like(ener, en), ener)
    elif kind == "rand":
        # G-RAND: log-uniform density in [0.1, 100] from a seed (per cell counter)
        idx = (torch.arange(y0, y1, device="cpu", dtype=torch.int64).unsqueeze(1) * n
               + torch.arange(n, dtype=torch.int64).unsqueeze(0)).numpy().ravel()
        u = (uniform_pm1(idx.size, seed=1234, offset=0, index=idx) + 1.0) * 0.5
        dens = torch.from_numpy(np.power(10.0, -1.0 + 3.0 * u).reshape(y1 - y0, n)).to(device)
    return dens, ener, dx, dy


def _coefs(n, ny, y0, y1, device, kind, kconst):
    """Face coefficients for rows [y0,y1): Kw, Ke, Ks, Kn (each (y1-y0, n)),
    zero on domain faces."""
    h = y1 - y0
    xs = torch.arange(n, device=device).unsqueeze(0).expand(h, n)
    ys = torch.arange(y0, y1, device=device).unsqueeze(1).expand(h, n)
    if kind == "const":
        one = torch.full((h, n), float(kconst), dtype=torch.float64, device=device)
        Kw = Ke = Ks = Kn = one
    else:
        lo, hi = max(y0 - 1, 0), min(y1 + 1, ny)
        dens, _, dx, dy = _fields(n, lo, hi, device, kind, ny)
        rx = DT / (dx * dx)
        ry = DT / (dy * dy)
        off = y0 - lo
        d = dens[off:off + h]
        below = dens[off - 1:off - 1 + h] if off == 1 else torch.cat([d[:1], d[:-1]])
        above = dens[off + 1:off + 1 + h] if (off + h) < dens.shape[0] else torch.cat([d[1:], d[-1:]])

        def face(d1, d2, r):
            return (r * (d1 + d2)) / ((2.0 * d1) * d2)

        left = torch.cat([d[:, :1], d[:, :-1]], dim=1)
        right = torch.cat([d[:, 1:], d[:, -1:]], dim=1)
        Kw, Ke = face(d, left, rx), face(d, right, rx)
        Ks, Kn = face(d, below, ry), face(d, above, ry)
    zero = torch.zeros((h, n), dtype=torch.float64, device=device)
    Kw = torch.where(xs > 0, Kw, zero)
    Ke = torch.where(xs < n - 1, Ke, zero)
    Ks = torch.where(ys > 0, Ks, zero)
    Kn = torch.where(ys < ny - 1, Kn, zero)
    return Kw, Ke, Ks, Kn


def strip_csr(n: int, y0: int, y1: int, ny: int | None = None, kind: str = "tea", kconst: float = 1.0,
              device="cpu", col_offset: int = 0, halo: bool = False):
    """CSR rows for grid rows [y0, y1) of an n x ny grid.

    Column indices are global flat indices minus (y0*n) plus col_offset, i.e.
    relative to a vector whose entry col_offset holds cell (0, y0).  With
    halo=True the neighbours in rows y0-1 / y1 (owned by other ranks) are
    referenced (they must exist in the extended vector); otherwise the caller
    owns the whole grid.  Returns (val f64 [5N], col int64 [5N], rowptr int64 [N+1]).
    """
    ny = n if ny is None else ny
    h = y1 - y0
    N = h * n
    Kw, Ke, Ks, Kn = _coefs(n, ny, y0, y1, device, kind, kconst)
    diag = (((1.0 + Kw) + Ke) + Ks) + Kn
    i = torch.arange(N, dtype=torch.int64, device=device).reshape(h, n) + col_offset
    xs = torch.arange(n, device=device).unsqueeze(0).expand(h, n)
    ys = torch.arange(y0, y1, device=device).unsqueeze(1).expand(h, n)
    has_s = ys > 0
    has_n = ys < ny - 1
    has_w = xs > 0
    has_e = xs < n - 1
    zero = torch.zeros((h, n), dtype=torch.float64, device=device)
    vals = torch.stack([torch.where(has_s, -Ks, zero), torch.where(has_w, -Kw, zero), diag,
                        torch.where(has_e, -Ke, zero), torch.where(has_n, -Kn, zero)], dim=-1)
    cols = torch.stack([torch.where(has_s, i - n, i), torch.where(has_w, i - 1, i), i,
                        torch.where(has_e, i + 1, i), torch.where(has_n, i + n, i)], dim=-1)
    # +0.0 (not -0.0) for out-of-grid neighbours
    vals = torch.where(vals == 0, torch.zeros_like(vals), vals)
    rowptr = torch.arange(0, 5 * N + 1, 5, dtype=torch.int64, device=device)
    return vals.reshape(-1).contiguous(), cols.reshape(-1).contiguous(), rowptr


def tealeaf_csr(n: int, device="cpu"):
    """Full n x n G-TEA matrix (single owner)."""
    return strip_csr(n, 0, n, device=device)


def const_k_csr(n: int, k: float, device="cpu"):
    """G-CONST: A = I + K * L_Neumann (PIN-9/10)."""
    return strip_csr(n, 0, n, kind="const", kconst=k, device=device)


def tealeaf_rhs(n: int, y0: int = 0, y1: int | None = None, ny: int | None = None, device="cpu"):
    """b = x0 = energy * density for grid rows [y0, y1)."""
    y1 = n if y1 is None else y1
    dens, ener, _, _ = _fields(n, y0, y1, device, "tea", ny)
    return (ener * dens).reshape(-1).contiguous()


# ------------------------------------------------------------------ splitmix64
_G = np.uint64(0x9E3779B97F4A7C15)


def splitmix64(index: np.ndarray, seed: int) -> np.ndarray:
    """Counter-based splitmix64: output k = mix(seed + (k+1)*golden)."""
    with np.errstate(over="ignore"):
        z = np.uint64(seed) + (np.asarray(index, dtype=np.uint64) + np.uint64(1)) * _G
        z = (z ^ (z >> np.uint64(30))) * np.uint64(0xBF58476D1CE4E5B9)
        z = (z ^ (z >> np.uint64(27))) * np.uint64(0x94D049BB133111EB)
        return z ^ (z >> np.uint64(31))


def uniform_pm1(n: int, seed: int, offset: int = 0, index=None) -> np.ndarray:
    """n uniforms in [-1, 1) from splitmix64 (53-bit mantissa)."""
    idx = np.arange(offset, offset + n, dtype=np.uint64) if index is None else np.asarray(index, np.uint64)
    u = (splitmix64(idx, seed) >> np.uint64(11)).astype(np.float64) * (1.0 / 9007199254740992.0)
    return 2.0 * u - 1.0


def fault_positions(seed: int, count: int, nbits_total: int) -> np.ndarray:
    """count bit positions uniform over [0, nbits_total) (O10).  Rejection-free
    modulo mapping of splitmix64 outputs (bias < 2^-40 for the sizes used)."""
    r = splitmix64(np.arange(count, dtype=np.uint64), seed)
    return (r % np.uint64(nbits_total)).astype(np.int64)


def chunk_plan(n: int, ny: int | None = None, max_cols: int = 1 << 24, chunk_rows: int | None = None,
               halo: bool = False):
    """Row-block chunks (reading R7 / S§8(c) O11) of an n x ny grid so that each
    chunk's column window [(y0-1)*n, (y1+1)*n) fits the 24-bit element index and
    its nnz fits 28-bit rowptr entries.  Returns [(y0, y1, col_base)].
    halo=True: the grid is one rank's strip of a larger grid (multi-GPU), so
    ghost rows exist above and below every chunk, also at the strip's edges."""
    ny = n if ny is None else ny

    def plan(rows):
        out = []
        for y0 in range(0, ny, rows):
            y1 = min(ny, y0 + rows)
            out.append((y0, y1, max(0, (y0 - 1) * n)))
        return out

    def fits(pl):
        def window(y0, y1, cb):
            return (y1 - y0 + 2) * n if halo else min(ny, y1 + 1) * n - cb
        return all(window(y0, y1, cb) <= max_cols and 5 * (y1 - y0) * n <= (1 << 28) - 1 for (y0, y1, cb) in pl)

    if chunk_rows is not None:
        return plan(chunk_rows)
    # fewest chunks: an even split into multiples of 8 grid rows (the SpMV tile
    # height), so the chunked SpMV pays the fewest launch tails
    for k in range(1, ny + 1):
        rows = -(-ny // k)
        rows = min(ny, -(-rows // 8) * 8)
        if fits(plan(rows)):
            return plan(rows)
    return plan(1)


def chunk_csr(n: int, y0: int, y1: int, col_base: int, ny: int | None = None, device="cpu", kind: str = "tea"):
    """CSR of grid rows [y0, y1) with column indices relative to col_base
    (global index - col_base), for a chunk that reads the global vector."""
    return strip_csr(n, y0, y1, ny=ny, kind=kind, device=device, col_offset=y0 * n - col_base)
