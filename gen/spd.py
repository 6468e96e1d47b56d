"""G-SPD: general (non-stencil) sparse SPD matrices for the gather path
(S§8(f) f4: "general SPD CSR through the gather path"; the paper claims its
techniques apply beyond TeaLeaf).

A = I + L(W): the weighted Laplacian of a random undirected graph plus the
identity, so A is symmetric, strictly diagonally dominant with a positive
diagonal, hence SPD.  Node i links to `deg` random partners (splitmix64), so
row lengths vary (1 + the node's degree, >= deg + 1 >= 4 for E-CRC).  Columns
are sorted within each row.  Holds no method arithmetic: only the matrix
recipe and random numbers.
"""
from __future__ import annotations

import numpy as np

from .tealeaf import splitmix64


def random_spd_csr(n: int, deg: int = 4, seed: int = 1, wmax: float = 2.0):
    """(val f64[nnz], col u32[nnz], rowptr u32[n+1]) of I + L(W) on n nodes."""
    assert n > deg
    src = np.repeat(np.arange(n, dtype=np.int64), deg)
    r = splitmix64(np.arange(n * deg, dtype=np.uint64), seed)
    dst = ((src + 1 + (r % np.uint64(n - 1)).astype(np.int64)) % n)   # never a self loop
    w = (splitmix64(np.arange(n * deg, dtype=np.uint64), seed + 7) >> np.uint64(11)).astype(np.float64)
    w = 0.05 + w * (wmax / 9007199254740992.0)
    # symmetrise: keep each undirected pair once (first occurrence wins)
    a, b = np.minimum(src, dst), np.maximum(src, dst)
    key = a * n + b
    _, first = np.unique(key, return_index=True)
    a, b, w = a[first], b[first], w[first]
    rows = np.concatenate([a, b])
    cols = np.concatenate([b, a])
    vals = np.concatenate([-w, -w])
    diag = np.ones(n)
    np.add.at(diag, a, w)
    np.add.at(diag, b, w)
    rows = np.concatenate([rows, np.arange(n)])
    cols = np.concatenate([cols, np.arange(n)])
    vals = np.concatenate([vals, diag])
    order = np.lexsort((cols, rows))
    rows, cols, vals = rows[order], cols[order], vals[order]
    rowptr = np.zeros(n + 1, dtype=np.uint32)
    np.add.at(rowptr, rows + 1, 1)
    rowptr = np.cumsum(rowptr).astype(np.uint32)
    return vals.astype(np.float64), cols.astype(np.uint32), rowptr
