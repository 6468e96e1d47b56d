"""Shared helpers for the GPU parity tests: build the same seeded problem on
both sides (oracle on the host, libabft.so on the device) from gen/."""
from __future__ import annotations

import numpy as np
import torch

import gen
import oracle as orc


def tea(n: int, kind: str = "tea"):
    if kind == "tea":
        v, c, r = gen.tealeaf_csr(n)
    else:
        v, c, r = gen.const_k_csr(n, 0.7)
    return v.numpy(), c.numpy().astype(np.uint32), r.numpy().astype(np.uint32)


def gpu_matrix(abft, ctx, v, c, r, nrows, ncols, es, rs, row_base=0, col_base=0, stencil_n=0):
    A = abft.Matrix(torch.from_numpy(v).cuda(), torch.from_numpy(c.view(np.int32)).cuda(),
                    torch.from_numpy(r.view(np.int32)).cuda(), nrows, ncols, es, rs, row_base=row_base,
                    col_base=col_base, stencil_n=stencil_n)
    st = A.encode(ctx)
    return A, st


def oracle_matrix(v, c, r, nrows, ncols, es, rs, row_base=0, col_base=0):
    A = orc.Matrix(v, c, r, nrows, ncols, es, rs, row_base=row_base, col_base=col_base)
    st = A.encode()
    return A, st


def gpu_vec_from_words(abft, words: np.ndarray, n: int, scheme: int):
    t = torch.from_numpy(words.view(np.int64).copy()).cuda()
    return abft.Vector(t.view(torch.float64), n, scheme)


def words_of(vec) -> np.ndarray:
    return vec.data.view(torch.int64).cpu().numpy().view(np.uint64)


def col_words(A) -> np.ndarray:
    return A.col.cpu().numpy().view(np.uint32)


def rowptr_words(A) -> np.ndarray:
    return A.rowptr.cpu().numpy().view(np.uint32)


def val_words(A) -> np.ndarray:
    return A.val.view(torch.int64).cpu().numpy().view(np.uint64)
