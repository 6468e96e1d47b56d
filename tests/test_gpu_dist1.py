"""The multi-GPU code path of the library (abft_cg_solve_dist: halo-extended
vectors, RED-1 subtree root + DUE flag all-gathered over NCCL, top-of-tree
combine kernel, DUE all-gather after calc_p) run with ONE rank on one GPU —
the only multi-GPU configuration this round's single-GPU boxes allow.  It must
reproduce the single-GPU solve and the oracle bit-exactly."""
import numpy as np
import pytest
import torch

import gen
import oracle as orc
from gpu_helpers import gpu_vec_from_words, words_of

pytestmark = pytest.mark.gpu


@pytest.fixture(scope="module")
def abft():
    from paper_conf_cluster_pawelczakmpm17_b200 import build
    build.build()
    from paper_conf_cluster_pawelczakmpm17_b200 import abft as A
    return A


@pytest.mark.parametrize("n,stencil", [(32, 0), (256, 256)])
@pytest.mark.parametrize("policy", [0, 1])
def test_dist_one_rank_matches_single(abft, n, stencil, policy):
    ctx = abft.Context(0)
    d = abft.Dist(0, 1, 0)
    S = orc.SECDED64
    N = n * n
    h = n
    v, c, r = gen.strip_csr(n, 0, n, ny=n, col_offset=h)
    v, c, r = v.numpy(), c.numpy().astype(np.uint32), r.numpy().astype(np.uint32)
    Ag = abft.Matrix(torch.from_numpy(v).cuda(), torch.from_numpy(c.view(np.int32)).cuda(),
                     torch.from_numpy(r.view(np.int32)).cuda(), N, N + 2 * h, S, S, row_base=h, col_base=0,
                     stencil_n=stencil)
    assert Ag.encode(ctx) == 0
    b = gen.tealeaf_rhs(n).numpy()
    bo = orc.vec_encode(b, S)
    ext = np.zeros(N + 2 * h, dtype=np.uint64)
    be, xe = ext.copy(), ext.copy()
    be[h:h + N] = bo[:N]
    xe[h:h + N] = bo[:N]
    xe[h + 77] ^= np.uint64(1 << 9)                       # one single flip in x0
    vecs = [gpu_vec_from_words(abft, a, N + 2 * h, S) for a in (be, xe)]
    vecs += [abft.Vector.empty(N + 2 * h, S) for _ in range(3)]
    cnt = abft.Counters()
    res = d.cg_solve(ctx, Ag, h, *vecs, tol=1e-10, max_iters=60, due_policy=policy, counts=cnt, poll_every=8)
    # oracle, plain single-process matrix
    v0, c0, r0 = gen.tealeaf_csr(n)
    Ao = orc.Matrix(v0.numpy(), c0.numpy().astype(np.uint32), r0.numpy().astype(np.uint32), N, N, S, S)
    Ao.encode()
    xo = bo.copy()
    xo[77] ^= np.uint64(1 << 9)
    ro, po, wo = (np.zeros_like(bo) for _ in range(3))
    cnt_o = orc.new_counts()
    st, res_o = orc.cg_solve(Ao, bo.copy(), xo, ro, po, wo, S, 1e-10, 60, policy, cnt_o)
    assert res.iters == res_o.iters and res.status == st
    assert np.array_equal(words_of(vecs[1])[h:h + N], xo[:N])
    assert np.array_equal(cnt.read(), cnt_o)
    d.close()
