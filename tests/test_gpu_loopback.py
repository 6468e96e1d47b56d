"""The product's multi-rank CG path (cg_run with P > 1: halo exchange of
encoded p, interior/boundary SpMV split that overlaps it, per-rank RED-1
subtree roots all-gathered and combined by the same top of the tree, DUE
consensus under policy abort, CUDA graph of the whole iteration) executed on
ONE GPU through the in-library loopback transport (abft_dist_init_loopback):
P = 2, 4, 8 virtual ranks, each a horizontal strip of the grid with one ghost
grid row above / below (§V-A, "spatially
decomposed regular grid").

Checked against the single-process oracle CG: equal iteration count and status,
bit-identical x on every strip (RED-1 makes the dots independent of P), and
fault counters that sum to the single-process counts (owner rule: a flipped
halo cell is corrected in registers by the neighbour, counted once by its
owner)."""
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


def _oracle(n, S, vflips, eflips, policy, max_iters, interval=1):
    N = n * n
    v, c, r = gen.tealeaf_csr(n)
    Ao = orc.Matrix(v.numpy(), c.numpy().astype(np.uint32), r.numpy().astype(np.uint32), N, N, S, S)
    assert Ao.encode() == 0
    for (e, bit) in eflips:
        Ao.val[e] ^= np.uint64(1 << bit)
    b = gen.tealeaf_rhs(n).numpy()
    bo = orc.vec_encode(b, S)
    xo = bo.copy()
    for (i, bits) in vflips:
        for bit in bits:
            xo[i] ^= np.uint64(1 << bit)
    ro, po, wo = (np.zeros_like(bo) for _ in range(3))
    cnt = orc.new_counts()
    st, res = orc.cg_solve(Ao, bo, xo, ro, po, wo, S, 1e-10, max_iters, policy, cnt, check_interval=interval)
    return st, res, xo[:N], cnt


def _loopback(abft, n, P, S, stencil, vflips, eflips, policy, max_iters, interval=1, poll=8, sr=False, peer=False):
    rows = n // P
    h = n
    ctxs, As, vecs, cnts = [], [], [], []
    b = gen.tealeaf_rhs(n).numpy()
    bo = orc.vec_encode(b, S)
    for q in range(P):
        y0, y1 = q * rows, (q + 1) * rows
        Nl = rows * n
        v, c, r = gen.strip_csr(n, y0, y1, ny=n, col_offset=h)
        v, c, r = v.numpy(), c.numpy().astype(np.uint32), r.numpy().astype(np.uint32)
        ctx = abft.Context(0)
        A = abft.Matrix(torch.from_numpy(v).cuda(), torch.from_numpy(c.view(np.int32)).cuda(),
                        torch.from_numpy(r.view(np.int32)).cuda(), Nl, Nl + 2 * h, S, S, row_base=h, col_base=0,
                        stencil_n=stencil)
        assert A.encode(ctx) == 0
        for (e, bit) in eflips:   # global element index -> owner strip
            if y0 * n * 5 <= e < y1 * n * 5:
                abft.inject_bitflip(ctx, A.val, 64 * (e - y0 * n * 5) + bit)
        be = np.zeros(Nl + 2 * h, dtype=np.uint64)
        be[h:h + Nl] = bo[y0 * n:y1 * n]
        xe = be.copy()
        for (i, bits) in vflips:
            if y0 * n <= i < y1 * n:
                for bit in bits:
                    xe[h + i - y0 * n] ^= np.uint64(1 << bit)
        vs = [gpu_vec_from_words(abft, a, Nl + 2 * h, S) for a in (be, xe)]
        vs += [abft.Vector.empty(Nl + 2 * h, S) for _ in range(4 if sr else 3)]
        ctxs.append(ctx)
        As.append(A)
        vecs.append(vs)
        cnts.append(abft.Counters())
    d = abft.Loopback(P, 0)
    if peer:
        d.set_peer_halo(True)
    if sr:
        res = d.cg_solve_sr(ctxs, As, h, vecs, tol=1e-10, max_iters=max_iters, due_policy=policy, counts=cnts,
                            poll_every=poll)
    else:
        res = d.cg_solve(ctxs, As, h, vecs, tol=1e-10, max_iters=max_iters, due_policy=policy, counts=cnts,
                         poll_every=poll, check_interval=interval)
    torch.cuda.synchronize()
    x = np.concatenate([words_of(vecs[q][1])[h:h + rows * n] for q in range(P)])
    cnt = sum(c.read() for c in cnts)
    d.close()
    return res, x, cnt


CASES = [(64, 0, 2), (64, 0, 4), (64, 0, 8), (256, 256, 2), (256, 256, 4), (256, 256, 8)]


@pytest.mark.parametrize("n,stencil,P", CASES)
@pytest.mark.parametrize("policy", [0, 1])
def test_loopback_cg_matches_oracle(abft, n, stencil, P, policy):
    S = orc.SECDED64
    rows = n // P
    # single flips in x0 at strip boundaries (halo cells of the neighbours) and
    # inside a strip, plus element-value flips in two strips
    vflips = [((rows - 1) * n + 5, [9]), (rows * n + 7, [40]), (rows * n // 2 + 3, [0]), (n * n - 1, [63])]
    eflips = [(5 * (rows * n - 2) + 4, 17), (5 * (n * n // 2 + 11) + 2, 60)]
    st, res_o, xo, cnt_o = _oracle(n, S, vflips, eflips, policy, 400)
    res, x, cnt = _loopback(abft, n, P, S, stencil, vflips, eflips, policy, 400)
    assert st == 0
    for q in range(P):
        assert res[q].iters == res_o.iters and res[q].status == st, (q, res[q].iters, res_o.iters)
        assert res[q].rrn == res_o.rrn and res[q].rr0 == res_o.rr0
    assert np.array_equal(x, xo)
    assert np.array_equal(cnt, cnt_o), (cnt, cnt_o)
    assert cnt[orc.VEC, S, orc.COR] == len(vflips) and cnt[orc.ELEM, S, orc.COR] == len(eflips)


@pytest.mark.parametrize("n,stencil,P", [(64, 0, 4), (256, 256, 4), (256, 256, 8)])
@pytest.mark.parametrize("policy", [0, 1])
def test_loopback_due_consensus(abft, n, stencil, P, policy):
    """A same-word double flip (DUE) in one strip's halo row of x0: under
    policy abort every rank stops after the same iteration with ABFT_E_DUE
    (all-gathered DUE flags); under continue the masked stored bits are used
    on both sides of the halo and the solve matches the oracle."""
    S = orc.SECDED64
    rows = n // P
    vflips = [(2 * rows * n - 3, [20, 33])]
    st, res_o, xo, cnt_o = _oracle(n, S, vflips, [], policy, 400)
    res, x, cnt = _loopback(abft, n, P, S, stencil, vflips, [], policy, 400)
    for q in range(P):
        assert res[q].iters == res_o.iters and res[q].status == st
    if policy == 0:
        assert st == orc.E_DUE
    assert np.array_equal(x, xo)
    assert np.array_equal(cnt, cnt_o)


@pytest.mark.parametrize("P", [2, 4])
def test_loopback_interval_and_maxiters(abft, P):
    """Interval checking and a max_iters stop through the loopback:
    the final detection-only sweep's DUE flags are all-gathered too."""
    n = 256
    S = orc.SECDED64
    st, res_o, xo, cnt_o = _oracle(n, S, [], [(5 * 1000 + 1, 3)], 1, 37, interval=4)
    res, x, cnt = _loopback(abft, n, P, S, n, [], [(5 * 1000 + 1, 3)], 1, 37, interval=4)
    for q in range(P):
        assert res[q].iters == res_o.iters == 37 and res[q].status == st
    assert np.array_equal(x, xo)
    assert np.array_equal(cnt, cnt_o)


def test_loopback_graph_vs_direct(abft):
    """poll_every larger than the solve (direct issue only) vs small polls (CUDA
    graph replays of the multi-rank iteration): identical results."""
    n, P, S = 256, 4, orc.SECDED64
    r1, x1, c1 = _loopback(abft, n, P, S, n, [], [], 1, 60, poll=1000)
    r2, x2, c2 = _loopback(abft, n, P, S, n, [], [], 1, 60, poll=4)
    assert [r.iters for r in r1] == [r.iters for r in r2]
    assert np.array_equal(x1, x2) and np.array_equal(c1, c2)


@pytest.mark.parametrize("n,stencil,P", [(64, 0, 4), (256, 256, 2), (256, 256, 8)])
@pytest.mark.parametrize("policy", [0, 1])
def test_loopback_single_reduction_cg(abft, n, stencil, P, policy):
    """Single-reduction CG on P strips: r's halo before the
    SpMV, ONE all-gather of (w.r root, DUE flag, r.r root) per iteration;
    bit-identical to the single-process oracle or_cg_solve_sr."""
    S = orc.SECDED64
    N = n * n
    rows = n // P
    vflips = [((rows - 1) * n + 5, [9]), (rows * n + 7, [40])]
    v, c, r = gen.tealeaf_csr(n)
    Ao = orc.Matrix(v.numpy(), c.numpy().astype(np.uint32), r.numpy().astype(np.uint32), N, N, S, S)
    assert Ao.encode() == 0
    bo = orc.vec_encode(gen.tealeaf_rhs(n).numpy(), S)
    xo = bo.copy()
    for (i, bits) in vflips:
        for bit in bits:
            xo[i] ^= np.uint64(1 << bit)
    ro, po, wo, so = (np.zeros_like(bo) for _ in range(4))
    cnt_o = orc.new_counts()
    st, res_o = orc.cg_solve_sr(Ao, bo.copy(), xo, ro, po, wo, so, S, 1e-10, 400, policy, cnt_o)
    res, x, cnt = _loopback(abft, n, P, S, stencil, vflips, [], policy, 400, sr=True)
    for q in range(P):
        assert res[q].iters == res_o.iters and res[q].status == st and res[q].rrn == res_o.rrn
    assert np.array_equal(x, xo[:N])
    assert np.array_equal(cnt, cnt_o)


@pytest.mark.parametrize("n,stencil,P", [(64, 0, 2), (64, 0, 8), (256, 256, 2), (256, 256, 4), (256, 256, 8)])
@pytest.mark.parametrize("policy", [0, 1])
def test_loopback_peer_halo_matches_oracle(abft, n, stencil, P, policy):
    """Peer-memory halos (abft_dist_set_peer_halo): calc_p stores p's boundary
    rows straight into the neighbours' ghost rows and the SpMV waits on arrival
    flags — iterations, residuals, x and counters bit-exact against the
    single-domain oracle, flips in halo cells included (tiled strips: the wait
    overlaps the interior tile rows on the comm stream)."""
    S = orc.SECDED64
    rows = n // P
    vflips = [((rows - 1) * n + 5, [9]), (rows * n + 7, [40]), (rows * n // 2 + 3, [0]), (n * n - 1, [63])]
    eflips = [(5 * (rows * n - 2) + 4, 17), (5 * (n * n // 2 + 11) + 2, 60)]
    st, res_o, xo, cnt_o = _oracle(n, S, vflips, eflips, policy, 400)
    l0 = abft.launch_count()
    res, x, cnt = _loopback(abft, n, P, S, stencil, vflips, eflips, policy, 400, peer=True)
    l_peer = abft.launch_count() - l0
    assert st == 0
    for q in range(P):
        assert res[q].iters == res_o.iters and res[q].status == st, (q, res[q].iters, res_o.iters)
        assert res[q].rrn == res_o.rrn and res[q].rr0 == res_o.rr0
    assert np.array_equal(x, xo)
    assert np.array_equal(cnt, cnt_o), (cnt, cnt_o)
    # the halo step ran as flag waits (one kernel per rank and iteration), not copies
    l0 = abft.launch_count()
    _loopback(abft, n, P, S, stencil, vflips, eflips, policy, 400)
    l_copy = abft.launch_count() - l0
    assert l_peer - l_copy >= P * res_o.iters, (l_peer, l_copy)


@pytest.mark.parametrize("P", [2, 4])
@pytest.mark.parametrize("policy", [0, 1])
def test_loopback_peer_halo_due(abft, P, policy):
    """A same-word double flip (DUE) in a halo row of x0 with peer halos:
    the DUE consensus and the statuses / counters match the oracle."""
    n, S = 256, orc.SECDED64
    rows = n // P
    vflips = [(rows * n + 3, [5, 6])]
    st, res_o, xo, cnt_o = _oracle(n, S, vflips, [], policy, 60)
    res, x, cnt = _loopback(abft, n, P, S, n, vflips, [], policy, 60, peer=True)
    for q in range(P):
        assert res[q].iters == res_o.iters and res[q].status == st
    if policy == 0:
        assert st == orc.E_DUE
    assert np.array_equal(x, xo)
    assert np.array_equal(cnt, cnt_o)
