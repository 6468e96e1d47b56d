"""The CG solvers with programmatic dependent launch ON (abft_ctx_set_pdl,
DESIGN.md §6.2) — the configuration bench.py times — bit-exact against the
oracle exactly as without it.  PDL lets a kernel's pre-wait part (matrix
loads; the SpMV's `in` window TMA when the host marks `in` final, early_in)
overlap its predecessor, so these re-run the CG parity tests of the other
modules on a PDL context: tiled CG to convergence at 512^2 with flips,
scheduled mid-solve faults (the injection kernel sits before the SpMV, so the
early window is off), DUE abort inside graph replays, the single-reduction CG,
PPCG (whose init copies p right before iteration 1), Chebyshev and the fused
calc_p arrangement.
"""
import pytest

import test_gpu_cheby as tch
import test_gpu_faults as tfa
import test_gpu_fused as tfu
import test_gpu_geometry as tge
import test_gpu_ppcg as tpp
import test_gpu_sr as tsr

pytestmark = pytest.mark.gpu
orc = tfa.orc


@pytest.fixture(scope="module")
def abft():
    from paper_conf_cluster_pawelczakmpm17_b200 import abft as a
    return a


@pytest.fixture(scope="module")
def pctx(abft):
    import torch
    torch.cuda.set_device(0)
    c = abft.Context(0)
    c.set_pdl(True)
    return c


def test_pdl_tiled_cg_512_converged(abft, pctx):
    tge.test_tiled_cg_512_converged(abft, pctx)


@pytest.mark.parametrize("stencil", [0, 256])
def test_pdl_scheduled_singles(abft, pctx, stencil):
    tfa.test_config2_schemes_mid_solve_singles(abft, pctx, stencil)


@pytest.mark.parametrize("t,k", [(orc.F_P, 13), (orc.F_X, 9), (orc.F_VAL, 21)])
def test_pdl_due_abort_in_graph(abft, pctx, t, k):
    tfa.test_due_abort_mid_solve_in_graph(abft, pctx, t, k)


@pytest.mark.parametrize("vs", ["SED", "SECDED64", "CRC32C"])
def test_pdl_sr_parity(abft, pctx, vs):
    tsr.test_sr_parity(abft, pctx, vs, 256, 256, 45)


@pytest.mark.parametrize("vs", ["SECDED64", "SECDED128"])
def test_pdl_ppcg_parity(abft, pctx, vs):
    tpp.test_ppcg_parity(abft, pctx, vs, 256, 256, 12, 3)


def test_pdl_cheby_parity(abft, pctx):
    tch.test_cheby_parity(abft, pctx, "SECDED64", 256, 256, 60)


@pytest.mark.parametrize("fused", [True, False])
def test_pdl_fused_cg_parity(abft, pctx, fused):
    tfu.test_fused_cg_parity(abft, pctx, "SECDED64", 41, fused)
