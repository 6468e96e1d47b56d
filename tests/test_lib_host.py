"""CPU-side checks of the CUDA library (no GPU needed):

* libabft.so loads and exports every function include/abft.h declares;
* the exact __host__ __device__ codec functions the kernels use agree with the
  oracle bit for bit (encode) and outcome for outcome (check) on every single-
  and double-bit flip of random codewords of every SECDED instance.
"""
import itertools
import os
import re

import numpy as np
import pytest

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


@pytest.fixture(scope="module")
def lib():
    from paper_conf_cluster_pawelczakmpm17_b200 import build
    build.build()
    from paper_conf_cluster_pawelczakmpm17_b200 import abft
    return abft


def test_exports_every_header_symbol(lib):
    hdr = open(os.path.join(ROOT, "include", "abft.h")).read()
    hdr = re.sub(r"/\*.*?\*/", "", hdr, flags=re.S)
    declared = set(re.findall(r"\b(abft_[a-z0-9_]+)\s*\(", hdr))
    assert declared, "no declarations parsed"
    import ctypes
    so = ctypes.CDLL(lib._SO)
    missing = [s for s in declared if not hasattr(so, s)]
    assert not missing, missing
    assert declared <= set(lib.HEADER_SYMBOLS)


def _rand_words(orc, inst, rng):
    nb = orc.inst_nbits(inst)
    w = rng.integers(0, 2**32, size=nb // 32, dtype=np.uint64).astype(np.uint32)
    if inst in (orc.I_R_SECDED64, orc.I_R_SECDED128):
        w &= np.uint32(0x0FFFFFFF)
    if inst == orc.I_V_SECDED64:
        w[0] &= np.uint32(0xFFFFFF00)
    if inst == orc.I_V_SECDED128:
        w[0] &= np.uint32(0xFFFFFFE0)
        w[2] &= np.uint32(0xFFFFFFE0)
    if inst == orc.I_E_SECDED:
        w[2] &= np.uint32(0x00FFFFFF)
    return w


@pytest.mark.parametrize("inst_name", ["I_E_SECDED", "I_V_SECDED64", "I_R_SECDED64", "I_R_SECDED128",
                                       "I_V_SECDED128"])
def test_host_codec_matches_oracle(lib, orc, inst_name):
    inst = getattr(orc, inst_name)
    nb = orc.inst_nbits(inst)
    rng = np.random.default_rng(100 + inst)
    for _ in range(3):
        data = _rand_words(orc, inst, rng)
        cw_o = orc.secded_encode(inst, data)
        cw_g = np.array(lib.codec_host_encode(inst, list(data)), dtype=np.uint32)
        assert np.array_equal(cw_o, cw_g), (inst_name, [hex(x) for x in cw_o], [hex(x) for x in cw_g])
        assert lib.codec_host_check(inst, list(cw_g)) == orc.CLEAN
        for b in range(nb):
            w = cw_g.copy()
            w[b // 32] ^= np.uint32(1 << (b % 32))
            lst = list(w)
            o = lib.codec_host_check(inst, lst)
            assert o == orc.CORRECTED and np.array_equal(np.array(lst, dtype=np.uint32), cw_g), (inst_name, b)
        pairs = list(itertools.combinations(range(nb), 2))
        for idx in rng.choice(len(pairs), 300, replace=False):
            a, b = pairs[idx]
            w = cw_g.copy()
            w[a // 32] ^= np.uint32(1 << (a % 32))
            w[b // 32] ^= np.uint32(1 << (b % 32))
            assert lib.codec_host_check(inst, list(w)) == orc.DUE


def test_host_pair_fast_check_matches_oracle(lib, orc):
    """The tiled SpMV's pair-packed E-SECDED fast check (codec e96_acc2, host
    hook inst 5) says 'clean' exactly when the oracle finds both codewords
    clean: every single flip of either codeword, random doubles within one and
    across both, and random 3-flip patterns."""
    rng = np.random.default_rng(77)
    inst = orc.I_E_SECDED
    for _ in range(20):
        cws = []
        for _ in range(2):
            data = _rand_words(orc, inst, rng)
            cws.append(orc.secded_encode(inst, data))
        both = np.concatenate(cws)
        assert lib.codec_host_check(5, list(both)) == orc.CLEAN
        patterns = [[b] for b in range(192)]
        patterns += [list(rng.choice(192, 2, replace=False)) for _ in range(200)]
        patterns += [list(rng.choice(192, 3, replace=False)) for _ in range(100)]
        for pat in patterns:
            w = both.copy()
            for b in pat:
                w[b // 32] ^= np.uint32(1 << (b % 32))
            ref = [orc.secded_check(inst, w[3 * k:3 * k + 3].copy()) for k in range(2)]
            clean = all(o[0] == orc.CLEAN for o in ref)
            assert (lib.codec_host_check(5, list(w)) == orc.CLEAN) == clean, pat


def test_host_pair_window_check_matches_oracle(lib, orc):
    """The decoded window's pair-packed V-SECDED64 fast check (codec v64_acc2,
    host hook inst 6) says 'clean' exactly when the oracle finds both codewords
    clean (singles of either word, random doubles and triples)."""
    rng = np.random.default_rng(78)
    inst = orc.I_V_SECDED64
    for _ in range(20):
        both = np.concatenate([orc.secded_encode(inst, _rand_words(orc, inst, rng)) for _ in range(2)])
        assert lib.codec_host_check(6, list(both)) == orc.CLEAN
        patterns = [[b] for b in range(128)]
        patterns += [list(rng.choice(128, 2, replace=False)) for _ in range(200)]
        patterns += [list(rng.choice(128, 3, replace=False)) for _ in range(100)]
        for pat in patterns:
            w = both.copy()
            for b in pat:
                w[b // 32] ^= np.uint32(1 << (b % 32))
            clean = all(orc.secded_check(inst, w[2 * k:2 * k + 2].copy())[0] == orc.CLEAN for k in range(2))
            assert (lib.codec_host_check(6, list(w)) == orc.CLEAN) == clean, pat
