"""Pins of the oracle's codes against what the paper and
mathematics fix — not against the oracle itself.

* SED detects every odd flip set and misses every even one (PIN-1).
* Every SECDED instance: each single flip gives q=1 and a syndrome that locates
  exactly that bit, each double flip gives q=0, s!=0 (Hamming 1950
  [ref 11], PIN-2); brute force over all reserved patterns finds exactly one
  codeword and it is the encoder's (uniqueness of systematic encoding).
* CRC32C matches RFC 3720 B.4 check values and has HD >= 6 at our codeword
  lengths (PIN-4/5).
* Textbook instances reproduce the survey's independent self-check vectors.
"""
import itertools
import json
import math
import os
import struct

import numpy as np
import pytest

GOLD = os.path.join(os.path.dirname(__file__), "golden")


def _f(s):
    return {"pi": math.pi}.get(s, None) if s == "pi" else float(s)


def _bits(x: float) -> int:
    return struct.unpack("<Q", struct.pack("<d", x))[0]


def _h(s):
    return int(s, 16)


INSTANCES = None


def _instances(orc):
    return [orc.I_E_SECDED, orc.I_V_SECDED64, orc.I_R_SECDED64, orc.I_R_SECDED128, orc.I_V_SECDED128]


def _random_codeword(orc, inst, rng):
    nb = orc.inst_nbits(inst)
    w = rng.integers(0, 2**32, size=nb // 32, dtype=np.uint64).astype(np.uint32)
    if inst == orc.I_R_SECDED64:
        w &= np.uint32(0x0FFFFFFF)
    if inst == orc.I_R_SECDED128:
        w &= np.uint32(0x0FFFFFFF)
    if inst == orc.I_V_SECDED128:
        w[2] &= np.uint32(0xFFFFFFE0)
    return orc.secded_encode(inst, w)


# ------------------------------------------------------------------ SED (PIN-1)
def test_sed_vector_exhaustive_1_2_flips(orc):
    enc = orc.vec_encode(np.array([math.pi]), orc.SED)
    base = int(enc[0])
    for a in range(64):
        w = np.array([base ^ (1 << a)], dtype=np.uint64)
        cnt = orc.new_counts()
        orc.vec_check(w, 1, orc.SED, cnt)
        assert cnt[orc.VEC, orc.SED, orc.UNC] == 1
    for a, b in itertools.combinations(range(64), 2):
        w = np.array([base ^ (1 << a) ^ (1 << b)], dtype=np.uint64)
        cnt = orc.new_counts()
        orc.vec_check(w, 1, orc.SED, cnt)
        assert cnt.sum() == 0  # even flips are invisible to parity


def test_sed_element_and_rowptr_parity(orc):
    val = np.array([1.5, -2.25], dtype=np.float64)
    col = np.array([3, 0x7FFFFFFF], dtype=np.uint32)
    rp = np.array([0, 1, 2], dtype=np.uint32)
    A = orc.Matrix(val, col, rp, 2, 2**31, orc.SED, orc.SED)
    assert A.encode() == orc.OK
    for e in range(2):
        words = [int(A.val[e]) & 0xFFFFFFFF, int(A.val[e]) >> 32, int(A.col[e])]
        assert sum(bin(x).count("1") for x in words) % 2 == 0
    for x in A.rowptr[:3]:
        assert bin(int(x)).count("1") % 2 == 0
    # single flip anywhere in the 96-bit element -> one DUE
    for bit in range(96):
        B = orc.Matrix(val, col, rp, 2, 2**31, orc.SED, orc.SED)
        B.encode()
        if bit < 64:
            B.val[0] ^= np.uint64(1 << bit)
        else:
            B.col[0] ^= np.uint32(1 << (bit - 64))
        cnt = orc.new_counts()
        B.check(cnt)
        assert cnt[orc.ELEM, orc.SED, orc.UNC] == 1


# --------------------------------------------------------------- SECDED (PIN-2)
@pytest.mark.parametrize("inst_name", ["I_E_SECDED", "I_V_SECDED64", "I_R_SECDED64", "I_R_SECDED128",
                                       "I_V_SECDED128"])
def test_secded_single_and_double_exhaustive(orc, inst_name):
    inst = getattr(orc, inst_name)
    rng = np.random.default_rng(7)
    nb = orc.inst_nbits(inst)
    cols = orc.inst_columns(inst)
    assert len(set(cols)) == nb and cols.count(0) == 1
    for trial in range(2):
        cw = _random_codeword(orc, inst, rng)
        s, q = orc.secded_syndrome(inst, cw)
        assert (s, q) == (0, 0)
        for b in range(nb):
            w = cw.copy()
            w[b // 32] ^= np.uint32(1 << (b % 32))
            s, q = orc.secded_syndrome(inst, w)
            assert q == 1
            out, bit = orc.secded_check(inst, w)
            assert out == orc.CORRECTED and bit == b
            assert np.array_equal(w, cw)
        for a, b in itertools.combinations(range(nb), 2):
            w = cw.copy()
            w[a // 32] ^= np.uint32(1 << (a % 32))
            w[b // 32] ^= np.uint32(1 << (b % 32))
            s, q = orc.secded_syndrome(inst, w)
            assert q == 0 and s != 0
            out, _ = orc.secded_check(inst, w)
            assert out == orc.DUE


@pytest.mark.parametrize("inst_name", ["I_E_SECDED", "I_V_SECDED64", "I_R_SECDED64", "I_R_SECDED128",
                                       "I_V_SECDED128"])
def test_secded_encode_unique_by_brute_force(orc, inst_name):
    """The encoder output is the ONLY assignment of the reserved bits with
    q=0, s=0 (found by enumerating all 2^nres patterns)."""
    inst = getattr(orc, inst_name)
    res = orc.inst_reserved(inst)
    rng = np.random.default_rng(11)
    for _ in range(3):
        cw = _random_codeword(orc, inst, rng)
        sols = []
        for pat in range(1 << len(res)):
            w = cw.copy()
            for k, b in enumerate(res):
                bitv = (pat >> k) & 1
                w[b // 32] = np.uint32((int(w[b // 32]) & ~(1 << (b % 32))) | (bitv << (b % 32)))
            if orc.secded_syndrome(inst, w) == (0, 0):
                sols.append(w.copy())
        assert len(sols) == 1 and np.array_equal(sols[0], cw)


@pytest.mark.parametrize("inst_name", ["I_E_SECDED", "I_V_SECDED64", "I_R_SECDED64", "I_R_SECDED128",
                                       "I_V_SECDED128"])
def test_secded_zero_and_linearity(orc, inst_name):
    """PIN-3: enc(0) = 0 and enc(a xor b) = enc(a) xor enc(b) (linear code)."""
    inst = getattr(orc, inst_name)
    nb = orc.inst_nbits(inst)
    z = orc.secded_encode(inst, np.zeros(nb // 32, dtype=np.uint32))
    assert not z.any()
    rng = np.random.default_rng(3)
    a = _random_codeword(orc, inst, rng)
    b = _random_codeword(orc, inst, rng)
    assert np.array_equal(orc.secded_encode(inst, a ^ b), a ^ b)


def test_folded_layout_structure(orc):
    """The folded-index layouts: s[0:5] of a single flip in a
    plain data bit is that bit's index within its 32-bit word — the property the
    GPU's bit-sliced syndrome relies on.  Checked on the oracle's syndrome."""
    for inst, data_words in [(orc.I_V_SECDED64, [(0, range(8, 32)), (1, range(32))]),
                             (orc.I_E_SECDED, [(0, range(32)), (1, range(31)), (2, range(24))])]:
        nb = orc.inst_nbits(inst)
        for wi, js in data_words:
            for j in js:
                w = np.zeros(nb // 32, dtype=np.uint32)
                w[wi] = np.uint32(1 << j)
                s, q = orc.secded_syndrome(inst, w)
                assert q == 1 and (s & 31) == j


# -------------------------------------------------------------- CRC32C (PIN-4/5)
def test_crc32c_rfc3720_values(orc):
    g = json.load(open(os.path.join(GOLD, "crc32c_rfc3720.json")))
    assert orc.crc32c(b"123456789") == _h(g["check_123456789"])
    assert orc.crc32c(bytes(32)) == _h(g["zeros32"])
    assert orc.crc32c(bytes([0xFF] * 32)) == _h(g["ones32"])
    assert orc.crc32c(bytes(range(32))) == _h(g["inc32"])
    assert orc.crc32c(bytes(range(31, -1, -1))) == _h(g["dec32"])


def test_crc32c_x_plus_1_factor():
    # G(x) = x^32 + 0x1EDC6F41 terms: an even number of terms <=> (x+1) | G
    assert (bin(0x1EDC6F41).count("1") + 1) % 2 == 0


@pytest.mark.parametrize("nbytes", [32, 60])
def test_crc32c_hamming_distance_ge_6(orc, nbytes):
    """No error pattern of weight <= 4 is missed at the V/R (256-bit message)
    and E (60-byte row) lengths; with the (x+1) factor every odd weight is
    caught, so HD >= 6."""
    rng = np.random.default_rng(5)
    msg = bytes(rng.integers(0, 256, nbytes, dtype=np.uint8))
    base = orc.crc32c(msg)
    nb = 8 * nbytes
    syn = []
    for b in range(nb):
        m = bytearray(msg)
        m[b // 8] ^= 1 << (b % 8)
        syn.append(orc.crc32c(bytes(m)) ^ base)
    # the CRC field itself is also part of the codeword: its bits have syndromes 1<<k
    syn += [1 << k for k in range(32)]
    S = set(syn)
    assert 0 not in S and len(S) == len(syn)                 # weight 1, 2 (same CRC field)
    pairs = {}
    n = len(syn)
    for i in range(n):
        si = syn[i]
        for j in range(i + 1, n):
            x = si ^ syn[j]
            assert x not in S                                 # weight 3
            assert x not in pairs                             # weight 4 (and 2)
            pairs[x] = (i, j)


# ---------------------------------------------------------- survey SSV pins
def _ssv():
    return json.load(open(os.path.join(GOLD, "survey_ssv.json")))


def _val(s):
    return math.pi if s == "pi" else float(s)


def test_ssv_v_sed(orc):
    for v, hexs in _ssv()["v_sed"]:
        assert int(orc.vec_encode(np.array([_val(v)]), orc.SED)[0]) == _h(hexs)


def test_ssv_v_secded64_masked_rounding(orc):
    for v, m in _ssv()["v_secded64_masked"]:
        enc = orc.vec_encode(np.array([_val(v)]), orc.SECDED64)
        assert orc.vec_masked(enc, 1, orc.SECDED64)[0] == m


def test_ssv_v_secded128(orc):
    for vals, hexs in _ssv()["v_secded128"]:
        enc = orc.vec_encode(np.array([_val(x) for x in vals]), orc.SECDED128)
        assert [int(x) for x in enc] == [_h(h) for h in hexs]


def _rowptr_group(orc, entries, scheme):
    n = len(entries) - 1
    val = np.zeros(max(entries[-1], 1), dtype=np.float64)
    col = np.zeros(max(entries[-1], 1), dtype=np.uint32)
    A = orc.Matrix(val, col, np.array(entries, dtype=np.uint32), n, 1, orc.NONE, scheme)
    A.nnz = int(entries[-1])
    # encode only the rowptr: nnz must match the last entry for padding
    A.encode()
    return [int(x) for x in A.rowptr[:len(entries)]]


def test_ssv_r_secded64(orc):
    for ents, hexs in _ssv()["r_secded64"]:
        w = orc.secded_encode(orc.I_R_SECDED64, np.array(ents, dtype=np.uint32))
        assert [int(x) for x in w] == [_h(h) for h in hexs]


def test_ssv_r_secded128(orc):
    for ents, hexs in _ssv()["r_secded128"]:
        w = orc.secded_encode(orc.I_R_SECDED128, np.array(ents, dtype=np.uint32))
        assert [int(x) for x in w] == [_h(h) for h in hexs]


def test_ssv_v_crc(orc):
    g = _ssv()["v_crc"]
    enc = orc.vec_encode(np.array([_val(x) for x in g["values"]]), orc.CRC32C)
    assert [int(x) for x in enc] == [_h(h) for h in g["stored"]]


def test_ssv_r_crc(orc):
    g = _ssv()["r_crc"]
    ents = g["values"]
    # a 7-row matrix whose rowptr is exactly these 8 entries (nnz = 35)
    val = np.ones(35)
    col = np.zeros(35, dtype=np.uint32)
    A = orc.Matrix(val, col, np.array(ents, dtype=np.uint32), 7, 1, orc.NONE, orc.CRC32C)
    assert A.encode() == orc.OK
    assert [int(x) for x in A.rowptr[:8]] == [_h(h) for h in g["stored"]]


def test_ssv_e_crc(orc):
    g = _ssv()["e_crc"]
    n, i = g["n"], g["row"]
    cols = [i - n, i - 1, i, i + 1, i + n]
    A = orc.Matrix(np.array(g["vals"]), np.array(cols, dtype=np.uint32), np.array([0, 5], dtype=np.uint32), 1,
                   n * n, orc.CRC32C, orc.NONE)
    assert A.encode() == orc.OK
    assert [int(x) for x in A.col] == [_h(h) for h in g["stored_cols"]]


# ------------------------------------------------------------- capacity (PIN-6/7)
def test_capacity_edges(orc):
    one = np.array([1.0])
    rp = np.array([0, 1], dtype=np.uint32)
    ok = orc.Matrix(one, np.array([2**24 - 1], dtype=np.uint32), rp, 1, 2**24, orc.SECDED64, orc.SECDED64)
    assert ok.encode() == orc.OK
    bad = orc.Matrix(one, np.array([2**24], dtype=np.uint32), rp, 1, 2**24 + 1, orc.SECDED64, orc.SECDED64)
    assert bad.encode() == orc.E_RANGE
    sed = orc.Matrix(one, np.array([2**31 - 1], dtype=np.uint32), rp, 1, 2**31, orc.SED, orc.SED)
    assert sed.encode() == orc.OK
    # CRC rows need >= 4 entries
    crc = orc.Matrix(np.ones(3), np.array([0, 1, 2], dtype=np.uint32), np.array([0, 3], dtype=np.uint32), 1, 3,
                     orc.CRC32C, orc.NONE)
    assert crc.encode() == orc.E_SHAPE


def test_zero_storage_overhead(orc):
    """protected buffers have the unprotected byte size (+ < G padding)."""
    for n in [1, 7, 1024, 1025]:
        for s, g in [(orc.NONE, 1), (orc.SED, 1), (orc.SECDED64, 1), (orc.SECDED128, 2), (orc.CRC32C, 4)]:
            p = orc.vec_padded_len(n, s)
            assert n <= p < n + g
        for s, g in [(orc.SED, 1), (orc.SECDED64, 2), (orc.SECDED128, 4), (orc.CRC32C, 8)]:
            p = orc.rowptr_padded_len(n, s)
            assert n + 1 <= p < n + 1 + g


def test_rounding_rule(orc):
    """round half away from zero at 2^k ulp; Inf/NaN truncated."""
    one = _bits(1.0)
    assert orc.round_k(one + 0x7F, 8) == one
    assert orc.round_k(one + 0x80, 8) == one + 0x100
    neg = _bits(-1.0)
    assert orc.round_k(neg + 0x80, 8) == neg + 0x100        # magnitude rounds up
    inf = _bits(float("inf"))
    assert orc.round_k(inf, 8) == inf
    nan = 0x7FF80000000000FF
    assert orc.round_k(nan, 8) == 0x7FF8000000000000
    mx = 0x7FEFFFFFFFFFFFFF                                  # largest finite -> Inf allowed
    assert orc.round_k(mx, 8) == inf
