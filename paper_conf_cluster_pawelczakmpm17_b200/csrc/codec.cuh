// codec.cuh — device (and host-testable) ABFT codecs for sm_100a.
//
// Implements DESIGN.md §3 (restating PAPER.md §IV P:196-284 and §VI
// P:352-451): SED parity, SECDED syndrome+parity with single-bit correction
// (P:230-238), CRC32C detection, the 96-bit CSR element code in the
// column's spare top byte, row-pointer codes in the top bits
// and vector codes in the low mantissa bits.
//
// The two hot instances (E-SECDED: every CSR element, V-SECDED64: every vector
// access) use the folded-index layout of DESIGN.md §3.2, so the 5 "index" rows
// of the syndrome of a container are the bit-sliced superset-sum (Moebius)
// transform of ONE 32-bit fold register: 10 LOP3/SHF instead of 5 POPC
// (POPC issues at 16/clk/SM on B200 vs 64/clk/SM for LOP3; measured,
// tools/microbench/pipes.cu).  The fast path only decides "clean?"; locating
// and correcting a flip is a cold, divergent path ("correction happens very
// infrequently, unlike error detection").
//
// Every function is __host__ __device__ so the exact same code is unit-tested
// on the host against the oracle (abft_codec_host_* in capi.cu).
#pragma once
#include <stdint.h>

#if defined(__CUDACC__)
#define ABFT_HD __host__ __device__ __forceinline__
#else
#define ABFT_HD inline
#endif

namespace abft {

enum Scheme { NONE = 0, SED = 1, SECDED64 = 2, SECDED128 = 3, CRC32C = 4, NSCHEME = 5 };
enum Target { T_ELEM = 0, T_ROWPTR = 1, T_VEC = 2, NTARGET = 3 };
enum Outcome { CLEAN = 0, CORRECTED = 1, DUE = 2 };

// ------------------------------------------------------------ bit helpers
ABFT_HD int popc32(uint32_t x) {
#if defined(__CUDA_ARCH__)
  return __popc(x);
#else
  return __builtin_popcount(x);
#endif
}
ABFT_HD int popc64(uint64_t x) {
#if defined(__CUDA_ARCH__)
  return __popcll(x);
#else
  return __builtin_popcountll(x);
#endif
}
// PRMT: result byte i = byte sel_i of the 8-byte pair {y:x}.
ABFT_HD uint32_t byte_perm(uint32_t x, uint32_t y, uint32_t s) {
#if defined(__CUDA_ARCH__)
  return __byte_perm(x, y, s);
#else
  uint64_t v = ((uint64_t)y << 32) | x;
  uint32_t r = 0;
  for (int i = 0; i < 4; i++) r |= (uint32_t)((v >> (8 * ((s >> (4 * i)) & 7))) & 0xFF) << (8 * i);
  return r;
#endif
}
// LOP3 with an explicit truth table (a = 0xF0, b = 0xCC, c = 0xAA): ptxas does
// not always merge a mask-and-combine into one LOP3 on its own.
template <uint32_t LUT>
ABFT_HD uint32_t lop3(uint32_t a, uint32_t b, uint32_t c) {
#if defined(__CUDA_ARCH__)
  uint32_t r;
  asm("lop3.b32 %0, %1, %2, %3, %4;" : "=r"(r) : "r"(a), "r"(b), "r"(c), "n"(LUT));
  return r;
#else
  uint32_t r = 0;
  for (int i = 0; i < 8; i++)
    if ((LUT >> i) & 1u) r |= ((i & 4) ? a : ~a) & ((i & 2) ? b : ~b) & ((i & 1) ? c : ~c);
  return r;
#endif
}
ABFT_HD uint32_t lo32(uint64_t u) { return (uint32_t)u; }
ABFT_HD uint32_t hi32(uint64_t u) { return (uint32_t)(u >> 32); }
ABFT_HD uint64_t mk64(uint32_t lo, uint32_t hi) { return ((uint64_t)hi << 32) | lo; }

// Subset-sum (Moebius / zeta) transform of a 32-bit fold register:
// R[i] = XOR_{j subset of i} D[j].  Then R[31] = parity(D) and, for k = 0..4,
// R[31 - 2^k] = parity of the bits whose index has bit k CLEAR, i.e.
// R[31] ^ R[31 - 2^k] = bit k of (XOR of the indices of the set bits of D).
// Only left shifts: ptxas emits IMAD.SHL (FMA pipe) for them, so the 10-op
// transform splits across the ALU and FMA pipes (measured faster on sm_100a,
// tools/microbench/codec.cu).
constexpr ABFT_HD uint32_t moebius32(uint32_t d) {
  d ^= (d << 1) & 0xAAAAAAAAu;
  d ^= (d << 2) & 0xCCCCCCCCu;
  d ^= (d << 4) & 0xF0F0F0F0u;
  d ^= (d << 8) & 0xFF00FF00u;
  d ^= (d << 16) & 0xFFFF0000u;
  return d;
}
// R bits {31, 30, 29, 27, 23, 15}: all zero <=> parity 0 and index syndrome 0
constexpr uint32_t MOEB_SYN_MASK = 0xE8808000u;
// "any syndrome or parity bit set" over OR-accumulated Moebius registers and
// code-row popcounts of several codewords
ABFT_HD bool syn_bad(uint32_t acc_r, uint32_t acc_p) { return ((acc_r & MOEB_SYN_MASK) | (acc_p & 1u)) != 0u; }
// q and the 5-bit index syndrome from a Moebius register
ABFT_HD int moeb_q(uint32_t r) { return (int)(r >> 31); }
ABFT_HD int moeb_index(uint32_t r) {
  const uint32_t q = r >> 31;
  return (int)(((r >> 30) & 1) ^ q) | (int)((((r >> 29) & 1) ^ q) << 1) | (int)((((r >> 27) & 1) ^ q) << 2) |
         (int)((((r >> 23) & 1) ^ q) << 3) | (int)((((r >> 15) & 1) ^ q) << 4);
}
// inverse: the Moebius-register bits a (q, index syndrome) pair produces
constexpr ABFT_HD uint32_t moeb_bits(int q, int idx) {
  uint32_t r = (uint32_t)q << 31;
  r |= (uint32_t)(q ^ (idx & 1)) << 30;
  r |= (uint32_t)(q ^ ((idx >> 1) & 1)) << 29;
  r |= (uint32_t)(q ^ ((idx >> 2) & 1)) << 27;
  r |= (uint32_t)(q ^ ((idx >> 3) & 1)) << 23;
  r |= (uint32_t)(q ^ ((idx >> 4) & 1)) << 15;
  return r;
}

// ------------------------------------------------------ layout tables
// A layout = the H column of every container bit (DESIGN.md §3.2/§3.3).
struct Layout {
  int nbits;
  int r;          // syndrome bits
  int col[128];
  int nres;       // reserved bits (checks + parity)
  int res[16];
};

// E-SECDED.  A = val[0:32], B = val[32:64], C = col.
constexpr Layout make_e96() {
  Layout L{};
  L.nbits = 96; L.r = 7; L.nres = 8;
  for (int j = 0; j < 32; j++) L.col[j] = j;
  for (int j = 0; j < 31; j++) L.col[32 + j] = j | 32;
  L.col[63] = 31 | 96;
  for (int j = 0; j < 24; j++) L.col[64 + j] = j | 64;
  const int pos[8] = {8, 17, 26, 27, 28, 29, 30, 31};
  const int code[8] = {3, 3, 3, 3, 3, 2, 2, 1};
  for (int t = 0; t < 8; t++) { L.col[88 + t] = pos[t] | (code[t] << 5); L.res[t] = 88 + t; }
  return L;
}
// V-SECDED64.  A = bits 0..31 (reserved A[0:8]), B = bits 32..63.
constexpr Layout make_v64() {
  Layout L{};
  L.nbits = 64; L.r = 7; L.nres = 8;
  for (int j = 8; j < 32; j++) L.col[j] = j;
  for (int j = 0; j < 32; j++) L.col[32 + j] = j | 32;
  const int pos[8] = {0, 9, 18, 3, 4, 5, 6, 7};
  const int code[8] = {0, 2, 2, 2, 0, 0, 0, 3};
  for (int t = 0; t < 8; t++) { L.col[t] = pos[t] | (code[t] << 5); L.res[t] = t; }
  return L;
}
// Textbook extended Hamming: c_k at position 2^k, P at 0, the
// remaining bits (forced-zero included) numbered 3,5,6,7,9,... in container order.
constexpr Layout make_textbook(int nbits, int r, const int* cpos, int ppos) {
  Layout L{};
  L.nbits = nbits; L.r = r; L.nres = r + 1;
  bool is_res[128] = {};
  for (int k = 0; k < r; k++) { is_res[cpos[k]] = true; L.col[cpos[k]] = 1 << k; L.res[k] = cpos[k]; }
  is_res[ppos] = true; L.col[ppos] = 0; L.res[r] = ppos;
  int p = 3;
  for (int b = 0; b < nbits; b++) {
    if (is_res[b]) continue;
    while ((p & (p - 1)) == 0) p++;
    L.col[b] = p++;
  }
  return L;
}
constexpr int kR64C[7] = {28, 29, 30, 31, 60, 61, 62};
constexpr int kR128C[8] = {28, 29, 30, 31, 60, 61, 62, 63};
constexpr int kV128C[8] = {0, 1, 2, 3, 4, 64, 65, 66};
constexpr Layout kE96 = make_e96();
constexpr Layout kV64 = make_v64();
constexpr Layout kR64 = make_textbook(64, 7, kR64C, 63);
constexpr Layout kR128 = make_textbook(128, 8, kR128C, 92);
constexpr Layout kV128 = make_textbook(128, 8, kV128C, 67);

// mask of container word w whose bits have syndrome row k set (k == r: all bits)
constexpr uint32_t row_mask(const Layout& L, int k, int w) {
  uint32_t m = 0;
  for (int j = 0; j < 32; j++) {
    int b = 32 * w + j;
    if (b >= L.nbits) break;
    if (k == L.r || ((L.col[b] >> k) & 1)) m |= 1u << j;
  }
  return m;
}
// Per-instance row masks + reserved positions (constant bank on the device:
// LOP3 reads c[] operands directly, warp-uniform indices broadcast).
struct MaskTable { uint32_t m[9][4]; int res[9]; };
constexpr MaskTable make_masks(const Layout& L) {
  MaskTable T{};
  for (int k = 0; k <= L.r; k++)
    for (int w = 0; w < 4; w++) T.m[k][w] = row_mask(L, k, w);
  for (int k = 0; k < L.nres && k < 9; k++) T.res[k] = L.res[k];
  return T;
}
#if defined(__CUDACC__)
static __constant__ MaskTable c_mt_r64 = make_masks(kR64);
static __constant__ MaskTable c_mt_r128 = make_masks(kR128);
static __constant__ MaskTable c_mt_v128 = make_masks(kV128);
#endif
constexpr MaskTable h_mt_r64 = make_masks(kR64);
constexpr MaskTable h_mt_r128 = make_masks(kR128);
constexpr MaskTable h_mt_v128 = make_masks(kV128);

// Column -> container bit (-1: not a column).  Only used on the cold path.
struct ColMap { int16_t bit[256]; };
constexpr ColMap make_colmap(const Layout& L) {
  ColMap M{};
  for (int i = 0; i < 256; i++) M.bit[i] = -1;
  for (int b = 0; b < L.nbits; b++) M.bit[L.col[b]] = (int16_t)b;
  return M;
}

#if defined(__CUDACC__)
static __constant__ ColMap c_map_e96 = make_colmap(kE96);
static __constant__ ColMap c_map_v64 = make_colmap(kV64);
static __constant__ ColMap c_map_r64 = make_colmap(kR64);
static __constant__ ColMap c_map_r128 = make_colmap(kR128);
static __constant__ ColMap c_map_v128 = make_colmap(kV128);
#endif
constexpr ColMap h_map_e96 = make_colmap(kE96);
constexpr ColMap h_map_v64 = make_colmap(kV64);
constexpr ColMap h_map_r64 = make_colmap(kR64);
constexpr ColMap h_map_r128 = make_colmap(kR128);
constexpr ColMap h_map_v128 = make_colmap(kV128);

#if defined(__CUDA_ARCH__)
#define ABFT_MAP(name) c_map_##name
#define ABFT_MT(name) c_mt_##name
#else
#define ABFT_MAP(name) h_map_##name
#define ABFT_MT(name) h_mt_##name
#endif

// Generic syndrome over NW 32-bit words via masked POPC (textbook instances):
// s = sum_k parity(w & mask_k) << k, q = parity(all).
template <int NW, int R>
ABFT_HD void generic_syndrome(const MaskTable& M, const uint32_t* w, int& s, int& q) {
  s = 0;
#pragma unroll
  for (int k = 0; k < R; k++) {
    uint32_t t = 0;
#pragma unroll
    for (int i = 0; i < NW; i++) t ^= w[i] & M.m[k][i];
    s |= (popc32(t) & 1) << k;
  }
  uint32_t t = 0;
#pragma unroll
  for (int i = 0; i < NW; i++) t ^= w[i];
  q = popc32(t) & 1;
}

// Locate + correct given (s, q) (cold path).  Returns outcome, *word = index
// of the corrected 32-bit word (for the scrub CAS).
template <int NW>
ABFT_HD int secded_resolve(const ColMap& M, uint32_t* w, int s, int q, int* word) {
  if (q == 0 && s == 0) return CLEAN;
  if (q == 0) return DUE;
  int b = M.bit[s];
  if (b < 0 || b >= 32 * NW) return DUE;
  w[b >> 5] ^= 1u << (b & 31);
  if (word) *word = b >> 5;
  return CORRECTED;
}

// ======================================================== vectors (f64)
// reserved LSBs per scheme
ABFT_HD int vec_k(int s) { return s == SED ? 1 : s == SECDED64 ? 8 : s == SECDED128 ? 5 : s == CRC32C ? 8 : 0; }
ABFT_HD int vec_group(int s) { return s == SECDED128 ? 2 : s == CRC32C ? 4 : 1; }
ABFT_HD uint64_t vec_keep(int s) { int k = vec_k(s); return k ? ~((1ull << k) - 1ull) : ~0ull; }

// round_k: + 2^(k-1), clear k LSBs; Inf/NaN truncated (R11/R12)
ABFT_HD uint64_t round_k(uint64_t u, int k) {
  if (k == 0) return u;
  uint64_t keep = ~((1ull << k) - 1ull);
  if (((u >> 52) & 0x7FF) == 0x7FF) return u & keep;
  return (u + (1ull << (k - 1))) & keep;
}

// ---- V-SED: even parity of the 64-bit pattern, parity bit = bit 0
ABFT_HD bool vsed_clean(uint64_t u) { return (popc64(u) & 1) == 0; }
ABFT_HD uint64_t vsed_encode(uint64_t rounded) {
  uint64_t d = rounded & ~1ull;
  return d | (uint64_t)(popc64(d) & 1);
}

// ---- V-SECDED64 (folded).  Fold register: A with A1, A2 moved to fold
// positions 9 and 18 (one PRMT copies byte 0 into bytes 1 and 2).
ABFT_HD uint32_t v64_fold(uint32_t a, uint32_t b) {
  uint32_t t = byte_perm(a, 0u, 0x4004u);           // [0, a.b0, a.b0, 0]
  return lop3<0x78>(lop3<0x6C>(a, b, ~0x6u), t, 0x00040200u);   // (a & ~6) ^ b ^ (t & mask)
}
// Returns nonzero iff the codeword is NOT clean (fast path).
ABFT_HD void v64_acc(uint32_t a, uint32_t b, uint32_t& acc_r, uint32_t& acc_p) {
  acc_r |= moebius32(v64_fold(a, b));
  acc_p |= (uint32_t)(popc32(b ^ (a & 0x80u)) | popc32(a & 0x8Eu));
}
// Two V-SECDED64 codewords at once (the decoded SpMV window's slot pairs):
// the fold registers' 4-step Moebius shared as in e96_acc2, par(lo) of each
// fold and the two code rows by POPC.  Nonzero (acc_u & MOEB2_SYN_MASK, or
// acc_p bit 0) iff either codeword fails v64_bad.
ABFT_HD void v64_acc2(uint32_t a1, uint32_t b1, uint32_t a2, uint32_t b2, uint32_t& acc_u, uint32_t& acc_p);
ABFT_HD uint32_t v64_bad(uint32_t a, uint32_t b) {
  uint32_t r = moebius32(v64_fold(a, b));
  uint32_t s56 = (uint32_t)(popc32(b ^ (a & 0x80u)) | popc32(a & 0x8Eu)) & 1u;
  return (r & MOEB_SYN_MASK) | s56;
}
ABFT_HD void v64_syndrome(uint32_t a, uint32_t b, int& s, int& q) {
  uint32_t r = moebius32(v64_fold(a, b));
  s = moeb_index(r) | ((popc32(b ^ (a & 0x80u)) & 1) << 5) | ((popc32(a & 0x8Eu) & 1) << 6);
  q = moeb_q(r);
}
// Slow path: correct in place; returns outcome, *word = 0/1 for the half fixed.
ABFT_HD int v64_correct(uint64_t& u, int* word) {
  uint32_t w[2] = {lo32(u), hi32(u)};
  int s, q;
  v64_syndrome(w[0], w[1], s, q);
  int o = secded_resolve<2>(ABFT_MAP(v64), w, s, q, word);
  if (o == CORRECTED) u = mk64(w[0], w[1]);
  return o;
}
// Encoder LUT: index = ((R & MOEB_SYN_MASK) | s5) * 0x10000805 >> 25, a
// bijection of the 7 data-syndrome bits (q, s0..s5) onto 0..127 (found by
// search); s6 of the data part is always 0 because no data bit of V-SECDED64
// has code bit 1.
constexpr uint32_t V64_LUT_MUL = 0x10000805u;
constexpr ABFT_HD uint32_t v64_lut_index(uint32_t r, uint32_t s5) {
  return (((r & MOEB_SYN_MASK) | (s5 & 1u)) * V64_LUT_MUL) >> 25;
}
struct V64Lut { uint8_t r[128]; };
constexpr V64Lut make_v64_lut() {
  // For every reserved byte whose own s6 is 0, its syndrome (q,s0..s5) is the
  // data syndrome it cancels; record it under that syndrome's index.
  V64Lut T{};
  for (int r = 0; r < 256; r++) {
    int s = 0, q = 0;
    for (int b = 0; b < 8; b++) if ((r >> b) & 1) { s ^= kV64.col[b]; q ^= 1; }
    if ((s >> 6) & 1) continue;
    T.r[v64_lut_index(moeb_bits(q, s & 31), (uint32_t)((s >> 5) & 1))] = (uint8_t)r;
  }
  return T;
}
constexpr V64Lut h_v64_lut = make_v64_lut();
#if defined(__CUDACC__)
static __constant__ V64Lut c_v64_lut = make_v64_lut();
#endif
// Encode with a LUT pointer (shared-memory copy on the device: 128 B = one word
// per bank, conflict-free for any index pattern).
ABFT_HD uint64_t v64_encode_lut(uint64_t rounded, const uint8_t* lut) {
  uint32_t a = lo32(rounded) & ~0xFFu, b = hi32(rounded);
  uint32_t r = moebius32(a ^ b);
  uint32_t idx = v64_lut_index(r, (uint32_t)popc32(b));
  return mk64(a | lut[idx], b);
}

// ---- V-SECDED128 (textbook, pair of doubles; 5 LSBs each)
ABFT_HD void v128_syndrome(const uint32_t* w, int& s, int& q) { generic_syndrome<4, 8>(ABFT_MT(v128), w, s, q); }
ABFT_HD void v128_encode(uint64_t* d) {   // d[0..1] already rounded (low 5 bits zero)
  uint32_t w[4] = {lo32(d[0]) & ~0x1Fu, hi32(d[0]), lo32(d[1]) & ~0x1Fu, hi32(d[1])};
  int s, q;
  v128_syndrome(w, s, q);
  // c_k (unit columns) = s bit k, P = q ^ parity(c): textbook systematic encode
#pragma unroll
  for (int k = 0; k < 8; k++) {
    int b = ABFT_MT(v128).res[k];
    w[b >> 5] |= (uint32_t)((s >> k) & 1) << (b & 31);
  }
  int pc = popc32((uint32_t)s) & 1;
  w[2] |= (uint32_t)(q ^ pc) << (67 - 64);
  d[0] = mk64(w[0], w[1]);
  d[1] = mk64(w[2], w[3]);
}
// Fast "not clean?" test of a pair (bit 0 of the result set <=> q or some
// syndrome bit is 1): OR of the 9 row popcounts, masks as immediates.
ABFT_HD uint32_t v128_acc(uint64_t d0, uint64_t d1) {
  constexpr MaskTable M = h_mt_v128;
  const uint32_t w[4] = {lo32(d0), hi32(d0), lo32(d1), hi32(d1)};
  uint32_t acc = (uint32_t)popc32(w[0] ^ w[1] ^ w[2] ^ w[3]);
#pragma unroll
  for (int k = 0; k < 8; k++) {
    uint32_t t = 0;
#pragma unroll
    for (int i = 0; i < 4; i++)
      if (M.m[k][i]) t ^= w[i] & M.m[k][i];
    acc |= (uint32_t)popc32(t);
  }
  return acc;
}
ABFT_HD int v128_check(uint64_t* d, int* word) {
  uint32_t w[4] = {lo32(d[0]), hi32(d[0]), lo32(d[1]), hi32(d[1])};
  int s, q;
  v128_syndrome(w, s, q);
  if (!s && !q) return CLEAN;
  int o = secded_resolve<4>(ABFT_MAP(v128), w, s, q, word);
  if (o == CORRECTED) { d[0] = mk64(w[0], w[1]); d[1] = mk64(w[2], w[3]); }
  return o;
}

// ---- CRC32C (bit-parallel by nibble tables would go here; plain bitwise
// for the detection-only sweep instances)
ABFT_HD uint32_t crc32c_update(uint32_t crc, uint32_t byte) {
  crc ^= byte;
  for (int k = 0; k < 8; k++) crc = (crc >> 1) ^ (0x82F63B78u & (0u - (crc & 1u)));
  return crc;
}
ABFT_HD uint32_t crc32c_u32(uint32_t crc, uint32_t v) {
  for (int i = 0; i < 4; i++) crc = crc32c_update(crc, (v >> (8 * i)) & 0xFF);
  return crc;
}
// V-CRC over 4 doubles (low bytes zeroed in the message)
ABFT_HD uint32_t vcrc_compute(const uint64_t* d) {
  uint32_t c = 0xFFFFFFFFu;
  for (int i = 0; i < 4; i++) {
    c = crc32c_u32(c, lo32(d[i]) & ~0xFFu);
    c = crc32c_u32(c, hi32(d[i]));
  }
  return c ^ 0xFFFFFFFFu;
}
ABFT_HD void vcrc_encode(uint64_t* d) {
  for (int i = 0; i < 4; i++) d[i] &= ~0xFFull;
  uint32_t c = vcrc_compute(d);
  for (int i = 0; i < 4; i++) d[i] |= (uint64_t)((c >> (8 * i)) & 0xFF);
}
ABFT_HD bool vcrc_clean(const uint64_t* d) {
  uint32_t st = 0;
  for (int i = 0; i < 4; i++) st |= (uint32_t)(d[i] & 0xFF) << (8 * i);
  return st == vcrc_compute(d);
}

// ---- CRC32C single-bit correction, 1EC4ED;
// optional pair correction, 2EC3ED (crc_locate2 below).
// CRC32C is affine in the message, so a failing codeword's syndrome
// syn = stored CRC ^ recomputed CRC depends only on the error pattern: a flip
// of stored CRC bit t gives 1 << t; a flip of message bit i (bytes LSB-first,
// i = 8 * byte + bit) of an M-bit message gives the register that a single 1
// at position i leaves after the remaining M-1-i zero bits, i.e.
// step0^(M-1-i)(poly).  Within CRC32C's HD-6 range (message + 32 <= 5243
// bits) all these syndromes are distinct and no pattern of 2..4
// flips shares one, so a match corrects exactly one bit and anything else is
// a DUE (1EC4ED).  This runs only on the cold (failed-check) path.
constexpr int CRC_NO_FIX = -1000;
constexpr int CRC_HD6_MAX_BITS = 5243;
ABFT_HD int ctz32(uint32_t x) {
#if defined(__CUDA_ARCH__)
  return __ffs((int)x) - 1;
#else
  return __builtin_ctz(x);
#endif
}
// >= 0: message bit index; -1 - t: stored CRC bit t; CRC_NO_FIX: no single-bit explanation.
ABFT_HD int crc_locate(uint32_t syn, int mbits) {
  if (syn == 0u || mbits + 32 > CRC_HD6_MAX_BITS) return CRC_NO_FIX;
  if ((syn & (syn - 1u)) == 0u) return -1 - ctz32(syn);
  uint32_t v = 0x82F63B78u;   // syndrome of the last message bit
  for (int i = mbits - 1; i >= 0; i--) {
    if (v == syn) return i;
    v = (v >> 1) ^ (0x82F63B78u & (0u - (v & 1u)));
  }
  return CRC_NO_FIX;
}
// 2EC3ED (reading R9b): when no single flip explains syn, the
// unique pair of positions (message bits and / or stored CRC bits) whose
// syndromes XOR to syn; with HD 6 a weight-2 error is unique and a weight-3
// one never matches.  Returns 2 with pos[0..1] (encoded as crc_locate) or 0.
// O(M^2) register steps: cold path only.
ABFT_HD int crc_locate2(uint32_t syn, int mbits, int* pos) {
  if (syn == 0u || mbits + 32 > CRC_HD6_MAX_BITS) return 0;
  const uint32_t P = 0x82F63B78u;
  if (popc32(syn) == 2) {   // two stored CRC bits
    pos[0] = -1 - ctz32(syn);
    pos[1] = -1 - ctz32(syn & (syn - 1u));
    return 2;
  }
  uint32_t vi = P;   // S(i) for i = mbits-1 .. 0
  for (int i = mbits - 1; i >= 0; i--) {
    const uint32_t t = syn ^ vi;
    if ((t & (t - 1u)) == 0u) {   // message bit i + stored CRC bit
      pos[0] = i;
      pos[1] = -1 - ctz32(t);
      return 2;
    }
    uint32_t vj = vi;
    for (int j = i - 1; j >= 0; j--) {
      vj = (vj >> 1) ^ (P & (0u - (vj & 1u)));
      if (vj == t) { pos[0] = i; pos[1] = j; return 2; }
    }
    vi = (vi >> 1) ^ (P & (0u - (vi & 1u)));
  }
  return 0;
}
// CRC32C correction capability of a launch (1 = 1EC4ED, 2 = 2EC3ED): cfg is
// the context's device int[4] flag block (cfg[1], set by
// abft_ctx_set_crc_correction); read only on the cold path.
ABFT_HD int crc_t_of(const int* cfg) { return (cfg && cfg[1] == 2) ? 2 : 1; }
// Positions of a failing CRC codeword to flip: 1 (1EC), 2 (2EC) or 0 (DUE).
ABFT_HD int crc_fix_positions(uint32_t syn, int mbits, const int* cfg, int* pos) {
  const int r = crc_locate(syn, mbits);
  if (r != CRC_NO_FIX) { pos[0] = r; return 1; }
  if (crc_t_of(cfg) == 2) return crc_locate2(syn, mbits, pos);
  return 0;
}
// V-CRC quad: check, locate and correct in place (1 or 2 bits); *word = 32-bit
// word index of the (first) corrected bit in the group.
ABFT_HD int vcrc_check_fix(uint64_t* d, int* word, const int* cfg = nullptr) {
  uint32_t st = 0;
  for (int i = 0; i < 4; i++) st |= (uint32_t)(d[i] & 0xFF) << (8 * i);
  const uint32_t syn = st ^ vcrc_compute(d);
  if (!syn) return CLEAN;
  int pos[2];
  const int np = crc_fix_positions(syn, 256, cfg, pos);
  if (np == 0) return DUE;
  int bits[2];
  for (int q = 0; q < np; q++) {
    const int r = pos[q];
    if (r < 0) bits[q] = 64 * ((-1 - r) >> 3) + ((-1 - r) & 7);   // CRC byte t/8 = low byte of double t/8
    else {
      const int byte = r >> 3, bb = byte & 7;
      if (bb == 0) return DUE;                    // zeroed message byte: not a stored bit
      bits[q] = 64 * (byte >> 3) + 8 * bb + (r & 7);
    }
  }
  for (int q = 0; q < np; q++) d[bits[q] >> 6] ^= 1ull << (bits[q] & 63);
  if (word) *word = bits[0] >> 5;
  return CORRECTED;
}

// Generic vector group encode / check (G = vec_group(S) consecutive values).
template <int S>
ABFT_HD void vec_encode_group(uint64_t* d, const uint8_t* v64lut) {
  if (S == SED) d[0] = vsed_encode(d[0]);
  else if (S == SECDED64) d[0] = v64_encode_lut(d[0], v64lut);
  else if (S == SECDED128) v128_encode(d);
  else if (S == CRC32C) vcrc_encode(d);
}
// Returns outcome; corrects d in place; *word = 32-bit word (within the group)
// that was corrected.
template <int S>
ABFT_HD int vec_check_group(uint64_t* d, int* word, const int* cfg = nullptr) {
  if (S == SED) return vsed_clean(d[0]) ? CLEAN : DUE;
  if (S == SECDED64) {
    if (!v64_bad(lo32(d[0]), hi32(d[0]))) return CLEAN;
    return v64_correct(d[0], word);
  }
  if (S == SECDED128) return v128_check(d, word);
  if (S == CRC32C) return vcrc_check_fix(d, word, cfg);
  return CLEAN;
}

// ======================================================== CSR elements
ABFT_HD uint32_t col_keep(int s) { return s == NONE ? 0xFFFFFFFFu : s == SED ? 0x7FFFFFFFu : 0x00FFFFFFu; }
ABFT_HD uint64_t col_limit(int s) { return s == NONE ? 0xFFFFFFFFull : s == SED ? 0x7FFFFFFFull : 0x00FFFFFFull; }

// ---- E-SECDED (folded).  Fold register: A ^ B ^ C with C24, C25 moved to fold
// positions 8 and 17 (PRMT copies col's top byte into bytes 1 and 2).
ABFT_HD uint32_t e96_fold(uint32_t a, uint32_t b, uint32_t c) {
  // t = [0, c.b3, c.b3, c.b3]; XOR-ing t & 0x03020100 removes C24/C25 from
  // fold positions 24/25 and inserts them at 8/17 (PRMT + 2 LOP3).
  uint32_t t = byte_perm(c, 0u, 0x3334u);
  return lop3<0x78>(lop3<0x96>(a, b, c), t, 0x03020100u);   // (a ^ b ^ c) ^ (t & mask)
}
// Accumulating fast check (OR the Moebius registers and the code-row popcounts
// of several codewords, test once with syn_bad): one branch per row / step.
// Code rows: s5 = parity(b ^ (c & 0x9F000000)), s6 = parity(b[31] | c[0:31]).
ABFT_HD void e96_acc(uint32_t a, uint32_t b, uint32_t c, uint32_t& acc_r, uint32_t& acc_p) {
  acc_r |= moebius32(e96_fold(a, b, c));
  acc_p |= (uint32_t)(popc32(lop3<0x78>(b, c, 0x9F000000u)) | popc32(lop3<0xE4>(b, c, 0x80000000u)));
}

// Two E-SECDED codewords at once (the hot path's element pairs): the five
// index-syndrome bits and the overall parity of a fold F are parities of its
// 16-bit halves' XOR u = lo ^ hi (R31, R30, R29, R27, R23 = the 4-step
// Moebius transform of u at bits 15, 14, 13, 11, 7) plus par(lo) (R15).  The
// two codewords' u share one register, so the 4 Moebius steps run once for
// both; par(lo) of each is a POPC next to the code-row POPCs.  OR-accumulates
// into acc_u (test with MOEB2_SYN_MASK) and acc_p (bit 0): nonzero iff either
// codeword's syndrome or parity is nonzero — exactly e96_bad of each.
constexpr uint32_t MOEB2_SYN_MASK = 0xE880E880u;
ABFT_HD void e96_acc2(uint32_t a1, uint32_t b1, uint32_t c1, uint32_t a2, uint32_t b2, uint32_t c2, uint32_t& acc_u,
                      uint32_t& acc_p) {
  const uint32_t f1 = e96_fold(a1, b1, c1), f2 = e96_fold(a2, b2, c2);
  const uint32_t x = byte_perm(f1, f2, 0x5410u), y = byte_perm(f1, f2, 0x7632u);   // lo halves, hi halves
  uint32_t u = x ^ y;
  u ^= (u << 1) & 0xAAAAAAAAu;
  u ^= (u << 2) & 0xCCCCCCCCu;
  u ^= (u << 4) & 0xF0F0F0F0u;
  u ^= (u << 8) & 0xFF00FF00u;
  acc_u |= u;
  acc_p |= (uint32_t)(popc32(x & 0xFFFFu) | popc32(x >> 16) | popc32(lop3<0x78>(b1, c1, 0x9F000000u)) |
                      popc32(lop3<0xE4>(b1, c1, 0x80000000u)) | popc32(lop3<0x78>(b2, c2, 0x9F000000u)) |
                      popc32(lop3<0xE4>(b2, c2, 0x80000000u)));
}

ABFT_HD void v64_acc2(uint32_t a1, uint32_t b1, uint32_t a2, uint32_t b2, uint32_t& acc_u, uint32_t& acc_p) {
  const uint32_t f1 = v64_fold(a1, b1), f2 = v64_fold(a2, b2);
  const uint32_t x = byte_perm(f1, f2, 0x5410u), y = byte_perm(f1, f2, 0x7632u);
  uint32_t u = x ^ y;
  u ^= (u << 1) & 0xAAAAAAAAu;
  u ^= (u << 2) & 0xCCCCCCCCu;
  u ^= (u << 4) & 0xF0F0F0F0u;
  u ^= (u << 8) & 0xFF00FF00u;
  acc_u |= u;
  acc_p |= (uint32_t)(popc32(x & 0xFFFFu) | popc32(x >> 16) | popc32(b1 ^ (a1 & 0x80u)) | popc32(a1 & 0x8Eu) |
                      popc32(b2 ^ (a2 & 0x80u)) | popc32(a2 & 0x8Eu));
}

ABFT_HD uint32_t e96_bad(uint32_t a, uint32_t b, uint32_t c) {
  uint32_t r = 0, p = 0;
  e96_acc(a, b, c, r, p);
  return syn_bad(r, p) ? 1u : 0u;
}
ABFT_HD void e96_syndrome(uint32_t a, uint32_t b, uint32_t c, int& s, int& q) {
  uint32_t r = moebius32(e96_fold(a, b, c));
  s = moeb_index(r) | ((popc32(b ^ (c & 0x9F000000u)) & 1) << 5) |
      ((popc32((c & 0x7FFFFFFFu) ^ (b & 0x80000000u)) & 1) << 6);
  q = moeb_q(r);
}
ABFT_HD int e96_correct(uint64_t& v, uint32_t& c, int* word) {
  uint32_t w[3] = {lo32(v), hi32(v), c};
  int s, q;
  e96_syndrome(w[0], w[1], w[2], s, q);
  int o = secded_resolve<3>(ABFT_MAP(e96), w, s, q, word);
  if (o == CORRECTED) { v = mk64(w[0], w[1]); c = w[2]; }
  return o;
}
// Encode (cold, once per solve): solve the 8 reserved bits by trying the 256
// patterns' syndromes against the data syndrome (table built on first use).
struct E96Enc { uint8_t r[256]; };
constexpr E96Enc make_e96_enc() {
  E96Enc T{};
  for (int r = 0; r < 256; r++) {
    int s = 0, q = 0;
    for (int t = 0; t < 8; t++) if ((r >> t) & 1) { s ^= kE96.col[88 + t]; q ^= 1; }
    T.r[(s | (q << 7)) & 255] = (uint8_t)r;
  }
  return T;
}
constexpr E96Enc h_e96_enc = make_e96_enc();
#if defined(__CUDACC__)
static __constant__ E96Enc c_e96_enc = make_e96_enc();
#endif
ABFT_HD uint32_t e96_encode_col(uint64_t v, uint32_t col24) {
  uint32_t c = col24 & 0x00FFFFFFu;
  int s, q;
  e96_syndrome(lo32(v), hi32(v), c, s, q);
#if defined(__CUDA_ARCH__)
  uint32_t r = c_e96_enc.r[(s | (q << 7)) & 255];
#else
  uint32_t r = h_e96_enc.r[(s | (q << 7)) & 255];
#endif
  return c | (r << 24);
}

ABFT_HD uint32_t esed_encode_col(uint64_t v, uint32_t col31) {
  uint32_t c = col31 & 0x7FFFFFFFu;
  uint32_t p = (uint32_t)((popc64(v) + popc32(c)) & 1);
  return c | (p << 31);
}
ABFT_HD bool esed_clean(uint64_t v, uint32_t c) { return ((popc64(v) + popc32(c)) & 1) == 0; }

// Element check for the non-CRC element schemes: corrects in place.
template <int ES>
ABFT_HD int elem_check(uint64_t& v, uint32_t& c, int* word) {
  if (ES == SED) return esed_clean(v, c) ? CLEAN : DUE;
  if (ES == SECDED64 || ES == SECDED128) {
    if (!e96_bad(lo32(v), hi32(v), c)) return CLEAN;
    return e96_correct(v, c, word);
  }
  return CLEAN;
}

// E-CRC over one row's entries (message: val LE, col LE with top byte zeroed
// for entries 0..3).
ABFT_HD uint32_t ecrc_update(uint32_t crc, uint64_t v, uint32_t c, int k) {
  crc = crc32c_u32(crc, lo32(v));
  crc = crc32c_u32(crc, hi32(v));
  return crc32c_u32(crc, k < 4 ? (c & 0x00FFFFFFu) : c);
}

// ======================================================== row pointers
ABFT_HD int rp_group(int s) { return s == SECDED64 ? 2 : s == SECDED128 ? 4 : s == CRC32C ? 8 : 1; }
ABFT_HD uint32_t rp_keep(int s) { return s == NONE ? 0xFFFFFFFFu : s == SED ? 0x7FFFFFFFu : 0x0FFFFFFFu; }
ABFT_HD uint64_t rp_limit(int s) { return s == NONE ? 0xFFFFFFFFull : s == SED ? 0x7FFFFFFFull : 0x0FFFFFFFull; }

ABFT_HD uint32_t rcrc_compute(const uint32_t* e) {
  uint32_t c = 0xFFFFFFFFu;
  for (int i = 0; i < 8; i++) c = crc32c_u32(c, e[i] & 0x0FFFFFFFu);
  return c ^ 0xFFFFFFFFu;
}

template <int RS>
ABFT_HD void rp_encode_group(uint32_t* e) {
  if (RS == SED) {
    uint32_t d = e[0] & 0x7FFFFFFFu;
    e[0] = d | ((uint32_t)(popc32(d) & 1) << 31);
  } else if (RS == SECDED64 || RS == SECDED128) {
    constexpr int NW = (RS == SECDED64) ? 2 : 4;
    constexpr int R = (RS == SECDED64) ? 7 : 8;
    const MaskTable& M = (RS == SECDED64) ? ABFT_MT(r64) : ABFT_MT(r128);
#pragma unroll
    for (int i = 0; i < NW; i++) e[i] &= 0x0FFFFFFFu;
    int s, q;
    generic_syndrome<NW, R>(M, e, s, q);
#pragma unroll
    for (int k = 0; k < R; k++) { int b = M.res[k]; e[b >> 5] |= (uint32_t)((s >> k) & 1) << (b & 31); }
    int b = M.res[R];
    e[b >> 5] |= (uint32_t)(q ^ (popc32((uint32_t)s) & 1)) << (b & 31);
  } else if (RS == CRC32C) {
    for (int i = 0; i < 8; i++) e[i] &= 0x0FFFFFFFu;
    uint32_t c = rcrc_compute(e);
    for (int i = 0; i < 8; i++) e[i] |= ((c >> (4 * i)) & 0xFu) << 28;
  }
}

// OR-accumulable fast check of a rowptr group: bit 0 of the result is set
// iff the group is not clean (parity rows' popcounts OR-ed).
template <int RS>
ABFT_HD uint32_t rp_acc(const uint32_t* e) {
  if (RS == SED) return (uint32_t)popc32(e[0]);
  if (RS == SECDED64 || RS == SECDED128) {
    constexpr int NW = (RS == SECDED64) ? 2 : 4;
    constexpr int R = (RS == SECDED64) ? 7 : 8;
    constexpr MaskTable M = (RS == SECDED64) ? h_mt_r64 : h_mt_r128;   // masks as immediates
    uint32_t q = 0;
#pragma unroll
    for (int i = 0; i < NW; i++) q ^= e[i];
    uint32_t acc = (uint32_t)popc32(q);
#pragma unroll
    for (int k = 0; k < R; k++) {
      uint32_t t = 0;
#pragma unroll
      for (int i = 0; i < NW; i++) t ^= e[i] & M.m[k][i];
      acc |= (uint32_t)popc32(t);
    }
    return acc;
  }
  if (RS == CRC32C) {
    uint32_t st = 0;
    for (int i = 0; i < 8; i++) st |= (e[i] >> 28) << (4 * i);
    return st == rcrc_compute(e) ? 0u : 1u;
  }
  return 0u;
}

// Fast-path check of a rowptr group; corrects in place.
template <int RS>
ABFT_HD int rp_check_group(uint32_t* e, int* word, const int* cfg = nullptr) {
  if (RS == SED) return (popc32(e[0]) & 1) ? DUE : CLEAN;
  if (RS == SECDED64) {
    int s, q;
    generic_syndrome<2, 7>(ABFT_MT(r64), e, s, q);
    if (!s && !q) return CLEAN;
    return secded_resolve<2>(ABFT_MAP(r64), e, s, q, word);
  }
  if (RS == SECDED128) {
    int s, q;
    generic_syndrome<4, 8>(ABFT_MT(r128), e, s, q);
    if (!s && !q) return CLEAN;
    return secded_resolve<4>(ABFT_MAP(r128), e, s, q, word);
  }
  if (RS == CRC32C) {   // R-CRC octet, 1EC4ED (see crc_locate)
    uint32_t st = 0;
    for (int i = 0; i < 8; i++) st |= (e[i] >> 28) << (4 * i);
    const uint32_t syn = st ^ rcrc_compute(e);
    if (!syn) return CLEAN;
    int pos[2];
    const int np = crc_fix_positions(syn, 256, cfg, pos);
    if (np == 0) return DUE;
    int ent[2], bit[2];
    for (int q = 0; q < np; q++) {
      const int r = pos[q];
      if (r < 0) { ent[q] = (-1 - r) >> 2; bit[q] = 28 + ((-1 - r) & 3); }   // CRC nibble t/4 = bits 28..31 of entry t/4
      else {
        ent[q] = r >> 5;            // 4 message bytes per entry
        bit[q] = r & 31;
        if (bit[q] >= 28) return DUE;   // masked-out top nibble: not a message bit
      }
    }
    for (int q = 0; q < np; q++) e[ent[q]] ^= 1u << bit[q];
    if (word) *word = ent[0];
    return CORRECTED;
  }
  return CLEAN;
}

}  // namespace abft
