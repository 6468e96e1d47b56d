// kernels_impl.cuh — device helpers and kernel templates shared by the kernel
// translation units (kernels.cu, spmv_es*.cu).
#pragma once
#include <cuda.h>
#include <cuda_runtime.h>
#include <stdint.h>

#include "codec.cuh"
#include "internal.h"

namespace abft {

// Host: launch k with the programmatic-stream-serialization attribute when the
// CG driver turned PDL on (set_pdl), else a plain launch.
extern thread_local bool g_pdl;   // per host thread: one solve's PdlGuard never leaks into another thread's launches
template <typename... KArgs, typename... Args>
static inline void launch_k(void (*k)(KArgs...), dim3 grid, dim3 block, size_t smem, cudaStream_t s, Args... args) {
  if (!g_pdl) {
    k<<<grid, block, smem, s>>>(args...);
    return;
  }
  cudaLaunchConfig_t cfg{};
  cfg.gridDim = grid;
  cfg.blockDim = block;
  cfg.dynamicSmemBytes = smem;
  cfg.stream = s;
  cudaLaunchAttribute at[1];
  at[0].id = cudaLaunchAttributeProgrammaticStreamSerialization;
  at[0].val.programmaticStreamSerializationAllowed = 1;
  cfg.attrs = at;
  cfg.numAttrs = 1;
  cudaLaunchKernelEx(&cfg, k, args...);
}

// --------------------------------------------------------------- helpers
__host__ __device__ constexpr int vgrp(int s) { return s == SECDED128 ? 2 : s == CRC32C ? 4 : 1; }
__host__ __device__ constexpr int rgrp(int s) { return s == SECDED64 ? 2 : s == SECDED128 ? 4 : s == CRC32C ? 8 : 1; }
__host__ __device__ constexpr int vk(int s) { return s == SED ? 1 : s == SECDED64 ? 8 : s == SECDED128 ? 5 : s == CRC32C ? 8 : 0; }
__host__ __device__ constexpr uint64_t vkeep(int s) { return vk(s) ? ~((1ull << vk(s)) - 1ull) : ~0ull; }

static __device__ __forceinline__ double as_d(uint64_t u) { return __longlong_as_double((long long)u); }
static __device__ __forceinline__ uint64_t as_u(double d) { return (uint64_t)__double_as_longlong(d); }
static __device__ __forceinline__ uint64_t shfl64(uint64_t v, int src) {
  uint32_t lo = __shfl_sync(0xffffffffu, (uint32_t)v, src);
  uint32_t hi = __shfl_sync(0xffffffffu, (uint32_t)(v >> 32), src);
  return mk64(lo, hi);
}
// Programmatic dependent launch (PDL): everything before
// pdl_wait() may only read data no kernel of the previous two launches writes
// (the matrix; vectors last written >= 2 kernels earlier); pdl_trigger() comes
// right after the wait, so a kernel's pre-wait part overlaps only its direct
// predecessor.  Both are no-ops for launches without the PDL attribute.
static __device__ __forceinline__ void pdl_wait() { asm volatile("griddepcontrol.wait;" ::: "memory"); }
static __device__ __forceinline__ void pdl_trigger() { asm volatile("griddepcontrol.launch_dependents;" ::: "memory"); }
static __device__ __forceinline__ uint64_t ldg64(const uint64_t* p) { return (uint64_t)__ldg((const unsigned long long*)p); }

static __device__ __forceinline__ void cnt_add(DevCounts* c, int t, int s, int o) {
  if (!c) return;
  atomicAdd(&c->v[t][s][0], 1ull);
  atomicAdd(&c->v[t][s][o == CORRECTED ? 1 : 2], 1ull);
}
static __device__ __forceinline__ void cnt_range(DevCounts* c, int t, int s) {
  if (c) atomicAdd(&c->v[t][s][3], 1ull);
}
// Scrub one 32-bit word; returns true iff this thread's CAS replaced it (the
// winner counts the correction: exactly-once counting).
static __device__ __forceinline__ bool scrub32(uint32_t* addr, uint32_t oldw, uint32_t neww) {
  return atomicCAS((unsigned int*)addr, oldw, neww) == oldw;
}
// Scrub every 32-bit word of a corrected group that changed (one for a single
// flip, up to two for a CRC32C 2EC3ED pair); the winner of the first CAS counts.
static __device__ __noinline__ bool scrub_group32(uint32_t* a32, const uint64_t* oldv, const uint64_t* newv, int G) {
  bool first = true, won = false;
  for (int w = 0; w < 2 * G; w++) {
    const uint32_t ow = (w & 1) ? hi32(oldv[w >> 1]) : lo32(oldv[w >> 1]);
    const uint32_t nw = (w & 1) ? hi32(newv[w >> 1]) : lo32(newv[w >> 1]);
    if (ow == nw) continue;
    const bool ok = scrub32(a32 + w, ow, nw);
    if (first) won = ok;
    first = false;
  }
  return won;
}
static __device__ __noinline__ bool scrub_entries32(uint32_t* a32, const uint32_t* oldv, const uint32_t* newv, int G) {
  bool first = true, won = false;
  for (int w = 0; w < G; w++) {
    if (oldv[w] == newv[w]) continue;
    const bool ok = scrub32(a32 + w, oldv[w], newv[w]);
    if (first) won = ok;
    first = false;
  }
  return won;
}

static __device__ __forceinline__ void load_lut(uint8_t* s_lut) {
  if (threadIdx.x < 32) reinterpret_cast<uint32_t*>(s_lut)[threadIdx.x] = reinterpret_cast<const uint32_t*>(&c_v64_lut)[threadIdx.x];
}

// ====================================== CRC32C tables in shared memory (§3.5)
// Table-driven CRC32C: the plain bit-serial division costs 8 shift/XOR steps per
// byte; slicing-by-4 does a 32-bit word with 4 SMEM lookups.
constexpr uint32_t VCRC_ZERO = 0x8A9136AAu;   // CRC32C of 32 zero bytes (RFC 3720 check value, PIN-4)
constexpr int CRC_SLICE_WORDS = 4 * 256;
constexpr int CRC_VPOS_WORDS = 4 * 7 * 256;
static __device__ __forceinline__ void smem_fill(uint32_t* dst, const uint32_t* src, int nwords) {
  for (int i = 4 * (int)threadIdx.x; i < nwords; i += 4 * (int)blockDim.x)
    *reinterpret_cast<uint4*>(dst + i) = __ldg(reinterpret_cast<const uint4*>(src + i));
}
// one little-endian 32-bit message word through the reflected CRC register
static __device__ __forceinline__ uint32_t crc_word(uint32_t c, uint32_t w, const uint32_t* T) {
  c ^= w;
  return T[768 + (c & 0xFFu)] ^ T[512 + ((c >> 8) & 0xFFu)] ^ T[256 + ((c >> 16) & 0xFFu)] ^ T[c >> 24];
}
// R-CRC octet: bit 0 set <=> stored nibbles != CRC of the masked entries
static __device__ __forceinline__ uint32_t rcrc_acc_tab(const uint32_t* e, const uint32_t* T) {
  uint32_t c = 0xFFFFFFFFu, st = 0;
#pragma unroll
  for (int i = 0; i < 8; i++) {
    c = crc_word(c, e[i] & 0x0FFFFFFFu, T);
    st |= (e[i] >> 28) << (4 * i);
  }
  return (c ^ 0xFFFFFFFFu) != st ? 1u : 0u;
}

// ================================== lane-split group vector codecs (G = 2, 4)
// In every warp-wide vector access lane l holds index base + l, so the 2 / 4
// words of an aligned group sit in adjacent lanes.
static __device__ __forceinline__ uint64_t shfl_xor64(uint64_t v, int m) {
  const uint32_t lo = __shfl_xor_sync(0xffffffffu, (uint32_t)v, m);
  const uint32_t hi = __shfl_xor_sync(0xffffffffu, (uint32_t)(v >> 32), m);
  return mk64(lo, hi);
}
// V-SECDED128 "pair gather": lanes 2m, 2m+1 hold the halves of group A in w0
// (pass k) and of group B in w1 (pass k+32); after one exchange the even lane
// holds A and the odd lane B whole (d0 = first double, d1 = second), so each
// lane runs the textbook code with immediate masks.
static __device__ __forceinline__ void pair_gather(uint64_t w0, uint64_t w1, int lane, uint64_t& d0, uint64_t& d1) {
  const bool odd = lane & 1;
  const uint64_t r = shfl_xor64(odd ? w0 : w1, 1);
  d0 = odd ? r : w0;
  d1 = odd ? w1 : r;
}
static __device__ __forceinline__ void pair_scatter(uint64_t d0, uint64_t d1, int lane, uint64_t& w0, uint64_t& w1) {
  const bool odd = lane & 1;
  const uint64_t r = shfl_xor64(odd ? d0 : d1, 1);
  w0 = odd ? r : d0;
  w1 = odd ? d1 : r;
}
// V-CRC (G = 4): CRC32C is affine in the message, crc(m) = L(m) ^ crc(0^32), so
// each lane adds the linear part of its double's 7 message bytes (position
// tables vp = vpos[lane & 3]) and the group XORs 4 partials.
static __device__ __forceinline__ uint32_t vcrc_lin(uint64_t w, const uint32_t* vp) {
  const uint32_t lo = lo32(w), hi = hi32(w);
  return vp[(lo >> 8) & 0xFFu] ^ vp[256 + ((lo >> 16) & 0xFFu)] ^ vp[512 + (lo >> 24)] ^ vp[768 + (hi & 0xFFu)] ^
         vp[1024 + ((hi >> 8) & 0xFFu)] ^ vp[1280 + ((hi >> 16) & 0xFFu)] ^ vp[1536 + (hi >> 24)];
}
static __device__ __forceinline__ uint32_t xor4(uint32_t p) {
  p ^= __shfl_xor_sync(0xffffffffu, p, 1);
  return p ^ __shfl_xor_sync(0xffffffffu, p, 2);
}
static __device__ __forceinline__ const uint32_t* vcrc_tab(const uint8_t* cs, int lane) {
  return reinterpret_cast<const uint32_t*>(cs) + (lane & 3) * 7 * 256;
}
static __device__ __forceinline__ bool vcrc_bad_lane(uint64_t w, const uint32_t* vp, int lane) {
  return xor4(vcrc_lin(w, vp) ^ ((lo32(w) & 0xFFu) << (8 * (lane & 3)))) != VCRC_ZERO;
}
static __device__ __forceinline__ uint64_t vcrc_encode_lane(uint64_t rounded, const uint32_t* vp, int lane) {
  const uint64_t d = rounded & ~0xFFull;
  const uint32_t crc = xor4(vcrc_lin(d, vp)) ^ VCRC_ZERO;
  return d | ((crc >> (8 * (lane & 3))) & 0xFFu);
}
// Whole warp, G > 1 schemes: does any group holding w0 (pass k) or w1 (pass
// k+32) fail its check?  cs: V-CRC position tables in SMEM (CRC32C).
template <int VS>
__device__ __forceinline__ bool gbad2(uint64_t w0, uint64_t w1, int lane, const uint8_t* cs) {
  if (VS == SECDED128) {
    uint64_t d0, d1;
    pair_gather(w0, w1, lane, d0, d1);
    return (v128_acc(d0, d1) & 1u) != 0u;
  }
  const uint32_t* vp = vcrc_tab(cs, lane);
  return vcrc_bad_lane(w0, vp, lane) | vcrc_bad_lane(w1, vp, lane);
}
// Whole warp, G > 1 schemes: encode the rounded values r0 (pass k), r1 (pass k+32).
template <int VS>
__device__ __forceinline__ void genc2(uint64_t r0, uint64_t r1, int lane, const uint8_t* cs, uint64_t& e0,
                                      uint64_t& e1) {
  if (VS == SECDED128) {
    uint64_t d[2];
    pair_gather(r0, r1, lane, d[0], d[1]);
    v128_encode(d);
    pair_scatter(d[0], d[1], lane, e0, e1);
  } else {
    const uint32_t* vp = vcrc_tab(cs, lane);
    e0 = vcrc_encode_lane(r0, vp, lane);
    e1 = vcrc_encode_lane(r1, vp, lane);
  }
}

// Matrix check mode of this SpMV access.
static __device__ __forceinline__ int spmv_mode(const SpmvArgs& a) {
  if (a.check_interval > 1) {
    const int64_t acc = a.state ? (int64_t)a.state->iters + 1 : 0;   // init = access 0
    return (acc % a.check_interval) ? MODE_RANGE : MODE_DETECT;
  }
  return a.check_mode;
}


// Cold path of a single-codeword vector check (G = 1 schemes).
template <int VS>
__device__ __noinline__ uint64_t v1_fix(uint64_t w, uint64_t* addr, bool owner, DevCounts* cnt, int* due) {
  uint64_t d = w;
  int word = 0;
  int o = (VS == SECDED64) ? v64_correct(d, &word) : DUE;
  if (o == CORRECTED) {
    if (owner) {
      uint32_t oldw = word ? hi32(w) : lo32(w), neww = word ? hi32(d) : lo32(d);
      if (scrub32(reinterpret_cast<uint32_t*>(addr) + word, oldw, neww)) cnt_add(cnt, T_VEC, VS, CORRECTED);
    }
    return d;
  }
  if (owner) { cnt_add(cnt, T_VEC, VS, DUE); *due = 1; }
  return w;
}
// Check one G=1 codeword: returns the (corrected) stored word.
template <int VS>
__device__ __forceinline__ uint64_t v1_check(uint64_t w, uint64_t* addr, bool owner, DevCounts* cnt, int* due) {
  if (VS == SED) { if (!vsed_clean(w)) return v1_fix<VS>(w, addr, owner, cnt, due); }
  if (VS == SECDED64) { if (v64_bad(lo32(w), hi32(w))) return v1_fix<VS>(w, addr, owner, cnt, due); }
  return w;
}

// Group check (G = 2, 4): lanes [lead, lead+G) hold the group's words; the
// leader checks, counts and scrubs, then broadcasts the corrected words.
// Must be called by the full warp.
template <int VS>
__device__ uint64_t vg_check(uint64_t my, uint64_t* group_addr, int lane, bool active, bool owner, DevCounts* cnt,
                             int* due) {
  constexpr int G = vgrp(VS);
  const int lead = lane & ~(G - 1);
  uint64_t d[G];
#pragma unroll
  for (int t = 0; t < G; t++) d[t] = shfl64(my, lead + t);
  if (lane == lead && active) {
    uint64_t o0[G];
#pragma unroll
    for (int t = 0; t < G; t++) o0[t] = d[t];
    int word = 0;
    int o = vec_check_group<VS>(d, &word, due);
    if (o == CORRECTED) {
      if (owner && scrub_group32(reinterpret_cast<uint32_t*>(group_addr), o0, d, G))
        cnt_add(cnt, T_VEC, VS, CORRECTED);
    } else if (o == DUE) {
#pragma unroll
      for (int t = 0; t < G; t++) d[t] = o0[t];
      if (owner) { cnt_add(cnt, T_VEC, VS, DUE); *due = 1; }
    }
  }
  uint64_t res = my;
#pragma unroll
  for (int t = 0; t < G; t++) {
    uint64_t v = shfl64(d[t], lead);
    if ((lane & (G - 1)) == t) res = v;
  }
  return res;
}

// Encode: each lane passes its rounded value; returns its encoded word.
template <int VS>
__device__ __forceinline__ uint64_t v_encode(uint64_t rounded, int lane, const uint8_t* lut) {
  constexpr int G = vgrp(VS);
  if (G == 1) {
    uint64_t d[1] = {rounded};
    vec_encode_group<VS>(d, lut);
    return d[0];
  } else {
    const int lead = lane & ~(G - 1);
    uint64_t d[G > 1 ? G : 1];
#pragma unroll
    for (int t = 0; t < G; t++) d[t] = shfl64(rounded, lead + t);
    if (lane == lead) vec_encode_group<VS>(d, lut);
    uint64_t res = 0;
#pragma unroll
    for (int t = 0; t < G; t++) {
      uint64_t v = shfl64(d[t], lead);
      if ((lane & (G - 1)) == t) res = v;
    }
    return res;
  }
}

// Warp-uniform vector access for one pass: load my word (if idx < npad), check
// as owner, return the corrected stored word.
template <int VS>
__device__ __forceinline__ uint64_t v_load_check(uint64_t* v, int64_t idx, int64_t npad, int lane, bool owner,
                                                 DevCounts* cnt, int* due) {
  constexpr int G = vgrp(VS);
  const bool in = idx < npad;
  uint64_t w = in ? ldg64(v + idx) : 0ull;
  if (VS == NONE) return w;
  if (G == 1) return in ? v1_check<VS>(w, v + idx, owner, cnt, due) : w;
  const int64_t gidx = idx & ~(int64_t)(G - 1);
  return vg_check<VS>(w, v + gidx, lane, in, owner && in, cnt, due);
}

// Non-owner gather of in[idx] (any lane, no shuffles): returns the masked value.
template <int VS>
__device__ __forceinline__ double gather_in(const uint64_t* in, int64_t idx, const int* cfg = nullptr) {
  constexpr int G = vgrp(VS);
  if (G == 1) {
    uint64_t w = ldg64(in + idx);
    if (VS == SED) return as_d(w & vkeep(VS));
    if (VS == SECDED64) {
      if (v64_bad(lo32(w), hi32(w))) {
        uint64_t d = w;
        if (v64_correct(d, nullptr) == CORRECTED) w = d;
      }
    }
    return as_d(w & vkeep(VS));
  } else {
    const int64_t g = idx & ~(int64_t)(G - 1);
    uint64_t d[G];
#pragma unroll
    for (int t = 0; t < G; t++) d[t] = ldg64(in + g + t);
    uint64_t o0 = d[idx - g];
    int o = vec_check_group<VS>(d, nullptr, cfg);
    uint64_t w = (o == CORRECTED) ? d[idx - g] : o0;
    return as_d(w & vkeep(VS));
  }
}

// Fused calc_p (non-owner): p_k[idx] = round(fma(beta, p_{k-1}[idx], r[idx]))
// from the checked (corrected in registers, not counted) operands — the
// masked value of the word the unfused calc_p would have stored (G = 1).
template <int VS>
__device__ __forceinline__ double gather_fused(const uint64_t* pprev, const uint64_t* r, double beta, int64_t idx) {
  const double pn = fma(beta, gather_in<VS>(pprev, idx), gather_in<VS>(r, idx));
  return as_d(round_k(as_u(pn), vk(VS)));
}

// ============================================================ rowptr pass
// Decode the rowptr groups covering entries [pb, pb+32] into srp (per warp),
// checking them (owner = the pass holding row min(gG, nrows-1)), then return
// this lane's start/end.
template <int RS>
__device__ __forceinline__ void rowptr_pass(const SpmvArgs& a, int64_t pb, int lane, uint32_t* srp, uint32_t& start,
                                            uint32_t& end, int mode) {
  constexpr int G = rgrp(RS);
  if (RS == NONE) {
    const int64_t e = pb + lane;
    start = (e <= a.nrows) ? __ldg(a.rowptr + e) : 0u;
    end = (e + 1 <= a.nrows) ? __ldg(a.rowptr + e + 1) : 0u;
    return;
  }
  constexpr int NG = 32 / G + 1;
  for (int gl = lane; gl < NG; gl += 32) {  // NG = 33 for G = 1: lane 0 takes the extra group
    const int64_t g = pb / G + gl;
    if (g * G > a.nrows) continue;
    uint32_t e[G];
    uint32_t* gp = a.rowptr + g * G;
    if (G == 1) e[0] = __ldg(gp);
    else if (G == 2) { uint2 u = __ldg(reinterpret_cast<const uint2*>(gp)); e[0] = u.x; e[1 % G] = u.y; }
    else {
#pragma unroll
      for (int q = 0; q < G; q += 4) {
        uint4 u = __ldg(reinterpret_cast<const uint4*>(gp + q));
        e[q] = u.x; e[(q + 1) % G] = u.y; e[(q + 2) % G] = u.z; e[(q + 3) % G] = u.w;
      }
    }
    uint32_t o0[G];
#pragma unroll
    for (int t = 0; t < G; t++) o0[t] = e[t];
    int word = 0;
    int o = (mode == MODE_RANGE) ? CLEAN : rp_check_group<RS>(e, &word, a.due);
    if (o == CORRECTED && mode == MODE_DETECT) o = DUE;   // interval mode: detection only
    if (o != CLEAN) {
      int64_t own = g * G < a.nrows ? g * G : a.nrows - 1;
      bool owner = own >= pb && own < pb + 32;
      if (o == CORRECTED) {
        if (owner && scrub_entries32(gp, o0, e, G)) cnt_add(a.counts, T_ROWPTR, RS, CORRECTED);
      } else {
#pragma unroll
        for (int t = 0; t < G; t++) e[t] = o0[t];
        if (owner) { cnt_add(a.counts, T_ROWPTR, RS, DUE); *a.due = 1; }
      }
    }
#pragma unroll
    for (int t = 0; t < G; t++) srp[gl * G + t] = e[t] & rp_keep(RS);
  }
  __syncwarp();
  start = srp[lane];
  end = srp[lane + 1];
  __syncwarp();
}

// Cold path of an element check: correct, scrub (winner counts), or DUE.
template <int ES>
__device__ __noinline__ int elem_fix(uint64_t& v, uint32_t& c, uint64_t* vaddr, uint32_t* caddr, DevCounts* cnt,
                                     int* due, int mode) {
  uint64_t v0 = v;
  uint32_t c0 = c;
  int word = 0;
  int o = (ES == SED) ? DUE : e96_correct(v, c, &word);
  if (o == CORRECTED && mode == MODE_DETECT) o = DUE;   // interval mode: detection only
  if (o == CORRECTED) {
    bool won;
    if (word == 2) won = scrub32(caddr, c0, c);
    else won = scrub32(reinterpret_cast<uint32_t*>(vaddr) + word, word ? hi32(v0) : lo32(v0), word ? hi32(v) : lo32(v));
    if (won) cnt_add(cnt, T_ELEM, ES, CORRECTED);
  } else {
    v = v0;
    c = c0;
    cnt_add(cnt, T_ELEM, ES, DUE);
    *due = 1;
  }
  return o;
}

// E-CRC row codeword [start, start+len) failed its check:
// recompute from global memory, locate a single flipped bit (1EC4ED,
// crc_locate) or, with 2EC3ED enabled (cfg, reading R9b), a flipped pair, and,
// per `how`: 1 scrub it (32-bit CAS per changed word; the first CAS's winner
// counts the correction), 0 count it without writing (check_all count-only),
// 2 report a DUE (detection only: interval mode).  Anything else is
// a DUE (counted at every access).  Returns CLEAN (someone else already
// scrubbed it), CORRECTED (read the row from global memory again) or DUE (use
// the stored bits).  fix_addr / fix_bit [2] receive the located bits (null
// when none) for count-only callers to apply.
static __device__ __noinline__ int ecrc_fix(uint64_t* val, uint32_t* col, uint32_t start, uint32_t len, int how,
                                            DevCounts* cnt, int* due, uint32_t** fix_addr = nullptr,
                                            int* fix_bit = nullptr) {
  int o = DUE;
  uint32_t* addr[2] = {nullptr, nullptr};
  int bit[2] = {0, 0}, np = 0;
  if (len >= 4) {
    uint32_t crc = 0xFFFFFFFFu, st = 0;
    for (uint32_t j = 0; j < len; j++) {
      const uint32_t c = *(volatile uint32_t*)(col + start + j);
      const uint64_t v = *(volatile uint64_t*)(val + start + j);
      if (j < 4) st |= (c >> 24) << (8 * j);
      crc = ecrc_update(crc, v, c, (int)j);
    }
    const uint32_t syn = st ^ crc ^ 0xFFFFFFFFu;
    if (!syn) return CLEAN;
    int pos[2];
    np = crc_fix_positions(syn, 96 * (int)len, due, pos);
    o = np ? CORRECTED : DUE;
    for (int q = 0; q < np && o == CORRECTED; q++) {
      const int r = pos[q];
      if (r < 0) {   // stored CRC byte t/8 = col[31:24] of entry t/8
        addr[q] = col + start + ((-1 - r) >> 3);
        bit[q] = 24 + ((-1 - r) & 7);
      } else {       // message: per entry 8 bytes val LE, 4 bytes col LE (top byte zeroed for entries 0..3)
        const int byte = r >> 3, k = byte / 12, bb = byte - 12 * k;
        if (bb < 8) {
          addr[q] = reinterpret_cast<uint32_t*>(val + start + k) + (bb >> 2);
          bit[q] = 8 * (bb & 3) + (r & 7);
        } else if (!(k < 4 && bb == 11)) {
          addr[q] = col + start + k;
          bit[q] = 8 * (bb - 8) + (r & 7);
        } else {
          o = DUE;   // a zeroed message byte: not a stored bit
        }
      }
    }
  }
  if (o == CORRECTED && how == 2) o = DUE;
  if (fix_addr)
    for (int q = 0; q < 2; q++) {
      fix_addr[q] = (o == CORRECTED && q < np) ? addr[q] : nullptr;
      fix_bit[q] = bit[q];
    }
  if (o == CORRECTED) {
    if (how == 1) {
      bool won = false;
      for (int q = 0; q < np; q++) {
        const uint32_t w = *(volatile uint32_t*)addr[q];
        const bool ok = scrub32(addr[q], w, w ^ (1u << bit[q]));
        if (q == 0) won = ok;
      }
      if (won) cnt_add(cnt, T_ELEM, CRC32C, CORRECTED);
    } else {
      cnt_add(cnt, T_ELEM, CRC32C, CORRECTED);
    }
  } else {
    cnt_add(cnt, T_ELEM, CRC32C, DUE);
    *due = 1;
  }
  return o;
}

// ================================================================ SpMV (a3)
// DOT: 0 no dot, 1 in.out, 2 in.out and in.in (single-reduction CG)
template <int ES, int RS, int VS, int DOT>
__global__ void __launch_bounds__(256) k_spmv(SpmvArgs a) {
  __shared__ __align__(16) uint8_t s_lut[128];
  __shared__ uint32_t s_rp[8][40];
  if (VS == SECDED64) load_lut(s_lut);
  __syncthreads();
  pdl_wait();
  pdl_trigger();
  if (a.state && a.state->stop) return;
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  const int64_t rb = (int64_t)blockIdx.x * 8 + warp;
  const int64_t nrb = (a.nrows + 255) >> 8;
  if (rb >= nrb) return;
  double dot = 0.0, dot2 = 0.0;
  const uint32_t ckeep = col_keep(ES);
  const int mode = spmv_mode(a);
  for (int k = 0; k < 8; k++) {
    const int64_t pb = rb * 256 + k * 32;
    if (pb >= a.nrows) break;
    const int64_t i = pb + lane;
    const bool valid = i < a.nrows;
    uint32_t start, end;
    rowptr_pass<RS>(a, pb, lane, s_rp[warp], start, end, mode);
    // own codeword of `in` (checked once, counted here: DESIGN.md §3.8)
    const int64_t own = a.row_base + i;
    const int64_t own_lim = (vgrp(VS) == 1 && !valid) ? 0 : a.npad_in;
    const uint64_t pw_own = v_load_check<VS>(a.in, own, own_lim, lane, valid, a.counts, a.due);
    const double p_own = as_d(pw_own & vkeep(VS));
    double acc = 0.0;
    if (valid) {
      const bool ok = (start <= end) && ((int64_t)end <= a.nnz);
      if (RS != NONE && !ok) {
        cnt_range(a.counts, T_ROWPTR, RS);
        *a.due = 1;
      } else {
        bool fixed = false;   // E-CRC row corrected in global memory: read it without the read-only path
        if (ES == CRC32C && mode != MODE_RANGE) {   // the row is the codeword: check it first (1EC4ED)
          uint32_t crc = 0xFFFFFFFFu, crc_st = 0;
          for (uint32_t j = start; j < end; j++) {
            const uint32_t c = __ldg(a.col + j);
            if (j - start < 4) crc_st |= (c >> 24) << (8 * (j - start));
            crc = ecrc_update(crc, ldg64(a.val + j), c, (int)(j - start));
          }
          if (end - start < 4 || (crc ^ 0xFFFFFFFFu) != crc_st)
            fixed = ecrc_fix(a.val, a.col, start, end - start, mode == MODE_DETECT ? 2 : 1, a.counts, a.due) != DUE;
        }
        for (uint32_t j = start; j < end; j++) {
          uint64_t v = fixed ? *(volatile uint64_t*)(a.val + j) : ldg64(a.val + j);
          uint32_t c = fixed ? *(volatile uint32_t*)(a.col + j) : __ldg(a.col + j);
          if (ES != NONE && ES != CRC32C && mode != MODE_RANGE) {
            bool bad = (ES == SED) ? !esed_clean(v, c) : (e96_bad(lo32(v), hi32(v), c) != 0);
            if (bad) elem_fix<ES>(v, c, a.val + j, a.col + j, a.counts, a.due, mode);
          }
          const uint32_t cm = c & ckeep;
          if (ES != NONE && (int64_t)cm >= a.ncols) {
            cnt_range(a.counts, T_ELEM, ES);
            *a.due = 1;
            continue;
          }
          const int64_t idx = a.col_base + cm;
          const double x = (idx == own) ? p_own : gather_in<VS>(a.in, idx, a.due);
          acc = fma(as_d(v), x, acc);
        }
      }
    }
    // write-buffered output (whole codewords)
    // npad_out = local rows this chunk may write (nrows, + vector padding for the last chunk)
    const uint64_t rounded = valid ? round_k(as_u(acc), vk(VS)) : 0ull;
    const uint64_t enc = v_encode<VS>(rounded, lane, s_lut);
    if (i < a.npad_out) a.out[own] = enc;
    if (DOT && valid) dot = fma(p_own, as_d(enc & vkeep(VS)), dot);
    if (DOT == 2 && valid) dot2 = fma(p_own, p_own, dot2);
  }
  if (DOT) {
#pragma unroll
    for (int off = 16; off >= 1; off >>= 1) dot = dot + __shfl_xor_sync(0xffffffffu, dot, off);
    if (lane == 0) a.partials[a.rb_offset + rb] = dot;
  }
  if (DOT == 2) {
#pragma unroll
    for (int off = 16; off >= 1; off >>= 1) dot2 = dot2 + __shfl_xor_sync(0xffffffffu, dot2, off);
    if (lane == 0) a.partials2[a.rb_offset + rb] = dot2;
  }
}

// ====================================================== tiled stencil SpMV (a3)
// Fast path for 5-point-stencil matrices (stencil_n = n, n % 256 == 0,
// nrows % n == 0, nnz == 5 nrows, G = 1 vector scheme).  A CTA owns a tile of
// TILE_TY grid rows x 256 cells; warp w owns grid row w of the tile = one
// reduction block, processed as 8 passes of 32 rows.
//  0. thread 0 is the CTA's TMA producer: the (val, col) element streams of one
//     pass of all TILE_TY warps form a 2-D box [TILE_TY grid rows][160
//     elements] of the matrix viewed as [ny][5n] (tensor maps built on the
//     host), so ONE pair of cp.async.bulk.tensor copies per pass feeds the
//     whole CTA through a TILE_NST-stage full/empty mbarrier ring.  The box
//     position assumes the stencil layout rowptr[i] = 5i; every row compares
//     its decoded rowptr with that assumption and reads global memory instead
//     whenever it disagrees, so results never depend on the guess;
//  1. each warp decodes its segment's 257 rowptr entries into SMEM (one check
//     per group; owner counts);
//  2. the CTA stages the decoded `in` window (tile + one halo row above/below
//     + one halo cell left/right) in SMEM: every codeword of the tile is
//     checked ONCE here (owner: counted + scrubbed), halo codewords are
//     checked without counting.  This is the paper's "multiple ECC element and
//     multi-iteration aware" SpMV cache in B200 form; like the
//     paper's caches, the decoded copies in SMEM are outside the software trust
//     boundary;
//  3. per pass each lane checks/corrects its row's elements from the stage,
//     gathers neighbours from the window whenever col-row is one of {0, +-1,
//     +-n} (anything else takes the global gather path, so results never
//     depend on the stencil hint), encodes w, and releases the stage.
// val / col element streams ([ny][5n] boxes); vin / vcur: the SpMV input
// vector (and the fused path's p_cur) viewed as [rows][n/2][2] doubles, one
// box = the tile's decoded-window rows (has_vmaps = 0: not built)
struct TileMaps { CUtensorMap val, col, vin, vcur; int has_vmaps; };

constexpr int TILE_TY = 8;
// window row: x = tx0-2 .. tx0+261 (one TMA box of 132 double pairs); the
// tile's own cells sit at slots TILE_WX0 .. TILE_WX0+255
constexpr int TILE_WX0 = 2;
// (x = tx0-2 .. tx0+261: 132 double pairs per row, so any two rows start on a
// 128-byte boundary, as TMA destinations must)
constexpr int TILE_WW = 256 + 8;
constexpr int TILE_PE = 160;                                   // elements per warp per pass (32 rows x 5)
#ifndef ABFT_TILE_NST
#define ABFT_TILE_NST 3
#endif
constexpr int TILE_NST = ABFT_TILE_NST;                        // pipeline stages
constexpr int TILE_STAGE_VAL = TILE_TY * TILE_PE * 8;          // 10240
constexpr int TILE_STAGE = TILE_STAGE_VAL + TILE_TY * TILE_PE * 4;   // + 5120
constexpr int TILE_WIN_BYTES = (TILE_TY + 2) * TILE_WW * 8;    // 21120
constexpr int TILE_RP = 264;                                   // rowptr entries staged per warp
// SMEM layout (tile_off_*): stages, window, row pointers, mbarriers, CRC tables
// ABFT_CRC_SLICE_SMEM = 0: the tiled SpMV reads the 4 KB slicing tables of
// E-CRC / R-CRC through L1 instead of staging them in SMEM (keeps 3 CTAs per
// SM for CRC32C matrices)
#ifndef ABFT_CRC_SLICE_SMEM
#define ABFT_CRC_SLICE_SMEM 1
#endif
// dynamic SMEM of one tile kernel: + slicing tables (E-CRC / R-CRC), + V-CRC position tables
// E-CRC / R-CRC instantiations run 2 stages: their 4 KB of slicing tables
// would otherwise push the CTA past 76 KB (2 CTAs per SM instead of 3, the
// range-only accesses of interval mode then +13 %, r2n / r2o)
#ifndef ABFT_CRC_NST
#define ABFT_CRC_NST 2
#endif
template <int ES, int RS>
constexpr int tile_nst() { return (ES == CRC32C || RS == CRC32C) ? ABFT_CRC_NST : TILE_NST; }
constexpr int tile_off_win(int nst) { return nst * TILE_STAGE; }
constexpr int tile_off_rp(int nst) { return tile_off_win(nst) + TILE_WIN_BYTES; }
constexpr int tile_off_bar(int nst) { return tile_off_rp(nst) + TILE_TY * TILE_RP * 4; }
constexpr int tile_off_crc(int nst) { return tile_off_bar(nst) + 64; }
template <int ES, int RS, int VS>
constexpr int tile_smem() {
  return tile_off_crc(tile_nst<ES, RS>()) + 128 +
         ((ABFT_CRC_SLICE_SMEM && (ES == CRC32C || RS == CRC32C)) ? 4 * CRC_SLICE_WORDS : 0) +
         (VS == CRC32C ? 4 * CRC_VPOS_WORDS : 0);
}

static __device__ __forceinline__ uint32_t smem_u32(const void* p) { return (uint32_t)__cvta_generic_to_shared(p); }
static __device__ __forceinline__ void mbar_init(uint64_t* bar, uint32_t count) {
  asm volatile("mbarrier.init.shared::cta.b64 [%0], %1;" ::"r"(smem_u32(bar)), "r"(count) : "memory");
}
static __device__ __forceinline__ void mbar_expect_tx(uint64_t* bar, uint32_t bytes) {
  asm volatile("mbarrier.arrive.expect_tx.shared::cta.b64 _, [%0], %1;" ::"r"(smem_u32(bar)), "r"(bytes) : "memory");
}
static __device__ __forceinline__ void mbar_arrive(uint64_t* bar) {
  asm volatile("mbarrier.arrive.shared::cta.b64 _, [%0];" ::"r"(smem_u32(bar)) : "memory");
}
static __device__ __forceinline__ void mbar_wait(uint64_t* bar, uint32_t parity) {
  asm volatile(
      "{\n .reg .pred P1;\n WAIT_%=:\n mbarrier.try_wait.parity.shared::cta.b64 P1, [%0], %1;\n @!P1 bra WAIT_%=;\n}\n" ::"r"(
          smem_u32(bar)),
      "r"(parity)
      : "memory");
}
static __device__ __forceinline__ void tma_2d(void* dst, const CUtensorMap* map, int x, int y, uint64_t* bar) {
  asm volatile(
      "cp.async.bulk.tensor.2d.shared::cluster.global.tile.mbarrier::complete_tx::bytes [%0], [%1, {%2, %3}], [%4];" ::"r"(
          smem_u32(dst)),
      "l"(reinterpret_cast<uint64_t>(map)), "r"(x), "r"(y), "r"(smem_u32(bar))
      : "memory");
}
static __device__ __forceinline__ void tma_3d(void* dst, const CUtensorMap* map, int x, int y, int z, uint64_t* bar) {
  asm volatile(
      "cp.async.bulk.tensor.3d.shared::cluster.global.tile.mbarrier::complete_tx::bytes [%0], [%1, {%2, %3, %4}], [%5];" ::"r"(
          smem_u32(dst)),
      "l"(reinterpret_cast<uint64_t>(map)), "r"(x), "r"(y), "r"(z), "r"(smem_u32(bar))
      : "memory");
}
// Producer: the element boxes of pass k of the tile (tx0, ty0) into stage buffer `stage`.
static __device__ __forceinline__ void tile_produce(const TileMaps& tm, uint8_t* stage, uint64_t* full, int64_t tx0,
                                                    int64_t ty0, int k) {
  mbar_expect_tx(full, TILE_STAGE);
  const int x = (int)(5 * (tx0 + 32 * k)), y = (int)ty0;
  tma_2d(stage, &tm.val, x, y, full);
  tma_2d(stage + TILE_STAGE_VAL, &tm.col, x, y, full);
}

// One row, general case: check/correct its elements (from the stage or
// global), gather, fma chain.  Also the cold path of the 5-entry fast path
// below.  sval/scol hold elements [s0, s1) of the chunk (if staged).
template <int ES, int RS, int VS>
static __device__ __noinline__ double tile_row(const SpmvArgs& a, uint32_t start, uint32_t end, const uint64_t* sval,
                                                 const uint32_t* scol, bool staged, const double* win, int oslot,
                                                 double p_own, int64_t own, uint32_t s0, uint32_t s1, int mode) {
  double acc = 0.0;
  const bool ok = (start <= end) && ((int64_t)end <= a.nnz);
  // a corrupted (DUE) rowptr entry can put this row outside the staged range:
  // read it from global memory then
  staged = staged && start >= s0 && end <= s1;
  if (RS != NONE && !ok) {
    cnt_range(a.counts, T_ROWPTR, RS);
    *a.due = 1;
    return 0.0;
  }
  const uint32_t ckeep = col_keep(ES);
  const int64_t n = a.stencil_n;
  const uint32_t len = end - start;
  bool fixed = false;   // E-CRC row corrected in global memory: read it from there, past the read-only path
  if (ES == CRC32C && mode != MODE_RANGE) {   // the row is the codeword: check it first (1EC4ED)
    uint32_t crc = 0xFFFFFFFFu, crc_st = 0;
    for (uint32_t j = 0; j < len; j++) {
      const uint64_t v = staged ? sval[start + j - s0] : ldg64(a.val + start + j);
      const uint32_t c = staged ? scol[start + j - s0] : __ldg(a.col + start + j);
      if (j < 4) crc_st |= (c >> 24) << (8 * j);
      crc = ecrc_update(crc, v, c, (int)j);
    }
    if (len < 4 || (crc ^ 0xFFFFFFFFu) != crc_st) {
      fixed = ecrc_fix(a.val, a.col, start, len, mode == MODE_DETECT ? 2 : 1, a.counts, a.due) != DUE;
      staged = staged && !fixed;
    }
  }
  for (uint32_t j = 0; j < len; j++) {
    uint64_t v;
    uint32_t c;
    if (staged) {
      v = sval[start + j - s0];
      c = scol[start + j - s0];
    } else if (fixed) {
      v = *(volatile uint64_t*)(a.val + start + j);
      c = *(volatile uint32_t*)(a.col + start + j);
    } else {
      v = ldg64(a.val + start + j);
      c = __ldg(a.col + start + j);
    }
    if (ES != NONE && ES != CRC32C && mode != MODE_RANGE) {
      bool bad = (ES == SED) ? !esed_clean(v, c) : (e96_bad(lo32(v), hi32(v), c) != 0);
      if (bad) elem_fix<ES>(v, c, a.val + start + j, a.col + start + j, a.counts, a.due, mode);
    }
    const uint32_t cm = c & ckeep;
    if (ES != NONE && (int64_t)cm >= a.ncols) {
      cnt_range(a.counts, T_ELEM, ES);
      *a.due = 1;
      continue;
    }
    const int64_t rel = a.col_base + (int64_t)cm - own;
    double x;
    if (rel == 0) x = p_own;
    else if (rel == 1) x = win[oslot + 1];
    else if (rel == -1) x = win[oslot - 1];
    else if (rel == n) x = win[oslot + TILE_WW];
    else if (rel == -n) x = win[oslot - TILE_WW];
    else x = a.fz ? gather_fused<VS>(a.in, a.r_f, a.beta_f, own + rel) : gather_in<VS>(a.in, own + rel, a.due);
    acc = fma(as_d(v), x, acc);
  }
  return acc;
}

// E-SECDED fast check of the stencil rows' elements in pairs (codec e96_acc2)
#ifndef ABFT_PAIR_E
#define ABFT_PAIR_E 1
#endif
// V-SECDED64 fast check of the decoded window in slot pairs (codec v64_acc2)
#ifndef ABFT_PAIR_W
#define ABFT_PAIR_W 1
#endif
// 5-entry stencil rows (the TeaLeaf layout, reading R16) at the assumed
// position start = s0 + 5 lane: straight-line code, one uniform branch for
// "any element needs correction / any index is not the canonical stencil
// neighbour or in range / rowptr disagrees" -> tile_row (identical semantics,
// so counts and results do not depend on which path ran).
template <int ES, int RS, int VS>
static __device__ __forceinline__ double tile_row5(const SpmvArgs& a, const SpmvArgs& sa, uint32_t start, uint32_t end,
                                                   const uint64_t* sval, const uint32_t* scol, const double* win,
                                                   int oslot, double p_own, int64_t own, uint32_t s0, int lane,
                                                   int mode, const uint32_t* crc_slice) {
  const uint32_t s1 = s0 + TILE_PE;
  if (start != s0 + 5u * (uint32_t)lane || end != start + 5u)
    return tile_row<ES, RS, VS>(sa, start, end, sval, scol, true, win, oslot, p_own, own, s0, s1, mode);
  const int n32 = (int)a.stencil_n;
  const int own_col = (int)(own - a.col_base);
  const uint32_t ckeep = col_keep(ES);
  uint64_t v[5];
  uint32_t c[5];
#pragma unroll
  for (int t = 0; t < 5; t++) {
    v[t] = sval[5 * lane + t];
    c[t] = scol[5 * lane + t];
  }
  uint32_t acc_r = 0, acc_p = 0, acc_u = 0;
  if (mode != MODE_RANGE) {   // uniform: interval mode's unchecked accesses skip the codec
    if (ES == CRC32C) {       // E-CRC over the row, slicing-by-4 tables
      uint32_t crc = 0xFFFFFFFFu, st = 0;
#pragma unroll
      for (int t = 0; t < 5; t++) {
        crc = crc_word(crc, lo32(v[t]), crc_slice);
        crc = crc_word(crc, hi32(v[t]), crc_slice);
        crc = crc_word(crc, t < 4 ? (c[t] & 0x00FFFFFFu) : c[t], crc_slice);
        if (t < 4) st |= (c[t] >> 24) << (8 * t);
      }
      acc_p = ((crc ^ 0xFFFFFFFFu) != st) ? 1u : 0u;
    }
    if ((ES == SECDED64 || ES == SECDED128) && ABFT_PAIR_E) {   // elements (0,1), (2,3) pair-packed, 4 alone
      e96_acc2(lo32(v[0]), hi32(v[0]), c[0], lo32(v[1]), hi32(v[1]), c[1], acc_u, acc_p);
      e96_acc2(lo32(v[2]), hi32(v[2]), c[2], lo32(v[3]), hi32(v[3]), c[3], acc_u, acc_p);
      e96_acc(lo32(v[4]), hi32(v[4]), c[4], acc_r, acc_p);
    } else {
#pragma unroll
      for (int t = 0; t < 5; t++) {
        if (ES == SED) acc_p |= (uint32_t)(popc64(v[t]) + popc32(c[t]));
        else if (ES == SECDED64 || ES == SECDED128) e96_acc(lo32(v[t]), hi32(v[t]), c[t], acc_r, acc_p);
      }
    }
  }
  // canonical stencil neighbours [i-n, i-1, i, i+1, i+n] or the row itself (R16)
  int d[5];
  uint32_t cmax = 0;
#pragma unroll
  for (int t = 0; t < 5; t++) {
    const uint32_t cm = c[t] & ckeep;
    cmax = max(cmax, cm);
    d[t] = (int)cm - own_col;
  }
  const bool canon = (d[0] == 0 || d[0] == -n32) && ((unsigned)(d[1] + 1) <= 1u) && d[2] == 0 &&
                     ((unsigned)d[3] <= 1u) && (d[4] == 0 || d[4] == n32);
  const bool in_range = (ES == NONE) || cmax < (uint32_t)a.ncols;
  if ((ES != NONE && (syn_bad(acc_r, acc_p) || (acc_u & MOEB2_SYN_MASK) != 0u)) || !canon || !in_range)
    return tile_row<ES, RS, VS>(sa, start, end, sval, scol, true, win, oslot, p_own, own, s0, s1, mode);
  // slot offsets: d itself for +-1 / 0, +-window width for +-n
  const int o0 = d[0] ? -TILE_WW : 0, o4 = d[4] ? TILE_WW : 0;
  double acc = fma(as_d(v[0]), win[oslot + o0], 0.0);
  acc = fma(as_d(v[1]), win[oslot + d[1]], acc);
  acc = fma(as_d(v[2]), p_own, acc);
  acc = fma(as_d(v[3]), win[oslot + d[3]], acc);
  acc = fma(as_d(v[4]), win[oslot + o4], acc);
  return acc;
}

#ifndef ABFT_TILE_MINB
#define ABFT_TILE_MINB 3
#endif
// decoded-window variant knob: 1 = every slot of the thread loaded and checked
// with one OR-accumulated branch; 0 (default) = the per-slot loop with a branch
// per codeword (measured faster on the same box: 0.2561 vs 0.2623 ms, r2k)
#ifndef ABFT_RP_AFTER_WAIT
#define ABFT_RP_AFTER_WAIT 0
#endif
// window TMA before the PDL wait when the host marks `in` final (early_in)
#ifndef ABFT_EARLY_WIN
#define ABFT_EARLY_WIN 1
#endif
#ifndef ABFT_WIN_ACC
#define ABFT_WIN_ACC 0
#endif
template <int ES, int RS, int VS, int DOT, bool FUSED = false>
__global__ void __launch_bounds__(256, ABFT_TILE_MINB) k_spmv_tile(const SpmvArgs a, const __grid_constant__ TileMaps tm) {
  static_assert(!FUSED || (vgrp(VS) == 1 && DOT), "fused calc_p: G = 1 vector schemes, CG SpMV only");
  extern __shared__ uint8_t s_raw[];
  __shared__ __align__(16) uint8_t s_lut[128];
  // the cold row path takes the arguments by reference: give it a SMEM copy so
  // the kernel parameters are never spilled to local memory
  __shared__ SpmvArgs s_args;
  uint8_t* s_dyn = s_raw + ((128u - (smem_u32(s_raw) & 127u)) & 127u);
  constexpr int NST = tile_nst<ES, RS>();   // pipeline stages of this instantiation
  double* s_win = reinterpret_cast<double*>(s_dyn + tile_off_win(NST));
  uint64_t* full = reinterpret_cast<uint64_t*>(s_dyn + tile_off_bar(NST));
  uint64_t* empty = full + NST;
  uint64_t* winbar = empty + NST;   // the TMA-staged `in` window
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  uint32_t* srp = reinterpret_cast<uint32_t*>(s_dyn + tile_off_rp(NST)) + warp * TILE_RP;
  constexpr bool SLICE = ABFT_CRC_SLICE_SMEM && (ES == CRC32C || RS == CRC32C);
  const uint32_t* s_slice = SLICE ? reinterpret_cast<const uint32_t*>(s_dyn + tile_off_crc(NST)) : &a.crc->slice[0][0];
  uint8_t* s_vpos = s_dyn + tile_off_crc(NST) + (SLICE ? 4 * CRC_SLICE_WORDS : 0);
  const int64_t n = a.stencil_n;
  const int64_t ny = a.nrows / n;
  const int64_t tiles_x = n >> 8;
  const int64_t tx0 = (blockIdx.x % tiles_x) << 8;
  const int64_t ty0 = ((int64_t)(blockIdx.x / tiles_x) + a.ty_lo) * TILE_TY;
  // ---- 0. producer: barriers, then the first NST passes in flight (the
  // matrix: loaded before the PDL grid dependency resolves)
  if (threadIdx.x == 0) {
#pragma unroll
    for (int s = 0; s < NST; s++) {
      mbar_init(&full[s], 1);
      mbar_init(&empty[s], TILE_TY);
    }
    mbar_init(winbar, 1);
    asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
#pragma unroll
    for (int k = 0; k < NST; k++) tile_produce(tm, s_dyn + k * TILE_STAGE, &full[k], tx0, ty0, k);
    if (ABFT_EARLY_WIN && !FUSED && a.early_in && vgrp(VS) == 1 && tm.has_vmaps) {   // `in` is final already
      mbar_expect_tx(winbar, TILE_WIN_BYTES);
      tma_3d(s_win, &tm.vin, 0, (int)(tx0 / 2 - 1), (int)(a.row_base / n + ty0 - 1), winbar);
    }
  }
  if (VS == SECDED64) load_lut(s_lut);
  // E-CRC / R-CRC slicing tables: only range-checked accesses (interval mode)
  // never read them, so a known-range launch skips the 4 KB fill; interval
  // launches learn their mode after the PDL wait and fill below if checked
  if (SLICE && a.check_interval <= 1 && a.check_mode != MODE_RANGE)
    smem_fill(const_cast<uint32_t*>(s_slice), &a.crc->slice[0][0], CRC_SLICE_WORDS);
  if (VS == CRC32C) smem_fill(reinterpret_cast<uint32_t*>(s_vpos), &a.crc->vpos[0][0][0], CRC_VPOS_WORDS);
  const uint8_t* cs = (VS == CRC32C) ? s_vpos : s_lut;   // vector codec tables
  const int64_t gy = ty0 + warp;
  const bool has_seg = gy < ny;
  const int64_t rowseg = gy * n + tx0;
  // ---- 1. rowptr of the segment (entries rowseg .. rowseg+256): loads first
  // (matrix, before the grid dependency), checks after it
  constexpr int G = rgrp(RS);
  constexpr int NG = 256 / G + 1;
  constexpr int PER = (NG + 31) / 32;
  uint32_t e[PER][G];
  if (has_seg) {
#pragma unroll
    for (int q = 0; q < PER; q++) {  // all loads first (latency overlapped)
      const int gl = lane + 32 * q;
      const uint32_t* gp = a.rowptr + (rowseg / G + gl) * G;
      if (gl < NG) {
        if (G == 1) e[q][0] = __ldg(gp);
        else if (G == 2) { uint2 u = __ldg(reinterpret_cast<const uint2*>(gp)); e[q][0] = u.x; e[q][1 % G] = u.y; }
        else {
#pragma unroll
          for (int t = 0; t < G; t += 4) {
            uint4 u = __ldg(reinterpret_cast<const uint4*>(gp + t));
            e[q][t] = u.x; e[q][(t + 1) % G] = u.y; e[q][(t + 2) % G] = u.z; e[q][(t + 3) % G] = u.w;
          }
        }
      }
    }
  }
  // the fast check of the loaded groups is pure arithmetic on matrix data;
  // R-CRC needs the SMEM tables, so it waits for the barrier.  ABFT_RP_AFTER_WAIT
  // = 0 (default): computed before the PDL wait (overlapping the previous
  // kernel's tail under PDL); 1: after the wait, once the CG state's stop flag
  // load is in flight (measured 0.2335 vs 0.2316 ms standalone, equal in the
  // CG loop, r2m)
  constexpr bool EARLY_RP = (RS != CRC32C);
  uint32_t rp_fast = 0;
  if (EARLY_RP && !ABFT_RP_AFTER_WAIT && has_seg) {
#pragma unroll
    for (int q = 0; q < PER; q++)
      if (RS != NONE && lane + 32 * q < NG) rp_fast |= rp_acc<RS>(e[q]);
  }
  pdl_wait();   // the previous kernel's writes (p / r, CG state, counters) are visible from here
  pdl_trigger();
  // the CG state's stop flag: loaded first, its latency overlapping the
  // rowptr check, the window TMA issue and the CTA barrier below
  const int stop_v = a.state ? *(volatile const int*)&a.state->stop : 0;
  if (EARLY_RP && ABFT_RP_AFTER_WAIT && has_seg) {
#pragma unroll
    for (int q = 0; q < PER; q++)
      if (RS != NONE && lane + 32 * q < NG) rp_fast |= rp_acc<RS>(e[q]);
  }
  // fused calc_p: iteration 1 multiplies by p_cur as init
  // wrote it; later iterations build p_cur from (in = p_{k-1}, r) in the window
  const bool fz = FUSED && a.state->iters > 0;
  uint64_t* const pin = (FUSED && !fz) ? a.p_cur : a.in;
  // G = 1, not building p_k: the raw `in` window arrives by one TMA box
  // (out-of-range rows / columns zero-filled = encoded +0.0) and is decoded in
  // place.  Unfused, it is issued right here, before the CG-state load below,
  // so the window's latency overlaps it (a stopped solve drains it).
  const bool tma_win = vgrp(VS) == 1 && !(FUSED && fz) && tm.has_vmaps;
  const bool win_issued = ABFT_EARLY_WIN && !FUSED && a.early_in;
  if (tma_win && !win_issued && threadIdx.x == 0) {
    mbar_expect_tx(winbar, TILE_WIN_BYTES);
    tma_3d(s_win, (FUSED && !fz) ? &tm.vcur : &tm.vin, 0, (int)(tx0 / 2 - 1), (int)(a.row_base / n + ty0 - 1), winbar);
  }
  if (threadIdx.x == 0) {
    s_args = a;
    if (FUSED) {
      s_args.in = pin;
      s_args.fz = fz ? 1 : 0;
      s_args.beta_f = fz ? a.state->beta : 0.0;
    }
  }
  const int mode = spmv_mode(a);
  if (SLICE && a.check_interval > 1 && mode != MODE_RANGE)
    smem_fill(const_cast<uint32_t*>(s_slice), &a.crc->slice[0][0], CRC_SLICE_WORDS);
  // every warp waits on winbar / the stage barriers below: thread 0's
  // mbarrier.init (and the SMEM tables) must be visible to the whole CTA first
  __syncthreads();
  if (has_seg) {
    if (!stop_v) {
      uint32_t acc = 0;
      if (mode != MODE_RANGE) {
        if (EARLY_RP) {
          acc = rp_fast;
        } else {
#pragma unroll
          for (int q = 0; q < PER; q++)
            if (RS != NONE && lane + 32 * q < NG) acc |= rcrc_acc_tab(e[q], s_slice);
        }
      }
      if (RS != NONE && (acc & 1u)) {  // cold: locate, correct, count (owner), per group
#pragma unroll
        for (int q = 0; q < PER; q++) {
          const int gl = lane + 32 * q;
          if (gl >= NG) continue;
          const int64_t g = rowseg / G + gl;
          uint32_t* gp = a.rowptr + g * G;
          // the codec works on a copy: taking e[q]'s address would put the whole
          // e[][] array (the hot prologue's rowptr loads) in local memory
          uint32_t c[G];
#pragma unroll
          for (int t = 0; t < G; t++) c[t] = e[q][t];
          int word = 0;
          int o = rp_check_group<RS>(c, &word, a.due);
          if (o == CORRECTED && mode == MODE_DETECT) o = DUE;   // interval mode: detection only
          if (o != CLEAN) {
            const int64_t own = g * G < a.nrows ? g * G : a.nrows - 1;
            const bool owner = own >= rowseg && own < rowseg + 256;
            if (o == CORRECTED) {
              uint32_t ov[G];   // (a copy: indexing e[q] would move it to local memory)
#pragma unroll
              for (int t = 0; t < G; t++) ov[t] = e[q][t];
              if (owner && scrub_entries32(gp, ov, c, G)) cnt_add(a.counts, T_ROWPTR, RS, CORRECTED);
#pragma unroll
              for (int t = 0; t < G; t++) e[q][t] = c[t];
            } else if (owner) {   // DUE: e keeps the stored bits
              cnt_add(a.counts, T_ROWPTR, RS, DUE);
              *a.due = 1;
            }
          }
        }
      }
#pragma unroll
      for (int q = 0; q < PER; q++) {
        const int gl = lane + 32 * q;
        if (gl >= NG) continue;
#pragma unroll
        for (int t = 0; t < G; t++) if (gl * G + t < TILE_RP) srp[gl * G + t] = e[q][t] & rp_keep(RS);
      }
    }
  }
  if (stop_v) {  // uniform per grid: drain the producer's copies before the CTA exits
    if (threadIdx.x == 0) {
      for (int s = 0; s < NST; s++) mbar_wait(&full[s], 0u);
      if (tma_win) mbar_wait(winbar, 0u);
    }
    return;
  }
  // ---- 2. decoded `in` window: rows ty0-1 .. ty0+TILE_TY, x = tx0-2 .. tx0+261
  const int64_t win0 = a.row_base + (ty0 - 1) * n + tx0 - TILE_WX0;   // in-index of slot (0,0)
  constexpr int WPER = (TILE_WW + 31) / 32;                             // 9 slots per lane per window row
  constexpr int VG = vgrp(VS);
  if (tma_win) {
    mbar_wait(winbar, 0);
    // every codeword of the tile is checked ONCE here (owner: counted + scrubbed),
    // halo codewords are checked without counting
    constexpr int WS = (TILE_TY + 2) * TILE_WW;
    const uint64_t* raw = reinterpret_cast<const uint64_t*>(s_win);
#if ABFT_WIN_ACC
    // fast path: all of this thread's slots loaded, their checks OR-accumulated,
    // one uniform branch; the cold path re-reads the raw words (not yet overwritten)
    constexpr int WQ = (WS + 255) / 256;
    uint64_t wv[WQ];
#pragma unroll
    for (int q = 0; q < WQ; q++) {
      const int sl = threadIdx.x + 256 * q;
      wv[q] = (q < WQ - 1 || sl < WS) ? raw[sl] : 0ull;
    }
    uint32_t wacc_r = 0, wacc_p = 0;
#pragma unroll
    for (int q = 0; q < WQ; q++) {
      if (VS == SED) wacc_p |= (uint32_t)popc64(wv[q]);
      if (VS == SECDED64) v64_acc(lo32(wv[q]), hi32(wv[q]), wacc_r, wacc_p);
    }
    if (!(VS != NONE && syn_bad(wacc_r, wacc_p))) {
#pragma unroll
      for (int q = 0; q < WQ; q++) {
        const int sl = threadIdx.x + 256 * q;
        if (q < WQ - 1 || sl < WS) s_win[sl] = as_d(wv[q] & vkeep(VS));
      }
    } else
#endif
#if ABFT_PAIR_W
    if (VS == SECDED64) {   // slot pairs (sl, sl + 256): one shared fast check, the per-slot path when it fails
      auto slot = [&](int sl, uint64_t w) {
        if (v64_bad(lo32(w), hi32(w))) {
          const int wy = sl / TILE_WW, j = sl - wy * TILE_WW;
          const int64_t idx = win0 + (int64_t)wy * n + j;
          const bool owner = wy >= 1 && wy <= TILE_TY && ty0 + wy - 1 < ny && j >= TILE_WX0 && j < TILE_WX0 + 256;
          w = v1_check<VS>(w, pin + idx, owner, a.counts, a.due);
        }
        s_win[sl] = as_d(w & vkeep(VS));
      };
#pragma unroll 1
      for (int sl = threadIdx.x; sl < WS; sl += 512) {
        const bool two = sl + 256 < WS;
        uint64_t w0 = raw[sl], w1 = two ? raw[sl + 256] : 0ull;   // zero is a clean codeword
        uint32_t au = 0, ap = 0;
        v64_acc2(lo32(w0), hi32(w0), lo32(w1), hi32(w1), au, ap);
        if (((au & MOEB2_SYN_MASK) | (ap & 1u)) == 0u) {
          s_win[sl] = as_d(w0 & vkeep(VS));
          if (two) s_win[sl + 256] = as_d(w1 & vkeep(VS));
        } else {   // cold
          slot(sl, w0);
          if (two) slot(sl + 256, w1);
        }
      }
    } else
#endif
#pragma unroll 1
    for (int sl = threadIdx.x; sl < WS; sl += 256) {
      uint64_t w = raw[sl];
      const bool bad = (VS == SED) ? !vsed_clean(w) : (VS == SECDED64) ? (v64_bad(lo32(w), hi32(w)) != 0u) : false;
      if (VS != NONE && bad) {   // cold: only real codewords fail (zero fill is clean)
        const int wy = sl / TILE_WW, j = sl - wy * TILE_WW;
        const int64_t idx = win0 + (int64_t)wy * n + j;
        const bool owner = wy >= 1 && wy <= TILE_TY && ty0 + wy - 1 < ny && j >= TILE_WX0 && j < TILE_WX0 + 256;
        w = v1_check<VS>(w, pin + idx, owner, a.counts, a.due);
      }
      s_win[sl] = as_d(w & vkeep(VS));
    }
    // grid-edge tiles: the x = -1 / x = n slots hold the linearly adjacent
    // entries (in-index +-1: the previous row's last / next row's first cell),
    // as the plain gather in[col] would read them for a column i -+ 1
    const bool eL = tx0 == 0, eR = tx0 + 256 == n;
    if (eL || eR) {
      __syncthreads();
      const int t = threadIdx.x;
      int wy = -1, j = 0;
      if (eL && t < TILE_TY + 2) { wy = t; j = TILE_WX0 - 1; }
      else if (eR && t >= 32 && t < 32 + TILE_TY + 2) { wy = t - 32; j = TILE_WX0 + 256; }
      if (wy >= 0) {
        const int64_t idx = win0 + (int64_t)wy * n + j;
        const uint64_t w = (idx >= 0 && idx < a.npad_in) ? v1_check<VS>(ldg64(pin + idx), pin + idx, false, a.counts, a.due)
                                                         : 0ull;
        s_win[wy * TILE_WW + j] = as_d(w & vkeep(VS));
      }
    }
  } else if (VG > 1) {  // G = 2 / 4: load aligned groups (lane 0 at tx0 - G), lane-split fast check
    for (int wy = warp; wy < TILE_TY + 2; wy += 8) {
      const int64_t a0 = win0 + (int64_t)wy * n + TILE_WX0 - VG;     // in-index of lane 0's word, aligned to G
      const bool row_own = wy >= 1 && wy <= TILE_TY && ty0 + wy - 1 < ny;
      double* dst = s_win + wy * TILE_WW;
      uint64_t wv[WPER];
      bool ok[WPER];
#pragma unroll
      for (int q = 0; q < WPER; q++) {
        const int64_t idx = a0 + 32 * q + lane;
        ok[q] = idx >= 0 && idx < a.npad_in;   // identical across a group (npad_in is a multiple of G)
        wv[q] = ok[q] ? ldg64(pin + idx) : 0ull;
      }
      bool bad = false;
      if (VS == SECDED128) {   // zero groups are clean
#pragma unroll
        for (int q = 0; q + 1 < WPER; q += 2) bad |= gbad2<VS>(wv[q], wv[q + 1], lane, cs);
        bad |= gbad2<VS>(wv[WPER - 1], 0ull, lane, cs);
      } else {
        const uint32_t* vp = vcrc_tab(cs, lane);
#pragma unroll
        for (int q = 0; q < WPER; q++) {
          const bool b = vcrc_bad_lane(wv[q], vp, lane);   // every lane: shuffles inside
          bad |= ok[q] & b;
        }
      }
      if (__any_sync(0xffffffffu, bad)) {   // cold: locate / correct per group (owner counts + scrubs)
#pragma unroll 1
        for (int q = 0; q < WPER; q++) {
          const int slot = 32 * q + lane + TILE_WX0 - VG;
          const bool owner = row_own && slot >= TILE_WX0 && slot < TILE_WX0 + 256;   // groups never straddle the tile edge
          wv[q] = vg_check<VS>(wv[q], pin + (a0 + 32 * q + (lane & ~(VG - 1))), lane, ok[q], owner && ok[q],
                               a.counts, a.due);
        }
      }
#pragma unroll
      for (int q = 0; q < WPER; q++) {
        const int slot = 32 * q + lane + TILE_WX0 - VG;
        if (slot >= 0 && slot < TILE_WW) dst[slot] = as_d(wv[q] & vkeep(VS));
      }
    }
  } else if (FUSED && fz) {
    // fused calc_p window (G = 1): every slot is p_k = round(fma(beta, p_{k-1},
    // r)) of the checked operands (the masked value of the word calc_p would
    // store); the tile's own cells (calc_p's owners) count and scrub, halo
    // cells are recomputed without counting.  enc(p_k) of the own cells is
    // stored to p_cur in the pass loop (off this latency-exposed phase).
    const double beta = a.state->beta;
    for (int wy = warp; wy < TILE_TY + 2; wy += 8) {
      const int64_t rbase = win0 + (int64_t)wy * n;
      const bool row_in = rbase >= 0 && rbase + TILE_WW <= a.npad_in;
      double* dst = s_win + wy * TILE_WW;
      uint64_t pv[WPER], rv[WPER];
#pragma unroll
      for (int q = 0; q < WPER; q++) {
        const int wx = lane + 32 * q;
        const int64_t idx = rbase + wx;
        const bool ok = wx < TILE_WW && (row_in || (idx >= 0 && idx < a.npad_in));
        pv[q] = ok ? ldg64(pin + idx) : 0ull;
        rv[q] = ok ? ldg64(a.r_f + idx) : 0ull;
      }
      uint32_t acc_r = 0, acc_p = 0;
#pragma unroll
      for (int q = 0; q < WPER; q++) {   // OR-accumulated fast check; zero (out-of-range) words are clean
        const int wx = lane + 32 * q;
        if (VS == SED) acc_p |= (uint32_t)(popc64(pv[q]) | popc64(rv[q]));
        if (VS == SECDED64) {
          v64_acc(lo32(pv[q]), hi32(pv[q]), acc_r, acc_p);
          v64_acc(lo32(rv[q]), hi32(rv[q]), acc_r, acc_p);
        }
        if (wx < TILE_WW) {
          const int64_t idx = rbase + wx;
          const bool ok = row_in || (idx >= 0 && idx < a.npad_in);
          const double pn = fma(beta, as_d(pv[q] & vkeep(VS)), as_d(rv[q] & vkeep(VS)));
          dst[wx] = ok ? as_d(round_k(as_u(pn), vk(VS))) : 0.0;
        }
      }
      if (VS != NONE && syn_bad(acc_r, acc_p)) {  // cold: reload, correct (owner counts + scrubs), recompute
        const bool row_own = wy >= 1 && wy <= TILE_TY && ty0 + wy - 1 < ny;
        for (int q = 0; q < WPER; q++) {
          const int wx = lane + 32 * q;
          const int64_t idx = rbase + wx;
          if (wx >= TILE_WW || idx < 0 || idx >= a.npad_in) continue;
          const bool owner = row_own && wx >= TILE_WX0 && wx < TILE_WX0 + 256;
          const uint64_t rw = v1_check<VS>(ldg64(a.r_f + idx), a.r_f + idx, owner, a.counts, a.due);
          const uint64_t pw = v1_check<VS>(ldg64(pin + idx), pin + idx, owner, a.counts, a.due);
          const double pn = fma(beta, as_d(pw & vkeep(VS)), as_d(rw & vkeep(VS)));
          dst[wx] = as_d(round_k(as_u(pn), vk(VS)));
        }
      }
    }
  } else
  for (int wy = warp; wy < TILE_TY + 2; wy += 8) {   // G = 1 without vector tensor maps
    const int64_t rbase = win0 + (int64_t)wy * n;                 // in-index of (wy, 0)
    const bool row_in = rbase >= 0 && rbase + TILE_WW <= a.npad_in;  // uniform: no per-slot bounds
    const bool row_own = wy >= 1 && wy <= TILE_TY && ty0 + wy - 1 < ny;
    const uint64_t* src = pin + rbase;
    double* dst = s_win + wy * TILE_WW;
    uint64_t wv[WPER];
#pragma unroll
    for (int q = 0; q < WPER; q++) {
      const int wx = lane + 32 * q;
      const int64_t idx = rbase + wx;
      const bool ok = wx < TILE_WW && (row_in || (idx >= 0 && idx < a.npad_in));
      wv[q] = ok ? ldg64(src + wx) : 0ull;
    }
    uint32_t badm = 0;
#pragma unroll
    for (int q = 0; q < WPER; q++) {
      const int wx = lane + 32 * q;
      if (VS == SED) badm |= (vsed_clean(wv[q]) ? 0u : 1u) << q;
      if (VS == SECDED64) badm |= (v64_bad(lo32(wv[q]), hi32(wv[q])) ? 1u : 0u) << q;
      if (wx < TILE_WW) dst[wx] = as_d(wv[q] & vkeep(VS));
    }
    if (VS != NONE && badm) {  // cold: reload, correct (owner counts + scrubs), overwrite
      for (int q = 0; q < WPER; q++) {
        if (!((badm >> q) & 1u)) continue;
        const int wx = lane + 32 * q;
        const int64_t idx = rbase + wx;
        if (wx >= TILE_WW || idx < 0 || idx >= a.npad_in) continue;
        const bool owner = row_own && wx >= TILE_WX0 && wx < TILE_WX0 + 256;
        const uint64_t w = v1_check<VS>(ldg64(src + wx), pin + idx, owner, a.counts, a.due);
        dst[wx] = as_d(w & vkeep(VS));
      }
    }
  }
  __syncthreads();
  // ---- 3. passes (every warp takes part in the stage protocol)
  double dot = 0.0, dot2 = 0.0;
  uint64_t acc_prev = 0;   // SECDED128: rounded result of the even pass awaiting its pair
  double p_prev = 0.0;
  const uint32_t seg_e = (uint32_t)(5 * rowseg);   // assumed element start of the segment
// pass-loop unroll: 8 (full) measured 0.2525 vs 0.2573 ms (r2l, same box):
// the stage index / phase / address arithmetic of every pass folds away
#ifndef ABFT_TILE_UNROLL
#define ABFT_TILE_UNROLL 8
#endif
  // (G > 1 vector codecs and the CRC element / rowptr codecs spill at 80
  // registers when the 8 passes are unrolled: they keep the rolled loop)
  constexpr int kPassUnroll = (vgrp(VS) == 1 && ES != CRC32C && RS != CRC32C) ? ABFT_TILE_UNROLL : 1;
#pragma unroll kPassUnroll
  for (int k = 0; k < 8; k++) {
    const int st = k % NST;
    const uint32_t ph = (uint32_t)((k / NST) & 1);
    uint8_t* stage = s_dyn + st * TILE_STAGE;
    mbar_wait(&full[st], ph);
    if (has_seg) {
      const uint64_t* sval = reinterpret_cast<const uint64_t*>(stage) + warp * TILE_PE;
      const uint32_t* scol = reinterpret_cast<const uint32_t*>(stage + TILE_STAGE_VAL) + warp * TILE_PE;
      const uint32_t start = srp[32 * k + lane], end = srp[32 * k + lane + 1];
      const int oslot = (warp + 1) * TILE_WW + k * 32 + lane + TILE_WX0;
      const double p_own = s_win[oslot];
      const int64_t own = a.row_base + rowseg + k * 32 + lane;
      const double acc = tile_row5<ES, RS, VS>(a, s_args, start, end, sval, scol, s_win, oslot, p_own, own,
                                               seg_e + 160u * k, lane, mode, s_slice);
      const uint64_t rounded = round_k(as_u(acc), vk(VS));
      if (VS == SECDED128) {   // encode pass pairs (k-1, k): pair gather
        if ((k & 1) == 0) {
          acc_prev = rounded;
          p_prev = p_own;
        } else {
          uint64_t e0, e1;
          genc2<VS>(acc_prev, rounded, lane, cs, e0, e1);
          a.out[own - 32] = e0;
          a.out[own] = e1;
          if (DOT) {
            dot = fma(p_prev, as_d(e0 & vkeep(VS)), dot);
            dot = fma(p_own, as_d(e1 & vkeep(VS)), dot);
          }
          if (DOT == 2) {
            dot2 = fma(p_prev, p_prev, dot2);
            dot2 = fma(p_own, p_own, dot2);
          }
        }
      } else {
        const uint64_t enc = (VS == CRC32C) ? vcrc_encode_lane(rounded, vcrc_tab(cs, lane), lane)
                                            : v_encode<VS>(rounded, lane, s_lut);
        a.out[own] = enc;
        if (FUSED && fz) a.p_cur[own] = v_encode<VS>(as_u(p_own), lane, s_lut);   // enc(p_k), own cell
        // enc & vkeep == rounded: the encoders only fill the k bits round_k cleared
        if (DOT) dot = fma(p_own, as_d(rounded), dot);
        if (DOT == 2) dot2 = fma(p_own, p_own, dot2);
      }
    }
    __syncwarp();
    if (lane == 0) mbar_arrive(&empty[st]);
    if (k + NST < 8 && threadIdx.x == 0) {  // refill the stage once every warp released it
      mbar_wait(&empty[st], ph);
      tile_produce(tm, stage, &full[st], tx0, ty0, k + NST);
    }
  }
  if (DOT && has_seg) {
#pragma unroll
    for (int off = 16; off >= 1; off >>= 1) dot = dot + __shfl_xor_sync(0xffffffffu, dot, off);
    if (lane == 0) a.partials[a.rb_offset + (rowseg >> 8)] = dot;
  }
  if (DOT == 2 && has_seg) {
#pragma unroll
    for (int off = 16; off >= 1; off >>= 1) dot2 = dot2 + __shfl_xor_sync(0xffffffffu, dot2, off);
    if (lane == 0) a.partials2[a.rb_offset + (rowseg >> 8)] = dot2;
  }
}

// ============================================================= BLAS-1 (a4, a5, a2)
// Full-RB fast paths: two passes per step, so each lane has 8 (calc_ur) / 4
// (calc_p) independent 8-byte loads in flight, and all addressing is pointer +
// immediate offset.  Lane l still visits rows l, l+32, ... in ascending order
// (RED-1).  G = 1 schemes check each word in its lane; G = 2 / 4 schemes use
// the lane-split group codecs (pair gather / V-CRC partials), the pass pair
// (k, k+32) being exactly what the SECDED128 pair gather needs.
// BLAS-1 V-SECDED64 fast checks in pairs (codec v64_acc2): off — calc_ur
// measured 0.1537 vs 0.1347 ms with it (r2o)
#ifndef ABFT_PAIR_V
#define ABFT_PAIR_V 0
#endif
// OR-accumulated fast check of up to 8 G=1 codewords (zero words are clean in
// every scheme): true iff any of them needs the per-word cold path.
template <int VS>
__device__ __forceinline__ bool vacc_bad(uint64_t w0, uint64_t w1, uint64_t w2, uint64_t w3, uint64_t w4, uint64_t w5,
                                         uint64_t w6, uint64_t w7) {
  if (VS == SED) return ((popc64(w0) | popc64(w1) | popc64(w2) | popc64(w3) | popc64(w4) | popc64(w5) |
                          popc64(w6) | popc64(w7)) & 1) != 0;
  if (VS == SECDED64 && ABFT_PAIR_V) {   // pair-packed fast checks (codec v64_acc2); zero words fold away
    uint32_t u = 0, p = 0;
    v64_acc2(lo32(w0), hi32(w0), lo32(w1), hi32(w1), u, p);
    v64_acc2(lo32(w2), hi32(w2), lo32(w3), hi32(w3), u, p);
    v64_acc2(lo32(w4), hi32(w4), lo32(w5), hi32(w5), u, p);
    v64_acc2(lo32(w6), hi32(w6), lo32(w7), hi32(w7), u, p);
    return ((u & MOEB2_SYN_MASK) | (p & 1u)) != 0u;
  }
  if (VS == SECDED64) {
    uint32_t r = 0, p = 0;
    v64_acc(lo32(w0), hi32(w0), r, p);
    v64_acc(lo32(w1), hi32(w1), r, p);
    v64_acc(lo32(w2), hi32(w2), r, p);
    v64_acc(lo32(w3), hi32(w3), r, p);
    v64_acc(lo32(w4), hi32(w4), r, p);
    v64_acc(lo32(w5), hi32(w5), r, p);
    v64_acc(lo32(w6), hi32(w6), r, p);
    v64_acc(lo32(w7), hi32(w7), r, p);
    return syn_bad(r, p);
  }
  return false;
}
// Check the words w0 (this lane's row of pass k at addr) and w1 (pass k+32):
// fast test, then (warp-uniform cold branch) locate / correct / count per group.
template <int VS>
__device__ __forceinline__ void vcheck2(uint64_t& w0, uint64_t& w1, uint64_t* addr, const VecArgs& a, int lane,
                                        const uint8_t* cs, bool any_bad) {
  constexpr int G = vgrp(VS);
  if (G == 1) {
    if (any_bad) {
      w0 = v1_check<VS>(w0, addr, true, a.counts, a.due);
      w1 = v1_check<VS>(w1, addr + 32, true, a.counts, a.due);
    }
  } else if (__any_sync(0xffffffffu, any_bad)) {
    w0 = vg_check<VS>(w0, addr - (lane & (G - 1)), lane, true, true, a.counts, a.due);
    w1 = vg_check<VS>(w1, addr + 32 - (lane & (G - 1)), lane, true, true, a.counts, a.due);
  }
}
// Encode two rounded values (rows of pass k and k+32).
template <int VS>
__device__ __forceinline__ void venc2(uint64_t r0, uint64_t r1, int lane, const uint8_t* cs, uint64_t& e0,
                                      uint64_t& e1) {
  if (vgrp(VS) == 1) {
    e0 = v_encode<VS>(r0, lane, cs);
    e1 = v_encode<VS>(r1, lane, cs);
  } else {
    genc2<VS>(r0, r1, lane, cs, e0, e1);
  }
}

template <int VS>
struct UrStep { uint64_t x0, x1, p0, p1, r0, r1, w0, w1; };
template <int VS>
__device__ __forceinline__ void ur_load(const uint64_t* X, const uint64_t* P, const uint64_t* R, const uint64_t* W, int k,
                                        UrStep<VS>& s) {
  s.x0 = ldg64(X + k); s.x1 = ldg64(X + k + 32); s.p0 = ldg64(P + k); s.p1 = ldg64(P + k + 32);
  s.r0 = ldg64(R + k); s.r1 = ldg64(R + k + 32); s.w0 = ldg64(W + k); s.w1 = ldg64(W + k + 32);
}
template <int VS>
__device__ __forceinline__ void ur_step(const VecArgs& a, uint64_t* X, uint64_t* P, uint64_t* R, uint64_t* W, int k,
                                        const UrStep<VS>& s, double alpha, int lane, const uint8_t* cs, double& dot);
// Full RB of calc_ur; step 0's loads were issued by the caller before the
// kernel's barrier / stop check so their latency overlaps the state loads.
template <int VS>
__device__ __forceinline__ double ur_full(const VecArgs& a, int64_t base, int lane, double alpha, const uint8_t* cs,
                                          UrStep<VS> s) {
  uint64_t* X = a.x + base + lane;
  uint64_t* P = a.p + base + lane;
  uint64_t* R = a.r + base + lane;
  uint64_t* W = a.w + base + lane;
  double dot = 0.0;
  ur_step<VS>(a, X, P, R, W, 0, s, alpha, lane, cs, dot);
#pragma unroll 1
  for (int k = 64; k < 256; k += 64) {
    ur_load<VS>(X, P, R, W, k, s);
    ur_step<VS>(a, X, P, R, W, k, s, alpha, lane, cs, dot);
  }
  return dot;
}
template <int VS>
__device__ __forceinline__ void ur_step(const VecArgs& a, uint64_t* X, uint64_t* P, uint64_t* R, uint64_t* W, int k,
                                        const UrStep<VS>& s, double alpha, int lane, const uint8_t* cs, double& dot) {
  const uint64_t keep = vkeep(VS);
  uint64_t x0 = s.x0, x1 = s.x1, p0 = s.p0, p1 = s.p1, r0 = s.r0, r1 = s.r1, w0 = s.w0, w1 = s.w1;
  if (vgrp(VS) == 1) {
    if (vacc_bad<VS>(x0, x1, p0, p1, r0, r1, w0, w1)) {  // cold: locate per word
      vcheck2<VS>(x0, x1, X + k, a, lane, cs, true);
      vcheck2<VS>(p0, p1, P + k, a, lane, cs, true);
      vcheck2<VS>(r0, r1, R + k, a, lane, cs, true);
      vcheck2<VS>(w0, w1, W + k, a, lane, cs, true);
    }
  } else {
    const bool bad = gbad2<VS>(x0, x1, lane, cs) | gbad2<VS>(p0, p1, lane, cs) | gbad2<VS>(r0, r1, lane, cs) |
                     gbad2<VS>(w0, w1, lane, cs);
    if (__any_sync(0xffffffffu, bad)) {  // cold, warp-uniform: locate per group
      vcheck2<VS>(x0, x1, X + k, a, lane, cs, true);
      vcheck2<VS>(p0, p1, P + k, a, lane, cs, true);
      vcheck2<VS>(r0, r1, R + k, a, lane, cs, true);
      vcheck2<VS>(w0, w1, W + k, a, lane, cs, true);
    }
  }
  const double xn0 = fma(alpha, as_d(p0 & keep), as_d(x0 & keep));
  const double xn1 = fma(alpha, as_d(p1 & keep), as_d(x1 & keep));
  const double rn0 = fma(-alpha, as_d(w0 & keep), as_d(r0 & keep));
  const double rn1 = fma(-alpha, as_d(w1 & keep), as_d(r1 & keep));
  uint64_t xe0, xe1, re0, re1;
  venc2<VS>(round_k(as_u(xn0), vk(VS)), round_k(as_u(xn1), vk(VS)), lane, cs, xe0, xe1);
  venc2<VS>(round_k(as_u(rn0), vk(VS)), round_k(as_u(rn1), vk(VS)), lane, cs, re0, re1);
  X[k] = xe0; X[k + 32] = xe1;
  R[k] = re0; R[k + 32] = re1;
  const double m0 = as_d(re0 & keep), m1 = as_d(re1 & keep);
  dot = fma(m0, m0, dot);
  dot = fma(m1, m1, dot);
}
// peer-memory halo: the encoded word of local row i also goes to the
// neighbour ghost row that mirrors it (VecArgs.halo_up / halo_dn)
__device__ __forceinline__ void halo_store(const VecArgs& a, int64_t i, uint64_t e) {
  if (a.halo_up && i < a.halo_n) a.halo_up[i] = e;
  if (a.halo_dn && i >= a.n - a.halo_n && i < a.n) a.halo_dn[i - (a.n - a.halo_n)] = e;
}
template <int VS>
__device__ __forceinline__ void p_step(const VecArgs& a, uint64_t* P, uint64_t* R, int k, uint64_t r0, uint64_t r1,
                                       uint64_t p0, uint64_t p1, double beta, int lane, const uint8_t* cs,
                                       int64_t row0 = 0, bool edge = false) {
  const uint64_t keep = vkeep(VS);
  if (vgrp(VS) == 1) {
    if (vacc_bad<VS>(r0, r1, p0, p1, 0ull, 0ull, 0ull, 0ull)) {  // cold: locate per word
      vcheck2<VS>(r0, r1, R + k, a, lane, cs, true);
      vcheck2<VS>(p0, p1, P + k, a, lane, cs, true);
    }
  } else {
    const bool bad = gbad2<VS>(r0, r1, lane, cs) | gbad2<VS>(p0, p1, lane, cs);
    if (__any_sync(0xffffffffu, bad)) {
      vcheck2<VS>(r0, r1, R + k, a, lane, cs, true);
      vcheck2<VS>(p0, p1, P + k, a, lane, cs, true);
    }
  }
  const double n0 = fma(beta, as_d(p0 & keep), as_d(r0 & keep));
  const double n1 = fma(beta, as_d(p1 & keep), as_d(r1 & keep));
  uint64_t e0, e1;
  venc2<VS>(round_k(as_u(n0), vk(VS)), round_k(as_u(n1), vk(VS)), lane, cs, e0, e1);
  P[k] = e0;
  P[k + 32] = e1;
  if (edge) {   // warp-uniform: this RB holds rows of the first / last grid row of the strip
    halo_store(a, row0 + k, e0);
    halo_store(a, row0 + k + 32, e1);
  }
}
// 0 (default): calc_p's end-of-iteration logic runs in a one-thread kernel
// after it (measured r2c: protected calc_p 0.0758 -> 0.0723 ms at 4096^2);
// 1: in calc_p's last CTA (per-CTA fence + ticket)
#ifndef ABFT_P_TICKET
#define ABFT_P_TICKET 0
#endif
#ifndef ABFT_P_UNROLL
#define ABFT_P_UNROLL 0
#endif
#ifndef ABFT_P_PREFETCH
#define ABFT_P_PREFETCH 1
#endif
// Full RB of calc_p; step 0's words were loaded by the caller ahead of the
// barrier / stop check.
template <int VS>
__device__ __forceinline__ void p_full(const VecArgs& a, int64_t base, int lane, double beta, const uint8_t* cs,
                                       uint64_t r0, uint64_t r1, uint64_t p0, uint64_t p1) {
  uint64_t* P = a.p + base + lane;
  uint64_t* R = a.r + base + lane;
  const bool edge = a.halo_n > 0 && (base < a.halo_n || base + 256 > a.n - a.halo_n);
  const int64_t row0 = base + lane;
#if ABFT_P_PREFETCH == 2
  // every word of the RB in flight at once (16 loads per lane), then the steps
  uint64_t rr[8], pp[8];
  rr[0] = r0; rr[1] = r1; pp[0] = p0; pp[1] = p1;
#pragma unroll
  for (int j = 1; j < 4; j++) {
    rr[2 * j] = ldg64(R + 64 * j); rr[2 * j + 1] = ldg64(R + 64 * j + 32);
    pp[2 * j] = ldg64(P + 64 * j); pp[2 * j + 1] = ldg64(P + 64 * j + 32);
  }
#pragma unroll
  for (int j = 0; j < 4; j++)
    p_step<VS>(a, P, R, 64 * j, rr[2 * j], rr[2 * j + 1], pp[2 * j], pp[2 * j + 1], beta, lane, cs, row0, edge);
#elif ABFT_P_PREFETCH
  // Register double buffer: step k+64's four words are in flight while step k
  // decodes / encodes (the codec ALU otherwise serialises with the next loads).
#if ABFT_P_UNROLL
#pragma unroll
#else
#pragma unroll 1
#endif
  for (int k = 0; k < 256; k += 64) {
    uint64_t nr0 = 0, nr1 = 0, np0 = 0, np1 = 0;
    if (k + 64 < 256) {
      nr0 = ldg64(R + k + 64); nr1 = ldg64(R + k + 96);
      np0 = ldg64(P + k + 64); np1 = ldg64(P + k + 96);
    }
    p_step<VS>(a, P, R, k, r0, r1, p0, p1, beta, lane, cs, row0, edge);
    r0 = nr0; r1 = nr1; p0 = np0; p1 = np1;
  }
#else
  p_step<VS>(a, P, R, 0, r0, r1, p0, p1, beta, lane, cs, row0, edge);
#pragma unroll 1
  for (int k = 64; k < 256; k += 64)
    p_step<VS>(a, P, R, k, ldg64(R + k), ldg64(R + k + 32), ldg64(P + k), ldg64(P + k + 32), beta, lane, cs, row0,
               edge);
#endif
}

// Codec tables of the BLAS-1 / SpMV kernels in shared memory: the V-SECDED64
// encoder LUT (128 B) or the V-CRC position tables (28 KB, dynamic).
template <int VS>
constexpr size_t vec_dyn_smem() { return VS == CRC32C ? sizeof(uint32_t) * CRC_VPOS_WORDS : 0; }
template <int VS>
__device__ __forceinline__ const uint8_t* vec_codec_smem(uint8_t* s_lut, uint8_t* s_dyn, const CrcTables* crc) {
  if (VS == SECDED64) { load_lut(s_lut); return s_lut; }
  if (VS == CRC32C) {
    smem_fill(reinterpret_cast<uint32_t*>(s_dyn), &crc->vpos[0][0][0], CRC_VPOS_WORDS);
    return s_dyn;
  }
  return s_lut;
}

template <int VS>
#ifndef ABFT_UR_MINB
#define ABFT_UR_MINB 5
#endif
#ifndef ABFT_P_MINB
#define ABFT_P_MINB 6
#endif
__global__ void __launch_bounds__(256, vgrp(VS) > 1 ? 3 : ABFT_UR_MINB) k_calc_ur(VecArgs a) {
  __shared__ __align__(16) uint8_t s_lut[128];
  extern __shared__ __align__(16) uint8_t s_dyn_v[];
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  const int64_t rb = (int64_t)blockIdx.x * 8 + warp;
  const bool full = rb * 256 + 256 <= a.n;
  UrStep<VS> s0{};
  if (full)  // issue step 0 first: its latency overlaps the state loads and the barrier
    ur_load<VS>(a.x + rb * 256 + lane, a.p + rb * 256 + lane, a.r + rb * 256 + lane, a.w + rb * 256 + lane, 0, s0);
  pdl_wait();   // alpha / stop from the pw reduction
  pdl_trigger();
  const int stop = a.state->stop;
  const double alpha = a.state->alpha;
  const uint8_t* cs = vec_codec_smem<VS>(s_lut, s_dyn_v, a.crc);
  __syncthreads();
  if (stop) return;
  if (rb * 256 >= a.n) return;
  double dot = 0.0;
  if (full) {
    dot = ur_full<VS>(a, rb * 256, lane, alpha, cs, s0);
  } else for (int k = 0; k < 8; k++) {
    const int64_t pb = rb * 256 + k * 32;
    if (pb >= a.n) break;
    const int64_t i = pb + lane;
    const bool valid = i < a.n;
    const int64_t lim = a.npad;
    uint64_t xw = v_load_check<VS>(a.x, i, lim, lane, true, a.counts, a.due);
    uint64_t pw = v_load_check<VS>(a.p, i, lim, lane, true, a.counts, a.due);
    uint64_t rw = v_load_check<VS>(a.r, i, lim, lane, true, a.counts, a.due);
    uint64_t ww = v_load_check<VS>(a.w, i, lim, lane, true, a.counts, a.due);
    const uint64_t keep = vkeep(VS);
    double X = fma(alpha, as_d(pw & keep), as_d(xw & keep));
    double R = fma(-alpha, as_d(ww & keep), as_d(rw & keep));
    uint64_t xe = v_encode<VS>(valid ? round_k(as_u(X), vk(VS)) : 0ull, lane, s_lut);
    uint64_t re = v_encode<VS>(valid ? round_k(as_u(R), vk(VS)) : 0ull, lane, s_lut);
    if (i < a.npad) { a.x[i] = xe; a.r[i] = re; }
    if (valid) { double rm = as_d(re & keep); dot = fma(rm, rm, dot); }
  }
#pragma unroll
  for (int off = 16; off >= 1; off >>= 1) dot = dot + __shfl_xor_sync(0xffffffffu, dot, off);
  if (lane == 0) a.partials[rb] = dot;
}

template <int VS>
__global__ void __launch_bounds__(256, vgrp(VS) > 1 ? 4 : ABFT_P_MINB) k_calc_p(VecArgs a) {
  __shared__ __align__(16) uint8_t s_lut[128];
  extern __shared__ __align__(16) uint8_t s_dyn_v[];
#if ABFT_P_TICKET
  __shared__ bool s_last;
#endif
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  const int64_t rb = (int64_t)blockIdx.x * 8 + warp;
  const bool full = rb * 256 + 256 <= a.n;
  uint64_t r0 = 0, r1 = 0, p0 = 0, p1 = 0;
  if (full) {  // issue step 0 first: its latency overlaps the state loads and the barrier
    const uint64_t* R = a.r + rb * 256 + lane;
    const uint64_t* P = a.p + rb * 256 + lane;
    r0 = ldg64(R); r1 = ldg64(R + 32); p0 = ldg64(P); p1 = ldg64(P + 32);
  }
  pdl_wait();   // beta / stop from the rrn reduction
  pdl_trigger();
  const int stop = a.state->stop;
  const double beta = a.state->beta;
  const uint8_t* cs = vec_codec_smem<VS>(s_lut, s_dyn_v, a.crc);
  __syncthreads();
  if (stop) return;
  if (full) {
    p_full<VS>(a, rb * 256, lane, beta, cs, r0, r1, p0, p1);
  } else if (rb * 256 < a.n) {
    for (int k = 0; k < 8; k++) {
      const int64_t pb = rb * 256 + k * 32;
      if (pb >= a.n) break;
      const int64_t i = pb + lane;
      const bool valid = i < a.n;
      const int64_t lim = a.npad;
      uint64_t rw = v_load_check<VS>(a.r, i, lim, lane, true, a.counts, a.due);
      uint64_t pw = v_load_check<VS>(a.p, i, lim, lane, true, a.counts, a.due);
      const uint64_t keep = vkeep(VS);
      double P = fma(beta, as_d(pw & keep), as_d(rw & keep));
      uint64_t pe = v_encode<VS>(valid ? round_k(as_u(P), vk(VS)) : 0ull, lane, s_lut);
      if (i < a.npad) a.p[i] = pe;
      if (a.halo_n > 0) halo_store(a, i, pe);
    }
  }
#if ABFT_P_TICKET
  // last block finishes the iteration: DUE policy and max_iters
  __syncthreads();
  if (threadIdx.x == 0) {
    __threadfence();
    unsigned t = atomicAdd(&a.state->ticket_p, 1u);
    s_last = (t == gridDim.x - 1);
  }
  __syncthreads();
  if (s_last && threadIdx.x == 0) {
    __threadfence();
    CgState* st = a.state;
    st->ticket_p = 0;
    volatile int* due = a.due;
    // multi-GPU runs take the DUE decision in k_due_combine after an all-gather
    if (!st->dist && st->abort_policy && *due) { st->stop = 1; st->status = ABFT_E_DUE; }
    else if (st->iters >= st->max_iters) { st->stop = 1; st->status = ABFT_E_NOT_CONVERGED; }
    st->rro = st->rrn;
  }
#endif
}
// calc_p staged by bulk copies (a5, G = 1 vector schemes): a persistent grid
// (CP_CTAS_PER_SM CTAs per SM) walks the vector in stages of CP_STAGE rows;
// thread 0 keeps CP_NST stages of r and p in flight (two 1-D
// cp.async.bulk copies into SMEM per stage, an mbarrier each), so the codec
// work of one stage never stalls the loads of the next.  Each row is checked
// (owner: counts + scrub), p = enc(round(fma(beta, p, r))) stored back, and
// the peer-memory halo rows mirrored — word for word what k_calc_p does.
constexpr int CP_STAGE = 1024;   // rows per stage: 8 KB of r + 8 KB of p
constexpr int CP_NST = 3;
constexpr int CP_CTAS_PER_SM = 4;
constexpr int CP_SMEM = CP_NST * 2 * CP_STAGE * 8 + 128;
static __device__ __forceinline__ void bulk_g2s(void* dst, const void* src, uint32_t bytes, uint64_t* bar) {
  asm volatile("cp.async.bulk.shared::cluster.global.mbarrier::complete_tx::bytes [%0], [%1], %2, [%3];" ::"r"(
                   smem_u32(dst)),
               "l"(reinterpret_cast<uint64_t>(src)), "r"(bytes), "r"(smem_u32(bar))
               : "memory");
}
template <int VS>
__global__ void __launch_bounds__(256, CP_CTAS_PER_SM) k_calc_p_bulk(VecArgs a) {
  static_assert(vgrp(VS) == 1, "G = 1 vector schemes");
  extern __shared__ __align__(128) uint8_t s_cp[];
  __shared__ __align__(16) uint8_t s_lut[128];
  __shared__ __align__(8) uint64_t s_bar[CP_NST];
  uint64_t* sbuf = reinterpret_cast<uint64_t*>(s_cp + ((128u - (smem_u32(s_cp) & 127u)) & 127u));
  const int64_t nstage = a.n / CP_STAGE;   // host: n % CP_STAGE == 0
  const int64_t G = gridDim.x;
  const int64_t mine = nstage > blockIdx.x ? (nstage - blockIdx.x + G - 1) / G : 0;   // stages of this CTA
  auto issue = [&](int64_t j) {   // j-th stage of this CTA into ring slot j % CP_NST
    const int slot = (int)(j % CP_NST);
    const int64_t row = (blockIdx.x + j * G) * CP_STAGE;
    uint64_t* dst = sbuf + (int64_t)slot * 2 * CP_STAGE;
    mbar_expect_tx(&s_bar[slot], 2 * CP_STAGE * 8);
    bulk_g2s(dst, a.r + row, CP_STAGE * 8, &s_bar[slot]);
    bulk_g2s(dst + CP_STAGE, a.p + row, CP_STAGE * 8, &s_bar[slot]);
  };
  if (threadIdx.x == 0) {   // r and p were last written >= 2 kernels back: loaded before the PDL wait
    for (int k = 0; k < CP_NST; k++) mbar_init(&s_bar[k], 1);
    asm volatile("fence.mbarrier_init.release.cluster;" ::: "memory");
    for (int64_t j = 0; j < CP_NST && j < mine; j++) issue(j);
  }
  if (VS == SECDED64) load_lut(s_lut);
  pdl_wait();   // beta / stop from the rrn reduction
  pdl_trigger();
  const int stop = a.state->stop;
  const double beta = a.state->beta;
  __syncthreads();   // barriers initialised, LUT in place
  if (stop) {   // drain the copies in flight before the CTA exits
    if (threadIdx.x == 0)
      for (int64_t j = 0; j < CP_NST && j < mine; j++) mbar_wait(&s_bar[j], 0u);
    return;
  }
  const uint64_t keep = vkeep(VS);
  const int lane = threadIdx.x & 31;
  for (int64_t j = 0; j < mine; j++) {
    const int slot = (int)(j % CP_NST);
    mbar_wait(&s_bar[slot], (uint32_t)((j / CP_NST) & 1));
    const uint64_t* sr = sbuf + (int64_t)slot * 2 * CP_STAGE;
    const uint64_t* sp = sr + CP_STAGE;
    const int64_t row = (blockIdx.x + j * G) * CP_STAGE;
    uint64_t rv[4], pv[4];
#pragma unroll
    for (int t = 0; t < 4; t++) {
      rv[t] = sr[threadIdx.x + 256 * t];
      pv[t] = sp[threadIdx.x + 256 * t];
    }
    if (vacc_bad<VS>(rv[0], rv[1], rv[2], rv[3], pv[0], pv[1], pv[2], pv[3])) {   // cold: per word, owner
#pragma unroll 1
      for (int t = 0; t < 4; t++) {
        const int64_t i = row + threadIdx.x + 256 * t;
        rv[t] = v1_check<VS>(rv[t], a.r + i, true, a.counts, a.due);
        pv[t] = v1_check<VS>(pv[t], a.p + i, true, a.counts, a.due);
      }
    }
    const bool edge = a.halo_n > 0 && (row < a.halo_n || row + CP_STAGE > a.n - a.halo_n);
#pragma unroll
    for (int t = 0; t < 4; t++) {
      const int64_t i = row + threadIdx.x + 256 * t;
      const double P = fma(beta, as_d(pv[t] & keep), as_d(rv[t] & keep));
      const uint64_t e = v_encode<VS>(round_k(as_u(P), vk(VS)), lane, s_lut);
      a.p[i] = e;
      if (edge) halo_store(a, i, e);
    }
    __syncthreads();   // every thread is done with this slot
    if (threadIdx.x == 0 && j + CP_NST < mine) issue(j + CP_NST);
  }
}

// ABFT_P_TICKET = 0: the end-of-iteration logic runs in this one-thread kernel
// after calc_p instead of in calc_p's last block (no per-CTA fence + ticket).
static __global__ void k_post_p(CgState* st, const int* due, int* sig_up, int* sig_dn) {
  pdl_wait();
  pdl_trigger();
  if (st->stop) return;
  if (!st->dist && st->abort_policy && *((volatile const int*)due)) { st->stop = 1; st->status = ABFT_E_DUE; }
  else if (st->iters >= st->max_iters) { st->stop = 1; st->status = ABFT_E_NOT_CONVERGED; }
  if (!st->pcg) st->rro = st->rrn;
  if (sig_up || sig_dn) {
    // peer-memory halo: calc_p (the previous kernel, complete) stored this
    // iteration's boundary rows into the neighbours' ghost rows; publish them
    // system-wide, then raise the neighbours' arrival flags to the iteration
    __threadfence_system();
    if (sig_up) atomicExch_system(sig_up, st->iters);
    if (sig_dn) atomicExch_system(sig_dn, st->iters);
  }
}
// Peer-memory halo, consumer side: before the SpMV of iteration iters + 1
// (boundary tile rows), wait until both neighbours' calc_p of iteration
// `iters` has published p's ghost rows (flags[0]: from rank - 1, flags[1]: from
// rank + 1).  A stopped solve does not wait.
static __global__ void k_wait_halo(const int* flags, const CgState* st, int need_up, int need_dn) {
  const volatile CgState* vs = st;
  if (vs->stop) return;
  const int it = vs->iters;
  const volatile int* f = flags;
  while ((need_up && f[0] < it) || (need_dn && f[1] < it)) {
    if (vs->stop) return;
    __nanosleep(64);
  }
  __threadfence_system();   // acquire: the ghost rows are read after the flags
}

// Single-reduction CG update (S§8(f) f3): p = enc(fma(beta,
// p, r)); s = enc(fma(beta, s, w)); x = enc(fma(alpha, p', x)); r =
// enc(fma(-alpha, s', r)) with p', s' the masked NEW stored values.  Checks
// (owner: counts + scrubs) x, p, s, r, w; VecArgs.b carries s.
template <int VS>
__global__ void __launch_bounds__(256) k_calc_sr(VecArgs a) {
  __shared__ __align__(16) uint8_t s_lut[128];
  extern __shared__ __align__(16) uint8_t s_dyn_v[];
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  const int64_t rb = (int64_t)blockIdx.x * 8 + warp;
  pdl_wait();   // alpha / beta / stop from the reduction
  pdl_trigger();
  const int stop = a.state->stop;
  const double alpha = a.state->alpha, beta = a.state->beta;
  const uint8_t* cs = vec_codec_smem<VS>(s_lut, s_dyn_v, a.crc);
  (void)cs;
  __syncthreads();
  if (stop || rb * 256 >= a.n) return;
  uint64_t* const S = a.b;
  const uint64_t keep = vkeep(VS);
  for (int k = 0; k < 8; k++) {
    const int64_t pb = rb * 256 + k * 32;
    if (pb >= a.n) break;
    const int64_t i = pb + lane;
    const bool valid = i < a.n;
    const int64_t lim = a.npad;
    const uint64_t xw = v_load_check<VS>(a.x, i, lim, lane, true, a.counts, a.due);
    const uint64_t pw = v_load_check<VS>(a.p, i, lim, lane, true, a.counts, a.due);
    const uint64_t sw = v_load_check<VS>(S, i, lim, lane, true, a.counts, a.due);
    const uint64_t rw = v_load_check<VS>(a.r, i, lim, lane, true, a.counts, a.due);
    const uint64_t ww = v_load_check<VS>(a.w, i, lim, lane, true, a.counts, a.due);
    const uint64_t pr = valid ? round_k(as_u(fma(beta, as_d(pw & keep), as_d(rw & keep))), vk(VS)) : 0ull;
    const uint64_t sr = valid ? round_k(as_u(fma(beta, as_d(sw & keep), as_d(ww & keep))), vk(VS)) : 0ull;
    const uint64_t pe = v_encode<VS>(pr, lane, s_lut);
    const uint64_t se = v_encode<VS>(sr, lane, s_lut);
    const uint64_t xr = valid ? round_k(as_u(fma(alpha, as_d(pe & keep), as_d(xw & keep))), vk(VS)) : 0ull;
    const uint64_t rr = valid ? round_k(as_u(fma(-alpha, as_d(se & keep), as_d(rw & keep))), vk(VS)) : 0ull;
    const uint64_t xe = v_encode<VS>(xr, lane, s_lut);
    const uint64_t re = v_encode<VS>(rr, lane, s_lut);
    if (i < a.npad) { a.p[i] = pe; S[i] = se; a.x[i] = xe; a.r[i] = re; }
  }
}

// Chebyshev update (TeaLeaf tea_leaf_cheby, reading R32):
// r = enc(b - w); p = enc(r'/theta) (INIT) or enc(fma(alpha, p', beta r'));
// u = enc(u' + p'); RED-1 partials of r'.r'.  Checks b, w, (p), u; VecArgs.x is u.
// MODE 0 / 1: step / first step with the state's coefficients (abft_cheby_solve);
// MODE 2 / 3: step / first step from u = 0 with the given coefficients (PPCG).
template <int VS, int MODE>
__global__ void __launch_bounds__(256) k_cheb(VecArgs a, double c_alpha, double c_beta, double c_theta) {
  constexpr bool INIT = (MODE == 1 || MODE == 3), ZERO = (MODE == 3);
  __shared__ __align__(16) uint8_t s_lut[128];
  extern __shared__ __align__(16) uint8_t s_dyn_v[];
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  const int64_t rb = (int64_t)blockIdx.x * 8 + warp;
  pdl_wait();
  pdl_trigger();
  const int stop = a.state->stop;
  const double alpha = MODE >= 2 ? c_alpha : a.state->alpha, beta = MODE >= 2 ? c_beta : a.state->beta;
  const double theta = MODE >= 2 ? c_theta : a.state->ch_theta;
  const uint8_t* cs = vec_codec_smem<VS>(s_lut, s_dyn_v, a.crc);
  (void)cs;
  __syncthreads();
  if (stop || rb * 256 >= a.n) return;
  const uint64_t keep = vkeep(VS);
  double dot = 0.0;
  for (int k = 0; k < 8; k++) {
    const int64_t pb = rb * 256 + k * 32;
    if (pb >= a.n) break;
    const int64_t i = pb + lane;
    const bool valid = i < a.n;
    const int64_t lim = a.npad;
    const uint64_t bw = v_load_check<VS>(a.b, i, lim, lane, true, a.counts, a.due);
    const uint64_t ww = ZERO ? 0ull : v_load_check<VS>(a.w, i, lim, lane, true, a.counts, a.due);
    const uint64_t pw = INIT ? 0ull : v_load_check<VS>(a.p, i, lim, lane, true, a.counts, a.due);
    const uint64_t uw = ZERO ? 0ull : v_load_check<VS>(a.x, i, lim, lane, true, a.counts, a.due);
    const uint64_t rr = !valid ? 0ull
                        : ZERO ? round_k(bw & keep, vk(VS))
                               : round_k(as_u(__dsub_rn(as_d(bw & keep), as_d(ww & keep))), vk(VS));
    const uint64_t re = v_encode<VS>(rr, lane, s_lut);
    const double rm = as_d(re & keep);
    const double pn = INIT ? rm / theta : fma(alpha, as_d(pw & keep), __dmul_rn(beta, rm));
    const uint64_t pe = v_encode<VS>(valid ? round_k(as_u(pn), vk(VS)) : 0ull, lane, s_lut);
    const double un = ZERO ? as_d(pe & keep) : __dadd_rn(as_d(uw & keep), as_d(pe & keep));
    const uint64_t ue = v_encode<VS>(valid ? round_k(as_u(un), vk(VS)) : 0ull, lane, s_lut);
    if (i < a.npad) { a.r[i] = re; a.p[i] = pe; a.x[i] = ue; }
    if (valid) dot = fma(rm, rm, dot);
  }
#pragma unroll
  for (int off = 16; off >= 1; off >>= 1) dot = dot + __shfl_xor_sync(0xffffffffu, dot, off);
  if (lane == 0) a.partials[rb] = dot;
}

// Checked dot a.r . a.x over the masked stored values (PPCG's r.z; RED-1
// partials); both operands checked as their owner (O9).
template <int VS>
__global__ void __launch_bounds__(256) k_dot(VecArgs a) {
  __shared__ __align__(16) uint8_t s_lut[128];
  extern __shared__ __align__(16) uint8_t s_dyn_v[];
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  const int64_t rb = (int64_t)blockIdx.x * 8 + warp;
  pdl_wait();
  pdl_trigger();
  const int stop = a.state->stop;
  (void)vec_codec_smem<VS>(s_lut, s_dyn_v, a.crc);
  __syncthreads();
  if (stop || rb * 256 >= a.n) return;
  const uint64_t keep = vkeep(VS);
  double dot = 0.0;
  for (int k = 0; k < 8; k++) {
    const int64_t pb = rb * 256 + k * 32;
    if (pb >= a.n) break;
    const int64_t i = pb + lane;
    const uint64_t rw = v_load_check<VS>(a.r, i, a.npad, lane, true, a.counts, a.due);
    const uint64_t zw = v_load_check<VS>(a.x, i, a.npad, lane, true, a.counts, a.due);
    if (i < a.n) dot = fma(as_d(rw & keep), as_d(zw & keep), dot);
  }
#pragma unroll
  for (int off = 16; off >= 1; off >>= 1) dot = dot + __shfl_xor_sync(0xffffffffu, dot, off);
  if (lane == 0) a.partials[rb] = dot;
}
static __global__ void k_copy_running(uint64_t* dst, const uint64_t* src, int64_t npad, const CgState* st) {
  pdl_wait();
  pdl_trigger();
  if (st->stop) return;
  for (int64_t i = blockIdx.x * (int64_t)blockDim.x + threadIdx.x; i < npad; i += (int64_t)gridDim.x * blockDim.x)
    dst[i] = src[i];
}

// init (a2): r = enc(round(b - w)), p = r, rr0 partials
template <int VS>
__global__ void __launch_bounds__(256) k_init_r(VecArgs a) {
  __shared__ __align__(16) uint8_t s_lut[128];
  if (VS == SECDED64) load_lut(s_lut);
  __syncthreads();
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  const int64_t rb = (int64_t)blockIdx.x * 8 + warp;
  if (rb * 256 >= a.n) return;
  double dot = 0.0;
  for (int k = 0; k < 8; k++) {
    const int64_t pb = rb * 256 + k * 32;
    if (pb >= a.n) break;
    const int64_t i = pb + lane;
    const bool valid = i < a.n;
    const int64_t lim = a.npad;
    uint64_t bw = v_load_check<VS>(a.b, i, lim, lane, true, a.counts, a.due);
    uint64_t ww = v_load_check<VS>(a.w, i, lim, lane, true, a.counts, a.due);
    const uint64_t keep = vkeep(VS);
    double R = as_d(bw & keep) - as_d(ww & keep);
    uint64_t re = v_encode<VS>(valid ? round_k(as_u(R), vk(VS)) : 0ull, lane, s_lut);
    if (i < a.npad) { a.r[i] = re; a.p[i] = re; }
    if (valid) { double rm = as_d(re & keep); dot = fma(rm, rm, dot); }
  }
#pragma unroll
  for (int off = 16; off >= 1; off >>= 1) dot = dot + __shfl_xor_sync(0xffffffffu, dot, off);
  if (lane == 0) a.partials[rb] = dot;
}

// ============================================================ reduction (a6)
// Complete binary tree over the RB partials padded to a power of two: each
// block reduces an aligned subtree of <= 1024 leaves in shared memory, the
// last block (ticket) reduces the block roots and applies the CG scalar logic.
static __device__ __forceinline__ double tree_smem(double* s, int m) {
  // s[0..m) -> pairwise levels; m power of two; blockDim >= m/2
  for (; m > 1; m >>= 1) {
    double v = 0.0;
    const int t = threadIdx.x;
    if (t < m / 2) v = s[2 * t] + s[2 * t + 1];
    __syncthreads();
    if (t < m / 2) s[t] = v;
    __syncthreads();
  }
  return s[0];
}

// CG scalar logic applied by exactly one thread.
// Chebyshev step coefficients for the next step, rounded as
// written: no contraction into FMAs
static __device__ __forceinline__ void cheb_next(CgState* st) {
  const double rho_new = __ddiv_rn(1.0, __dsub_rn(__dmul_rn(2.0, st->ch_sigma), st->ch_rho));
  st->alpha = __dmul_rn(rho_new, st->ch_rho);
  st->beta = __ddiv_rn(__dmul_rn(2.0, rho_new), st->ch_delta);
  st->ch_rho = rho_new;
}
static __device__ void apply_op(int op, double res, CgState* st, bool dueflag) {
  if (op == 8) {  // Chebyshev init: rr0 of r = b - A u0
    st->rr0 = st->rro = st->rrn = res;
    if (st->abort_policy && dueflag) { st->stop = 1; st->status = ABFT_E_DUE; }
    else if (res == 0.0) { st->stop = 1; st->status = ABFT_OK; st->converged = 1; }
    else if (st->max_iters <= 0) { st->stop = 1; st->status = ABFT_OK; }
    else cheb_next(st);
    return;
  }
  if (op == 9) {  // Chebyshev step
    st->iters += 1;
    st->rrn = res;
    const bool conv = sqrt(res) <= st->tol * sqrt(st->rr0);
    if (st->abort_policy && dueflag) { st->stop = 1; st->status = ABFT_E_DUE; }
    else if (conv) { st->stop = 1; st->status = ABFT_OK; st->converged = 1; }
    else if (st->iters >= st->max_iters) { st->stop = 1; st->status = ABFT_E_NOT_CONVERGED; }
    else cheb_next(st);
    return;
  }
  if (op == 12) { st->rro = res; return; }   // PPCG init: rz = r.z
  if (op == 11) {                             // PPCG: beta = rz'/rz, rz = rz'
    st->beta = res / st->rro;
    st->rro = res;
    return;
  }
  if (op == 1) {  // rr0
    st->rr0 = st->rro = st->rrn = res;
    if (st->abort_policy && dueflag) { st->stop = 1; st->status = ABFT_E_DUE; }
    else if (res == 0.0) { st->stop = 1; st->status = ABFT_OK; st->converged = 1; }
    else if (st->max_iters <= 0) { st->stop = 1; st->status = ABFT_OK; }
  } else if (op == 2) {  // pw -> alpha
    st->pw = res;
    st->alpha = st->rro / res;
    st->iters += 1;
    if (st->alpha_log && st->iters <= CG_LOG) st->alpha_log[st->iters - 1] = st->alpha;
  } else if (op == 3) {  // rrn -> convergence, beta
    st->rrn = res;
    if (sqrt(res) <= st->tol * sqrt(st->rr0)) {
      st->stop = 1;
      st->converged = 1;
      st->status = (st->abort_policy && dueflag) ? ABFT_E_DUE : ABFT_OK;
    } else {
      st->beta = res / st->rro;
      if (st->beta_log && st->iters <= CG_LOG) st->beta_log[st->iters - 1] = st->beta;
      if (st->fused) {  // calc_p's last-block logic (k_calc_p), taken here: calc_p runs in the next SpMV
        st->rro = res;
        if (!st->dist && st->abort_policy && dueflag) { st->stop = 1; st->status = ABFT_E_DUE; st->pending_p = 1; }
        else if (st->iters >= st->max_iters) { st->stop = 1; st->status = ABFT_E_NOT_CONVERGED; st->pending_p = 1; }
      }
    }
  }
}

// Pairwise tree of m = 2^j values held by lanes 0..m-1 (m <= 32): butterfly
// over offsets 1..m/2 combines adjacent subtrees first; lane 0 gets the root.
static __device__ __forceinline__ double warp_tree(double v, int m) {
  for (int off = 1; off < m; off <<= 1) v = v + __shfl_xor_sync(0xffffffffu, v, off);
  return v;
}
// Tree over L = 2^j leaves src[0..L) (src[i] for i >= valid read as 0) by one warp.
static __device__ double warp_subtree(const double* src, int64_t L, int64_t valid, int lane) {
  if (L <= 32) {
    double v = (lane < L && lane < valid) ? __ldcg(src + lane) : 0.0;
    return warp_tree(v, (int)L);
  }
  const int per = (int)(L / 32);  // leaves per lane, power of two <= 32
  double t[32];
  for (int i = 0; i < per; i++) {
    const int64_t j = (int64_t)lane * per + i;
    t[i] = (j < valid) ? __ldcg(src + j) : 0.0;
  }
  for (int m = per; m > 1; m >>= 1)
    for (int i = 0; i < m / 2; i++) t[i] = t[2 * i] + t[2 * i + 1];
  return warp_tree(t[0], 32);
}
// Single-reduction CG scalar logic: g = r.r, d = w.r of the
// SpMV w = A r.  op 7: init (rr0); op 6: end of an iteration.
static __device__ void apply_op_sr(int op, double g, double d, CgState* st, bool dueflag) {
  if (op == 7) {
    st->rr0 = st->rro = st->rrn = g;
    st->pw = d;
    if (st->abort_policy && dueflag) { st->stop = 1; st->status = ABFT_E_DUE; }
    else if (g == 0.0) { st->stop = 1; st->status = ABFT_OK; st->converged = 1; }
    else if (st->max_iters <= 0) { st->stop = 1; st->status = ABFT_OK; }
    else { st->alpha = g / d; st->beta = 0.0; }
    return;
  }
  st->iters += 1;
  st->rrn = g;
  st->pw = d;
  const bool conv = sqrt(g) <= st->tol * sqrt(st->rr0);
  if (!conv) {
    const double beta = g / st->rro;
    st->alpha = g / (d - beta * g / st->alpha);
    st->beta = beta;
    st->rro = g;
  }
  if (st->abort_policy && dueflag) { st->stop = 1; st->status = ABFT_E_DUE; }
  else if (conv) { st->stop = 1; st->status = ABFT_OK; st->converged = 1; }
  else if (st->iters >= st->max_iters) { st->stop = 1; st->status = ABFT_E_NOT_CONVERGED; }
}

// ABFT_RED_PREFETCH (default 1): stop flag, CG state and DUE flag loaded at
// the start of k_reduce (their latency overlapping the subtree loads); the
// scalar logic runs on a register copy of the state
#ifndef ABFT_RED_PREFETCH
#define ABFT_RED_PREFETCH 1
#endif
// TWO: also reduce partials2 (second tree, same order) and apply the
// single-reduction CG logic (op 6 / 7) to both results.
template <bool TWO>
static __global__ void __launch_bounds__(256) k_reduce(const double* partials, int64_t nrb, int64_t leaves,
                                                       double* roots, uint32_t* ticket, int op, CgState* st,
                                                       double* out, const int* due, const double* partials2,
                                                       double* roots2) {
  // Block b reduces leaves [b*L, b*L+L): warp w the aligned sub-range of L/8
  // leaves (warp trees keep the pairwise order), then warp 0 combines the 8
  // warp roots; the last block (ticket) combines the block roots.
  __shared__ double s_w[8], s_w2[8];
  __shared__ bool s_last;
  pdl_wait();   // partials of the producing kernel
  pdl_trigger();
  const bool check_stop = st && op != 1 && op != 7 && op != 8 && op != 10;
#if ABFT_RED_PREFETCH
  // the stop flag, the CG state and the DUE flag are loaded now, in flight
  // while the subtree is reduced (thread 0: used by the last block)
  const int stopv = check_stop ? *(volatile const int*)&st->stop : 0;
  CgState loc;
  bool due_pre = false;
  if (threadIdx.x == 0) {
    if (st) loc = *st;
    due_pre = *((volatile const int*)due) != 0;
  }
#else
  if (check_stop && st->stop) return;
#endif
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  const int64_t base = (int64_t)blockIdx.x * leaves;
  const int nw = leaves >= 8 ? 8 : 1;
  const int64_t per = leaves / nw;
  double r = 0.0, r2 = 0.0;
  if (warp < nw) {
    r = warp_subtree(partials + base + warp * per, per, nrb - base - warp * per, lane);
    if (TWO) r2 = warp_subtree(partials2 + base + warp * per, per, nrb - base - warp * per, lane);
  }
#if ABFT_RED_PREFETCH
  if (stopv) return;   // uniform over the grid
#endif
  if (warp < nw && lane == 0) {
    s_w[warp] = r;
    if (TWO) s_w2[warp] = r2;
  }
  __syncthreads();
  double root = 0.0, root2 = 0.0;
  if (warp == 0) {
    root = warp_tree((lane < nw) ? s_w[lane] : 0.0, nw);
    if (TWO) root2 = warp_tree((lane < nw) ? s_w2[lane] : 0.0, nw);
  }
  if (gridDim.x > 1) {
    if (threadIdx.x == 0) {
      roots[blockIdx.x] = root;
      if (TWO) roots2[blockIdx.x] = root2;
      __threadfence();
      s_last = (atomicAdd(ticket, 1u) == gridDim.x - 1);
    }
    __syncthreads();
    if (!s_last || warp != 0) return;
    __threadfence();
    root = warp_subtree(roots, gridDim.x, gridDim.x, lane);
    if (TWO) root2 = warp_subtree(roots2, gridDim.x, gridDim.x, lane);
  }
  if (threadIdx.x != 0) return;
  if (gridDim.x > 1) *ticket = 0;
#if ABFT_RED_PREFETCH
  const bool dueflag = due_pre;
  CgState* const sp = &loc;   // the scalar logic on the register copy, written back once
#else
  const bool dueflag = *((volatile const int*)due) != 0;
  CgState* const sp = st;
#endif
  if (TWO && op == 10) { out[0] = root; out[1] = (double)(dueflag ? 1 : 0); out[2] = root2; return; }
  if (op == 0) { *out = root; return; }
  if (op == 4) { out[0] = root; out[1] = (double)(dueflag ? 1 : 0); out[2] = 0.0; return; }
  if (TWO) apply_op_sr(op, root2, root, sp, dueflag);
  else apply_op(op, root, sp, dueflag);
#if ABFT_RED_PREFETCH
  *st = loc;
#endif
}

// Cluster form of k_reduce (a6) for p2 <= RED_CL_MAX padded leaves: one thread
// block cluster of C <= 8 CTAs x nt threads; CTA c reduces the aligned subtree
// [c L, c L + L) (thread: lpt consecutive leaves pairwise, then the warp
// butterfly, then the warp roots in SMEM), and CTA 0 combines the C CTA roots
// through distributed shared memory — the same complete binary tree as
// k_reduce, with no global ticket, fence or roots array.  CTA 0's thread 0
// loads the CG state and the DUE flag (after pdl_wait) before the tree, so
// their latency overlaps it, and applies the scalar logic on a register copy.
constexpr int RED_CL_MAX = 8 * 512 * 16;
static __device__ __forceinline__ uint32_t cluster_ctarank() {
  uint32_t r;
  asm volatile("mov.u32 %0, %%cluster_ctarank;" : "=r"(r));
  return r;
}
static __device__ __forceinline__ void cluster_sync_all() {
  asm volatile("barrier.cluster.arrive.release.aligned;\n barrier.cluster.wait.acquire.aligned;" ::: "memory");
}
static __device__ __forceinline__ double ld_dsmem_f64(const double* local, uint32_t rank) {
  uint32_t a = smem_u32(local), ra;
  asm volatile("mapa.shared::cluster.u32 %0, %1, %2;" : "=r"(ra) : "r"(a), "r"(rank));
  double v;
  asm volatile("ld.shared::cluster.f64 %0, [%1];" : "=d"(v) : "r"(ra) : "memory");
  return v;
}
// one thread's lpt (power of two <= 16) consecutive leaves, pairwise
static __device__ __forceinline__ double thread_subtree(const double* src, int64_t j0, int lpt, int64_t valid) {
  double t[16];
#pragma unroll
  for (int i = 0; i < 16; i++)
    if (i < lpt) t[i] = (j0 + i < valid) ? __ldcg(src + j0 + i) : 0.0;
#pragma unroll
  for (int m = 16; m > 1; m >>= 1)
    if (m <= lpt) {
#pragma unroll
      for (int i = 0; i < m / 2; i++) t[i] = t[2 * i] + t[2 * i + 1];
    }
  return t[0];
}
template <bool TWO>
static __global__ void __launch_bounds__(512) k_reduce_cl(const double* partials, int64_t nrb, int nt, int lpt, int op,
                                                           CgState* st, double* out, const int* due,
                                                           const double* partials2) {
  __shared__ double s_w[16], s_w2[16];
  __shared__ double s_root[2];
  pdl_wait();   // partials of the producing kernel
  pdl_trigger();
  const uint32_t rank = cluster_ctarank();
  const bool fin = rank == 0 && threadIdx.x == 0;
  CgState loc;
  bool dueflag = false;
  if (fin) {   // the scalar logic's inputs, in flight while the tree is computed
    if (st) loc = *st;
    dueflag = *((volatile const int*)due) != 0;
  }
  const bool stopped = st && op != 1 && op != 7 && op != 8 && op != 10 && st->stop;
  const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
  // nt threads hold the CTA's leaves (blockDim.x = max(nt, 32): lanes >= nt
  // read past p2 >= nrb, i.e. zeros, and stay outside lane 0's nt-lane tree)
  const int64_t L = (int64_t)nt * lpt;
  const int64_t j0 = (int64_t)rank * L + (int64_t)threadIdx.x * lpt;
  double v = thread_subtree(partials, j0, lpt, nrb);
  double v2 = TWO ? thread_subtree(partials2, j0, lpt, nrb) : 0.0;
  if (stopped) return;   // uniform over the grid
  const int nw = (nt + 31) >> 5;
  const int wm = nt < 32 ? nt : 32;
  v = warp_tree(v, wm);
  if (TWO) v2 = warp_tree(v2, wm);
  if (lane == 0) { s_w[warp] = v; if (TWO) s_w2[warp] = v2; }
  __syncthreads();
  if (warp == 0) {
    v = warp_tree(lane < nw ? s_w[lane] : 0.0, nw);
    if (TWO) v2 = warp_tree(lane < nw ? s_w2[lane] : 0.0, nw);
    if (lane == 0) { s_root[0] = v; s_root[1] = v2; }
  }
  const uint32_t C = gridDim.x;   // one cluster spans the grid
  if (C > 1) {
    cluster_sync_all();   // every CTA root in its SMEM
    if (rank == 0 && warp == 0) {
      v = warp_tree(lane < (int)C ? ld_dsmem_f64(&s_root[0], lane) : 0.0, (int)C);
      if (TWO) v2 = warp_tree(lane < (int)C ? ld_dsmem_f64(&s_root[1], lane) : 0.0, (int)C);
    }
    cluster_sync_all();   // CTA 0 has read them: the others may exit
  }
  if (!fin) return;
  if (TWO && op == 10) { out[0] = v; out[1] = (double)(dueflag ? 1 : 0); out[2] = v2; return; }
  if (op == 0) { *out = v; return; }
  if (op == 4) { out[0] = v; out[1] = (double)(dueflag ? 1 : 0); out[2] = 0.0; return; }
  if (TWO) apply_op_sr(op, v2, v, &loc, dueflag);
  else apply_op(op, v, &loc, dueflag);
  *st = loc;
}

// Multi-GPU: combine the all-gathered (root, due) pairs of P ranks with the top
// of the RED-1 tree (identical on every rank) and apply the CG scalar logic.
static __global__ void k_combine(const double* gathered, int P, int op, CgState* st, int* due) {
  __shared__ double s[1024];
  if (op != 1 && st->stop) return;
  int m = 1;
  while (m < P) m <<= 1;
  for (int t = threadIdx.x; t < m; t += blockDim.x) s[t] = (t < P) ? gathered[GATHER_W * t] : 0.0;
  __syncthreads();
  double root = tree_smem(s, m);
  if (threadIdx.x != 0) return;
  int any = 0;
  for (int t = 0; t < P; t++) any |= gathered[GATHER_W * t + 1] != 0.0;
  if (any) *due = 1;
  apply_op(op, root, st, any != 0);
}
// Single-reduction CG, multi-rank: both roots' top of the tree (same order on
// every rank), then the SR scalar logic (op 6 / 7).
static __global__ void k_combine_sr(const double* gathered, int P, int op, CgState* st, int* due) {
  __shared__ double s[1024], s2[1024];
  if (op != 7 && st->stop) return;
  int m = 1;
  while (m < P) m <<= 1;
  for (int t = threadIdx.x; t < m; t += blockDim.x) {
    s[t] = (t < P) ? gathered[GATHER_W * t] : 0.0;
    s2[t] = (t < P) ? gathered[GATHER_W * t + 2] : 0.0;
  }
  __syncthreads();
  const double d = tree_smem(s, m);
  const double g = tree_smem(s2, m);
  if (threadIdx.x != 0) return;
  int any = 0;
  for (int t = 0; t < P; t++) any |= gathered[GATHER_W * t + 1] != 0.0;
  if (any) *due = 1;
  apply_op_sr(op, g, d, st, any != 0);
}
// Multi-GPU abort check after calc_p (policy abort only): gathered due flags.
static __global__ void k_due_combine(const double* gathered, int P, CgState* st, int* due) {
  int any = 0;
  for (int t = 0; t < P; t++) any |= gathered[GATHER_W * t + 1] != 0.0;
  if (any) *due = 1;
  if (st->stop && st->status != ABFT_E_NOT_CONVERGED) return;
  if (st->abort_policy && any) { st->stop = 1; st->status = ABFT_E_DUE; }
}
static __global__ void k_pack_due(double* out, const int* due) {
  out[1] = (double)(*((volatile const int*)due));
  out[0] = 0.0;
  out[2] = 0.0;
}

// ========================================================== vector encode / check
template <int VS>
__global__ void k_vec_encode(uint64_t* d, int64_t n, int64_t npad) {
  constexpr int G = vgrp(VS);
  const int64_t ng = npad / G;
  for (int64_t g = blockIdx.x * (int64_t)blockDim.x + threadIdx.x; g < ng; g += (int64_t)gridDim.x * blockDim.x) {
    uint64_t v[G];
#pragma unroll
    for (int t = 0; t < G; t++) {
      int64_t i = g * G + t;
      v[t] = (i < n) ? round_k(d[i], vk(VS)) : 0ull;
    }
#if 1
    if (VS == SECDED64) v[0] = v64_encode_lut(v[0], c_v64_lut.r);
    else vec_encode_group<VS>(v, nullptr);
#endif
#pragma unroll
    for (int t = 0; t < G; t++) d[g * G + t] = v[t];
  }
}

template <int VS>
__global__ void k_vec_check(uint64_t* d, int64_t n, int64_t npad, double* out, DevCounts* cnt, int* due, int scrub) {
  constexpr int G = vgrp(VS);
  const int64_t ng = npad / G;
  for (int64_t g = blockIdx.x * (int64_t)blockDim.x + threadIdx.x; g < ng; g += (int64_t)gridDim.x * blockDim.x) {
    uint64_t v[G], o0[G];
#pragma unroll
    for (int t = 0; t < G; t++) o0[t] = v[t] = d[g * G + t];
    int word = 0;
    int o = vec_check_group<VS>(v, &word, due);
    if (o == CORRECTED && scrub == 2) o = DUE;   // detection only
    if (o == CORRECTED) {
      bool won = true;
      if (scrub) won = scrub_group32(reinterpret_cast<uint32_t*>(d + g * G), o0, v, G);
      if (won) cnt_add(cnt, T_VEC, VS, CORRECTED);
    } else if (o == DUE) {
#pragma unroll
      for (int t = 0; t < G; t++) v[t] = o0[t];
      cnt_add(cnt, T_VEC, VS, DUE);
      *due = 1;
    }
    if (out) {
#pragma unroll
      for (int t = 0; t < G; t++) if (g * G + t < n) out[g * G + t] = as_d(v[t] & vkeep(VS));
    }
  }
}

// ============================================================ CSR encode (a0)
// flags[0] |= 1: col beyond capacity, |= 2: rowptr beyond capacity, |= 4: CRC row < 4 entries
template <int ES>
__global__ void k_encode_elems(const uint64_t* val, uint32_t* col, int64_t nnz, int64_t ncols, uint32_t* flags) {
  for (int64_t e = blockIdx.x * (int64_t)blockDim.x + threadIdx.x; e < nnz; e += (int64_t)gridDim.x * blockDim.x) {
    uint32_t c = col[e];
    if ((uint64_t)c > col_limit(ES) || (int64_t)c >= ncols) { atomicOr(flags, 1u); continue; }
    if (ES == SED) col[e] = esed_encode_col(val[e], c);
    else if (ES == SECDED64 || ES == SECDED128) col[e] = e96_encode_col(val[e], c);
  }
}
static __global__ void k_encode_ecrc(const uint64_t* val, uint32_t* col, const uint32_t* rowptr, int64_t nrows, uint32_t* flags) {
  for (int64_t i = blockIdx.x * (int64_t)blockDim.x + threadIdx.x; i < nrows; i += (int64_t)gridDim.x * blockDim.x) {
    uint32_t s = rowptr[i], t = rowptr[i + 1];
    if (t < s + 4) { atomicOr(flags, 4u); continue; }
    uint32_t crc = 0xFFFFFFFFu;
    for (uint32_t j = s; j < t; j++) {
      uint32_t c = col[j];
      if (j < s + 4) c &= 0x00FFFFFFu;
      crc = ecrc_update(crc, val[j], c, (int)(j - s));
    }
    crc ^= 0xFFFFFFFFu;
    for (int k = 0; k < 4; k++) col[s + k] = (col[s + k] & 0x00FFFFFFu) | (((crc >> (8 * k)) & 0xFFu) << 24);
  }
}
template <int RS>
__global__ void k_encode_rowptr(uint32_t* rowptr, int64_t nrows, int64_t nnz, int64_t len, uint32_t* flags) {
  constexpr int G = rgrp(RS);
  for (int64_t g = blockIdx.x * (int64_t)blockDim.x + threadIdx.x; g < len / G; g += (int64_t)gridDim.x * blockDim.x) {
    uint32_t e[G];
    for (int t = 0; t < G; t++) {
      int64_t i = g * G + t;
      e[t] = (i <= nrows) ? rowptr[i] : (uint32_t)nnz;
      if ((uint64_t)e[t] > rp_limit(RS)) atomicOr(flags, 2u);
    }
    if (RS != NONE) rp_encode_group<RS>(e);
    for (int t = 0; t < G; t++) rowptr[g * G + t] = e[t];
  }
}

// ============================================================ check_all (a7)
template <int ES>
__global__ void k_check_elems(uint64_t* val, uint32_t* col, int64_t nnz, int64_t ncols, DevCounts* cnt, int* due,
                              int scrub) {
  for (int64_t e = blockIdx.x * (int64_t)blockDim.x + threadIdx.x; e < nnz; e += (int64_t)gridDim.x * blockDim.x) {
    uint64_t v = val[e], v0 = v;
    uint32_t c = col[e], c0 = c;
    int word = 0;
    int o = CLEAN;
    if (ES == SED) o = esed_clean(v, c) ? CLEAN : DUE;
    else if (e96_bad(lo32(v), hi32(v), c)) o = e96_correct(v, c, &word);
    if (o == CORRECTED && scrub == 2) o = DUE;   // detection only (interval mode's final check)
    if (o == CORRECTED) {
      bool won = true;
      if (scrub) won = (word == 2) ? scrub32(col + e, c0, c)
                                   : scrub32(reinterpret_cast<uint32_t*>(val + e) + word, word ? hi32(v0) : lo32(v0),
                                             word ? hi32(v) : lo32(v));
      if (won) cnt_add(cnt, T_ELEM, ES, CORRECTED);
    } else if (o == DUE) {
      c = c0;
      cnt_add(cnt, T_ELEM, ES, DUE);
      *due = 1;
    }
    if ((int64_t)(c & col_keep(ES)) >= ncols) { cnt_range(cnt, T_ELEM, ES); *due = 1; }
  }
}
template <int RS>
__global__ void k_check_rowptr(uint32_t* rowptr, int64_t len, DevCounts* cnt, int* due, int scrub) {
  constexpr int G = rgrp(RS);
  for (int64_t g = blockIdx.x * (int64_t)blockDim.x + threadIdx.x; g < len / G; g += (int64_t)gridDim.x * blockDim.x) {
    uint32_t e[G], o0[G];
    for (int t = 0; t < G; t++) o0[t] = e[t] = rowptr[g * G + t];
    int word = 0;
    int o = rp_check_group<RS>(e, &word, due);
    if (o == CORRECTED && scrub == 2) o = DUE;   // detection only (interval mode's final check)
    if (o == CORRECTED) {
      bool won = scrub ? scrub_entries32(rowptr + g * G, o0, e, G) : true;
      if (won) cnt_add(cnt, T_ROWPTR, RS, CORRECTED);
    } else if (o == DUE) {
      cnt_add(cnt, T_ROWPTR, RS, DUE);
      *due = 1;
    }
  }
}
// rowptr entry idx, its group checked and corrected in registers (a DUE group
// gives its stored bits), masked.
template <int RS>
__device__ uint32_t rp_decoded(const uint32_t* rowptr, int64_t idx, bool detect_only, const int* cfg) {
  constexpr int G = rgrp(RS);
  uint32_t e[G];
  const int64_t g0 = idx / G * G;
#pragma unroll
  for (int t = 0; t < G; t++) e[t] = rowptr[g0 + t];
  const uint32_t raw = e[idx - g0];
  uint32_t w = raw;
  if (RS != NONE && !detect_only) {   // detection only: a correctable group is a DUE (stored bits)
    int word = 0;
    if (rp_check_group<RS>(e, &word, cfg) == CORRECTED) {
#pragma unroll
      for (int t = 0; t < G; t++) if (t == idx - g0) w = e[t];
    }
  }
  return w & rp_keep(RS);
}
// Row pass of check_all: range check + E-CRC rows (after the rowptr pass scrubbed).
template <int ES, int RS>
__global__ void k_check_rows(uint64_t* val, uint32_t* col, const uint32_t* rowptr, int64_t nrows,
                             int64_t nnz, int64_t ncols, DevCounts* cnt, int* due, int scrub) {
  for (int64_t i = blockIdx.x * (int64_t)blockDim.x + threadIdx.x; i < nrows; i += (int64_t)gridDim.x * blockDim.x) {
    // decoded entries (corrected in registers, not counted: the rowptr pass
    // counts), so count-only sweeps see the same ranges as scrubbing ones
    const uint32_t s = rp_decoded<RS>(rowptr, i, scrub == 2, due), t = rp_decoded<RS>(rowptr, i + 1, scrub == 2, due);
    if (!(s <= t && (int64_t)t <= nnz)) {
      if (RS != NONE) { cnt_range(cnt, T_ROWPTR, RS); *due = 1; }
      continue;
    }
    if (ES == CRC32C) {
      bool bad = (t - s < 4);
      if (!bad) {
        uint32_t crc = 0xFFFFFFFFu, st = 0;
        for (uint32_t j = s; j < t; j++) {
          uint32_t c = col[j];
          if (j - s < 4) st |= (c >> 24) << (8 * (j - s));
          crc = ecrc_update(crc, val[j], c, (int)(j - s));
        }
        bad = (crc ^ 0xFFFFFFFFu) != st;
      }
      // scrub: 0 count only, 1 count + correct in place, 2 detection only
      uint32_t* fa[2] = {nullptr, nullptr};
      int fb[2] = {0, 0};
      if (bad) ecrc_fix(val, col, s, t - s, scrub == 1 ? 1 : scrub == 2 ? 2 : 0, cnt, due, fa, fb);
      // the row is the codeword: range-check its columns as decoded by it
      for (uint32_t j = s; j < t; j++) {
        uint32_t c = *(volatile uint32_t*)(col + j);
        for (int q = 0; q < 2; q++)
          if (fa[q] == col + j && scrub == 0) c ^= 1u << fb[q];
        if ((int64_t)(c & 0x00FFFFFFu) >= ncols) { cnt_range(cnt, T_ELEM, CRC32C); *due = 1; }
      }
    }
  }
}

static __global__ void k_inject(uint32_t* base, uint64_t bit) { atomicXor(base + (bit >> 5), 1u << (bit & 31)); }


}  // namespace abft
