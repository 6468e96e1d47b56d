// spmv_launch.cuh — host-side SpMV launch templates (tiled stencil fast path or
// generic CSR kernel), instantiated per element scheme in spmv_es_*.cu.
#pragma once
#include <cudaTypedefs.h>
#include <atomic>
#include <cstdlib>

#include "kernels_impl.cuh"

namespace abft {
namespace {
// Tiled path preconditions (host metadata; the kernel still checks every row's
// decoded rowptr against the assumed stencil layout).
static bool tile_ok(const SpmvArgs& a, int vs) {
  const int64_t n = a.stencil_n;
  return n > 0 && (n % 256) == 0 && (a.nrows % n) == 0 && a.npad_out >= a.nrows &&
         a.nnz == 5 * a.nrows && a.nnz < (int64_t(1) << 32) && (a.nrows / n) < (int64_t(1) << 31) &&
         (reinterpret_cast<uintptr_t>(a.val) & 15u) == 0 && (reinterpret_cast<uintptr_t>(a.col) & 15u) == 0;
}
// The driver's tensor-map encoder, resolved once through the runtime (no -lcuda).
static PFN_cuTensorMapEncodeTiled_v12000 tmap_encoder() {
  static const PFN_cuTensorMapEncodeTiled_v12000 fn = [] {   // thread-safe one-time lookup
    void* p = nullptr;
    cudaDriverEntryPointQueryResult q;
    if (cudaGetDriverEntryPoint("cuTensorMapEncodeTiled", &p, cudaEnableDefault, &q) == cudaSuccess &&
        q == cudaDriverEntryPointSuccess)
      return reinterpret_cast<PFN_cuTensorMapEncodeTiled_v12000>(p);
    return static_cast<PFN_cuTensorMapEncodeTiled_v12000>(nullptr);
  }();
  return fn;
}
// The chunk's element arrays viewed as [ny grid rows][5n elements]; box = one
// pass of all TILE_TY warps of a tile: [TILE_TY][TILE_PE].
static bool tile_maps(const SpmvArgs& a, TileMaps* m) {
  auto enc = tmap_encoder();
  if (!enc) return false;
  const int64_t n = a.stencil_n, ny = a.nrows / n;
  cuuint64_t dims[2] = {(cuuint64_t)(5 * n), (cuuint64_t)ny};
  cuuint32_t box[2] = {(cuuint32_t)TILE_PE, (cuuint32_t)TILE_TY};
  cuuint32_t estr[2] = {1, 1};
  cuuint64_t sv[1] = {(cuuint64_t)(5 * n * 8)}, sc[1] = {(cuuint64_t)(5 * n * 4)};
  CUresult r1 = enc(&m->val, CU_TENSOR_MAP_DATA_TYPE_UINT64, 2, a.val, dims, sv, box, estr,
                    CU_TENSOR_MAP_INTERLEAVE_NONE, CU_TENSOR_MAP_SWIZZLE_NONE, CU_TENSOR_MAP_L2_PROMOTION_L2_256B,
                    CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
  CUresult r2 = enc(&m->col, CU_TENSOR_MAP_DATA_TYPE_UINT32, 2, a.col, dims, sc, box, estr,
                    CU_TENSOR_MAP_INTERLEAVE_NONE, CU_TENSOR_MAP_SWIZZLE_NONE, CU_TENSOR_MAP_L2_PROMOTION_L2_256B,
                    CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
  if (r1 != CUDA_SUCCESS || r2 != CUDA_SUCCESS) return false;
  // the input vector (and p_cur) as [rows][n/2][2] doubles: one box = the
  // decoded window's TILE_TY+2 rows x 132 pairs (x = tx0-2 .. tx0+261)
  m->has_vmaps = 0;
  static const bool no_vmaps = [] { const char* e = getenv("ABFT_NO_VMAPS"); return e && e[0] == '1'; }();
  if (!no_vmaps && (a.npad_in % n) == 0 && (a.row_base % n) == 0 && (n % 2) == 0) {
    cuuint64_t vd[3] = {2, (cuuint64_t)(n / 2), (cuuint64_t)(a.npad_in / n)};
    cuuint64_t vs[2] = {16, (cuuint64_t)(n * 8)};
    cuuint32_t vb[3] = {2, (cuuint32_t)(TILE_WW / 2), (cuuint32_t)(TILE_TY + 2)};
    cuuint32_t ve[3] = {1, 1, 1};
    CUresult r3 = enc(&m->vin, CU_TENSOR_MAP_DATA_TYPE_UINT64, 3, a.in, vd, vs, vb, ve, CU_TENSOR_MAP_INTERLEAVE_NONE,
                      CU_TENSOR_MAP_SWIZZLE_NONE, CU_TENSOR_MAP_L2_PROMOTION_L2_256B, CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
    CUresult r4 = CUDA_SUCCESS;
    if (a.p_cur)
      r4 = enc(&m->vcur, CU_TENSOR_MAP_DATA_TYPE_UINT64, 3, a.p_cur, vd, vs, vb, ve, CU_TENSOR_MAP_INTERLEAVE_NONE,
               CU_TENSOR_MAP_SWIZZLE_NONE, CU_TENSOR_MAP_L2_PROMOTION_L2_256B, CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
    else
      m->vcur = m->vin;
    m->has_vmaps = (r3 == CUDA_SUCCESS && r4 == CUDA_SUCCESS) ? 1 : 0;
  }
  return true;
}
template <int ES, int RS, int VS, int DOT, bool FUSED = false>
static bool spmv_tile_launch(const SpmvArgs& a, cudaStream_t s) {
  TileMaps tm;
  if (!tile_maps(a, &tm)) return false;
  const size_t smem = tile_smem<ES, RS, VS>();
  // function attributes are per device: set them once per device (thread
  // safe), before first use there, so never inside a later CUDA-graph capture
  static std::atomic<uint64_t> attr_devs{0};
  int dev = 0;
  cudaGetDevice(&dev);
  const uint64_t bit = 1ull << (dev & 63);
  if (!(attr_devs.load(std::memory_order_acquire) & bit)) {
    cudaFuncSetAttribute(k_spmv_tile<ES, RS, VS, DOT, FUSED>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
    cudaFuncSetAttribute(k_spmv_tile<ES, RS, VS, DOT, FUSED>, cudaFuncAttributePreferredSharedMemoryCarveout, 100);
    attr_devs.fetch_or(bit, std::memory_order_release);
  }
  const int64_t ny = a.nrows / a.stencil_n;
  const int64_t nty = (ny + TILE_TY - 1) / TILE_TY;
  const int64_t lo = a.ty_lo, hi = a.ty_hi > 0 ? a.ty_hi : nty;
  const int64_t blocks = (a.stencil_n / 256) * (hi - lo);
  if (blocks <= 0) return true;
  // a launch without PDL starts after every earlier kernel of the stream has
  // finished, so its `in` window may always be fetched before the (no-op) wait
  SpmvArgs b = a;
  if (!g_pdl) b.early_in = 1;
  launch_k(k_spmv_tile<ES, RS, VS, DOT, FUSED>, (unsigned)blocks, 256, smem, s, b, tm);
  return true;
}
// Returns false only when a fused-calc_p launch (a.p_cur set) was requested
// and cannot run: the caller fails loudly, there is no unfused fallback here.
template <int ES, int RS, int VS>
static bool spmv3(const SpmvArgs& a, int dot, cudaStream_t s) {
  if (a.p_cur) {
    if constexpr (vgrp(VS) == 1) {
      return dot == 1 && tile_ok(a, VS) && spmv_tile_launch<ES, RS, VS, 1, true>(a, s);
    }
    return false;
  }
  if (tile_ok(a, VS)) {
    const bool ok = dot == 2   ? spmv_tile_launch<ES, RS, VS, 2>(a, s)
                    : dot == 1 ? spmv_tile_launch<ES, RS, VS, 1>(a, s)
                               : spmv_tile_launch<ES, RS, VS, 0>(a, s);
    if (ok) return true;
  }
  const int64_t nrb = (a.nrows + 255) / 256;
  const int blocks = (int)((nrb + 7) / 8);
  if (dot == 2) launch_k(k_spmv<ES, RS, VS, 2>, blocks, 256, 0, s, a);
  else if (dot == 1) launch_k(k_spmv<ES, RS, VS, 1>, blocks, 256, 0, s, a);
  else launch_k(k_spmv<ES, RS, VS, 0>, blocks, 256, 0, s, a);
  return true;
}
template <int ES, int RS>
static bool spmv2(const SpmvArgs& a, int vs, int dot, cudaStream_t s) {
  switch (vs) {
    case NONE: return spmv3<ES, RS, NONE>(a, dot, s);
    case SED: return spmv3<ES, RS, SED>(a, dot, s);
    case SECDED64: return spmv3<ES, RS, SECDED64>(a, dot, s);
    case SECDED128: return spmv3<ES, RS, SECDED128>(a, dot, s);
    default: return spmv3<ES, RS, CRC32C>(a, dot, s);
  }
}
template <int ES>
static bool spmv1(const SpmvArgs& a, int rs, int vs, int dot, cudaStream_t s) {
  switch (rs) {
    case NONE: return spmv2<ES, NONE>(a, vs, dot, s);
    case SED: return spmv2<ES, SED>(a, vs, dot, s);
    case SECDED64: return spmv2<ES, SECDED64>(a, vs, dot, s);
    case SECDED128: return spmv2<ES, SECDED128>(a, vs, dot, s);
    default: return spmv2<ES, CRC32C>(a, vs, dot, s);
  }
}

}  // namespace
}  // namespace abft
