// spmv_launch.cuh — host-side SpMV launch templates (tiled stencil fast path or
// generic CSR kernel), instantiated per element scheme in spmv_es_*.cu.
#pragma once
#include "kernels_impl.cuh"

namespace abft {
namespace {
static bool tile_ok(const SpmvArgs& a, int vs) {
  const int64_t n = a.stencil_n;
  return n > 0 && (n % 256) == 0 && (a.nrows % n) == 0 && vgrp(vs) == 1 && a.npad_out >= a.nrows;
}
template <int ES, int RS, int VS, bool DOT>
static void spmv_tile_launch(const SpmvArgs& a, cudaStream_t s) {
  const size_t smem = TILE_SMEM;
  static bool attr = false;
  if (!attr) {  // both variants at once: never inside a later CUDA-graph capture
    cudaFuncSetAttribute(k_spmv_tile<ES, RS, VS, true>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
    cudaFuncSetAttribute(k_spmv_tile<ES, RS, VS, false>, cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
    attr = true;
  }
  const int64_t ny = a.nrows / a.stencil_n;
  const int64_t blocks = (a.stencil_n / 256) * ((ny + TILE_TY - 1) / TILE_TY);
  k_spmv_tile<ES, RS, VS, DOT><<<(unsigned)blocks, 256, smem, s>>>(a);
}
template <int ES, int RS, int VS>
static void spmv3(const SpmvArgs& a, bool dot, cudaStream_t s) {
  if (vgrp(VS) == 1 && tile_ok(a, VS)) {
    if (dot) spmv_tile_launch<ES, RS, VS, true>(a, s);
    else spmv_tile_launch<ES, RS, VS, false>(a, s);
    return;
  }
  const int64_t nrb = (a.nrows + 255) / 256;
  const int blocks = (int)((nrb + 7) / 8);
  if (dot) k_spmv<ES, RS, VS, true><<<blocks, 256, 0, s>>>(a);
  else k_spmv<ES, RS, VS, false><<<blocks, 256, 0, s>>>(a);
}
template <int ES, int RS>
static void spmv2(const SpmvArgs& a, int vs, bool dot, cudaStream_t s) {
  switch (vs) {
    case NONE: spmv3<ES, RS, NONE>(a, dot, s); break;
    case SED: spmv3<ES, RS, SED>(a, dot, s); break;
    case SECDED64: spmv3<ES, RS, SECDED64>(a, dot, s); break;
    case SECDED128: spmv3<ES, RS, SECDED128>(a, dot, s); break;
    default: spmv3<ES, RS, CRC32C>(a, dot, s); break;
  }
}
template <int ES>
static void spmv1(const SpmvArgs& a, int rs, int vs, bool dot, cudaStream_t s) {
  switch (rs) {
    case NONE: spmv2<ES, NONE>(a, vs, dot, s); break;
    case SED: spmv2<ES, SED>(a, vs, dot, s); break;
    case SECDED64: spmv2<ES, SECDED64>(a, vs, dot, s); break;
    case SECDED128: spmv2<ES, SECDED128>(a, vs, dot, s); break;
    default: spmv2<ES, CRC32C>(a, vs, dot, s); break;
  }
}

}  // namespace
}  // namespace abft
