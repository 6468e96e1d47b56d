// spmv_es_none.cu — SpMV launcher instantiations for element scheme NONE
// (split out only so nvcc compiles the 25 (rowptr x vector) variants in parallel).
#include "spmv_launch.cuh"

namespace abft {

bool spmv_es_none(const SpmvArgs& a, int rs, int vs, int dot, cudaStream_t s) {
  return spmv1<NONE>(a, rs, vs, dot, s);
}

bool spmv_fusable(const SpmvArgs& a, int vs) {
  return (vs == NONE || vs == SED || vs == SECDED64) && tile_ok(a, vs) && tmap_encoder() != nullptr;
}

bool spmv_tileable(const SpmvArgs& a, int vs) { return tile_ok(a, vs) && tmap_encoder() != nullptr; }
int64_t spmv_tile_rows(const SpmvArgs& a) { return (a.nrows / a.stencil_n + TILE_TY - 1) / TILE_TY; }

}  // namespace abft
