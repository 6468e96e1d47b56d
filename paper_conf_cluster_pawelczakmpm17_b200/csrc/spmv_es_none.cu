// spmv_es_none.cu — SpMV launcher instantiations for element scheme NONE
// (split out only so nvcc compiles the 25 (rowptr x vector) variants in parallel).
#include "spmv_launch.cuh"

namespace abft {

void spmv_es_none(const SpmvArgs& a, int rs, int vs, bool dot, cudaStream_t s) {
  spmv1<NONE>(a, rs, vs, dot, s);
}

}  // namespace abft
