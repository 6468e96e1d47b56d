// spmv_es_sed.cu — SpMV launcher instantiations for element scheme SED
// (split out only so nvcc compiles the 25 (rowptr x vector) variants in parallel).
#include "spmv_launch.cuh"

namespace abft {

bool spmv_es_sed(const SpmvArgs& a, int rs, int vs, int dot, cudaStream_t s) {
  return spmv1<SED>(a, rs, vs, dot, s);
}

}  // namespace abft
