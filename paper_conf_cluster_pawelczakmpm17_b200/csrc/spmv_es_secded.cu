// spmv_es_secded.cu — SpMV launcher instantiations for element scheme SECDED64
// (split out only so nvcc compiles the 25 (rowptr x vector) variants in parallel).
#include "spmv_launch.cuh"

namespace abft {

bool spmv_es_secded(const SpmvArgs& a, int rs, int vs, int dot, cudaStream_t s) {
  return spmv1<SECDED64>(a, rs, vs, dot, s);
}

}  // namespace abft
