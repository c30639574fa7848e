// inst_k09.cu -- kernels and launch code for K = 9 (one K per unit: own constant bank, parallel build)
#include "launch.cuh"

namespace c2d {
template int single_entry<9>(const float *, int, int, int, const float *, float *, cudaStream_t, int,
                              const DevInfo &, const float *, int, long long, int);
template int multi_entry<9>(const float *, int, int, int, int, const float *, int, float *, cudaStream_t, int,
                             const DevInfo &);
}  // namespace c2d
