// inst_rect_kh12.cu -- rectangular-filter kernels with 12 filter rows (KW = 1..15), conv2d_single_rect
#include "launch.cuh"

namespace c2d {
template int rect_entry<12>(const float *, int, int, const float *, int, float *, cudaStream_t, const DevInfo &);
}  // namespace c2d
