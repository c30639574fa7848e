// inst_rect_kh08.cu -- rectangular-filter kernels with 8 filter rows (KW = 1..15), conv2d_single_rect
#include "launch.cuh"

namespace c2d {
template int rect_entry<8>(const float *, int, int, const float *, int, float *, cudaStream_t, const DevInfo &);
}  // namespace c2d
