/*
 * conv2d.h -- C ABI of the B200 (sm_100a) direct-convolution library libconv2d.so.
 *
 * The operation is the one Lu, Zhang & Wang, "Optimizing GPU Memory Transactions for Convolution
 * Operations" (IEEE Cluster 2020) accelerate: direct, stride-1, valid-mode fp32 2D convolution
 * (cross-correlation, no filter flip), for a single-channel image (Fig. 1 P:130-203,
 * Fig. 2 equations) and for multi-channel N x C x F convolution (Table I
 * P:335-352, naming P:350-352). The kernels behind these calls implement the paper's column reuse
 * (warp-shuffle exchange of overlapping input columns with static register indices, Alg. 1
 * P:243-254) and row reuse (each loaded input row multiplied by several filter rows,
 * Alg. 2), re-designed for sm_100a.
 *
 * Conventions shared by every entry point
 *   - All tensor pointers are DEVICE pointers (global memory of the current CUDA device), owned by
 *     the caller (except conv2d_single_host: host pointers). The library never frees or retains them
 *     after the call returns.
 *   - fp32, dense, row-major: no strides, no padding; every pointer must be 4-byte aligned. Any
 *     width and any 4-byte alignment is supported; 16-byte-aligned inputs with W % 4 == 0 take the
 *     vectorised (LDG.128) path.
 *   - `stream` is a cudaStream_t passed as void* (NULL = legacy default stream). Work is enqueued
 *     asynchronously on it; there is no host synchronisation. The calls are reentrant and
 *     thread-safe. Single-channel filters are staged (a stream-ordered device-to-device copy) into a
 *     per-K slot of the module's __constant__ bank; an event recorded behind each kernel orders the
 *     next overwrite of the slot, so concurrent calls on different streams never see each other's
 *     filter (same-K calls on different streams are serialised by that wait). Under CUDA-graph
 *     capture, and for small images (<= 512^2, or <= 1024^2 with K <= 5, where the staging copy
 *     would cost more than it saves), the filter is staged per CTA in shared memory instead.
 *     Multi-channel filters are staged per CTA in shared memory.
 *   - Return value: 0 when the work was enqueued. A negative CONV2D_E* code when an argument is
 *     invalid (nothing was launched) or the launch itself failed. Asynchronous execution errors
 *     surface at the caller's next synchronisation, as in CUDA.
 *   - Stride 1, no padding ("valid"): Ho = H-K+1, Wo = W-K+1. Square K x K filters, 1 <= K <= 15
 *     (R14). Every output element is written exactly once and never read.
 *   - Arithmetic: fp32 FMA, accumulated per output in filter-row / filter-column order (multi:
 *     filter-row, channel, filter-column). Exception: single-channel images with W <= 1024 and
 *     K >= 11 (when not captured into a graph) run the filter-row split kernel, which sums two
 *     partial results (filter rows [0, K/2) and [K/2, K)) -- same tolerance, not the same bits as the
 *     one-pass order. Results never depend on the band height or the row-band split. Acceptance vs the CPU oracle: |gpu - ref| <= 1e-5 *
 *     sum|x||w| per element (BASELINE.json north_star). No fast-math, denormals preserved.
 */
#ifndef CONV2D_B200_H
#define CONV2D_B200_H

#include <stdint.h>

#ifdef __cplusplus
extern "C" {
#endif

#define CONV2D_OK 0
#define CONV2D_ENULL (-1)     /* a tensor pointer is NULL */
#define CONV2D_ESHAPE (-2)    /* H<K, W<K, N/C/F<1, K<1, or an element count above 2^62 */
#define CONV2D_EK (-3)        /* K > 15 (K is a compile-time template parameter of the kernels) */
#define CONV2D_EOVERLAP (-4)  /* the output range overlaps the input or the filter range */
#define CONV2D_ECUDA (-5)     /* the kernel launch failed (cudaGetLastError after the launch) */
#define CONV2D_EALIGN (-6)    /* a tensor pointer is not 4-byte aligned */
#define CONV2D_EALLOC (-7)    /* device memory for a host-buffer call could not be allocated */

#define CONV2D_MAX_K 15

/*
 * Single-channel 2D image filtering.
 *   in   : H*W floats, row-major:        in[y*W + x]
 *   filt : K*K floats, row-major:        filt[i*K + j]
 *   out  : (H-K+1)*(W-K+1) floats, row-major, pitch W-K+1:
 *          out[y*(W-K+1) + x] = sum_{i<K} sum_{j<K} in[(y+i)*W + x+j] * filt[i*K + j]
 */
int conv2d_single(const float *in, int H, int W, const float *filt, int K, float *out, void *stream);

/*
 * Multi-channel 2D convolution (Table I; layout DESIGN.md R13).
 *   in   : N*C*H*W floats (NCHW)
 *   filt : F*C*K*K floats (FCKK == torch OIHW)
 *   out  : N*F*(H-K+1)*(W-K+1) floats (NFHoWo):
 *          out[n][f][y][x] = sum_{c<C} sum_{i<K} sum_{j<K} in[n][c][y+i][x+j] * filt[f][c][i][j]
 *   Kernel: the filter-blocked wide-lane kernel (a lane owns 8 output columns x FB = 8 or 4 filters;
 *   column reuse by warp shuffle). Each output sums its C*K*K terms in
 *   (filter row i, channel c, filter column j) order, one fmaf chain -- exact on integer data,
 *   independent of batch, tiling and F-block. The filters of one F-block (all C channels) are staged
 *   in shared memory (C*K*K*FB*4 bytes); when even FB = 4 does not fit, the round-1 kernel with one
 *   filter per warp takes over (C*K*ceil(K/4)*4*4 bytes: e.g. C <= 236 at K = 15, C <= 4843 at
 *   K = 3); larger C returns CONV2D_ESHAPE.
 */
int conv2d_multi(const float *in, int N, int C, int H, int W, const float *filt, int F, int K,
                 float *out, void *stream);

/*
 * A batch of N single-channel images filtered with one filter (image filtering of a batch; also the
 * unit the multi-GPU bench shards across ranks): the same operation as N conv2d_single calls on
 * in + n*H*W -> out + n*(H-K+1)*(W-K+1), n < N, in ONE launch (the warp tiles of all images form one
 * wave, so small images fill the GPU). Same layouts, ownership, stream semantics, errors and bits as
 * conv2d_single on each image (CONV2D_ESHAPE also for N < 1).
 */
int conv2d_single_batch(const float *in, int N, int H, int W, const float *filt, int K, float *out,
                        void *stream);

/*
 * Rectangular FH x FW filters (Table I's "FH x FW" filter columns): the same
 * valid, stride-1 cross-correlation with a non-square filter,
 *   filt : FH*FW floats, row-major:      filt[i*FW + j]
 *   out  : (H-FH+1)*(W-FW+1) floats:     out[y*(W-FW+1) + x] = sum_{i<FH} sum_{j<FW} in[(y+i)*W + x+j] * filt[i*FW + j]
 * 1 <= FH, FW <= 15 (CONV2D_EK above; CONV2D_ESHAPE for FH or FW < 1, H < FH, W < FW). FH == FW is
 * conv2d_single. The kernel is the wide-lane column + row reuse kernel with an FH-slot ring and an
 * FW-wide window (both compile-time), the filter staged per CTA in shared memory; each output sums in
 * filter-row, filter-column order (exact on integer data). Same layouts, ownership, stream semantics.
 */
int conv2d_single_rect(const float *in, int H, int W, const float *filt, int FH, int FW, float *out,
                       void *stream);

/*
 * Same as conv2d_single / conv2d_multi with an explicit tiling parameter (band_h <= 0: the library's
 * choice): conv2d_single_ex -- the output-row band height per warp; conv2d_multi_ex -- the warp-steps
 * per warp of the filter-blocked kernel (a warp-step = 32/SEG output-row segments). For tuning sweeps
 * and tests of the band / halo logic; the result is bitwise identical for every band_h (each
 * output's summation order does not depend on its tile).
 */
int conv2d_single_ex(const float *in, int H, int W, const float *filt, int K, float *out, void *stream,
                     int band_h);
int conv2d_multi_ex(const float *in, int N, int C, int H, int W, const float *filt, int F, int K,
                    float *out, void *stream, int band_h);

/*
 * Row-band call with a separate halo segment (BASELINE.json north_star "row-band
 * split ... with a (K-1)-row halo"): the same operation as conv2d_single on an image of
 * H + halo_rows rows whose first H rows are at `in` and whose last halo_rows rows are at `halo`, both
 * row-major with pitch W. Output: (H + halo_rows - K + 1) x (W - K + 1), dense row-major at `out`.
 * The kernels read the halo rows directly from `halo`, which may be another GPU's memory mapped into
 * this device's address space (CUDA IPC / symmetric memory over NVLink): a rank of a row-band
 * decomposition then computes its whole band in one launch, reading its neighbour's first K-1 rows
 * over NVLink, with no exchange step and no tail call. Outputs are bitwise equal to conv2d_single
 * on the concatenated rows (same kernels, same per-output summation order).
 * halo_rows == 0 (halo may be NULL) is conv2d_single. Errors as conv2d_single, plus CONV2D_ENULL for
 * a NULL halo with halo_rows > 0, CONV2D_ESHAPE for halo_rows < 0, and CONV2D_EOVERLAP if `out`
 * overlaps the halo rows. The halo memory must stay valid and unchanged until the work completes.
 */
int conv2d_single_halo(const float *in, int H, int W, const float *halo, int halo_rows, const float *filt,
                       int K, float *out, void *stream);

/*
 * Boundary and semantic variants of conv2d_single (the image-library semantics the
 * paper compares against). `mode` is a bitwise OR of
 *   CONV2D_PAD_ZERO      'same' output size H x W, input padded with zeros,
 *   CONV2D_PAD_REPLICATE 'same' output size H x W, input padded by repeating its edge elements,
 *                        (at most one PAD flag; padding: top/left (K-1)/2, bottom/right the rest --
 *                        torch.nn.functional.conv2d(padding='same') placement, also for even K),
 *   CONV2D_FLIP          true convolution: the filter is rotated by 180 degrees (NPP / ArrayFire /
 *                        scipy.signal.convolve2d orientation) instead of cross-correlation.
 * mode == 0 is conv2d_single. Without a PAD flag the output is (H-K+1) x (W-K+1) and H, W >= K is
 * required; with one, H, W >= 1. Same layouts, ownership, stream semantics and tolerance as
 * conv2d_single; the result is bitwise equal to conv2d_single on the padded image with the rotated
 * filter (the padding and the rotation are data movement done on the device into the library's
 * stream-ordered scratch pool; the convolution is the same per-K kernels).
 * Errors as conv2d_single, plus CONV2D_ESHAPE for an invalid mode and CONV2D_EALLOC when the scratch
 * pool cannot provide the padded image ((H+K-1) x (W+K-1) floats, row pitch rounded to 16 bytes).
 */
#define CONV2D_PAD_ZERO 1
#define CONV2D_PAD_REPLICATE 2
#define CONV2D_PAD_MASK 3
#define CONV2D_FLIP 4
int conv2d_single_pad(const float *in, int H, int W, const float *filt, int K, int mode, float *out,
                      void *stream);

/*
 * Baseline "direct convolution" of PAPER.md Fig. 1a: one thread per
 * output element, each thread loads its K*K inputs itself (no column or row reuse). Same arguments,
 * result and error codes as conv2d_single. Kept as the control for the memory-transaction evidence
 * (profiles/); not a performance path.
 */
int conv2d_single_direct(const float *in, int H, int W, const float *filt, int K, float *out,
                         void *stream);

/*
 * End-to-end single-channel call on HOST buffers (the user-facing path for data that lives in host
 * memory): same operation and result as conv2d_single, but in, filt and out are host pointers (pinned
 * memory -- cudaHostAlloc / cudaHostRegister -- lets the copies run asynchronously at full PCIe
 * speed; pageable memory works but the copies become synchronous).
 * The image is processed in row chunks through a three-stage pipeline on the current device: the
 * host->device copy of chunk i+1, the kernel of chunk i and the device->host copy of chunk i-1 run
 * concurrently (two internal copy streams plus `stream` for the kernels). Device memory for the image
 * is taken from the library's stream-ordered scratch pool (see conv2d_release_scratch) and returned
 * to it when the work completes. All work is ordered after the work already enqueued on `stream`, and
 * `stream` is ordered after all of it: synchronise `stream` before reading `out`.
 * chunk_rows <= 0 chooses ~8 MiB input chunks.
 */
int conv2d_single_host(const float *in, int H, int W, const float *filt, int K, float *out, void *stream,
                       int chunk_rows);

/*
 * Tensor-core variant of conv2d_multi for the large-C dense contraction (a separate, measured
 * variant: BASELINE.json north_star). Same arguments, layouts and result contract as
 * conv2d_multi; computed as an implicit GEMM (pixels x filters x C*K*K) on tcgen05 tensor cores with
 * the 3xTF32 split (a = a_hi + a_lo; A_hi B_hi + A_hi B_lo + A_lo B_hi, fp32 accumulation in TMEM),
 * within the same 1e-5 * sum|x||w| acceptance but NOT bitwise equal to conv2d_multi (different
 * summation order and per-product rounding). The filters are split into hi/lo tensor-core tiles in a
 * stream-ordered scratch buffer from the library's pool (2 * ceil(F/FN)*FN * ceil(C*K*K/32)*32 floats,
 * FN in {32, 64, 128, 256}); CONV2D_EALLOC if that fails. Limits: C*H*W < 2^31 and C*K*K <= 16384
 * (CONV2D_ESHAPE otherwise).
 */
int conv2d_multi_tc(const float *in, int N, int C, int H, int W, const float *filt, int F, int K, float *out,
                    void *stream);

/*
 * The library's stream-ordered scratch pool (conv2d_single_host buffers, conv2d_multi_tc filter
 * tiles) keeps freed memory for reuse by later calls, like a caching allocator. This call releases
 * the unused part of the current device's pool back to the driver (memory still in use by enqueued
 * work is kept). Returns 0, or CONV2D_ECUDA.
 */
int conv2d_release_scratch(void);

/* Human-readable text for a return code (static storage, never NULL). */
const char *conv2d_strerror(int code);

/* ABI version (major*100 + minor): 102 = conv2d_single_batch, 103 = conv2d_single_rect. */
int conv2d_version(void);

#ifdef __cplusplus
}
#endif

#endif /* CONV2D_B200_H */
