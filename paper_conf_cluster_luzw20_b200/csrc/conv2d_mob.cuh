// conv2d_mob.cuh -- multi-channel kernel blocked over filters ("filter-blocked wide lanes"), sm_100a.
//
// Same operation and the same per-output summation as k_conv2d_multi2 (conv2d_multi.cuh): out[n][f][y][x]
// = sum over filter row i, channel c, filter column j (in that order, one FMA chain per output) of
// in[n][c][y+i][x+j] * w[f][c][i][j] (Sec. II problem statement P:130-140; Table I).
// The two kernels give the same bits. What changes is which reuse carries the FMAs:
//   * a lane owns 8 CONTIGUOUS output columns (wide lanes) of ONE output row and FB filters: an
//     FB x 8 register block of accumulators (64 at FB = 8). Per input row (c, y+i) it loads its 8
//     columns + the halo quads (LDG.128, a1), assembles the 8+K-1 window with K-1 SEL + SHFL.IDX
//     (column reuse, Sec. II-A, Alg. 1, static register indices), then for every filter
//     column j fetches the FB filter values (c, i, j) as FB/4 broadcast LDS.128 and runs 8 x FB/2
//     FFMA2 (window value broadcast, filter pair, accumulator pair; fma.rn.f32x2 = two fmaf steps).
//   * Row reuse (Alg. 2) is NOT used here: with FB filters per lane each window already feeds 8*FB*K
//     FMAs, so one output row per lane keeps 8*FB accumulators instead of K*8*FB; the input rows a
//     neighbouring output row needs again come from L1/L2 (the whole configs[3] input is 77 MB, L2
//     126 MB). The shared-memory filter traffic per FMA halves against the 4-column kernel (one
//     LDS.128 broadcast feeds 8 columns x 4 filters), which was its bound (LSU 41%, configs[3]).
//   * Units: a unit = (image n, output row y, column block of 8*SEG columns); a warp is 32/SEG
//     segments of SEG lanes, each on its own unit, so narrow layers (54- or 218-column outputs) keep
//     their lanes busy: the units of all images of one F-block form one flat list, a warp-step is 32/SEG
//     consecutive units (a step may span two rows or two images: every lane computes its own
//     addresses), a warp runs L warp-steps and the 4 warps of a CTA interleave theirs (adjacent units
//     at the same time: shared L1 lines). All of a CTA's steps are in one F-block, staged once in
//     shared memory as [i][c][j][fb] (the streaming order, so the filter address only advances).
//   * The next input row (crossing into the next warp-step) is in flight in registers while the
//     current one is computed.
// EDGE 1: 16B-aligned rows (W % 4 == 0): quad loads clamped to the row's last quad (garbage reaches
// only outputs >= Wo, never stored); EDGE 2: misaligned rows, guarded scalar loads.
#pragma once

#include "conv2d_wide.cuh"

namespace c2d {

struct MobArgs {
  const float *in;
  const float *filt;  // F x C x K x K in global memory
  float *out;
  int N, C, H, W, F, Ho, Wo;
  int n_cb;            // column blocks of 8*SEG columns per output row
  int units_img;       // Ho * n_cb units per image
  int units;           // N * units_img units per F-block (< 2^31: checked by the launcher)
  int steps;           // warp-steps per F-block: ceil(units / (32/SEG))
  int L;               // warp-steps per warp
  int ctas_fb;         // CTAs per F-block: ceil(steps / (4L))
  int n_fb;            // F-blocks of FB filters
  int ovec;            // output rows: 2 = 16-byte aligned (vector stores), 1 = 8-byte aligned, 0 = scalar
};

template <int K, int FB, int SEG, int EDGE, int MINB, bool PFL1 = false>
__global__ void __launch_bounds__(kCtaWarps *kWarp, MINB) k_conv2d_mob(const MobArgs a) {
  static_assert(FB == 4 || FB == 8, "filter block");
  static_assert(SEG >= 4 && SEG <= kWarp, "segment");
  constexpr int SEGS = kWarp / SEG;
  constexpr int WN = WideCfg<K>::WN;
  extern __shared__ __align__(16) float smem[];
  // F-block fastest: the CTAs of all F-blocks on the same units run together and share the input rows
  // in L2 (F-block-major order re-read the configs[3] input 4.6x from DRAM: the output stream evicts it)
  const int cta = blockIdx.x / a.n_fb;
  const int fblk = blockIdx.x - cta * a.n_fb;
  const int f0 = fblk * FB;
  const int C = a.C;
  // stage the F-block as [i][c][j][fb]
  const int total = C * K * K * FB;
  for (int t = threadIdx.x; t < total; t += blockDim.x) {
    const int fb = t % FB;
    const int j = (t / FB) % K;
    const int c = (t / (FB * K)) % C;
    const int i = t / (FB * K * C);
    const int f = f0 + fb;
    smem[t] = (f < a.F) ? a.filt[((static_cast<size_t>(f) * C + c) * K + i) * K + j] : 0.f;
  }
  __syncthreads();
  const unsigned sbase = static_cast<unsigned>(__cvta_generic_to_shared(smem));
  const int warp = threadIdx.x >> 5;
  const int lane = threadIdx.x & (kWarp - 1);
  const int sl = lane & (SEG - 1);
  const int seg = lane / SEG;
  const int plane = a.H * a.W;  // < 2^31 (checked by the launcher)
  const int s0 = cta * kCtaWarps * a.L + warp;  // steps s0 + 4k, k < L
  if (s0 >= a.steps) return;
  const int nsteps = min(a.L, (a.steps - s0 + kCtaWarps - 1) / kCtaWarps);

  // unit of this lane at warp-step s: input row pointer (channel 0, row y), column x0, output index
  auto unit_of = [&](int s, int &roff, int &x0, long long &oidx, bool &valid) {
    int u = s * SEGS + seg;
    valid = u < a.units;
    if (!valid) u = a.units - 1;  // idle segment: recompute the last unit, never store
    const int n = u / a.units_img;
    const int r = u - n * a.units_img;
    const int y = r / a.n_cb;
    const int cb = r - y * a.n_cb;
    x0 = cb * kWideV * SEG;
    roff = (n * C * a.H + y) * a.W;  // < 2^31: N*C*H*W is checked by the launcher
    oidx = ((static_cast<long long>(n) * a.F + f0) * a.Ho + y) * a.Wo + x0 + kWideV * sl;
  };

  const int rows = K * C;  // (i, c) rows per unit
  const unsigned fstride = static_cast<unsigned>(K * FB * 4);
  const int fplane = a.Ho * a.Wo;

  // a6: FB output rows of 8 columns per lane for warp-step s
  auto store = [&](int s, const float2 (&acc)[FB / 2][kWideV]) {
    int rp_s;
    int x0_s;
    long long oidx;
    bool valid;
    unit_of(s, rp_s, x0_s, oidx, valid);
    if (!valid) return;
    const int xl = x0_s + kWideV * sl;  // first column of this lane
#pragma unroll
    for (int p = 0; p < FB / 2; ++p) {
#pragma unroll
      for (int h = 0; h < 2; ++h) {
        if (f0 + 2 * p + h < a.F) {
          float *o = a.out + oidx + static_cast<long long>(2 * p + h) * fplane;
          float v8[kWideV];
#pragma unroll
          for (int v = 0; v < kWideV; ++v) v8[v] = h ? acc[p][v].y : acc[p][v].x;
          if (xl + kWideV <= a.Wo && a.ovec == 2) {
            stg4(o, v8[0], v8[1], v8[2], v8[3]);
            stg4(o + 4, v8[4], v8[5], v8[6], v8[7]);
          } else if (xl + kWideV <= a.Wo && a.ovec == 1) {
#pragma unroll
            for (int v = 0; v < kWideV; v += 2)
              __stcs(reinterpret_cast<float2 *>(o + v), make_float2(v8[v], v8[v + 1]));
          } else {
#pragma unroll
            for (int v = 0; v < kWideV; ++v)
              if (xl + v < a.Wo) __stcs(o + v, v8[v]);
          }
        }
      }
    }
  };

  // The warp's row stream: steps k < nsteps, rows t = i*C + c of each (row t at rp + i*W + c*plane, its
  // filter values (i, c, j) at sbase + (t*K + j)*FB*4). Two register buffers in ping-pong: row t is
  // computed from one while row t+1 (the next step's row 0 after the last) lands in the other -- one
  // buffer copied at the loop edge made the compiler wait on the fresh load at the copy (23% of the
  // stall samples). Inside a step the fetch cursor advances with selects only, so a step's row pairs
  // are one branch-free block the scheduler can interleave (the next row's shuffles and filter loads
  // under the current row's FFMA2s).
  int frow;  // fetch cursor (element offset of its row in `in`): row, column, channel, row-in-step
  int fx0, fc = 0, ft = 0;
  int nrp;  // the unit of the fetch cursor's next warp-step (element offset)
  int nx0;
  {
    long long oi;
    bool vd;
    unit_of(s0, frow, fx0, oi, vd);
    nrp = frow;
    nx0 = fx0;
    if (nsteps > 1) unit_of(s0 + kCtaWarps, nrp, nx0, oi, vd);
  }
  // the fetch row's 64-bit base formed once per row (opaque to the compiler, which otherwise folds the
  // row offset into every quad's column offset and redoes the 64-bit scaling per load)
  // (K >= 5: configs[3] 49.7 -> 50.8 TFLOP/s; at K <= 4 it costs the L1-prefetch form its last registers)
  auto row_ptr = [&](int off) {
    const float *p = a.in + off;
    if constexpr (K >= 5) asm("" : "+l"(p));
    return p;
  };
  const int wrap = a.W - (C - 1) * plane;  // (i, C-1) -> (i+1, 0); |wrap| < 2^31 (checked by the launcher)
  auto advance = [&]() {
    const bool cw = fc + 1 < C;
    const int nr = frow + (cw ? plane : wrap);
    fc = cw ? fc + 1 : 0;
    const bool last = ++ft == rows;
    frow = last ? nrp : nr;
    fx0 = last ? nx0 : fx0;
    ft = last ? 0 : ft;
    if (PFL1) {  // the cursor's new row (two ahead of the compute) into L1 (many-channel layers miss L1)
      const float *pr = a.in + frow;
      asm volatile("prefetch.global.L1 [%0];" ::"l"(pr + min(fx0 + kWideV * sl, a.W - 4)));
      if (K > 1) asm volatile("prefetch.global.L1 [%0];" ::"l"(pr + min(fx0 + kWideV * SEG + kWideV * (sl & 1), a.W - 4)));
    }
  };

  float2 acc[FB / 2][kWideV];
#pragma unroll
  for (int p = 0; p < FB / 2; ++p)
#pragma unroll
    for (int v = 0; v < kWideV; ++v) acc[p][v] = make_float2(0.f, 0.f);
  unsigned fa = sbase;
  // a2-a5 for one row: window (column reuse), FB x 8 x K FMAs
  auto compute = [&](const WideRow &cur) {
    float w[WN];
    wide_window<K, SEG>(cur, w, lane);
#pragma unroll
    for (int j = 0; j < K; ++j) {
      float2 fp[FB / 2];
#pragma unroll
      for (int q = 0; q < FB / 4; ++q) {
        float f0v, f1v, f2v, f3v;
        lds4_at(fa + static_cast<unsigned>((j * FB + 4 * q) * 4), f0v, f1v, f2v, f3v);
        fp[2 * q] = make_float2(f0v, f1v);
        fp[2 * q + 1] = make_float2(f2v, f3v);
      }
#pragma unroll
      for (int p = 0; p < FB / 2; ++p)
#pragma unroll
        for (int v = 0; v < kWideV; ++v)
          acc[p][v] = __ffma2_rn(make_float2(w[v + j], w[v + j]), fp[p], acc[p][v]);
    }
    fa += fstride;
  };
  WideRow bufA, bufB;
  wide_load<K, EDGE, SEG>(bufA, row_ptr(frow), fx0, a.W, sl);
  advance();
  // one warp-step starting from buffer X (rows t, t+1 in pairs; an odd last row leaves the next
  // step's row 0 in the other buffer)
  auto step = [&](WideRow &X, WideRow &Y) {
    int t = 0;
#pragma unroll 1
    for (; t + 1 < rows; t += 2) {
      wide_load<K, EDGE, SEG>(Y, row_ptr(frow), fx0, a.W, sl);
      advance();
      compute(X);
      wide_load<K, EDGE, SEG>(X, row_ptr(frow), fx0, a.W, sl);
      advance();
      compute(Y);
    }
    if (t < rows) {
      wide_load<K, EDGE, SEG>(Y, row_ptr(frow), fx0, a.W, sl);
      advance();
      compute(X);
    }
  };
  bool fromA = true;
#pragma unroll 1
  for (int k = 0; k < nsteps; ++k) {
    if (fromA)
      step(bufA, bufB);
    else
      step(bufB, bufA);
    if (rows & 1) fromA = !fromA;
    store(s0 + k * kCtaWarps, acc);
#pragma unroll
    for (int p = 0; p < FB / 2; ++p)
#pragma unroll
      for (int v = 0; v < kWideV; ++v) acc[p][v] = make_float2(0.f, 0.f);
    fa = sbase;
    if (k + 2 < nsteps) {  // the fetch cursor is in step k+1 now: it next crosses into k+2
      long long oi;
      bool vd;
      unit_of(s0 + (k + 2) * kCtaWarps, nrp, nx0, oi, vd);
    }
  }
}

}  // namespace c2d
