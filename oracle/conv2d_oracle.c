/*
 * CPU ORACLE -- TEST INFRASTRUCTURE ONLY.
 *
 * Only tests/, __graft_entry__.smoke() and bench.py's cpu_baseline / --impl reference legs may load
 * this library. The product path (paper_conf_cluster_luzw20_b200/) never links, imports or calls it,
 * and shares no code, header, table or helper with it.
 *
 * What it computes: the textbook definition of the operation the paper accelerates -- direct,
 * stride-1, valid-mode 2D cross-correlation -- written out as plain nested loops:
 *
 *   single-channel (Fig. 1a "each thread calculates the convolution for
 *   one output element"; P:269-271 the Fig. 2 equations out_o = sum_i rowi_{o+i} . rowf_i,
 *   i.e. NO filter flip; P:291/P:299 IH-FH+1 outputs = valid mode):
 *       out[y][x] = fl32( sum_{i<K} sum_{j<K} (double)in[y+i][x+j] * (double)f[i][j] )
 *   multi-channel (Table I P:335-352 with the I/F/O x N/C/H/W naming of P:350-352;
 *   NCHW input, FCKK filters, NFHoWo output -- DESIGN.md reading R13):
 *       out[n][f][y][x] = fl32( sum_{c<C} sum_{i<K} sum_{j<K} in[n][c][y+i][x+j] * w[f][c][i][j] )
 *
 * Column reuse and row reuse only change which loads feed which FMA and in
 * what order; they are not approximations, so the oracle is that plain definition (R6).
 * Accumulation is in double (each fp32 x fp32 product is exact in double), in the fixed (c, i, j)
 * lexicographic order, rounded ONCE to fp32 by the C cast (round-to-nearest-even). Alongside, the
 * oracle returns bound = sum |x||w| (double), the scale of the 1e-5 * sum|x||w| acceptance test of
 * BASELINE.json north_star. Optionally the un-rounded double result is returned too (out64).
 *
 * Build: gcc -O2 -fopenmp -ffp-contract=off -fPIC -shared (no -ffast-math; OpenMP only splits the
 * independent output rows across host cores, never a single output's sum).
 */
#include <math.h>
#include <stdint.h>
#include <stddef.h>

#ifdef _OPENMP
#include <omp.h>
#endif

int oracle_num_threads(void)
{
#ifdef _OPENMP
    return omp_get_max_threads();
#else
    return 1;
#endif
}

/* One output element of the single-channel definition. */
static void single_point(const float *in, int64_t W, const float *f, int64_t K, int64_t y, int64_t x,
                         double *acc_out, double *bound_out)
{
    double acc = 0.0, b = 0.0;
    for (int64_t i = 0; i < K; ++i) {
        for (int64_t j = 0; j < K; ++j) {
            double p = (double)in[(y + i) * W + (x + j)] * (double)f[i * K + j];
            acc += p;
            b += fabs(p);
        }
    }
    *acc_out = acc;
    *bound_out = b;
}

/*
 * in: H*W row-major. f: K*K row-major. out: (H-K+1)*(W-K+1) row-major fp32 (may be NULL).
 * bound, out64: same shape, double (each may be NULL). Rows [y_begin, y_end) of the output only
 * (pass 0, H-K+1 for the whole image; the bench's bounded cpu_baseline sample uses a sub-range).
 */
void oracle_conv2d_single_rows(const float *in, int64_t H, int64_t W, const float *f, int64_t K,
                               int64_t y_begin, int64_t y_end, float *out, double *bound, double *out64)
{
    const int64_t Wo = W - K + 1;
    (void)H;
#pragma omp parallel for schedule(dynamic, 1)
    for (int64_t y = y_begin; y < y_end; ++y) {
        for (int64_t x = 0; x < Wo; ++x) {
            double acc, b;
            single_point(in, W, f, K, y, x, &acc, &b);
            const int64_t o = y * Wo + x;
            if (out) out[o] = (float)acc;
            if (bound) bound[o] = b;
            if (out64) out64[o] = acc;
        }
    }
}

void oracle_conv2d_single(const float *in, int64_t H, int64_t W, const float *f, int64_t K, float *out,
                          double *bound, double *out64)
{
    oracle_conv2d_single_rows(in, H, W, f, K, 0, H - K + 1, out, bound, out64);
}

/* Sampled outputs, one by one: points (ys[p], xs[p]) for p < npts. */
void oracle_conv2d_single_points(const float *in, int64_t H, int64_t W, const float *f, int64_t K,
                                 const int64_t *ys, const int64_t *xs, int64_t npts, float *out,
                                 double *bound)
{
    (void)H;
#pragma omp parallel for schedule(static)
    for (int64_t p = 0; p < npts; ++p) {
        double acc, b;
        single_point(in, W, f, K, ys[p], xs[p], &acc, &b);
        out[p] = (float)acc;
        if (bound) bound[p] = b;
    }
}

/*
 * Rectangular FH x FW filters (Table I lists filters as "FH x FW", P:338 --
 * every entry there is square, the variant is the image-library generalisation):
 *     out[y][x] = fl32( sum_{i<FH} sum_{j<FW} (double)in[y+i][x+j] * (double)f[i][j] )
 * in: H*W row-major. f: FH*FW row-major. out / bound / out64: (H-FH+1)*(W-FW+1) row-major (each may be
 * NULL). Same order and single rounding as the square definition above.
 */
void oracle_conv2d_single_rect(const float *in, int64_t H, int64_t W, const float *f, int64_t FH, int64_t FW,
                               float *out, double *bound, double *out64)
{
    const int64_t Ho = H - FH + 1, Wo = W - FW + 1;
#pragma omp parallel for schedule(dynamic, 1)
    for (int64_t y = 0; y < Ho; ++y) {
        for (int64_t x = 0; x < Wo; ++x) {
            double acc = 0.0, b = 0.0;
            for (int64_t i = 0; i < FH; ++i) {
                for (int64_t j = 0; j < FW; ++j) {
                    double p = (double)in[(y + i) * W + (x + j)] * (double)f[i * FW + j];
                    acc += p;
                    b += fabs(p);
                }
            }
            const int64_t o = y * Wo + x;
            if (out) out[o] = (float)acc;
            if (bound) bound[o] = b;
            if (out64) out64[o] = acc;
        }
    }
}

/* One output element of the multi-channel definition. */
static void multi_point(const float *in, int64_t C, int64_t H, int64_t W, const float *w, int64_t K,
                        int64_t n, int64_t f, int64_t y, int64_t x, double *acc_out, double *bound_out)
{
    double acc = 0.0, b = 0.0;
    for (int64_t c = 0; c < C; ++c) {
        const float *img = in + ((n * C + c) * H) * W;
        const float *flt = w + ((f * C + c) * K) * K;
        for (int64_t i = 0; i < K; ++i) {
            for (int64_t j = 0; j < K; ++j) {
                double p = (double)img[(y + i) * W + (x + j)] * (double)flt[i * K + j];
                acc += p;
                b += fabs(p);
            }
        }
    }
    *acc_out = acc;
    *bound_out = b;
}

/* in: N*C*H*W. w: F*C*K*K. out/bound/out64: N*F*Ho*Wo. Images [n_begin, n_end) only. */
void oracle_conv2d_multi_images(const float *in, int64_t N, int64_t C, int64_t H, int64_t W,
                                const float *w, int64_t F, int64_t K, int64_t n_begin, int64_t n_end,
                                float *out, double *bound, double *out64)
{
    const int64_t Ho = H - K + 1, Wo = W - K + 1;
    (void)N;
#pragma omp parallel for collapse(3) schedule(dynamic, 1)
    for (int64_t n = n_begin; n < n_end; ++n) {
        for (int64_t f = 0; f < F; ++f) {
            for (int64_t y = 0; y < Ho; ++y) {
                for (int64_t x = 0; x < Wo; ++x) {
                    double acc, b;
                    multi_point(in, C, H, W, w, K, n, f, y, x, &acc, &b);
                    const int64_t o = ((n * F + f) * Ho + y) * Wo + x;
                    if (out) out[o] = (float)acc;
                    if (bound) bound[o] = b;
                    if (out64) out64[o] = acc;
                }
            }
        }
    }
}

void oracle_conv2d_multi(const float *in, int64_t N, int64_t C, int64_t H, int64_t W, const float *w,
                         int64_t F, int64_t K, float *out, double *bound, double *out64)
{
    oracle_conv2d_multi_images(in, N, C, H, W, w, F, K, 0, N, out, bound, out64);
}

/* Sampled outputs (ns[p], fs[p], ys[p], xs[p]). */
void oracle_conv2d_multi_points(const float *in, int64_t N, int64_t C, int64_t H, int64_t W,
                                const float *w, int64_t F, int64_t K, const int64_t *ns,
                                const int64_t *fs, const int64_t *ys, const int64_t *xs, int64_t npts,
                                float *out, double *bound)
{
    (void)N;
    (void)F;
#pragma omp parallel for schedule(static)
    for (int64_t p = 0; p < npts; ++p) {
        double acc, b;
        multi_point(in, C, H, W, w, K, ns[p], fs[p], ys[p], xs[p], &acc, &b);
        out[p] = (float)acc;
        if (bound) bound[p] = b;
    }
}
