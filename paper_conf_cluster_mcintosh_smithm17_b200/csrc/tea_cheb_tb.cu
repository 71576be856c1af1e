// tea_cheb_tb.cu -- temporally blocked Chebyshev inner loop ("on-chip matrix powers").
//
// O'Leary's point 2 quoted by the paper: "the polynomial preconditioned
// algorithm is designed to use the matrix for several multiplications at a time", and the
// matrix-powers idea of Sec. IV.C.2 applied on chip instead of across ranks:
// one kernel performs M consecutive Chebyshev steps (DESIGN.md §4.3 recurrence)
//     z_i = cX X + cZ z_{i-2} + cR r - cA (A X),   X = z_{i-1} (or r at step 1)
// in a single pass through HBM. Per pass it reads z_{i-1}, z_{i-2}, r, Kx, Ky (the first
// pass: r [, w], Kx, Ky) and writes z_{i+M-2}, z_{i+M-1} (the last pass: z_s only, plus the
// fused r.z / r.r reductions) -- 7 streams for M steps instead of 6 M.
//
// Mapping: a warp owns a 64-column strip (32 lanes x double2) and marches down the rows.
// Step t lags the input by t rows: at row-iteration k the warp loads input row k and
// computes z_t at row k - t for t = 1..M. Each step keeps its last three rows in
// registers (the stencil window of the next step; its oldest row is also the z_{t-2}
// pointwise term of step t+2); x-neighbours come from warp shuffles. The pointwise
// operands Kx, Ky, r (and z_{i-2}) are needed M rows after they are loaded: they wait in
// per-thread shared-memory delay lines (each thread reads back only what it wrote, so no
// barriers). Every step loses one valid column per side (no edge loads): strips overlap
// and each produces 64 - 2*ceil_even(M) output columns. A CTA tile of ty output rows
// runs ty + 2M row-iterations (pipeline fill/drain).
//
// Single-block only (no extended bounds); blocks with neighbours use the per-step kernels.
#include "tea_internal.h"

namespace tea {

namespace {

__device__ __forceinline__ double2 ldg2c(const double *p) {
    return __ldg(reinterpret_cast<const double2 *>(p));
}
__device__ __forceinline__ void st2m(double *p, double2 v, bool a, bool b) {
    if (a && b) {
        *reinterpret_cast<double2 *>(p) = v;
    } else {
        if (a) p[0] = v.x;
        if (b) p[1] = v.y;
    }
}
__device__ __forceinline__ double wsum(double v) {
#pragma unroll
    for (int o = 16; o > 0; o >>= 1) v += __shfl_xor_sync(0xffffffffu, v, o);
    return v;
}

// Deterministic two-value grid reduction (same scheme as tea_kernels.cu).
__device__ bool grid_reduce2(double v0, double v1, double *partials, unsigned *ticket,
                             double *out0, double *out1) {
    __shared__ double sh[2][kWarps];
    __shared__ bool last;
    const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
    const int nblk = gridDim.x * gridDim.y * gridDim.z;
    const int bid = (blockIdx.z * gridDim.y + blockIdx.y) * gridDim.x + blockIdx.x;
    v0 = wsum(v0);
    v1 = wsum(v1);
    if (lane == 0) {
        sh[0][warp] = v0;
        sh[1][warp] = v1;
    }
    __syncthreads();
    if (threadIdx.x == 0) {
        double s0 = 0.0, s1 = 0.0;
        for (int w = 0; w < kWarps; ++w) {
            s0 += sh[0][w];
            s1 += sh[1][w];
        }
        partials[bid] = s0;
        partials[nblk + bid] = s1;
        __threadfence();
        last = (atomicAdd(ticket, 1u) == (unsigned)nblk - 1u);
    }
    __syncthreads();
    if (!last) return false;
    __threadfence();
    double t[2];
#pragma unroll
    for (int i = 0; i < 2; ++i) {
        double s = 0.0;
        for (int b = threadIdx.x; b < nblk; b += kThreads) s += __ldcg(partials + i * nblk + b);
        s = wsum(s);
        __syncthreads();
        if (lane == 0) sh[i][warp] = s;
        __syncthreads();
        double a = 0.0;
        for (int w = 0; w < kWarps; ++w) a += sh[i][w];
        t[i] = a;
    }
    *out0 = t[0];
    *out1 = t[1];
    if (threadIdx.x == 0) *ticket = 0u;
    return true;
}

__device__ bool grid_arrive2(unsigned *ticket) {
    __shared__ bool last;
    __syncthreads();
    if (threadIdx.x == 0) {
        __threadfence();
        last = (atomicAdd(ticket, 1u) == gridDim.x * gridDim.y * gridDim.z - 1u);
    }
    __syncthreads();
    if (last && threadIdx.x == 0) *ticket = 0u;
    return last;
}

}  // namespace

#ifndef TEA_TB_UNROLL
#define TEA_TB_UNROLL 1
#endif
constexpr int kTbUnroll = TEA_TB_UNROLL;  // measured: 2 (step t+1 of row k overlapping
                                          // step t of row k+1) costs registers, no gain

template <int M>
struct TbGeom {
    static constexpr int MR = (M + 1) & ~1;  // margin, even (double2 alignment)
    static constexpr int OW = kStrip - 2 * MR;  // output columns per warp strip
    static constexpr int D = M + 2;             // delay-line depth (rows)
};

#ifndef TEA_TB_MINB
#define TEA_TB_MINB 1
#endif
template <int M, bool FIRST, bool FUSE, bool LAST>
__global__ void __launch_bounds__(kThreads, TEA_TB_MINB)
    k_cheb_tb(const double *__restrict__ rin, const double *__restrict__ win,
              double *__restrict__ rout, const double *__restrict__ zin1,
              const double *__restrict__ zin2, double *__restrict__ zoutA,
              double *__restrict__ zoutB, const double *__restrict__ Kx,
              const double *__restrict__ Ky, KArgs a, Region R, int ty, int jlim, int step0,
              int restart) {
    using G = TbGeom<M>;
    constexpr int D = G::D;
    __shared__ double2 ringKx[D][kThreads], ringKy[D][kThreads], ringR[D][kThreads];
    __shared__ double2 ringZ2[2][kThreads];
    __shared__ double coef[4][M];

    Scalars *S = a.S;
    if (S->done) {
        if (LAST && blockIdx.x == 0 && blockIdx.y == 0 && blockIdx.z == 0 && threadIdx.x == 0 && a.set_cond &&
            a.cond)
            cudaGraphSetConditional(a.cond, 0u);
        return;
    }
    double alpha = 0.0;
    if (FUSE) {
        const double pw = S->red_pw;
        alpha = S->gam_old / pw;
        if (!(pw > 0.0) || !isfinite(alpha)) {
            if (grid_arrive2(&S->ticket) && threadIdx.x == 0) {
                S->done = 1;
                S->status = DS_BREAKDOWN;
                if (LAST && a.set_cond && a.cond) cudaGraphSetConditional(a.cond, 0u);
            }
            return;
        }
    }
    if (threadIdx.x < M) {
        const int i = step0 - 1 + threadIdx.x;
        coef[0][threadIdx.x] = S->cheb_cx[i];
        coef[1][threadIdx.x] = S->cheb_cz[i];
        coef[2][threadIdx.x] = S->cheb_cr[i];
        coef[3][threadIdx.x] = S->cheb_ca[i];
    }
    const double2 z0 = make_double2(0.0, 0.0);
    for (int d = 0; d < D; ++d) {
        ringKx[d][threadIdx.x] = z0;
        ringKy[d][threadIdx.x] = z0;
        ringR[d][threadIdx.x] = z0;
    }
    ringZ2[0][threadIdx.x] = z0;
    ringZ2[1][threadIdx.x] = z0;
    __syncthreads();

    const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5, tid = threadIdx.x;
    const int strip = blockIdx.x * kWarps + warp;
    const int jA = -G::MR + strip * G::OW + 2 * lane;
    const int kt0 = R.k0 + blockIdx.y * ty;
    const int kt1 = min(kt0 + ty, R.k1);
    const int pitch = a.pitch;
    const bool ld_ok = jA + 1 < jlim;  // inside the allocation
    // output columns: this strip's [MR, 64-MR) intersected with the region
    const int cA = 2 * lane, cB = 2 * lane + 1;
    const bool oA = cA >= G::MR && cA < kStrip - G::MR && jA >= R.j0 && jA < R.j1;
    const bool oB = cB >= G::MR && cB < kStrip - G::MR && jA + 1 >= R.j0 && jA + 1 < R.j1;

    // stencil windows: W[t] holds z_t rows (oldest, middle, newest); W[0] = input operand
    double2 W[M][3];
#pragma unroll
    for (int t = 0; t < M; ++t) W[t][0] = W[t][1] = W[t][2] = z0;
    double dot0 = 0.0, dot1 = 0.0;

    // prefetch registers for input row k
    double2 pX = z0, pW = z0, pZ2 = z0, pKx = z0, pKy = z0, pR = z0;
    auto load = [&](int k) {
        if (!ld_ok || kt0 >= kt1) return;
        const int o = k * pitch + jA;
        if (FIRST) {
            pX = ldg2c(rin + o);
            if (FUSE) pW = ldg2c(win + o);
        } else {
            pX = ldg2c(zin1 + o);
            pZ2 = ldg2c(zin2 + o);
            pR = ldg2c(rin + o);
        }
        pKx = ldg2c(Kx + o);
        pKy = ldg2c(Ky + o);
    };
    const int kbeg = kt0 - M, kend = kt1 + M;
    load(kbeg);
#pragma unroll(kTbUnroll)
    for (int k = kbeg; k < kend; ++k) {
        double2 X = pX, Wv = pW, Z2 = pZ2, KX = pKx, KY = pKy, RR = pR;
        if (k + 1 < kend) load(k + 1);
        double2 rk;
        if (FIRST) {
            if (FUSE) X = make_double2(X.x - alpha * Wv.x, X.y - alpha * Wv.y);
            rk = X;
            if (FUSE && k >= kt0 && k < kt1) st2m(rout + k * pitch + jA, X, oA, oB);
        } else {
            rk = RR;
        }
        const int slot = (k + 4 * D) % D;
        ringKx[slot][tid] = KX;
        ringKy[slot][tid] = KY;
        ringR[slot][tid] = rk;
        if (!FIRST) ringZ2[(k + 4) & 1][tid] = Z2;
        W[0][0] = W[0][1];
        W[0][1] = W[0][2];
        W[0][2] = X;
#pragma unroll
        for (int t = 1; t <= M; ++t) {
            const int q = k - t;
            const int sq = (q + 4 * D) % D, sq1 = (q + 1 + 4 * D) % D;
            const double2 kx = ringKx[sq][tid];
            const double2 kyc = ringKy[sq][tid];
            const double2 kyn = ringKy[sq1][tid];
            const double2 rq = ringR[sq][tid];
            double2 z2;
            if (t == 1) {
                z2 = FIRST ? z0 : ringZ2[(q + 4) & 1][tid];
            } else {
                z2 = W[t >= 2 ? t - 2 : 0][0];
            }
            const double2 xm = W[t - 1][0], xc = W[t - 1][1], xp = W[t - 1][2];
            double left = __shfl_up_sync(0xffffffffu, xc.y, 1);
            double right = __shfl_down_sync(0xffffffffu, xc.x, 1);
            double kxB = __shfl_down_sync(0xffffffffu, kx.x, 1);
            if (lane == 0) left = 0.0;
            if (lane == 31) {
                right = 0.0;
                kxB = 0.0;
            }
            double2 AX;
            AX.x = (1.0 + (kyn.x + kyc.x) + (kx.y + kx.x)) * xc.x - (kyn.x * xp.x + kyc.x * xm.x) -
                   (kx.y * xc.y + kx.x * left);
            AX.y = (1.0 + (kyn.y + kyc.y) + (kxB + kx.y)) * xc.y - (kyn.y * xp.y + kyc.y * xm.y) -
                   (kxB * right + kx.y * xc.x);
            const double cx = coef[0][t - 1], cz = coef[1][t - 1], cr = coef[2][t - 1],
                         ca = coef[3][t - 1];
            double2 zn;
            zn.x = cx * xc.x + cz * z2.x + cr * rq.x - ca * AX.x;
            zn.y = cx * xc.y + cz * z2.y + cr * rq.y - ca * AX.y;
            const bool rowout = q >= kt0 && q < kt1;
            if (t < M) {
                const int tt = t < M ? t : M - 1;
                W[tt][0] = W[tt][1];
                W[tt][1] = W[tt][2];
                W[tt][2] = zn;
                if (t == M - 1 && !LAST && rowout) st2m(zoutA + q * pitch + jA, zn, oA, oB);
            } else {
                if (rowout) {
                    st2m(zoutB + q * pitch + jA, zn, oA, oB);
                    if (LAST) {
                        if (oA) {
                            dot0 += rq.x * zn.x;
                            dot1 += rq.x * rq.x;
                        }
                        if (oB) {
                            dot0 += rq.y * zn.y;
                            dot1 += rq.y * rq.y;
                        }
                    }
                }
            }
        }
    }
    if (LAST) {
        double t0, t1;
        if (grid_reduce2(dot0, dot1, a.partials, &S->ticket, &t0, &t1)) {
            if (threadIdx.x == 0) {
                S->red_gam = t0;
                S->red_rr = t1;
                if (FUSE) S->alpha_prev = alpha;
                if (!restart) {
                    S->it += 1;
                    S->outer += 1;
                }
            }
        }
    } else if (FUSE) {
        if (blockIdx.x == 0 && blockIdx.y == 0 && blockIdx.z == 0 && threadIdx.x == 0) S->alpha_prev = alpha;
    }
}

int tb_out_cols(int M) {
    const int mr = (M + 1) & ~1;
    return kStrip - 2 * mr;
}

template <int M, bool FIRST, bool FUSE, bool LAST>
static void tb_launch(const KArgs &a, const Region &R, int ty, int jlim, int step0, bool restart,
                      const double *rin, const double *win, double *rout, const double *zin1,
                      const double *zin2, double *zoutA, double *zoutB, const double *kx,
                      const double *ky, cudaStream_t st) {
    using G = TbGeom<M>;
    const int width = R.j1;  // single block: R.j0 == 0
    const int nstrips = (width + G::OW - 1) / G::OW;
    dim3 grid((nstrips + kWarps - 1) / kWarps, (R.k1 - R.k0 + ty - 1) / ty);
    k_cheb_tb<M, FIRST, FUSE, LAST><<<grid, kThreads, 0, st>>>(
        rin, win, rout, zin1, zin2, zoutA, zoutB, kx, ky, a, R, ty, jlim, step0, restart ? 1 : 0);
}

template <int M>
static void tb_dispatch(const KArgs &a, const Region &R, int ty, int jlim, int step0, bool first,
                        bool fuse, bool last, bool restart, const double *rin, const double *win,
                        double *rout, const double *zin1, const double *zin2, double *zoutA,
                        double *zoutB, const double *kx, const double *ky, cudaStream_t st) {
#define TB(F, U, L)                                                                            \
    tb_launch<M, F, U, L>(a, R, ty, jlim, step0, restart, rin, win, rout, zin1, zin2, zoutA, \
                          zoutB, kx, ky, st)
    if (first) {
        if (fuse) {
            if (last) TB(true, true, true); else TB(true, true, false);
        } else {
            if (last) TB(true, false, true); else TB(true, false, false);
        }
    } else {
        if (last) TB(false, false, true); else TB(false, false, false);
    }
#undef TB
}

int tb_max_steps() { return 5; }

int tb_ctas(int M, int width, int height, int ty) {
    const int ow = tb_out_cols(M);
    const int nstrips = (width + ow - 1) / ow;
    return ((nstrips + kWarps - 1) / kWarps) * ((height + ty - 1) / ty);
}

void launch_cheb_tb(const KArgs &a, const Region &R, int M, int ty, int jlim, int step0,
                    bool first, bool fuse, bool last, bool restart, const double *rin,
                    const double *win, double *rout, const double *zin1, const double *zin2,
                    double *zoutA, double *zoutB, const double *kx, const double *ky,
                    cudaStream_t st) {
    switch (M) {
        case 1: tb_dispatch<1>(a, R, ty, jlim, step0, first, fuse, last, restart, rin, win, rout, zin1, zin2, zoutA, zoutB, kx, ky, st); break;
        case 2: tb_dispatch<2>(a, R, ty, jlim, step0, first, fuse, last, restart, rin, win, rout, zin1, zin2, zoutA, zoutB, kx, ky, st); break;
        case 3: tb_dispatch<3>(a, R, ty, jlim, step0, first, fuse, last, restart, rin, win, rout, zin1, zin2, zoutA, zoutB, kx, ky, st); break;
        case 4: tb_dispatch<4>(a, R, ty, jlim, step0, first, fuse, last, restart, rin, win, rout, zin1, zin2, zoutA, zoutB, kx, ky, st); break;
        default: tb_dispatch<5>(a, R, ty, jlim, step0, first, fuse, last, restart, rin, win, rout, zin1, zin2, zoutA, zoutB, kx, ky, st); break;
    }
}

}  // namespace tea
