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

#include <mutex>

namespace tea {

#ifndef TEA_TB_WARPS
#define TEA_TB_WARPS 4
#endif
// warps per CTA of the fused passes (each warp marches its own strip; CTAs only share the
// grid reduction). Smaller CTAs pack registers tighter: 138 registers allow 14 warps per SM
// but only 3 CTAs of 4 warps.
constexpr int kTbW = TEA_TB_WARPS;
constexpr int kTbT = 32 * kTbW;
#ifndef TEA_TB_TMEM
#define TEA_TB_TMEM 1  // Kx, Ky, r delay lines in tensor memory (see tm_st12)
#endif
#ifndef TEA_TB_CPA
#define TEA_TB_CPA 4  // rows of cp.async input staging ahead of the march (0: one register row)
#endif
#define TB_CPA (TEA_TB_CPA > 0)
#if TB_CPA && !TEA_TB_TMEM
#error "TEA_TB_CPA stages rows in the shared memory the rings would use: needs TEA_TB_TMEM"
#endif
constexpr int kTbNS = 5;  // staged streams per row (X, W or z_{i-2}, r, Kx, Ky)

// Chebyshev coefficients of the fused passes live in constant memory (one slot per
// context): uniform per-step scalars then cost LDC through the constant cache instead
// of shared-memory wavefronts on the L1TEX pipe the passes are bound by.
// Uploaded once per solve after the eigen-estimate (tb_coef_upload).
constexpr int kTbSlots = 16;
__constant__ double c_tb_coef[kTbSlots][4][kMaxS];
static_assert(offsetof(Scalars, cheb_cz) == offsetof(Scalars, cheb_cx) + kMaxS * sizeof(double) &&
                  offsetof(Scalars, cheb_ca) == offsetof(Scalars, cheb_cx) + 3 * kMaxS * sizeof(double),
              "folded coefficients must be contiguous [4][kMaxS]");
static std::mutex g_slot_mu;
static bool g_slot_used[kTbSlots];

int tb_slot_acquire() {
    std::lock_guard<std::mutex> g(g_slot_mu);
    for (int i = 0; i < kTbSlots; ++i)
        if (!g_slot_used[i]) {
            g_slot_used[i] = true;
            return i;
        }
    return -1;
}
void tb_slot_release(int slot) {
    if (slot < 0 || slot >= kTbSlots) return;
    std::lock_guard<std::mutex> g(g_slot_mu);
    g_slot_used[slot] = false;
}
cudaError_t tb_coef_upload(int slot, const Scalars *S, cudaStream_t st) {
    return cudaMemcpyToSymbolAsync(c_tb_coef, S->cheb_cx, sizeof(c_tb_coef[0]),
                                   sizeof(c_tb_coef[0]) * (size_t)slot, cudaMemcpyDeviceToDevice,
                                   st);
}

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
__device__ __forceinline__ void cp16(void *sdst, const double *gsrc) {
    asm volatile("cp.async.cg.shared.global [%0], [%1], 16;" ::"r"(
                     (uint32_t)__cvta_generic_to_shared(sdst)),
                 "l"(gsrc)
                 : "memory");
}
__device__ __forceinline__ void cp_commit() { asm volatile("cp.async.commit_group;" ::: "memory"); }
template <int N>
__device__ __forceinline__ void cp_wait() {
    asm volatile("cp.async.wait_group %0;" ::"n"(N) : "memory");
}
__device__ __forceinline__ double wsum(double v) {
#pragma unroll
    for (int o = 16; o > 0; o >>= 1) v += __shfl_xor_sync(0xffffffffu, v, o);
    return v;
}

// Tensor-memory (TMEM) delay lines (TEA_TB_TMEM): each thread owns one TMEM lane (warp w of
// the CTA reaches lanes 32(w%4)..32(w%4)+31) and keeps its Kx, Ky, r delay slots there --
// 16 32-bit columns per slot (Kx double2 in 0-3, Ky in 4-7, r in 8-11), 8 slots = 128
// columns per warp quarter. tcgen05.st / tcgen05.ld (.32x32b) run on the tensor-memory
// datapath, not on the L1TEX pipe that the shared-memory rings and the shuffles share
// (tools/tmem_probe.cu: ~165 B/clk/SM of TMEM reads vs ~110 of shared memory at 12 warps).
__device__ __forceinline__ uint32_t d_lo(double v) { return (uint32_t)__double_as_longlong(v); }
__device__ __forceinline__ uint32_t d_hi(double v) {
    return (uint32_t)((unsigned long long)__double_as_longlong(v) >> 32);
}
__device__ __forceinline__ double d_of(uint32_t lo, uint32_t hi) {
    return __longlong_as_double(((long long)hi << 32) | lo);
}
__device__ __forceinline__ void tm_st12(uint32_t a, double2 kx, double2 ky, double2 r) {
    asm volatile(
        "tcgen05.st.sync.aligned.32x32b.x8.b32 [%0], {%1, %2, %3, %4, %5, %6, %7, %8};\n\t"
        "tcgen05.st.sync.aligned.32x32b.x4.b32 [%9], {%10, %11, %12, %13};" ::"r"(a),
        "r"(d_lo(kx.x)), "r"(d_hi(kx.x)), "r"(d_lo(kx.y)), "r"(d_hi(kx.y)), "r"(d_lo(ky.x)),
        "r"(d_hi(ky.x)), "r"(d_lo(ky.y)), "r"(d_hi(ky.y)), "r"(a + 8u), "r"(d_lo(r.x)),
        "r"(d_hi(r.x)), "r"(d_lo(r.y)), "r"(d_hi(r.y))
        : "memory");
}
struct TmRow {
    uint32_t v[12];
};
__device__ __forceinline__ void tm_ld12(uint32_t a, TmRow &o) {
    asm volatile(
        "tcgen05.ld.sync.aligned.32x32b.x8.b32 {%0, %1, %2, %3, %4, %5, %6, %7}, [%12];\n\t"
        "tcgen05.ld.sync.aligned.32x32b.x4.b32 {%8, %9, %10, %11}, [%13];"
        : "=r"(o.v[0]), "=r"(o.v[1]), "=r"(o.v[2]), "=r"(o.v[3]), "=r"(o.v[4]), "=r"(o.v[5]),
          "=r"(o.v[6]), "=r"(o.v[7]), "=r"(o.v[8]), "=r"(o.v[9]), "=r"(o.v[10]), "=r"(o.v[11])
        : "r"(a), "r"(a + 8u)
        : "memory");
}
// wait for every outstanding tcgen05.ld; the registers are in/out operands so no use of
// them can be scheduled above the wait
__device__ __forceinline__ void tm_wait_ld(TmRow &o) {
    asm volatile("tcgen05.wait::ld.sync.aligned;"
                 : "+r"(o.v[0]), "+r"(o.v[1]), "+r"(o.v[2]), "+r"(o.v[3]), "+r"(o.v[4]),
                   "+r"(o.v[5]), "+r"(o.v[6]), "+r"(o.v[7]), "+r"(o.v[8]), "+r"(o.v[9]),
                   "+r"(o.v[10]), "+r"(o.v[11])
                 :
                 : "memory");
}
__device__ __forceinline__ void tm_wait_st() {
    asm volatile("tcgen05.wait::st.sync.aligned;" ::: "memory");
}
__device__ __forceinline__ double2 tm_get(const TmRow &o, int i) {
    return make_double2(d_of(o.v[4 * i], o.v[4 * i + 1]), d_of(o.v[4 * i + 2], o.v[4 * i + 3]));
}

// Deterministic two-value grid reduction (same scheme as tea_kernels.cu).
__device__ bool grid_reduce2(double v0, double v1, double *partials, unsigned *ticket,
                             double *out0, double *out1) {
    __shared__ double sh[2][kTbW];
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
        for (int w = 0; w < kTbW; ++w) {
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
        for (int b = threadIdx.x; b < nblk; b += kTbT) s += __ldcg(partials + i * nblk + b);
        s = wsum(s);
        __syncthreads();
        if (lane == 0) sh[i][warp] = s;
        __syncthreads();
        double a = 0.0;
        for (int w = 0; w < kTbW; ++w) a += sh[i][w];
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
#ifndef TEA_TB_UNROLL_L
#define TEA_TB_UNROLL_L 3
#endif
#ifndef TEA_TB_CPA_L
#define TEA_TB_CPA_L 2
#endif
// row-loop unroll and cp.async depth of the non-first passes (measured separately:
// profiles/r01g_tmem_cpa.txt; the first pass carries r, w and more registers)
constexpr int kTbUnrollL = TEA_TB_UNROLL_L;
constexpr int kTbCpaL = TEA_TB_CPA > 0 ? TEA_TB_CPA_L : 0;
static_assert(TEA_TB_CPA == 0 || (TEA_TB_CPA_L >= 1 && TEA_TB_CPA_L <= TEA_TB_CPA), "staging depth");

// dynamic shared memory of a pass: the Kx, Ky, r delay rings (depth 8, one double2 per
// thread and row)
// (TEA_TB_TMEM: the rings live in TMEM; the request then holds the cp.async row staging
// and caps residency at 4 CTAs per SM so 4 x kTmCols TMEM columns always fit)
constexpr size_t tb_smem_bytes() {
    return TEA_TB_CPA > 0 ? (sizeof(double2) * kTbNS * (TEA_TB_CPA + 1) * kTbT > 48u * 1024u
                                 ? sizeof(double2) * kTbNS * (TEA_TB_CPA + 1) * kTbT
                                 : 48u * 1024u)
                          : sizeof(double2) * 3 * 8 * kTbT;
}

template <int M>
struct TbGeom {
    static constexpr int MR = (M + 1) & ~1;  // margin, even (double2 alignment)
    static constexpr int OW = kStrip - 2 * MR;  // output columns per warp strip
    static constexpr int D = 8;  // delay-line depth (rows k-M-1..k fit for M <= 6); a power of
                                 // two so slots are (head - t) & 7, not a division
};

#ifndef TEA_TB_MINB
#define TEA_TB_MINB 1
#endif
#ifndef TEA_TB_REGLINES
#define TEA_TB_REGLINES 0  // 1: Kx, Ky and r lines in registers (measured slower: 225 regs,
                            // 2 CTAs/SM, 737 vs 660 us/outer, profiles/r01_tb_reglines.txt);
                            // 2: r only
#endif
#define TB_REG_K (TEA_TB_REGLINES == 1)
#ifndef TEA_TB_L2PF
#define TEA_TB_L2PF 0  // rows of L2 bulk-prefetch distance (0 = off; 3, 6, 10 measured
                       // slower: profiles/r01_tb_variants2.txt)
#endif
#define TB_REG_R (TEA_TB_REGLINES >= 1)
#if TEA_TB_TMEM && TEA_TB_REGLINES
#error "TEA_TB_TMEM replaces the delay lines; TEA_TB_REGLINES must be 0"
#endif
constexpr int kTmCols = 128;  // TMEM columns per CTA: 8 slots x 16 per warp quarter
template <int M, bool FIRST, bool FUSE, bool LAST>
__global__ void __launch_bounds__(kTbT, TEA_TB_MINB)
    k_cheb_tb(const double *__restrict__ rin, const double *__restrict__ win,
              double *__restrict__ rout, const double *__restrict__ zin1,
              const double *__restrict__ zin2, double *__restrict__ zoutA,
              double *__restrict__ zoutB, const double *__restrict__ Kx,
              const double *__restrict__ Ky, KArgs a, Region R, Region Dd, int ty, int jlim,
              int step0, int restart) {
    using G = TbGeom<M>;
    constexpr int D = G::D;
    static_assert(M <= 6, "delay lines hold M+2 rows");
    extern __shared__ double2 tb_smem[];
    double2(*ringKx)[kTbT] = reinterpret_cast<double2(*)[kTbT]>(tb_smem);
    double2(*ringKy)[kTbT] = ringKx + D;
    double2(*ringR)[kTbT] = ringKy + D;
    const double(*coef)[kMaxS] = c_tb_coef[a.coef_slot];

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
    const double2 z0 = make_double2(0.0, 0.0);
#if TEA_TB_TMEM
    static_assert(kTbW % 4 == 0 || kTbW < 4, "warp quarters");
    (void)ringKx;
    (void)ringKy;
    (void)ringR;
    // one warp allocates the CTA's TMEM columns; every warp then owns lanes 32(w%4).. and
    // a 128-column group per 4 warps. The dynamic shared memory request (tb_smem_bytes)
    // keeps at most 4 CTAs per SM, so 4 x kTmCols <= 512 columns always fit.
    __shared__ uint32_t tm_base_sh;
    constexpr int kTmAlloc = kTmCols * ((kTbW + 3) / 4);
    static_assert(kTmAlloc == 128 || kTmAlloc == 256, "TMEM allocation: power of two");
    if ((threadIdx.x >> 5) == 0) {
        asm volatile("tcgen05.alloc.cta_group::1.sync.aligned.shared::cta.b32 [%0], %1;" ::"r"(
                         (uint32_t)__cvta_generic_to_shared(&tm_base_sh)),
                     "n"(kTmAlloc)
                     : "memory");
        asm volatile("tcgen05.relinquish_alloc_permit.cta_group::1.sync.aligned;" ::: "memory");
    }
    asm volatile("tcgen05.fence::before_thread_sync;" ::: "memory");
    __syncthreads();
    asm volatile("tcgen05.fence::after_thread_sync;" ::: "memory");
    const uint32_t tm = tm_base_sh + ((uint32_t)(((threadIdx.x >> 5) & 3) * 32) << 16) +
                        (uint32_t)(((threadIdx.x >> 5) >> 2) * kTmCols);
    for (int d = 0; d < D; ++d) tm_st12(tm + 16u * d, z0, z0, z0);
#else
    for (int d = 0; d < D; ++d) {
        ringKx[d][threadIdx.x] = z0;
        ringKy[d][threadIdx.x] = z0;
        ringR[d][threadIdx.x] = z0;
    }
    __syncthreads();
#endif

    const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5, tid = threadIdx.x;
    (void)tid;
    const int strip = blockIdx.x * kTbW + warp;
    // strips tile the output region R (which may reach into the halo on sides with a
    // neighbour block: extended bounds); first strip starts MR before it
    const int jA = (R.j0 & ~1) - G::MR + strip * G::OW + 2 * lane;
    const int kt0 = R.k0 + blockIdx.y * ty;
    const int kt1 = min(kt0 + ty, R.k1);
    const int pitch = a.pitch;
    const bool ld_ok = jA + 1 < jlim;  // inside the allocation
    // output columns: this strip's [MR, 64-MR) intersected with the region
    const int cA = 2 * lane, cB = 2 * lane + 1;
    const bool oA = cA >= G::MR && cA < kStrip - G::MR && jA >= R.j0 && jA < R.j1;
    const bool oB = cB >= G::MR && cB < kStrip - G::MR && jA + 1 >= R.j0 && jA + 1 < R.j1;
    // dot products over owned cells only (D), whatever the extension of R
    const bool dA = oA && jA >= Dd.j0 && jA < Dd.j1, dB = oB && jA + 1 >= Dd.j0 && jA + 1 < Dd.j1;

    // stencil windows: W[t] holds z_t rows (oldest, middle, newest); W[0] = input operand
    double2 W[M][3];
#pragma unroll
    for (int t = 0; t < M; ++t) W[t][0] = W[t][1] = W[t][2] = z0;
    double dot0 = 0.0, dot1 = 0.0;

    // prefetch registers for input row k; running element offsets (no k*pitch products)
    double2 pX = z0, pW = z0, pZ2 = z0, pKx = z0, pKy = z0, pR = z0;
    const int kbeg = kt0 - M, kend = kt1 + M;
    long long orow = (long long)kbeg * pitch + jA;  // offset of (jA, k)
    auto load = [&](long long o) {
        if (!ld_ok) return;
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
#if TB_CPA
    // input rows staged TEA_TB_CPA rows ahead by cp.async into per-thread shared-memory slots
    // (each thread copies and later reads back only its own 16 B per stream, so no
    // barriers; slots the thread never fills stay zero). More bytes in flight per warp
    // than one prefetched register row: the one-row version stalled on the load of the
    // next row (ncu: 41% of stall samples on the first use of the prefetched row).
    constexpr int P = FIRST ? TEA_TB_CPA : kTbCpaL, NSL = P + 1;
    double2(*cpa)[kTbNS][kTbT] = reinterpret_cast<double2(*)[kTbNS][kTbT]>(tb_smem);
    for (int sl = 0; sl < NSL; ++sl)
#pragma unroll
        for (int q = 0; q < kTbNS; ++q) cpa[sl][q][threadIdx.x] = z0;
    auto issue = [&](long long o, int sl) {
        if (ld_ok) {
            if (FIRST) {
                cp16(&cpa[sl][0][threadIdx.x], rin + o);
                if (FUSE) cp16(&cpa[sl][1][threadIdx.x], win + o);
            } else {
                cp16(&cpa[sl][0][threadIdx.x], zin1 + o);
                cp16(&cpa[sl][1][threadIdx.x], zin2 + o);
                cp16(&cpa[sl][2][threadIdx.x], rin + o);
            }
            cp16(&cpa[sl][3][threadIdx.x], Kx + o);
            cp16(&cpa[sl][4][threadIdx.x], Ky + o);
        }
        cp_commit();  // one group per row, empty or not, so wait_group counts rows
    };
#pragma unroll
    for (int i = 0; i < P; ++i) {
        if (kt0 < kt1 && kbeg + i < kend)
            issue(orow + (long long)i * pitch, i);
        else
            cp_commit();
    }
    int cs = 0;  // slot of row k
#else
    if (kt0 < kt1) load(orow);
#endif
#if TEA_TB_L2PF
    // L2 prefetch TEA_TB_L2PF rows ahead through the TMA unit (one lane, no registers, no
    // L1TEX wavefronts): the one-row register prefetch then hits L2
    const int jA0 = __shfl_sync(0xffffffffu, jA, 0);
    int pfb = (jlim - jA0) * 8;
    pfb = pfb > kStrip * 8 ? kStrip * 8 : (pfb & ~15);
    auto l2pf = [&](const double *base, long long o) {
        asm volatile("cp.async.bulk.prefetch.L2.global [%0], %1;" ::"l"(base + o), "r"(pfb)
                     : "memory");
    };
#endif
    int head = 0;  // ring slot of row k
    double2 z2prev = z0;  // z_{i-2} input of the previous row (a one-row register delay)
#if TB_REG_K
    double2 rKx[M + 1], rKy[M + 1];
#pragma unroll
    for (int i = 0; i <= M; ++i) rKx[i] = rKy[i] = z0;
#endif
#if TB_REG_R
    double2 rR[M + 1];
#pragma unroll
    for (int i = 0; i <= M; ++i) rR[i] = z0;
#endif
    // the later passes (fewer live registers) unroll the row loop by the window period 3:
    // the W[t][*] rotation becomes register renaming instead of ~50 moves per row
    constexpr int UNR = FIRST ? kTbUnroll : kTbUnrollL;
#pragma unroll(UNR)
    for (int k = kbeg; k < kend; ++k, orow += pitch, head = (head + 1) & (D - 1)) {
#if TB_CPA
        cp_wait<P - 1>();  // row k's group (the oldest outstanding) has landed
        const double2 X0 = cpa[cs][0][threadIdx.x];
        const double2 KX = cpa[cs][3][threadIdx.x], KY = cpa[cs][4][threadIdx.x];
        double2 X = X0, Wv = z0, Z2 = z0, RR = z0;
        if (FIRST) {
            if (FUSE) Wv = cpa[cs][1][threadIdx.x];
        } else {
            Z2 = cpa[cs][1][threadIdx.x];
            RR = cpa[cs][2][threadIdx.x];
        }
        {
            // row k+P goes into the slot row k-1 used (read a full iteration ago)
            const int ns = cs == 0 ? P : cs - 1;
            if (kt0 < kt1 && k + P < kend)
                issue(orow + (long long)P * pitch, ns);
            else
                cp_commit();
            cs = cs == P ? 0 : cs + 1;
        }
#else
        double2 X = pX, Wv = pW, Z2 = pZ2, KX = pKx, KY = pKy, RR = pR;
        if (k + 1 < kend) load(orow + pitch);
#endif
#if TEA_TB_L2PF
        if (lane == 0 && pfb > 0 && k + TEA_TB_L2PF < kend) {
            const long long o = orow + (long long)TEA_TB_L2PF * pitch;
            if (FIRST) {
                l2pf(rin, o);
                if (FUSE) l2pf(win, o);
            } else {
                l2pf(zin1, o);
                l2pf(zin2, o);
                l2pf(rin, o);
            }
            l2pf(Kx, o);
            l2pf(Ky, o);
        }
#endif
        double2 rk;
        if (FIRST) {
            if (FUSE) X = make_double2(X.x - alpha * Wv.x, X.y - alpha * Wv.y);
            rk = X;
            if (FUSE && k >= kt0 && k < kt1) st2m(rout + orow, X, oA, oB);
        } else {
            rk = RR;
        }
        // delay lines: shared-memory rings, or register shift registers (index i holds
        // row k - i; the step loop is unrolled, so step t's lag t is a compile-time index)
#if TEA_TB_TMEM
        // the previous row's store must land before this row's loads read it back
        tm_wait_st();
        tm_st12(tm + 16u * head, KX, KY, rk);
        TmRow tmA;
        tm_ld12(tm + 16u * ((head - 1) & (D - 1)), tmA);
        tm_wait_ld(tmA);
        double2 ky_up = KY;  // Ky of row q+1 for step 1: this row's
#elif TB_REG_K
#pragma unroll
        for (int i = M; i > 0; --i) {
            rKx[i] = rKx[i - 1];
            rKy[i] = rKy[i - 1];
        }
        rKx[0] = KX;
        rKy[0] = KY;
#else
        ringKx[head][tid] = KX;
        ringKy[head][tid] = KY;
#endif
#if TEA_TB_TMEM
#elif TB_REG_R
#pragma unroll
        for (int i = M; i > 0; --i) rR[i] = rR[i - 1];
        rR[0] = rk;
#else
        ringR[head][tid] = rk;
#endif
        const double2 z2row = z2prev;  // z_{i-2} of row k-1
        if (!FIRST) z2prev = Z2;
        W[0][0] = W[0][1];
        W[0][1] = W[0][2];
        W[0][2] = X;
#pragma unroll
        for (int t = 1; t <= M; ++t) {
            const int q = k - t;
            const int sq = (head - t) & (D - 1), sq1 = (head - t + 1) & (D - 1);
#if TEA_TB_TMEM
            // slot of row q = k - t is in tmA; issue the next step's slot before computing
            const double2 kx = tm_get(tmA, 0), kyc = tm_get(tmA, 1), rq = tm_get(tmA, 2);
            const double2 kyn = ky_up;
            ky_up = kyc;
            TmRow tmB;
            if (t < M) tm_ld12(tm + 16u * ((head - t - 1) & (D - 1)), tmB);
#elif TB_REG_K
            const double2 kx = rKx[t], kyc = rKy[t], kyn = rKy[t - 1];
#else
            const double2 kx = ringKx[sq][tid];
            const double2 kyc = ringKy[sq][tid];
            const double2 kyn = ringKy[sq1][tid];
#endif
#if TEA_TB_TMEM
#elif TB_REG_R
            const double2 rq = rR[t];
#else
            const double2 rq = ringR[sq][tid];
#endif
            (void)sq;
            (void)sq1;
            double2 z2;
            if (t == 1) {
                z2 = FIRST ? z0 : z2row;
            } else {
                z2 = W[t >= 2 ? t - 2 : 0][0];
            }
            const double2 xm = W[t - 1][0], xc = W[t - 1][1], xp = W[t - 1][2];
            // lane 0's left and lane 31's right neighbours are outside the strip: the
            // shuffles return the lane's own (finite) value, which only pollutes the
            // overlap columns every step already discards -- no selects needed
            // x direction in flux form: A x = x + sum_faces K_f (x_c - x_f) (Listing 1
            // regrouped). gw = Kx_w (x_A - x_left) is formed by the lane that owns the face's
            // Kx; its east neighbour receives it as -(its east flux). Two shuffles of x and
            // one of the flux -- no shuffle of Kx.
            const double left = __shfl_up_sync(0xffffffffu, xc.y, 1);
            const double gw = kx.x * (xc.x - left);
            const double gm = kx.y * (xc.x - xc.y);
            const double ge = __shfl_down_sync(0xffffffffu, gw, 1);  // Kx_e (x_right - x_B)
            // Dependency order: xp (the "up" row) is the row step t-1 produced in THIS
            // row-iteration; everything else is older. Form the rest first, fold xp in last.
            const int ci = step0 - 2 + t;
            const double cx = coef[0][ci], cz = coef[1][ci], cr = coef[2][ci], ca = coef[3][ci];
            double2 AXo, base;  // A x without the up term; the step's x-independent part
            AXo.x = (1.0 + (kyn.x + kyc.x)) * xc.x - kyc.x * xm.x + (gw + gm);
            AXo.y = (1.0 + (kyn.y + kyc.y)) * xc.y - kyc.y * xm.y - (gm + ge);
            base.x = cx * xc.x + cz * z2.x + cr * rq.x;
            base.y = cx * xc.y + cz * z2.y + cr * rq.y;
            double2 zn;
            zn.x = fma(-ca, fma(-kyn.x, xp.x, AXo.x), base.x);
            zn.y = fma(-ca, fma(-kyn.y, xp.y, AXo.y), base.y);
            const bool rowout = q >= kt0 && q < kt1;
            if (t < M) {
                const int tt = t < M ? t : M - 1;
                W[tt][0] = W[tt][1];
                W[tt][1] = W[tt][2];
                W[tt][2] = zn;
                if (t == M - 1 && !LAST && rowout) st2m(zoutA + (orow - t * pitch), zn, oA, oB);
            } else {
                if (rowout) {
                    st2m(zoutB + (orow - t * pitch), zn, oA, oB);
                    if (LAST && q >= Dd.k0 && q < Dd.k1) {
                        if (dA) {
                            dot0 += rq.x * zn.x;
                            dot1 += rq.x * rq.x;
                        }
                        if (dB) {
                            dot0 += rq.y * zn.y;
                            dot1 += rq.y * rq.y;
                        }
                    }
                }
            }
#if TEA_TB_TMEM
            if (t < M) {
                tm_wait_ld(tmB);
                tmA = tmB;
            }
#endif
        }
    }
#if TEA_TB_TMEM
    asm volatile("tcgen05.fence::before_thread_sync;" ::: "memory");
    __syncthreads();
    if ((threadIdx.x >> 5) == 0)
        asm volatile("tcgen05.dealloc.cta_group::1.sync.aligned.b32 %0, %1;" ::"r"(tm_base_sh),
                     "n"(kTmAlloc)
                     : "memory");
#endif
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
static void tb_launch(const KArgs &a, const Region &R, const Region &Dd, int ty, int jlim,
                      int step0, bool restart,
                      const double *rin, const double *win, double *rout, const double *zin1,
                      const double *zin2, double *zoutA, double *zoutB, const double *kx,
                      const double *ky, cudaStream_t st) {
    using G = TbGeom<M>;
    const int width = R.j1 - (R.j0 & ~1);
    const int nstrips = (width + G::OW - 1) / G::OW;
    dim3 grid((nstrips + kTbW - 1) / kTbW, (R.k1 - R.k0 + ty - 1) / ty);
    constexpr size_t smem = tb_smem_bytes();
    static bool attr = false;  // per instantiation
    if (!attr) {
        cudaFuncSetAttribute(k_cheb_tb<M, FIRST, FUSE, LAST>,
                             cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
        attr = true;
    }
    k_cheb_tb<M, FIRST, FUSE, LAST><<<grid, kTbT, smem, st>>>(
        rin, win, rout, zin1, zin2, zoutA, zoutB, kx, ky, a, R, Dd, ty, jlim, step0, restart ? 1 : 0);
}

template <int M>
static void tb_dispatch(const KArgs &a, const Region &R, const Region &Dd, int ty, int jlim,
                        int step0, bool first,
                        bool fuse, bool last, bool restart, const double *rin, const double *win,
                        double *rout, const double *zin1, const double *zin2, double *zoutA,
                        double *zoutB, const double *kx, const double *ky, cudaStream_t st) {
#define TB(F, U, L)                                                                            \
    tb_launch<M, F, U, L>(a, R, Dd, ty, jlim, step0, restart, rin, win, rout, zin1, zin2, zoutA, \
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

// Rows per CTA tile: a CTA costs ~ (ty + 2M) row-iterations (pipeline fill/drain), all
// CTAs are alike, so a launch costs ~ waves x (ty + 2M) with waves = ceil(ctas / slots).
// Pick ty minimising that (slots = SMs x resident CTAs per SM of this kernel).
int tb_auto_rows(int M, int width, int height) {
    static int slots[8] = {};
    M = M < 1 ? 1 : (M > kTbMaxSteps ? kTbMaxSteps : M);
    if (!slots[M]) {
        int dev = 0, nsm = 148, per = 0;
        cudaGetDevice(&dev);
        cudaDeviceGetAttribute(&nsm, cudaDevAttrMultiProcessorCount, dev);
        const size_t smem = tb_smem_bytes();
        cudaError_t e = cudaSuccess;
        switch (M) {
#define OCC(m)                                                                                   \
    case m:                                                                                      \
        cudaFuncSetAttribute(k_cheb_tb<m, false, false, true>,                                   \
                             cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);            \
        e = cudaOccupancyMaxActiveBlocksPerMultiprocessor(&per, k_cheb_tb<m, false, false, true>, \
                                                          kTbT, smem);                       \
        break;
            OCC(1) OCC(2) OCC(3) OCC(4) OCC(5)
#undef OCC
        }
        if (e != cudaSuccess || per < 1) per = 1;
        slots[M] = nsm * per;
    }
    const int ow = tb_out_cols(M);
    const int gx = ((width + ow - 1) / ow + kTbW - 1) / kTbW;
    int best = height, bestc = 0x7fffffff;
    for (int w = 1; w <= 256; ++w) {
        const int tiles = (int)((long long)slots[M] * w / gx);
        if (tiles < 1) continue;
        const int ty = (height + tiles - 1) / tiles;
        const int waves = (int)(((long long)gx * ((height + ty - 1) / ty) + slots[M] - 1) / slots[M]);
        const long long cost = (long long)waves * (ty + 2 * M);
        if (cost < bestc) {
            bestc = (int)cost;
            best = ty;
        }
        if (ty <= 2 * M) break;
    }
    return best < 1 ? 1 : best;
}

int tb_ctas(int M, int width, int height, int ty) {
    const int ow = tb_out_cols(M);
    const int nstrips = (width + ow - 1) / ow;
    return ((nstrips + kTbW - 1) / kTbW) * ((height + ty - 1) / ty);
}

void launch_cheb_tb(const KArgs &a, const Region &R, const Region &Dd, int M, int ty, int jlim,
                    int step0,
                    bool first, bool fuse, bool last, bool restart, const double *rin,
                    const double *win, double *rout, const double *zin1, const double *zin2,
                    double *zoutA, double *zoutB, const double *kx, const double *ky,
                    cudaStream_t st) {
    switch (M) {
        case 1: tb_dispatch<1>(a, R, Dd, ty, jlim, step0, first, fuse, last, restart, rin, win, rout, zin1, zin2, zoutA, zoutB, kx, ky, st); break;
        case 2: tb_dispatch<2>(a, R, Dd, ty, jlim, step0, first, fuse, last, restart, rin, win, rout, zin1, zin2, zoutA, zoutB, kx, ky, st); break;
        case 3: tb_dispatch<3>(a, R, Dd, ty, jlim, step0, first, fuse, last, restart, rin, win, rout, zin1, zin2, zoutA, zoutB, kx, ky, st); break;
        case 4: tb_dispatch<4>(a, R, Dd, ty, jlim, step0, first, fuse, last, restart, rin, win, rout, zin1, zin2, zoutA, zoutB, kx, ky, st); break;
        default: tb_dispatch<5>(a, R, Dd, ty, jlim, step0, first, fuse, last, restart, rin, win, rout, zin1, zin2, zoutA, zoutB, kx, ky, st); break;
    }
}

}  // namespace tea
