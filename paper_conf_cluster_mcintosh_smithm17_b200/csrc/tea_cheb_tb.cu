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
// operands Kx, Ky, r and the diagonal of A are needed up to M rows after they are loaded:
// they wait in a per-thread ring of row slots in tensor memory (TMEM, tcgen05.st/ld), off
// the L1TEX pipe the shuffles use. Input rows arrive by cp.async into per-thread
// shared-memory slots P rows ahead of the march (bytes in flight). Every step loses one
// valid column per side (no edge loads): strips overlap and each produces
// 64 - 2*ceil_even(M) output columns. A CTA tile of ty output rows runs ty + 2M
// row-iterations (pipeline fill/drain). The region R may include extended bounds toward
// neighbour blocks (matrix powers across blocks).
#include "tea_internal.h"

#include <algorithm>
#include <cstdio>
#include <cstdlib>
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
#ifndef TEA_TB_CPA
#define TEA_TB_CPA 5  // rows of cp.async input staging ahead of the march (first pass): 4 -> 6
                      // rows, 184 -> 164 us at 4096^2 (profiles/r02_knobs_ab.txt); 6 -> 5: the
                      // 6 staging slots cycle with the 6-row unroll (compile-time slot indices,
                      // 48 fewer instructions per 6 rows; profiles/r02_cpa_ab.txt)
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

#ifndef TEA_TB_PSTORE
#define TEA_TB_PSTORE 1
#endif
// Store the lane's pair where a / b: predicated stores (one 16-B store, or one 8-B half at a
// region edge) instead of branches -- no reconvergence blocks in the row loop.
__device__ __forceinline__ void st2m(double *p, double2 v, bool a, bool b) {
#if TEA_TB_PSTORE
    const int ab = a && b, oa = a && !b, ob = b && !a;
    asm volatile(
        "{\n\t.reg .pred q0, q1, q2;\n\t"
        "setp.ne.s32 q0, %3, 0;\n\tsetp.ne.s32 q1, %4, 0;\n\tsetp.ne.s32 q2, %5, 0;\n\t"
        "@q0 st.global.v2.f64 [%0], {%1, %2};\n\t"
        "@q1 st.global.f64 [%0], %1;\n\t"
        "@q2 st.global.f64 [%0+8], %2;\n\t}" ::"l"(p),
        "d"(v.x), "d"(v.y), "r"(ab), "r"(oa), "r"(ob)
        : "memory");
#else
    if (a && b) {
        *reinterpret_cast<double2 *>(p) = v;
    } else {
        if (a) p[0] = v.x;
        if (b) p[1] = v.y;
    }
#endif
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

// Tensor-memory (TMEM) delay lines: each thread owns one TMEM lane (warp w of
// the CTA reaches lanes 32(w%4)..32(w%4)+31) and keeps its row slots there -- 16 32-bit
// columns per slot (Kx double2 in 0-3, Ky in 4-7, r in 8-11, diag(A) in 12-15), 8 slots =
// 128 columns per warp quarter. tcgen05.st / tcgen05.ld (.32x32b) run on the tensor-memory
// datapath, not on the L1TEX pipe that the shared-memory rings and the shuffles share
// (tools/tmem_probe.cu: ~165 B/clk/SM of TMEM reads vs ~110 of shared memory at 12 warps).
__device__ __forceinline__ uint32_t d_lo(double v) { return (uint32_t)__double_as_longlong(v); }
__device__ __forceinline__ uint32_t d_hi(double v) {
    return (uint32_t)((unsigned long long)__double_as_longlong(v) >> 32);
}
__device__ __forceinline__ double d_of(uint32_t lo, uint32_t hi) {
    return __longlong_as_double(((long long)hi << 32) | lo);
}
__device__ __forceinline__ void tm_st16(uint32_t a, double2 v0, double2 v1, double2 v2,
                                        double2 v3) {
    asm volatile(
        "tcgen05.st.sync.aligned.32x32b.x16.b32 [%0], {%1, %2, %3, %4, %5, %6, %7, %8, %9, "
        "%10, %11, %12, %13, %14, %15, %16};" ::"r"(a),
        "r"(d_lo(v0.x)), "r"(d_hi(v0.x)), "r"(d_lo(v0.y)), "r"(d_hi(v0.y)), "r"(d_lo(v1.x)),
        "r"(d_hi(v1.x)), "r"(d_lo(v1.y)), "r"(d_hi(v1.y)), "r"(d_lo(v2.x)), "r"(d_hi(v2.x)),
        "r"(d_lo(v2.y)), "r"(d_hi(v2.y)), "r"(d_lo(v3.x)), "r"(d_hi(v3.x)), "r"(d_lo(v3.y)),
        "r"(d_hi(v3.y))
        : "memory");
}
#ifndef TEA_TB_STX2
#define TEA_TB_STX2 1
#endif
// One double (an aligned register pair) into two TMEM columns: storing a row slot double by
// double needs no operand marshalling (the x8 / x4 forms want 8 / 4 consecutive registers:
// 16 register moves per row; with the warp-uniform base: 150.7/151.9 -> 148.8/149.8 us,
// profiles/r02_stx_ab.txt)
__device__ __forceinline__ void tm_st1(uint32_t a, double v) {
    asm volatile("tcgen05.st.sync.aligned.32x32b.x2.b32 [%0], {%1, %2};" ::"r"(a), "r"(d_lo(v)),
                 "r"(d_hi(v))
                 : "memory");
}
__device__ __forceinline__ void tm_st2x(uint32_t a, double2 v) {
    tm_st1(a, v.x);
    tm_st1(a + 2u, v.y);
}
#if !TEA_TB_STX2  // round 1: a row slot as one x8 + one x4 store, the diagonal as x4
__device__ __forceinline__ void tm_st12(uint32_t a, double2 v0, double2 v1, double2 v2) {
    asm volatile(
        "tcgen05.st.sync.aligned.32x32b.x8.b32 [%0], {%1, %2, %3, %4, %5, %6, %7, %8};\n\t"
        "tcgen05.st.sync.aligned.32x32b.x4.b32 [%9], {%10, %11, %12, %13};" ::"r"(a),
        "r"(d_lo(v0.x)), "r"(d_hi(v0.x)), "r"(d_lo(v0.y)), "r"(d_hi(v0.y)), "r"(d_lo(v1.x)),
        "r"(d_hi(v1.x)), "r"(d_lo(v1.y)), "r"(d_hi(v1.y)), "r"(a + 8u), "r"(d_lo(v2.x)),
        "r"(d_hi(v2.x)), "r"(d_lo(v2.y)), "r"(d_hi(v2.y))
        : "memory");
}
__device__ __forceinline__ void tm_st4(uint32_t a, double2 v) {
    asm volatile("tcgen05.st.sync.aligned.32x32b.x4.b32 [%0], {%1, %2, %3, %4};" ::"r"(a),
                 "r"(d_lo(v.x)), "r"(d_hi(v.x)), "r"(d_lo(v.y)), "r"(d_hi(v.y))
                 : "memory");
}
#endif
struct TmRow {
    uint32_t v[16];
};
__device__ __forceinline__ void tm_ld16(uint32_t a, TmRow &o) {
    asm volatile(
        "tcgen05.ld.sync.aligned.32x32b.x16.b32 {%0, %1, %2, %3, %4, %5, %6, %7, %8, %9, %10, "
        "%11, %12, %13, %14, %15}, [%16];"
        : "=r"(o.v[0]), "=r"(o.v[1]), "=r"(o.v[2]), "=r"(o.v[3]), "=r"(o.v[4]), "=r"(o.v[5]),
          "=r"(o.v[6]), "=r"(o.v[7]), "=r"(o.v[8]), "=r"(o.v[9]), "=r"(o.v[10]), "=r"(o.v[11]),
          "=r"(o.v[12]), "=r"(o.v[13]), "=r"(o.v[14]), "=r"(o.v[15])
        : "r"(a)
        : "memory");
}
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
                   "+r"(o.v[10]), "+r"(o.v[11]), "+r"(o.v[12]), "+r"(o.v[13]), "+r"(o.v[14]),
                   "+r"(o.v[15])
                 :
                 : "memory");
}
// no use of o's registers moves above this point (after a tm_wait_ld that covered its load)
__device__ __forceinline__ void tm_pin(TmRow &o) {
    asm volatile(""
                 : "+r"(o.v[0]), "+r"(o.v[1]), "+r"(o.v[2]), "+r"(o.v[3]), "+r"(o.v[4]),
                   "+r"(o.v[5]), "+r"(o.v[6]), "+r"(o.v[7]), "+r"(o.v[8]), "+r"(o.v[9]),
                   "+r"(o.v[10]), "+r"(o.v[11]), "+r"(o.v[12]), "+r"(o.v[13]), "+r"(o.v[14]),
                   "+r"(o.v[15])
                 :
                 : "memory");
}
__device__ __forceinline__ void tm_wait_st() {
    asm volatile("tcgen05.wait::st.sync.aligned;" ::: "memory");
}
__device__ __forceinline__ double2 tm_get(const TmRow &o, int i) {
    return make_double2(d_of(o.v[4 * i], o.v[4 * i + 1]), d_of(o.v[4 * i + 2], o.v[4 * i + 3]));
}

// Deterministic NV-value grid reduction (same scheme as tea_kernels.cu): fixed-order warp,
// CTA and partials sums; returns true in the last CTA, whose threads then hold the totals.
template <int NV>
__device__ bool grid_reduce_n(const double (&v)[NV], double *partials, unsigned *ticket,
                              double (&out)[NV]) {
    __shared__ double sh[NV][kTbW];
    __shared__ bool last;
    const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
    const int nblk = gridDim.x * gridDim.y * gridDim.z;
    const int bid = (blockIdx.z * gridDim.y + blockIdx.y) * gridDim.x + blockIdx.x;
#pragma unroll
    for (int i = 0; i < NV; ++i) {
        const double w = wsum(v[i]);
        if (lane == 0) sh[i][warp] = w;
    }
    __syncthreads();
    if (threadIdx.x == 0) {
#pragma unroll
        for (int i = 0; i < NV; ++i) {
            double s0 = 0.0;
            for (int w = 0; w < kTbW; ++w) s0 += sh[i][w];
            partials[i * nblk + bid] = s0;
        }
        __threadfence();
        last = (atomicAdd(ticket, 1u) == (unsigned)nblk - 1u);
    }
    __syncthreads();
    if (!last) return false;
    __threadfence();
#pragma unroll
    for (int i = 0; i < NV; ++i) {
        double s = 0.0;
        for (int b = threadIdx.x; b < nblk; b += kTbT) s += __ldcg(partials + i * nblk + b);
        s = wsum(s);
        __syncthreads();
        if (lane == 0) sh[i][warp] = s;
        __syncthreads();
        double a = 0.0;
        for (int w = 0; w < kTbW; ++w) a += sh[i][w];
        out[i] = a;
    }
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

#ifndef TEA_TB_CPA_L
#define TEA_TB_CPA_L 5  // later passes: 2 -> 5 rows (ncu: 11% of the last pass's stall samples on
                        // the staged-row LDS waiting for its cp.async; 147.7 -> 146.0 us)
#endif
// cp.async depth of the first pass (carries r, w and the update) and of the later passes,
// measured separately (profiles/r01g_tmem_cpa.txt, r02_knobs_ab.txt). The row loop is unrolled
// by a multiple of the window period 3 (TbGeom::UNR) so the W[t][*] rotation is register
// renaming instead of ~50 moves per row.
constexpr int kTbCpa = TEA_TB_CPA, kTbCpaL = TEA_TB_CPA_L;
static_assert(kTbCpa >= 1 && kTbCpaL >= 1 && kTbCpaL <= kTbCpa, "staging depth");

// dynamic shared memory of a pass: the cp.async row staging; at least 48 KB so at most 4
// CTAs are resident per SM and 4 x kTmCols TMEM columns always fit in the SM's 512
// staged (stream, row) slots of a pass: kTbNS streams (6 with UPD's p and u in a later pass)
// x (staging depth + 1) rows
template <bool FIRST, bool UPD>
__host__ __device__ constexpr int tb_slot_rows() {
    return ((UPD && !FIRST) ? 6 : kTbNS) * ((FIRST ? kTbCpa : kTbCpaL) + 1);
}
template <bool FIRST, bool UPD>
constexpr size_t tb_smem_bytes() {
    return sizeof(double2) * tb_slot_rows<FIRST, UPD>() * kTbT > 48u * 1024u
               ? sizeof(double2) * tb_slot_rows<FIRST, UPD>() * kTbT
               : 48u * 1024u;
}

#ifndef TEA_TB_RING6
#define TEA_TB_RING6 1
#endif
// Strip geometry: a warp's 64 columns output [SH, SH + OW); strips start SH before the
// region at a stride of OW. 1 (default): SH = MR = levels rounded up to even, OW = 64 - 2 MR
// (52 at 5 levels). 0: OW = 64 - 2 levels (54 at 5 levels: fewer redundant columns but 215 vs
// 184 us per first pass at 4096^2 -- strip starts at 8 offsets mod 128 B instead of 4,
// profiles/r02_knobs_ab.txt). 2: SH = 8, OW = 48: every strip starts on a 32-B sector, x1.33
// redundant work (slower). Sharing strip edges between the 4 warps of a CTA through shared
// memory (one CTA barrier per row; 244 of 256 columns) was bitwise equal but 274 vs 179 us:
// the barrier couples the warps' latency chains (profiles/r02_tb_share_ab.txt).
#ifndef TEA_TB_GEOM
#define TEA_TB_GEOM 1
#endif
template <int NL>  // NL = stencil levels of the pass
struct TbGeom {
    static constexpr int MR = (NL + 1) & ~1;  // >= NL, even (double2 loads)
    static constexpr int SH = TEA_TB_GEOM == 2 ? 8 : MR;
    static constexpr int OW = TEA_TB_GEOM == 0 ? kStrip - 2 * NL
                              : (TEA_TB_GEOM == 2 ? 48 : kStrip - 2 * MR);
    static_assert(SH >= NL && SH + OW <= kStrip - NL && OW % 2 == 0, "strip geometry");
    // TMEM ring depth: rows k-NL..k are live (NL + 1 slots). NL <= 5: 6 slots and the row
    // loop unrolled by 6 = 2 x the window period 3, so every slot index of the unrolled body
    // is a compile-time constant (no per-row address arithmetic or R2UR); NL = 6: 8 slots,
    // unrolled by 3 (TEA_TB_RING6 0: always 8 and 3, round 1)
    static constexpr int D = (TEA_TB_RING6 && NL <= 5) ? 6 : 8;
    static constexpr int UNR = D == 6 ? 6 : 3;
};

#ifndef TEA_TB_LDPAIR
#define TEA_TB_LDPAIR 0  // fetch two levels' TMEM slots per round trip in every pass
#endif
#ifndef TEA_TB_MINB_PRE
#define TEA_TB_MINB_PRE 2  // CPPCG1F's 6-level first pass: 2 CTAs/SM, no spills
#endif
#ifndef TEA_TB_FILL
#define TEA_TB_FILL 1  // skip the cone-exterior level-rows of the pipeline fill
#endif
#ifndef TEA_TB_MINB
#define TEA_TB_MINB 3
#endif
constexpr int kTmCols = 128;  // TMEM columns per 4 warps: 8 slots x 16 per warp quarter

// KG (tea_opts.kform): Kx points at g = 1/rho and the row's faces are formed
// as it arrives -- Kx(j) = hrx (g(j-1) + g(j)) with g(j-1) from the west lane (lane 0's
// west face is a margin column, polluted like its west operand), Ky(k) = hry (g(k-1) + g(k))
// with g(k-1) the previous row's -- one staged stream instead of two, same faces bit for bit.
//
// PRE / POST (single-reduction CPPCG in fused form, TEA_CPPCG1F, oracle ORA_CPPCG1F, reading
// R23): the first pass starts with the outer update -- level 0 forms p = z + beta p_old and
// writes p and u += alpha p, level 1 applies A to p and forms r' = r - alpha (A p) (written,
// and replacing r in the row's TMEM slot), then the M Chebyshev steps; the last pass ends with
// one more stencil level q = A z_s whose z_s . q joins r.z and r.r in ONE grid reduction.
// alpha and beta come from the previous reduction (Chronopoulos & Gear). Every level loses a
// column per side and lags a row: NL = M + PRE + POST <= 6 levels.
// UPD (CPPCG with faces from g, last pass): u += alpha p at the input rows, alpha = this
// iteration's (alpha_prev, set by the first pass) and p the direction the SpMV just wrote --
// the update the SpMV otherwise applies lazily, moved to the compute-bound last pass whose HBM
// bandwidth is idle (SpMV 7 -> 5 streams, this pass 5 -> 8).
template <int M, bool FIRST, bool FUSE, bool LAST, bool KG, bool PRE, bool POST, bool UPD = false>
__global__ void __launch_bounds__(kTbT, PRE ? TEA_TB_MINB_PRE : TEA_TB_MINB)
    k_cheb_tb(const double *__restrict__ rin, const double *__restrict__ win,
              double *__restrict__ rout, const double *__restrict__ zin1,
              const double *__restrict__ zin2, double *__restrict__ zoutA,
              double *__restrict__ zoutB, const double *__restrict__ Kx,
              const double *__restrict__ Ky, const double *__restrict__ pin,
              double *__restrict__ pout, double *__restrict__ uio, KArgs a, Region R,
              Region Dd, int ty, int jlim, int step0, int restart) {
    // POST with an odd level count: z.(A z) = sum z^2 + sum_faces K_f (z_i - z_j)^2 from the
    // last step's output itself (each face counted by its west / south cell, as that cell's
    // east / north face; an odd level count leaves the spare valid column east of the output
    // columns) -- no extra stencil level. Even: a stencil level q = A z_s after the last step.
    constexpr bool POSTF = POST && ((M + (PRE ? 1 : 0)) % 2 == 1);
    constexpr int NL = M + (PRE ? 1 : 0) + ((POST && !POSTF) ? 1 : 0);  // stencil levels
    constexpr int T0 = PRE ? 2 : 1;                         // level of the first Chebyshev step
    // paired TMEM slot fetches: CPPCG1F's last pass 168 -> 160 us at 4096^2, the CPPCG passes
    // unchanged or slower (profiles/r02_ldpair_ab.txt)
    constexpr bool kPair = TEA_TB_LDPAIR || POST;
    using G = TbGeom<NL>;
    constexpr int D = G::D;
    static_assert(NL <= 6, "the TMEM ring holds NL+2 rows");
    static_assert(!PRE || (FIRST && !FUSE && KG), "PRE: first pass, g faces, no FUSE update");
    static_assert(!POST || LAST, "POST: last pass");
    static_assert(!UPD || (LAST && KG && !PRE && !POST), "UPD: last pass, g faces");
    // staged streams per row: X, W / z_{i-2}, r, Kx (g), Ky -- UPD adds p and u
    constexpr int NS = (UPD && !FIRST) ? 6 : kTbNS;
    constexpr int PSL = FIRST ? 2 : 4, USL = FIRST ? 4 : 5;  // UPD's p / u slots
    static_assert(kTbW <= 4 || kTbW % 4 == 0, "warp quarters");
    extern __shared__ double2 tb_smem[];
    const double(*coef)[kMaxS] = c_tb_coef[a.coef_slot];

    Scalars *S = a.S;
    if (S->done) {
        if (LAST && blockIdx.x == 0 && blockIdx.y == 0 && blockIdx.z == 0 && threadIdx.x == 0 && a.set_cond &&
            a.cond)
            cudaGraphSetConditional(a.cond, 0u);
        return;
    }
    double alpha = 0.0, beta = 0.0;
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
    if (PRE) {
        const Cg1Coef cf = cg1_coef(S);  // stop test on r.r, limits, alpha, beta
        if (cf.state != 0) {
            if (grid_arrive2(&S->ticket) && threadIdx.x == 0) {
                cg1_finish(S, cf);
                if (LAST && a.set_cond && a.cond) cudaGraphSetConditional(a.cond, 0u);
            }
            return;
        }
        alpha = cf.alpha;
        beta = cf.beta;
    }
    // UPD: this iteration's alpha (FUSE computed it here; otherwise the first pass recorded it)
    const double ualpha = UPD ? (FUSE ? alpha : S->alpha_prev) : 0.0;
    trace_begin(a);
    const double2 z0 = make_double2(0.0, 0.0);
    // One warp allocates the CTA's TMEM columns; warp w then owns lanes 32(w%4).. and a
    // 128-column group per 4 warps: per thread a private ring of D row slots (tm_st16).
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
    // (broadcast from lane 0: a value the compiler knows is warp-uniform can stay in a
    // uniform register, so the TMEM operations need no per-use register->uniform moves)
    const uint32_t tm = __shfl_sync(0xffffffffu,
                                    tm_base_sh + ((uint32_t)(((threadIdx.x >> 5) & 3) * 32) << 16) +
                                        (uint32_t)(((threadIdx.x >> 5) >> 2) * kTmCols),
                                    0);
    for (int d = 0; d < D; ++d) tm_st16(tm + 16u * d, z0, z0, z0, z0);  // zero ring

    const int lane = threadIdx.x & 31, warp = threadIdx.x >> 5;
    const int strip = blockIdx.x * kTbW + warp;
    // strips tile the output region R (which may reach into the halo on sides with a
    // neighbour block: extended bounds); the first starts SH before it
    const int jA = (R.j0 & (TEA_TB_GEOM == 2 ? ~3 : ~1)) - G::SH + strip * G::OW + 2 * lane;
    const int kt0 = R.k0 + blockIdx.y * ty;
    const int kt1 = min(kt0 + ty, R.k1);
    const int pitch = a.pitch;
    const bool ld_ok = jA + 1 < jlim;  // inside the allocation
    // output columns: this strip's [SH, SH + OW) intersected with the region
    const int cA = 2 * lane, cB = 2 * lane + 1;
    const bool oA = cA >= G::SH && cA < G::SH + G::OW && jA >= R.j0 && jA < R.j1;
    const bool oB = cB >= G::SH && cB < G::SH + G::OW && jA + 1 >= R.j0 && jA + 1 < R.j1;
    // dot products over owned cells only (D), whatever the extension of R
    const bool dA = oA && jA >= Dd.j0 && jA < Dd.j1, dB = oB && jA + 1 >= Dd.j0 && jA + 1 < Dd.j1;

    // stencil windows: W[t] holds level t's rows (oldest, middle, newest); W[0] = input
    // operand (r, or p = z + beta p_old with PRE)
    double2 W[NL][3];
#pragma unroll
    for (int t = 0; t < NL; ++t) W[t][0] = W[t][1] = W[t][2] = z0;
    double dot0 = 0.0, dot1 = 0.0, dot2 = 0.0;  // r.z, r.r (LAST); z.(A z) (POST)

    // (POSTF: one more row-iteration, for the north face of the tile's last row)
    const int kbeg = kt0 - NL, kend = kt1 + NL + (POSTF ? 1 : 0);
    double2 zsp = z0;  // POSTF: the last step's previous row
    // offset of (jA, k), running (no k*pitch); 32-bit: the host runs the passes only on
    // fields of < 2^31 elements (tb_fits), so every address is one IMAD.WIDE
    int orow = kbeg * pitch + jA;
    // Input rows are staged P rows ahead by cp.async into per-thread shared-memory slots
    // (each thread copies and later reads back only its own 16 B per stream, so no
    // barriers; slots the thread never fills stay zero): P rows of bytes in flight per
    // warp. With one register-prefetched row the pass stalled on the load of the next row
    // (ncu: 41% of stall samples on its first use; profiles/r01g_tmem_cpa.txt).
    constexpr int P = FIRST ? kTbCpa : kTbCpaL, NSL = P + 1;
    static_assert(NS * NSL <= tb_slot_rows<FIRST, UPD>(), "staging fits the dynamic shared memory");
    double2(*cpa)[NS][kTbT] = reinterpret_cast<double2(*)[NS][kTbT]>(tb_smem);
    for (int sl = 0; sl < NSL; ++sl)
#pragma unroll
        for (int q = 0; q < NS; ++q) cpa[sl][q][threadIdx.x] = z0;
    auto issue = [&](int o, int sl) {
        if (ld_ok) {
            if (PRE) {  // z_s, p_old, r, g, u
                cp16(&cpa[sl][0][threadIdx.x], zin1 + o);
                cp16(&cpa[sl][1][threadIdx.x], pin + o);
                cp16(&cpa[sl][2][threadIdx.x], rin + o);
                cp16(&cpa[sl][4][threadIdx.x], uio + o);
            } else if (FIRST) {
                cp16(&cpa[sl][0][threadIdx.x], rin + o);
                if (FUSE) cp16(&cpa[sl][1][threadIdx.x], win + o);
            } else {
                cp16(&cpa[sl][0][threadIdx.x], zin1 + o);
                cp16(&cpa[sl][1][threadIdx.x], zin2 + o);
                cp16(&cpa[sl][2][threadIdx.x], rin + o);
            }
            cp16(&cpa[sl][3][threadIdx.x], Kx + o);
            if (!KG) cp16(&cpa[sl][4][threadIdx.x], Ky + o);
            if (UPD) {
                cp16(&cpa[sl][PSL][threadIdx.x], pin + o);
                cp16(&cpa[sl][USL][threadIdx.x], uio + o);
            }
        }
        cp_commit();  // one group per row, empty or not, so wait_group counts rows
    };
#pragma unroll
    for (int i = 0; i < P; ++i) {
        if (kt0 < kt1 && kbeg + i < kend)
            issue(orow + i * pitch, i);
        else
            cp_commit();
    }
    int cs = 0;    // staging slot of row k
    int head = 0;  // TMEM ring slot of row k
    double2 z2prev = z0;  // z_{i-2} input of the previous row (a one-row register delay)
    double2 gprev = z0;   // KG: g of the previous input row (row kbeg-1's only feeds the
                          // pipeline-fill rows every pass discards)
    const double hrx = a.hrx, hry = a.hry;
    constexpr int UNR = G::UNR;
    // One row-iteration: input row k, level t on row k - t. fi = k - kbeg during the pipeline
    // fill (TEA_TB_FILL), else large: level t's rows below kt0 - (NL - t) are outside the
    // tile's cone (no later level reads them) and are first needed at fi = 2t, so the first
    // 2 NL row-iterations skip their arithmetic -- NL (NL + 1) of the (ty + 2 NL) NL level-rows
    // a tile computed (30 of 985 at ty = 187; 30 of 240 on the ~38-row tiles of 2048 x 1024
    // blocks).
    auto row = [&](const int k, const int fi) {
        cp_wait<P - 1>();  // row k's group (the oldest outstanding) has landed
        double2 X = cpa[cs][0][threadIdx.x];
        double2 KX, KY;
        if (KG) {
            const double2 g = cpa[cs][3][threadIdx.x];
            const double gW = __shfl_up_sync(0xffffffffu, g.y, 1);
            // __dmul_rn: never contracted into an FMA with the faces' uses (the diagonal
            // sum below), so every face equals the stored one bit for bit
            KX.x = __dmul_rn(hrx, gW + g.x);
            KX.y = __dmul_rn(hrx, g.x + g.y);
            KY.x = __dmul_rn(hry, gprev.x + g.x);
            KY.y = __dmul_rn(hry, gprev.y + g.y);
            gprev = g;
        } else {
            KX = cpa[cs][3][threadIdx.x];
            KY = cpa[cs][4][threadIdx.x];
        }
        double2 Wv = z0, Z2 = z0, RR = z0, PO = z0, UU = z0;
        if (UPD) {
            PO = cpa[cs][PSL][threadIdx.x];
            UU = cpa[cs][USL][threadIdx.x];
        }
        if (PRE) {
            PO = cpa[cs][1][threadIdx.x];
            RR = cpa[cs][2][threadIdx.x];
            UU = cpa[cs][4][threadIdx.x];
        } else if (FIRST) {
            if (FUSE) Wv = cpa[cs][1][threadIdx.x];
        } else {
            Z2 = cpa[cs][1][threadIdx.x];
            RR = cpa[cs][2][threadIdx.x];
        }
        {
            // row k+P goes into the slot row k-1 used (read a full iteration ago)
            const int ns = cs == 0 ? P : cs - 1;
            if (kt0 < kt1 && k + P < kend)
                issue(orow + P * pitch, ns);
            else
                cp_commit();
            cs = cs == P ? 0 : cs + 1;
        }
        double2 rk;
        if (PRE) {
            // level 0: p = z + beta p_old; u += alpha p (pointwise, this row)
            X = make_double2(X.x + beta * PO.x, X.y + beta * PO.y);
            if (k >= kt0 && k < kt1) {
                st2m(pout + orow, X, oA, oB);
                st2m(uio + orow, make_double2(UU.x + alpha * X.x, UU.y + alpha * X.y), oA, oB);
            }
            rk = RR;  // r_old: the w level replaces it by r - alpha A p
        } else if (FIRST) {
            if (FUSE) X = make_double2(X.x - alpha * Wv.x, X.y - alpha * Wv.y);
            rk = X;
            if (FUSE && k >= kt0 && k < kt1) st2m(rout + orow, X, oA, oB);
        } else {
            rk = RR;
        }
        if (UPD && k >= kt0 && k < kt1 && k >= Dd.k0 && k < Dd.k1)  // owned cells only
            st2m(uio + orow, make_double2(UU.x + ualpha * PO.x, UU.y + ualpha * PO.y), dA, dB);
        // level t works on row q = k - t and needs that row's Kx, Ky, r (and Ky of row
        // q+1): they wait in this thread's TMEM ring. The previous row's stores must land
        // before this row's loads read them back.
        tm_wait_st();
#if TEA_TB_STX2
        tm_st2x(tm + 16u * head, KX);
        tm_st2x(tm + 16u * head + 4u, KY);
        tm_st2x(tm + 16u * head + 8u, rk);
#else
        tm_st12(tm + 16u * head, KX, KY, rk);
#endif
        TmRow tmA;
        tm_ld12(tm + 16u * ((head + D - 1) % D), tmA);  // row k-1: level 1's operands
        tm_wait_ld(tmA);
        double2 s_kx = tm_get(tmA, 0), s_ky = tm_get(tmA, 1), s_r = tm_get(tmA, 2), kyn = KY;
        // Row k-1 is completed now that its top faces (row k's Ky) are known: the diagonal
        // of A (Listing 1: 1 + the sum of the cell's four face coefficients) is formed once
        // per row here, not once per level, and joins the row's slot (columns 12-15).
        // Kx(jA+2) (the face east of cell B) is the east lane's Kx(jA): one shuffle per row
        // (lane 31's value only feeds the margin).
        const double kxE = __shfl_down_sync(0xffffffffu, s_kx.x, 1);
        double2 s_d;
        s_d.x = 1.0 + (s_kx.x + s_kx.y) + (s_ky.x + KY.x);
        s_d.y = 1.0 + (s_kx.y + kxE) + (s_ky.y + KY.y);
#if TEA_TB_STX2
        tm_st2x(tm + 16u * ((head + D - 1) % D) + 12u, s_d);
#else
        tm_st4(tm + 16u * ((head + D - 1) % D) + 12u, s_d);
#endif
        const double2 z2row = z2prev;  // z_{i-2} of row k-1
        if (!FIRST) z2prev = Z2;
        W[0][0] = W[0][1];
        W[0][1] = W[0][2];
        W[0][2] = X;
        TmRow tmC;  // kPair: the even level's slot, fetched with the odd level's
        (void)tmC;
#pragma unroll
        for (int t = 1; t <= NL; ++t) {
            const int q = k - t;
            // issue the next level's slot (row q-1) before computing this one
            TmRow tmB;
            if constexpr (kPair) {
            // odd levels fetch the next TWO levels' slots in one round trip (3 per row
            // instead of 5 at NL = 5); the second waits in tmC for the even level
            if (t < NL && t % 2 == 1) {
                tm_ld16(tm + 16u * ((head + 2 * D - t - 1) % D), tmB);
                if (t + 1 < NL) tm_ld16(tm + 16u * ((head + 2 * D - t - 2) % D), tmC);
            }
            } else {
            if (t < NL) tm_ld16(tm + 16u * ((head + 2 * D - t - 1) % D), tmB);
            }
            const double2 kx = s_kx, kyc = s_ky, rq = s_r;
            const double2 xm = W[t - 1][0], xc = W[t - 1][1], xp = W[t - 1][2];
            const double2 dg = s_d;
            // lane 0's left and lane 31's right neighbours are outside the strip: the
            // shuffles return the lane's own (finite) value, which only pollutes the
            // overlap columns every level already discards -- no selects needed.
            // West neighbour of cell A from the west lane; the east term of cell B,
            // Kx(jA+2) X(jA+2), is the east lane's own Kx(jA) X(jA) -- one product shuffled.
            // Dependency order: xp (the "up" row) is the row level t-1 produced in THIS
            // row-iteration; everything else is older. Form the rest first, fold xp in last.
            double2 zn = z0;
            if (fi >= 2 * t) {  // (fill: a compile-time constant per unrolled iteration)
            const double left = __shfl_up_sync(0xffffffffu, xc.y, 1);
            const double east = __shfl_down_sync(0xffffffffu, kx.x * xc.x, 1);
            double2 nb;  // sum_f K_f X_f - d X without the up face (Listing 1)
            nb.x = fma(-dg.x, xc.x, fma(kx.x, left, fma(kx.y, xc.y, kyc.x * xm.x)));
            nb.y = fma(-dg.y, xc.y, fma(kx.y, xc.x, fma(kyc.y, xm.y, east)));
            const bool rowout = q >= kt0 && q < kt1;
            if (PRE && t == 1) {
                // w = A p; r' = r - alpha w = r + alpha (sum_f K_f p_f - d p)
                zn.x = fma(alpha, fma(kyn.x, xp.x, nb.x), rq.x);
                zn.y = fma(alpha, fma(kyn.y, xp.y, nb.y), rq.y);
                tm_st2x(tm + 16u * ((head + D - 1) % D) + 8u, zn);  // row q's r is now r'
                if (rowout) st2m(rout + (orow - pitch), zn, oA, oB);
            } else if (POST && !POSTF && t == NL) {
                // q = A z_s at row q (xc = z_s): z_s . q, and r . z_s, r . r of the same row
                // (rq), over the owned cells
                if (rowout && q >= Dd.k0 && q < Dd.k1) {
                    const double mx = fma(kyn.x, xp.x, nb.x), my = fma(kyn.y, xp.y, nb.y);
                    if (dA) {
                        dot2 -= xc.x * mx;
                        dot0 += rq.x * xc.x;
                        dot1 += rq.x * rq.x;
                    }
                    if (dB) {
                        dot2 -= xc.y * my;
                        dot0 += rq.y * xc.y;
                        dot1 += rq.y * rq.y;
                    }
                }
            } else {
                // Chebyshev step j of this pass (DESIGN.md §4.3 recurrence):
                // z = cx X + cz z2 + cr r - ca (d X - sum_f K_f X_f)         (Listing 1)
                // The per-step coefficients only ever multiply vector registers (uniform
                // operands, nothing hoisted into vector registers).
                const int j = t - (PRE ? 1 : 0);
                const int ci = step0 - 2 + j;
                const double cx = coef[0][ci], cz = coef[1][ci], cr = coef[2][ci], ca = coef[3][ci];
                double2 z2 = z0;
                if (t == 1)
                    z2 = FIRST ? z0 : z2row;
                else if (!(FIRST && t == T0))
                    z2 = W[t >= 2 ? t - 2 : 0][0];
                double2 base;
                base.x = cx * xc.x;
                base.y = cx * xc.y;
                if (!(FIRST && t == T0)) {
                    base.x = fma(cz, z2.x, base.x);
                    base.y = fma(cz, z2.y, base.y);
                }
                base.x = fma(cr, rq.x, base.x);
                base.y = fma(cr, rq.y, base.y);
                // (folding ca into kyn to leave one dependent DFMA after xp costs a DMUL per
                // cell and measured slower: profiles/r01g_tmem_cpa.txt)
                zn.x = fma(ca, fma(kyn.x, xp.x, nb.x), base.x);
                zn.y = fma(ca, fma(kyn.y, xp.y, nb.y), base.y);
                if (j == M - 1 && !LAST && rowout) st2m(zoutA + (orow - t * pitch), zn, oA, oB);
                if (POSTF && j == M) {
                    // z.(A z) by faces, each face from its west / south cell: this row's
                    // z^2 and east faces, and the north face of the row below (kyc = Ky(q))
                    const double zE = __shfl_down_sync(0xffffffffu, zn.x, 1);
                    const double kE = __shfl_down_sync(0xffffffffu, kx.x, 1);
                    if (rowout && q >= Dd.k0 && q < Dd.k1) {
                        const double ea = zn.x - zn.y, eb = zn.y - zE;
                        if (dA) dot2 += fma(kx.y * ea, ea, zn.x * zn.x);
                        if (dB) dot2 += fma(kE * eb, eb, zn.y * zn.y);
                    }
                    const int qs = q - 1;
                    if (qs >= kt0 && qs < kt1 && qs >= Dd.k0 && qs < Dd.k1) {
                        const double na = zsp.x - zn.x, nb2 = zsp.y - zn.y;
                        if (dA) dot2 += kyc.x * na * na;
                        if (dB) dot2 += kyc.y * nb2 * nb2;
                    }
                    zsp = zn;
                }
                if (j == M && rowout) {
                    st2m(zoutB + (orow - t * pitch), zn, oA, oB);
                    if (LAST && !(POST && !POSTF) && q >= Dd.k0 && q < Dd.k1) {
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
            }  // fi >= 2t
            if (t < NL) {
                const int tt = t < NL ? t : NL - 1;
                W[tt][0] = W[tt][1];
                W[tt][1] = W[tt][2];
                W[tt][2] = zn;
                kyn = kyc;  // Ky of row q = the top faces of row q-1
                if constexpr (kPair) {
                if (t % 2 == 1) {
                    tm_wait_ld(tmB);
                    if (t + 1 < NL) tm_pin(tmC);
                    s_kx = tm_get(tmB, 0);
                    s_ky = tm_get(tmB, 1);
                    s_r = tm_get(tmB, 2);
                    s_d = tm_get(tmB, 3);
                } else {
                    s_kx = tm_get(tmC, 0);
                    s_ky = tm_get(tmC, 1);
                    s_r = tm_get(tmC, 2);
                    s_d = tm_get(tmC, 3);
                }
                } else {
                tm_wait_ld(tmB);
                s_kx = tm_get(tmB, 0);
                s_ky = tm_get(tmB, 1);
                s_r = tm_get(tmB, 2);
                s_d = tm_get(tmB, 3);
                }
            }
        }
    };
    int k = kbeg;
#if TEA_TB_FILL
    // the fill, fully unrolled (every fi, slot and window index a constant); a multiple of the
    // main loop's unroll, so the main loop starts on ring and staging slot 0 as before. A tile
    // shorter than the fill runs its extra row-iterations on rows past kend: nothing of them
    // is stored or summed (every store and dot is limited to rows < kt1).
    constexpr int kFill = (2 * NL + UNR - 1) / UNR * UNR;
#pragma unroll
    for (int i = 0; i < kFill; ++i, ++k, orow += pitch, head = head + 1 == D ? 0 : head + 1)
        row(k, i);
#endif
#pragma unroll(UNR)
    for (; k < kend; ++k, orow += pitch, head = head + 1 == D ? 0 : head + 1) row(k, 1 << 20);
    asm volatile("tcgen05.fence::before_thread_sync;" ::: "memory");
    __syncthreads();
    if ((threadIdx.x >> 5) == 0)
        asm volatile("tcgen05.dealloc.cta_group::1.sync.aligned.b32 %0, %1;" ::"r"(tm_base_sh),
                     "n"(kTmAlloc)
                     : "memory");
    if (LAST) {
        bool last;
        double tot[3] = {0.0, 0.0, 0.0};
        if (POST) {
            const double v[3] = {dot0, dot1, dot2};
            last = grid_reduce_n<3>(v, a.partials, &S->ticket, tot);
        } else {
            const double v[2] = {dot0, dot1};
            double t2[2];
            last = grid_reduce_n<2>(v, a.partials, &S->ticket, t2);
            tot[0] = t2[0];
            tot[1] = t2[1];
        }
        if (last && threadIdx.x == 0) {
            if (PRE) {  // this iteration's alpha, beta (before the new gamma replaces it)
                S->gam_old = S->red_gam;
                S->alpha_prev = alpha;
                S->beta_last = beta;
                S->fresh = 0;
            }
            S->red_gam = tot[0];
            S->red_rr = tot[1];
            if (POST) S->red_pw = tot[2];
            if (FUSE) S->alpha_prev = alpha;
            if (UPD) S->alpha_prev = 0.0;  // u is current: nothing pending for the SpMV
            if (!restart) {
                S->it += 1;
                S->outer += 1;
            }
        }
    } else if (PRE) {
        // every CTA has read the scalars (it arrived): the last one records this iteration's
        if (grid_arrive2(&S->ticket) && threadIdx.x == 0) {
            S->gam_old = S->red_gam;
            S->alpha_prev = alpha;
            S->beta_last = beta;
            S->fresh = 0;
        }
    } else if (FUSE) {
        if (blockIdx.x == 0 && blockIdx.y == 0 && blockIdx.z == 0 && threadIdx.x == 0) S->alpha_prev = alpha;
    }
    trace_end(a);
}

// output columns of one CTA of a pass with NL stencil levels
int tb_out_cols(int NL) {
    const int mr = (NL + 1) & ~1;
    const int ow = TEA_TB_GEOM == 0 ? kStrip - 2 * NL : (TEA_TB_GEOM == 2 ? 48 : kStrip - 2 * mr);
    return kTbW * ow;
}

template <int M, bool FIRST, bool FUSE, bool LAST, bool KG, bool PRE, bool POST, bool UPD = false>
static void tb_launch(const KArgs &a, const Region &R, const Region &Dd, int ty, int jlim,
                      int step0, bool restart, const TbArgs &f, cudaStream_t st) {
    constexpr int NL = M + (PRE ? 1 : 0) + ((POST && (M + (PRE ? 1 : 0)) % 2 == 0) ? 1 : 0);
    const int width = R.j1 - (R.j0 & (TEA_TB_GEOM == 2 ? ~3 : ~1));
    const int ow = tb_out_cols(NL);
    dim3 grid((width + ow - 1) / ow, (R.k1 - R.k0 + ty - 1) / ty);
    constexpr size_t smem = tb_smem_bytes<FIRST, UPD>();
    // > 48 KB of dynamic shared memory needs the attribute, set once per device
    static std::atomic<unsigned long long> attr{0ull};  // per instantiation: device bit mask
    const unsigned long long bit = 1ull << tea_device();
    if (!(attr.load() & bit)) {
        cudaFuncSetAttribute(k_cheb_tb<M, FIRST, FUSE, LAST, KG, PRE, POST, UPD>,
                             cudaFuncAttributeMaxDynamicSharedMemorySize, (int)smem);
        cudaFuncSetAttribute(k_cheb_tb<M, FIRST, FUSE, LAST, KG, PRE, POST, UPD>,
                             cudaFuncAttributePreferredSharedMemoryCarveout, 100);
        attr.fetch_or(bit);
    }
    k_cheb_tb<M, FIRST, FUSE, LAST, KG, PRE, POST, UPD><<<grid, kTbT, smem, st>>>(
        f.rin, f.win, f.rout, f.zin1, f.zin2, f.zoutA, f.zoutB, KG ? a.g : f.kx, f.ky, f.pin,
        f.pout, f.uio, a, R, Dd, ty, jlim, step0, restart ? 1 : 0);
}

template <int M>
static void tb_dispatch(const KArgs &a, const Region &R, const Region &Dd, int ty, int jlim,
                        int step0, bool first, bool fuse, bool last, bool restart, bool pre,
                        bool post, bool upd, const TbArgs &f, cudaStream_t st) {
    if (upd && last && a.g && !pre && !post) {  // CPPCG: u += alpha p in the last pass
        if (!first)
            tb_launch<M, false, false, true, true, false, false, true>(a, R, Dd, ty, jlim, step0, restart, f, st);
        else if (fuse)
            tb_launch<M, true, true, true, true, false, false, true>(a, R, Dd, ty, jlim, step0, restart, f, st);
        else
            tb_launch<M, true, false, true, true, false, false, true>(a, R, Dd, ty, jlim, step0, restart, f, st);
        return;
    }
#define TB(F, U, L)                                                                       \
    do {                                                                                  \
        if (a.g)                                                                          \
            tb_launch<M, F, U, L, true, false, false>(a, R, Dd, ty, jlim, step0, restart, f, st); \
        else                                                                              \
            tb_launch<M, F, U, L, false, false, false>(a, R, Dd, ty, jlim, step0, restart, f, st); \
    } while (0)
    if (pre || post) {
        // single-reduction CPPCG in fused form (faces from g only; at most 6 levels)
        if constexpr (M <= 4) {
            if (pre && post) {
                tb_launch<M, true, false, true, true, true, true>(a, R, Dd, ty, jlim, step0, restart, f, st);
                return;
            }
        }
        if constexpr (M <= 5) {
            if (pre && !post && first && !last) {
                tb_launch<M, true, false, false, true, true, false>(a, R, Dd, ty, jlim, step0, restart, f, st);
                return;
            }
            if (post && !pre && last) {
                if (first)
                    tb_launch<M, true, false, true, true, false, true>(a, R, Dd, ty, jlim, step0, restart, f, st);
                else
                    tb_launch<M, false, false, true, true, false, true>(a, R, Dd, ty, jlim, step0, restart, f, st);
                return;
            }
        }
        return;  // invalid combination (the host plans only the ones above)
    }
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

// Rows per CTA tile: a CTA costs ~ (ty + 2 NL) row-iterations (pipeline fill/drain); an SM
// holding n CTAs of a wave runs them at a rate that saturates at ~2 CTAs (tb_row_time): a
// launch costs the sum over its waves of (ty + 2 NL) x tb_row_time(CTAs on the busiest SM).
// This keeps 4096^2's full wave of 187-row tiles, ~36-row tiles at 2 CTAs per SM on 2048 x
// 1024 blocks (24-row tiles at 3 per SM: 26.8/29.9 vs 25.5/30.2 us) and 18-row tiles at
// 1024^2 (14.5/17.8 vs 17.5/20.1 us with 25). The occupancy is computed from the
// kernel's registers and shared memory: cudaOccupancyMaxActiveBlocksPerMultiprocessor reports
// 1 CTA per SM for these kernels while 3 are resident (ncu), which made every earlier plan a
// "3-wave" one.
// Relative row-iteration time of a fused-pass CTA when its SM holds n of them (round 2
// sweeps, profiles/r02_tbrows_model.txt): ~0.5 us with 2 CTAs per SM and ~0.7 us with 3 at
// 1965 MHz (1024^2, 2048^2, 2 x 4 blocks of 4096^2): an SM's throughput barely grows past 8
// warps, so a plan with one CTA less on the busiest SM can win with taller
// tiles. (Round 2a modelled n / (n + 1/2) on the average count: 25-row tiles at 1024^2, 8%
// slower than 18.)
static double tb_row_time(int n) { return n <= 1 ? 0.7 : (n == 2 ? 1.0 : 0.47 * n); }

int tb_auto_rows(int NL, int width, int height) {
    static std::atomic<int> slot_cache[kMaxDev][8];
    static std::atomic<int> sm_cache[kMaxDev];
    NL = NL < 1 ? 1 : (NL > 6 ? 6 : NL);
    const int dev = tea_device();
    int slots = slot_cache[dev][NL].load();
    if (!slots) {
        int nsm = 148, per = 0, smem_sm = 0;
        cudaDeviceGetAttribute(&nsm, cudaDevAttrMultiProcessorCount, dev);
        cudaDeviceGetAttribute(&smem_sm, cudaDevAttrMaxSharedMemoryPerMultiprocessor, dev);
        // (the larger of the first and later passes' staging: one plan serves both)
        const size_t smem = std::max(tb_smem_bytes<true, false>(), tb_smem_bytes<false, false>());
        cudaError_t e = cudaSuccess;
        // resident CTAs per SM from the kernel's registers and shared memory (the occupancy
        // API reports 1 for these kernels, round 2 probe -- ncu shows ~3 resident), capped
        // by the TMEM columns (512 per SM, 128 per CTA)
        cudaFuncAttributes fa{};
        switch (NL) {
#define OCC(m, POST)                                                                             \
    case (m + (POST ? 1 : 0)):                                                                   \
        e = cudaFuncGetAttributes(&fa, k_cheb_tb<m, false, false, true, true, false, POST>);     \
        break;
            OCC(1, false) OCC(2, false) OCC(3, false) OCC(4, false) OCC(5, false)
            case 6:  // CPPCG1F's first pass (PRE + 5 steps), compiled for 2 CTAs/SM
                e = cudaFuncGetAttributes(&fa, k_cheb_tb<5, true, false, false, true, true, false>);
                break;
#undef OCC
        }
        if (e == cudaSuccess && fa.numRegs > 0) {
            const int regs_cta = ((fa.numRegs * 32 + 255) / 256 * 256) * (kTbT / 32);
            const int by_regs = 65536 / regs_cta;
            const int by_smem = smem_sm / (int)(smem + fa.sharedSizeBytes + 1024);
            per = std::min(std::min(by_regs, by_smem), 512 / kTmCols);
        }
        if (e != cudaSuccess || per < 1) per = 1;
        slots = nsm * per;
        slot_cache[dev][NL].store(slots);
        if (std::getenv("TEA_DEBUG_PLAN"))
            fprintf(stderr, "tea: fused pass NL=%d: %d CTAs/SM (%s), %d SMs\n", NL, per,
                    cudaGetErrorString(e), nsm);
        sm_cache[dev].store(nsm);
    }
    return tb_plan_rows(NL, width, height, slots / std::max(1, sm_cache[dev].load()),
                        std::max(1, sm_cache[dev].load()));
}

// The cost model alone (host-only; tea_tb_plan exports it for tests): rows per tile for a
// pass of NL levels over width x height cells with `per` CTAs resident per SM on `nsm` SMs.
int tb_plan_rows(int NL, int width, int height, int per, int nsm) {
    NL = NL < 1 ? 1 : (NL > 6 ? 6 : NL);
    per = std::max(1, per);
    nsm = std::max(1, nsm);
    const int slots = per * nsm;
    const int ow = tb_out_cols(NL);
    const int gx = (width + ow - 1) / ow;
    int best = height;
    double bestc = 1e300;
    // tiles of at most 512 rows: taller ones leave the scheduler no CTAs to balance the SMs
    // with (16384^2: one wave of 3277-row tiles 2541 us vs waves of ~1261-row tiles 2382 us
    // per first pass, profiles/r02_blocks_ab.txt)
    for (int ty = std::max(1, height / 4096); ty <= std::min(height, 512); ++ty) {
        const long long ctas = (long long)gx * ((height + ty - 1) / ty);
        const long long full = ctas / slots, rest = ctas - full * slots;
        // a wave lasts as long as its busiest SM: (ty + 2 NL) row-iterations at the rate of
        // the CTA count that SM holds (ceil, not the average)
        const double cost =
            (ty + 2 * NL) * ((double)full * tb_row_time(slots / nsm) +
                             (rest ? tb_row_time((int)((rest + nsm - 1) / nsm)) : 0.0));
        if (cost < bestc - 1e-9) {
            bestc = cost;
            best = ty;
        }
    }
    return best < 1 ? 1 : best;
}

int tb_ctas(int NL, int width, int height, int ty) {
    const int ow = tb_out_cols(NL);
    return ((width + ow - 1) / ow) * ((height + ty - 1) / ty);
}

void launch_cheb_tb(const KArgs &a, const Region &R, const Region &Dd, int M, int ty, int jlim,
                    int step0, bool first, bool fuse, bool last, bool restart, bool pre,
                    bool post, bool upd, const TbArgs &f, cudaStream_t st) {
    switch (M) {
        case 1: tb_dispatch<1>(a, R, Dd, ty, jlim, step0, first, fuse, last, restart, pre, post, upd, f, st); break;
        case 2: tb_dispatch<2>(a, R, Dd, ty, jlim, step0, first, fuse, last, restart, pre, post, upd, f, st); break;
        case 3: tb_dispatch<3>(a, R, Dd, ty, jlim, step0, first, fuse, last, restart, pre, post, upd, f, st); break;
        case 4: tb_dispatch<4>(a, R, Dd, ty, jlim, step0, first, fuse, last, restart, pre, post, upd, f, st); break;
        default: tb_dispatch<5>(a, R, Dd, ty, jlim, step0, first, fuse, last, restart, pre, post, upd, f, st); break;
    }
}

}  // namespace tea
