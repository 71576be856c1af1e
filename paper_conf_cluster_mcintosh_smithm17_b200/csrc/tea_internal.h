// tea_internal.h -- internal types shared by the CUDA kernels and the host driver
// of the B200 TeaLeaf CG / CPPCG library (not part of the C ABI).
#pragma once

#include <cuda_runtime.h>
#include <cstddef>
#include <cstdint>
#include <atomic>

namespace tea {

// Per-device host caches (occupancy-derived tile plans, function attributes): a process may
// drive contexts on several GPUs, so every cache is indexed by the current device and
// filled idempotently (atomics: concurrent first uses compute the same value).
constexpr int kMaxDev = 64;
inline int tea_device() {
    int d = 0;
    cudaGetDevice(&d);
    return d < 0 ? 0 : (d >= kMaxDev ? kMaxDev - 1 : d);
}

constexpr int kMaxPre = 512;   // presteps cap (Lanczos history length)
constexpr int kMaxS = 64;      // Chebyshev inner steps cap
constexpr int kWarps = 4;      // warps per CTA in the stencil / pointwise kernels
constexpr int kThreads = 32 * kWarps;
constexpr int kStrip = 64;     // columns per warp (32 lanes x double2)
constexpr int kCtaCols = kWarps * kStrip;
constexpr int kTraceSlots = 32;  // (kernel class, bytes per launch) pairs timed in-graph

// Device-side solver state, one copy per local block (all copies evolve
// identically: every decision is taken from globally reduced scalars).
struct Scalars {
    // reduction slots: a kernel's last CTA writes the block-local sum; after the
    // cross-block combine / NCCL allreduce they hold the global sum
    double red_pw;    // p.w                        (eq (9))
    double red_gam;   // r.z (CG: r.r)              (CG numerator gamma)
    double red_rr;    // r.r                        (convergence, reading R5)
    double red_pad;
    // persistent state
    double gam_old;     // gamma of the current iterate (alpha numerator)
    double alpha_prev;  // alpha of the previous update, applied lazily to u
    double r0;          // ||r_0||
    double eps;
    double theta, eig_min, eig_max, ritz_min, ritz_max;
    double margin_lo, margin_hi;
    double beta_last;
    double cheb_sigma, cheb_delta, cheb_rho;  // stand-alone Chebyshev solver state
    int it;             // completed iterations (CG + presteps + outer)
    int it_limit;       // iteration limit of the current phase
    int done;           // phase finished (converged / limit / breakdown)
    int status;         // DS_* below
    int fresh;          // next spmv starts a new (P)CG sequence: beta = 0, no check
    int presteps;
    int outer;
    int max_iters;
    unsigned ticket;    // last-CTA ticket of the deterministic grid reduction
    int pad_[3];
    double cheb_a[kMaxS], cheb_b[kMaxS];                 // Saad 12.1 a_i, b_i
    double cheb_cx[kMaxS], cheb_cz[kMaxS], cheb_cr[kMaxS], cheb_ca[kMaxS];  // folded, §4.3
    double alpha_hist[kMaxPre], beta_hist[kMaxPre];
    // in-graph kernel timing (tea_opts.trace): per trace slot, the %globaltimer of the
    // current launch's start (CTA 0), the summed launch durations (ns), the launch count, and
    // the completion ticket. Launches that find the solve finished (no-ops) are not counted.
    unsigned long long trace_t0[kTraceSlots], trace_ns[kTraceSlots], trace_n[kTraceSlots];
    unsigned trace_ticket[kTraceSlots];
};

enum { DS_RUNNING = 0, DS_CONVERGED = 1, DS_LIMIT = 2, DS_BREAKDOWN = 3, DS_EIGFAIL = 4 };

// [j0,j1) x [k0,k1) in block-local cell coordinates (may reach into the halo)
struct Region {
    int j0, j1, k0, k1;
};

// Chronopoulos & Gear scalars of the single-reduction methods (CG1, CPPCG1, CPPCG1F), from the
// last reduction: red_gam = gamma_i, red_pw = delta_i, red_rr = r.r; gam_old = gamma_{i-1},
// alpha_prev = alpha_{i-1}; fresh marks i = 0 (beta = 0, alpha = gamma/delta).
struct Cg1Coef {
    double alpha, beta;
    int state;  // 0 run, 1 converged, 2 limit, 3 breakdown
};
__device__ __forceinline__ Cg1Coef cg1_coef(const Scalars *S) {
    Cg1Coef c{0.0, 0.0, 0};
    const double gam = S->red_gam, del = S->red_pw;
    // stop test on ||r|| (reading R5): red_rr = r.r (= gam for CG1, where z = r)
    if (!S->fresh && sqrt(S->red_rr) < S->eps * S->r0) {
        c.state = 1;
        return c;
    }
    if (S->it >= S->it_limit) {
        c.state = 2;
        return c;
    }
    double den = del;
    if (!S->fresh) {
        c.beta = gam / S->gam_old;
        den = del - c.beta * gam / S->alpha_prev;
    }
    c.alpha = gam / den;
    if (!(den > 0.0) || !isfinite(c.alpha)) c.state = 3;
    return c;
}
__device__ __forceinline__ void cg1_finish(Scalars *S, const Cg1Coef &c) {
    S->done = 1;
    S->status = c.state == 1 ? DS_CONVERGED : (c.state == 2 ? DS_LIMIT : DS_BREAKDOWN);
}

// Field indices inside a block's workspace.
enum Field {
    F_U0 = 0, F_U, F_KX, F_KY, F_KZ, F_R0, F_R1, F_P0, F_P1, F_W, F_Z0, F_Z1, F_Z2, F_Z3,
    F_COUNT,
    // block-Jacobi Thomas coefficients c'_i and 1/den_i: recomputed at the start of every
    // block-Jacobi solve into two fields that method never uses
    F_BJC = F_Z2, F_BJD = F_Z3
};

// Launch geometry of one stencil / pointwise launch.
struct Launch {
    dim3 grid;
    int jstart;  // even column of the first lane of CTA 0 / warp 0
    int ty;      // rows per CTA tile
};

// Kernel launchers (tea_kernels.cu). `orig` pointers address cell (0,0) of a
// field; element (j,k) is orig[k*pitch + j]. All take the block's Scalars and
// reduction scratch (partials) and run on `st`.
struct KArgs {
    int pitch;
    Scalars *S;
    double *partials;
    cudaGraphConditionalHandle cond;  // WHILE-loop handle (0 = none)
    int set_cond;                     // this launch may end the WHILE loop
    // 3D: planes of (rows x pitch), plane stride ps; nz == 1 is 2D
    const double *kz;
    long long ps;
    int nz;
    int coef_slot;  // constant-memory coefficient slot of the fused passes (tea_cheb_tb.cu)
    // 2D on-the-fly faces (tea_opts.kform): g = 1/rho (or rho) on the block
    // plus margin, ghost cells outside the mesh hold -g of their interior neighbour so the
    // physical-boundary faces come out exactly 0; Kx(j,k) = hrx (g(j-1,k) + g(j,k)),
    // Ky(j,k) = hry (g(j,k-1) + g(j,k)). g == nullptr: the kernels read the stored Kx, Ky.
    const double *g;
    double hrx, hry;
    int tslot;  // in-graph timing slot of this launch (tea_opts.trace), -1 = not traced
};

// In-graph kernel timing (tea_opts.trace): CTA 0 stamps the start, the last
// CTA to finish adds the launch's duration to its slot. trace_end must be reached by every
// thread of every CTA of a traced launch.
__device__ __forceinline__ unsigned long long tea_gtimer() {
    unsigned long long t;
    asm volatile("mov.u64 %0, %%globaltimer;" : "=l"(t));
    return t;
}
__device__ __forceinline__ void trace_begin(const KArgs &a) {
    if (a.tslot >= 0 && blockIdx.x == 0 && blockIdx.y == 0 && blockIdx.z == 0 &&
        threadIdx.x == 0) {
        a.S->trace_t0[a.tslot] = tea_gtimer();
        __threadfence();
    }
}
__device__ __forceinline__ void trace_end(const KArgs &a) {
    if (a.tslot < 0) return;
    __syncthreads();
    if (threadIdx.x == 0) {
        __threadfence();
        const unsigned n = gridDim.x * gridDim.y * gridDim.z;
        if (atomicAdd(&a.S->trace_ticket[a.tslot], 1u) == n - 1u) {
            const unsigned long long t1 = tea_gtimer();
            volatile unsigned long long *t0 = a.S->trace_t0;
            a.S->trace_ns[a.tslot] += t1 - t0[a.tslot];
            a.S->trace_n[a.tslot] += 1ull;
            a.S->trace_ticket[a.tslot] = 0u;
        }
    }
}

Launch plan_stencil(const Region &R, int ty_req, int ncta_target);
// 3D stencil geometry: CTA = 4 warps on 4 consecutive rows of one 64-column strip,
// marching tz planes (grid = strips x rows/4 x planes/tz).
Launch plan_stencil3(const Region &R, int nz, int tz_req);
int spmv_wave_rows(int width, int height);  // wave-fitted SpMV tile height (large blocks)
int max_ctas3(int width, int height, int nz);
Launch plan_pointwise(const Region &R, int ty_req, int ncta_target);
int max_ctas(int width, int height);

void launch_init_fields(const KArgs &a, const double *rho, const double *en, double *u0,
                        double *u, double *kx, double *ky, double *g, Region owned, Region all,
                        Region kxr, Region kyr, Region gall, double hrx, double hry,
                        int mean_mode, cudaStream_t st);
// 3D: Kx, Ky, Kz (rz = dt/dz^2) and u0 = u = rho e on the single block (planes [0, nz))
void launch_init_fields3(const KArgs &a, const double *rho, const double *en, double *u0,
                         double *u, double *kx, double *ky, double *kz, int nx, int ny, int nz,
                         double rx, double ry, double rz, int mean_mode, cudaStream_t st);
void launch_residual(const KArgs &a, const Launch &L, const Region &R, const double *u,
                     const double *kx, const double *ky, double *u0, double *r,
                     cudaStream_t st);
// lazy_u = false: no u += alpha_prev p_old (2D; the last fused pass does the update)
void launch_spmv(const KArgs &a, const Launch &L, const Region &R, const double *src,
                 const double *pin, double *pout, double *w, double *u, const double *kx,
                 const double *ky, cudaStream_t st, bool lazy_u = true);
void launch_update(const KArgs &a, const Launch &L, const Region &R, const double *w,
                   double *r, cudaStream_t st);
void launch_update_nodot(const KArgs &a, const Launch &L, const Region &R, const double *w,
                         double *r, cudaStream_t st);
// Chebyshev step i (1-based) of s: z_out = z1 + a_i (z1 - z2) + b_i (r - A z1)
// mode: 0 = first (z1 = r/theta, z2 = 0), 1 = second (z2 = r/theta), 2 = general.
// fuse_update: r_out = r_in - alpha w first (first step only, single block).
// last: also r.z_out and r.r over D; restart: do not advance the iteration count.
void launch_cheb(const KArgs &a, const Launch &L, const Region &R, const Region &D, int mode,
                 int step, bool last, bool fuse_update, bool restart, const double *rin,
                 const double *win, double *rout, const double *z1, const double *z2,
                 double *zout, const double *kx, const double *ky, cudaStream_t st);
void launch_eig_setup(const KArgs &a, int s, cudaStream_t st);
void launch_scalars(const KArgs &a, int mode, double eps, int it_limit, int max_iters,
                    double mlo, double mhi, cudaStream_t st);
void launch_combine(Scalars *const *S_dev_list, int nblocks, int nvals, int first_slot,
                    cudaStream_t st);
void launch_mask_done(Scalars *S, int first, int nvals, bool zero, cudaStream_t st);
// direct in-process halo exchange (k_xcopy): box e copies src block's field fld at
// (sj0.., sk0..) into dst block's field fld at (dj0.., dk0..), w x h cells
struct XCopy {
    int src, dst, fld, sj0, sk0, dj0, dk0, w, h;
};
constexpr int kXMaxBlocks = 64;
struct XFields {
    double *f[kXMaxBlocks][2];
    int pitch[kXMaxBlocks];
};
void launch_xcopy(const XCopy *desc, int n, const XFields &F, cudaStream_t st);
void launch_pack(const double *const *fields, int nf, int pitch, const int *boxes,
                 int nbox, double *buf, cudaStream_t st);
void launch_unpack(double *const *fields, int nf, int pitch, const int *boxes, int nbox,
                   const double *buf, cudaStream_t st);

enum { SC_BEGIN = 0, SC_R0 = 1, SC_PHASE2 = 2 };

// Block-Jacobi (tea_kernels.cu): Thomas coefficients once; per iteration
// r -= alpha w (update) then z = M^{-1} r on 4-row strips, r.z and r.r.
void launch_bj_setup(const KArgs &a, const Region &R, const double *kx, const double *ky,
                     double *bjc, double *bjd, cudaStream_t st);
void launch_bj(const KArgs &a, const Region &R, bool update, bool sets_cond, const double *w,
               double *r, double *z, const double *ky, const double *bjc, const double *bjd,
               cudaStream_t st);

// Stand-alone Jacobi / Chebyshev iteration: u_k -> u_{k+1} (into uprev_out), ||r_k||^2.
void launch_stat(const KArgs &a, const Launch &L, const Region &R, bool cheb, const double *uin,
                 const double *u0, double *uprev_out, const double *kx, const double *ky,
                 cudaStream_t st);

// Single-reduction (Chronopoulos-Gear) CG. Fused single-block iteration: reads r, w, s
// (ping-pong) and p, u; writes r', w', s', p, u; one reduction (r.r, w.r).
void launch_cg1(const KArgs &a, const Launch &L, const Region &R, const double *rin,
                const double *win, const double *sin, double *rout, double *wout, double *sout,
                double *p, double *u, const double *kx, const double *ky, cudaStream_t st);
// Multi-block: pointwise update (s, p, u, r) then w = A r with the dots.
// z == nullptr: CG1 (p = r + b p, counts the iteration); else CPPCG1 (p = z + b p)
void launch_cg1_update(const KArgs &a, const Launch &L, const Region &R, const double *w,
                       double *s, double *p, double *u, double *r, cudaStream_t st,
                       const double *z = nullptr);
// pw_only: w = A r and red_pw = r.w only (CPPCG1's q = A z, del = z.q)
void launch_cg1_w(const KArgs &a, const Launch &L, const Region &R, const double *r, double *w,
                  const double *kx, const double *ky, cudaStream_t st, bool pw_only = false);

// Single-reduction CPPCG, fused form (CPPCG1F): the outer update as one stencil pass
// (p = z + b p on R + ring, w = A p, r -= a w, u += a p), where the fused passes do not.
// r on R (may be extended toward neighbour blocks), u on D (the owned cells)
void launch_cg1f_pre(const KArgs &a, const Launch &L, const Region &R, const Region &D,
                     const double *z, const double *pin, double *pout, double *r, double *u,
                     const double *kx, const double *ky, cudaStream_t st);

// Temporally blocked Chebyshev passes (tea_cheb_tb.cu).
constexpr int kTbMaxSteps = 5;
struct TbArgs {
    const double *rin = nullptr, *win = nullptr;    // r (in), w (FUSE update)
    double *rout = nullptr;                         // r' (FUSE / PRE)
    const double *zin1 = nullptr, *zin2 = nullptr;  // z_{i-1}, z_{i-2} (later passes; PRE: z_s)
    double *zoutA = nullptr, *zoutB = nullptr;      // z_{last-1}, z_last
    const double *kx = nullptr, *ky = nullptr;      // stored faces (kform -1)
    const double *pin = nullptr;                    // PRE: p_old
    double *pout = nullptr, *uio = nullptr;         // PRE: p, u (in place)
};
int tb_out_cols(int levels);
int tb_ctas(int levels, int width, int height, int ty);
int tb_auto_rows(int levels, int width, int height);
int tb_plan_rows(int levels, int width, int height, int ctas_per_sm, int nsm);
int tb_slot_acquire();  // -1: none free (the context then uses per-step kernels)
void tb_slot_release(int slot);
cudaError_t tb_coef_upload(int slot, const Scalars *S, cudaStream_t st);
// M Chebyshev steps in one pass; pre: the CPPCG1F outer update first (first pass, g faces),
// post: q = A z_s and z_s.q after the last step (last pass, g faces); upd: u += alpha p in
// the last pass (CPPCG, g faces; the SpMV then runs without its lazy u update)
void launch_cheb_tb(const KArgs &a, const Region &R, const Region &Dd, int M, int ty, int jlim,
                    int step0, bool first, bool fuse, bool last, bool restart, bool pre,
                    bool post, bool upd, const TbArgs &f, cudaStream_t st);

// Persistent single-launch CG / CPPCG solve of one 2D block (tea_kernels.cu, k_persist):
// phases separated by grid-wide barriers of a cooperative launch.
struct PersistArgs {
    KArgs a;
    Region R;  // owned cells
    int jstart, ty, gx, ntiles;  // stencil tiling (plan_stencil)
    int s, two_phase;            // inner steps; 1 = CPPCG (presteps, eigen-estimate, PCG)
    const double *kx, *ky;
    double *u0, *u, *w;
    double *r[2], *p[2], *z[3];
    double *part;  // 2 x 3 x gridDim.x reduction partials
};
int persist_ctas(int ntiles);  // co-resident CTAs for a tiling of ntiles (<= ntiles)
cudaError_t launch_persist(const PersistArgs &P, int ctas, cudaStream_t st);

}  // namespace tea
