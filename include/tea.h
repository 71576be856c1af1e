/*
 * tea.h -- C ABI of the B200-native TeaLeaf CG / CPPCG hot path.
 *
 * One implicit timestep of 2D heat conduction (Sec. II):
 * solve (I + dt L) u^{n+1} = u^n with the matrix-free 5-point operator of
 * Listing 1 (L349-367), by CG (Sec. III.A) or by Chebyshev
 * polynomially preconditioned CG, CPPCG (Sec. III.B-D), on a mesh that
 * may be split into px x py rectangular blocks (Sec. IV.A) exchanging
 * halos of depth d (matrix powers, Sec. IV.C.2).
 *
 * All compute runs in hand-written sm_100a CUDA kernels inside this library.
 * Caller memory in the signatures is plain pointers: HOST pointers for the
 * global input/output fields, a DEVICE pointer for the workspace (the caller,
 * e.g. PyTorch, owns it; the library never frees it).
 *
 * Global field layout (density, energy, u_host): nx*ny doubles, row-major,
 * x fastest: cell (j,k) at index k*nx + j, j in [0,nx), k in [0,ny).
 *
 * Errors: every call returns a tea_status. Negative = failure; the context is
 * then unusable except for tea_last_error() and tea_finalize(). A positive
 * TEA_NOT_CONVERGED means max_iters was reached; the fields are valid.
 * Not thread-safe per context. All calls on one context must come from one host
 * thread; different contexts are independent.
 */
#ifndef TEA_H
#define TEA_H

#include <stddef.h>

#ifdef __cplusplus
extern "C" {
#endif

#define TEA_ABI_VERSION 5

typedef enum {
    TEA_OK = 0,
    TEA_NOT_CONVERGED = 1,
    TEA_ERR_ARG = -1,       /* bad argument: sizes, decomposition, depth, workspace   */
    TEA_ERR_CUDA = -2,      /* CUDA runtime error (message in tea_last_error)          */
    TEA_ERR_NCCL = -3,      /* NCCL error; in multi-process runs also an asynchronous
                               NCCL error or no completion within TEA_NCCL_TIMEOUT_S seconds
                               (environment, default 600) -- a dead or stalled peer: the
                               host waits poll ncclCommGetAsyncError and abort the comm  */
    TEA_ERR_BREAKDOWN = -4, /* p.w <= 0, non-finite scalar, or bad eigen-estimate      */
    TEA_ERR_STATE = -5      /* call out of order / context already failed             */
} tea_status;

/* TEA_BJCG: CG preconditioned by block Jacobi on 4-cell strips along y, each a
 * tridiagonal block of A solved by the Thomas algorithm, strips truncated at the mesh
 * edge and at block boundaries (Sec. IV.C.1). Halo depth 1:
 * block Jacobi does not combine with matrix powers.                    */
/* TEA_CG1: single-reduction CG (Chronopoulos & Gear): r.r and (A r).r in ONE global
 * reduction per iteration, s = A p carried by recurrence -- the restructuring the
 * paper names as future work. Same iterates as CG in
 * exact arithmetic; one fused kernel per iteration on a single block.             */
/* TEA_CPPCG1: single-reduction CPPCG: the same presteps, eigen-estimate and Chebyshev
 * preconditioner B(A) as TEA_CPPCG, with the outer PCG in Chronopoulos & Gear's form:
 * q = A z and s = A p carried by recurrence, so r.z, z.q and r.r form ONE global
 * reduction per outer iteration instead of two (P:L817-821 applied to CPPCG; SURVEY
 * NEXT-2). Same iterates as CPPCG in exact arithmetic; one more matvec per outer
 * iteration (q = A z) and a separate pointwise update, so on one GPU it moves more bytes
 * than TEA_CPPCG -- its point is the halved allreduce count across ranks.            */
/* TEA_JACOBI / TEA_CHEBY: the stand-alone solvers TeaLeaf ships beside CG
 * (SURVEY NEXT-4): point Jacobi u += D^{-1} (u^n - A u), and the Chebyshev
 * iteration (Saad Alg. 12.1) on the interval estimated from `presteps` CG iterations
 * (as CPPCG). One stencil pass per iteration; the stop test uses the true residual of
 * the iterate before the last update (reading R19). Chebyshev "cannot cope with some
 * condition numbers": max_iters bounds it.                          */
/* TEA_CPPCG1F: single-reduction CPPCG in fused form (reading R23): the scalars of TEA_CPPCG1
 * (one reduction of z.q, r.z, r.r per outer iteration) with w = A p applied
 * instead of carried by recurrence. On one block with the fused passes an outer iteration is
 * TWO kernels: the first pass does the outer update (p = z + beta p, u += alpha p,
 * r -= alpha A p) and the first Chebyshev steps, the last pass the last steps and q = A z
 * with the three dot products -- 15 fp64 streams (TEA_CPPCG: 3 kernels, 18 streams; TEA_CPPCG1:
 * 4 kernels, 22). Same iterates as CPPCG in exact arithmetic; s + 2 matvecs per outer
 * iteration. 2D fused passes; 3D (and d < s + 1 blocks) by one kernel per step.       */
typedef enum {
    TEA_CG = 0, TEA_CPPCG = 1, TEA_BJCG = 2, TEA_CG1 = 3, TEA_JACOBI = 4, TEA_CHEBY = 5,
    TEA_CPPCG1 = 6, TEA_CPPCG1F = 7
} tea_method;

typedef struct tea_ctx tea_ctx; /* opaque, library-owned */

/* Mesh: nx x ny (x nz) cells on [xmin,xmax] x [ymin,ymax] (x [zmin,zmax]);
 * dx = (xmax-xmin)/nx, ...; rx = dt/dx^2, ry = dt/dy^2 (BASELINE.json north_star),
 * rz = dt/dz^2. nz <= 1: the 2D 5-point problem (Listing 1); nz > 1: the 3D 7-point
 * problem (reading R20) -- single block, methods CG, CPPCG,
 * CG1, JACOBI, CHEBY. 3D host arrays are nx*ny*nz, index (l*ny + k)*nx + j.        */
typedef struct {
    int nx, ny;
    double xmin, xmax, ymin, ymax;
    int nz;
    double zmin, zmax;
} tea_mesh;

/* Decomposition: px x py blocks, block b = by*px + bx owns the
 * columns/rows given by an even split with the remainder on low-index blocks.
 * The blocks are shared by `nranks` processes (one process per GPU): rank r
 * owns blocks [r*B, (r+1)*B), B = px*py/nranks; multi-process runs need B = 1
 * (TEA_ERR_ARG otherwise). nranks == 1 with px*py > 1 runs every block in this
 * process on one GPU, halos by an on-device copy kernel; with the environment
 * variable TEA_NCCL_SELF=1 they go through a 1-rank NCCL communicator instead
 * (send/recv to self, allreduce, chunked graphs: the multi-process code path on
 * one GPU, bitwise the same results; a diagnostic).
 * halo_depth d >= 1: matrix-powers depth of the CPPCG inner loop.
 * nccl_id: 128-byte ncclUniqueId from tea_get_nccl_id() on rank 0, broadcast by
 * the caller; NULL when nranks == 1. Pass NULL for `dist` to get 1x1, d = 1.  */
typedef struct {
    int rank, nranks;
    int px, py;
    int halo_depth;
    const void *nccl_id;
} tea_dist;

/* Solver options (DESIGN.md readings). Pass NULL for the defaults in brackets. */
typedef struct {
    int presteps;           /* CG iterations before CPPCG switches (R6)        [30]   */
    double eig_margin_lo;   /* lambda_min = lo * min Ritz value (R8)           [0.95] */
    double eig_margin_hi;   /* lambda_max = hi * max Ritz value (R8)           [1.05] */
    int mean_mode;          /* face coefficient: 0 rx*mean(1/rho) (R1), 1 rx*mean(rho) [0] */
    int loop_mode;          /* 0 device WHILE graph, 1 chunked graphs, 2 eager  [0]    */
    int check_interval;     /* iterations per chunk in loop_mode 1/2 (0 = auto) [0]    */
    int profile;            /* 1: eager launches timed per kernel (tea_kernel_times)[0]*/
    int tile_rows;          /* rows per CTA tile of the stencil kernels, 0 = auto [0]  */
    int tb_steps;           /* Chebyshev steps fused per HBM pass (on-chip matrix
                               powers): 0 = auto (5 for 2D blocks >= 4e5 cells with
                               one block or d >= s + 1, else 1), 1 = one kernel per
                               step, 2..5 = at most that many                [0]   */
    int tb_rows;            /* output rows per CTA tile of the fused passes, 0 = auto */
    int persist;            /* whole solve in ONE cooperative launch (grid-wide barriers
                               between the phases; single 2D block, CG / CPPCG, one
                               process, loop_mode 0): 1 = on, -1 = off, 0 = auto:
                               on for CG blocks <= TEA_PERSIST_AUTO_CG cells and
                               CPPCG blocks <= TEA_PERSIST_AUTO_CPPCG cells, where it
                               measured faster              [0] */
    int overlap;            /* with neighbour blocks and the fused passes (d >= s + 1):
                               the residual's halo exchange runs on a second stream while
                               the first pass computes the block interior that needs no
                               halo cell; the frame follows the exchange (SURVEY §8(e)
                               "Overlap"). 1 = on, -1 = off, 0 = auto:
                               on when the halo crosses processes (nranks > 1; with all
                               blocks in one process the copies are on-device and the
                               split only adds launches: measured 383 vs 341 ms per
                               4096^2 timestep in 2 x 4). Never while profiling. Results
                               are bitwise identical either way.                [0] */
    int kform;              /* face coefficients in the 2D SpMV and the fused Chebyshev
                               passes: 1 = formed on the fly from ONE stream g = 1/rho
                               (mean_mode 1: g = rho) as K = (r/2)(g_L + g_R) (reading
                               R1 written out; one fp64 stream instead of the two
                               stored Kx, Ky: 8 -> 7 and 7/6 -> 6/5 streams), -1 =
                               stored Kx, Ky, 0 = auto (on). Every kernel's K is
                               bitwise the same either way (the stored faces are
                               computed by the same expression). [0] */
    int trace;              /* 1: in-graph kernel timing. Every hot-path kernel launch
                               (in any loop mode, inside the CUDA graphs too) stamps
                               %globaltimer at its start (CTA 0) and adds its duration,
                               taken by the last CTA to finish, to a per-(kernel class,
                               algorithmic bytes) slot on the device; launches that find
                               the solve finished (no-ops) and the finalising u update are
                               not counted. Read with tea_trace_read(). Costs one
                               atomicAdd per CTA per launch. 0 = off               [0] */
} tea_opts;
#define TEA_PERSIST_AUTO_CG (1024.0 * 1024.0)
#define TEA_PERSIST_AUTO_CPPCG (512.0 * 512.0)

/* Per-solve statistics. */
typedef struct {
    int iterations;    /* CG iterations (CG) or presteps + outer iterations (CPPCG)  */
    int presteps;      /* CG iterations run before switching to CPPCG                */
    int outer;         /* CPPCG outer iterations                                     */
    int inner_matvecs; /* matvecs inside the Chebyshev preconditioner                */
    int matvecs;       /* all applications of A (incl. the initial residual)         */
    int status;        /* tea_status of the solve                                    */
    double r0;         /* ||u^n - A u^n||_2                                           */
    double rnorm;      /* ||r||_2 at exit (recursively updated residual)              */
    double eig_min, eig_max;   /* preconditioner interval (after margins)            */
    double ritz_min, ritz_max; /* raw Lanczos extreme Ritz values                    */
    double seconds;    /* device time of the solve (CUDA events, this rank)          */
} tea_stats;

/* Kernel ids for tea_kernel_times(). */
enum {
    TEA_K_INIT = 0, TEA_K_RESIDUAL, TEA_K_SPMV, TEA_K_UPDATE, TEA_K_CHEB_FIRST,
    TEA_K_CHEB_STEP, TEA_K_CHEB_LAST, TEA_K_EIG, TEA_K_PACK, TEA_K_UNPACK, TEA_K_SCALAR,
    TEA_K_TB_FIRST, TEA_K_TB_MID, TEA_K_TB_LAST, /* fused multi-step Chebyshev passes */
    TEA_K_BJ,                                     /* block-Jacobi update + strip solves  */
    TEA_K_CG1, TEA_K_CG1W,                        /* single-reduction CG: fused / A r    */
    TEA_K_STAT,                                   /* Jacobi / Chebyshev iteration        */
    TEA_K_PERSIST,                                /* whole solve, one cooperative launch */
    TEA_K_COUNT
};

/* Library version string and ABI version. */
const char *tea_version(void);
int tea_abi_version(void);

/* Write a fresh ncclUniqueId (128 bytes) into id128. Call on rank 0 only. */
tea_status tea_get_nccl_id(void *id128);

/* Device workspace bytes this rank needs for `mesh` and `dist` (NULL = 1 block). */
tea_status tea_workspace_bytes(const tea_mesh *mesh, const tea_dist *dist, size_t *bytes);

/* Create a context. Reads this rank's blocks (plus a margin) of the HOST global
 * arrays `density` and `energy` (both nx*ny, see layout above), builds
 * u^0 = density*energy (reading R4) and the face coefficients Kx, Ky scaled by
 * rx, ry (reading R1/R2/R3). `d_workspace` is a DEVICE buffer of at
 * least tea_workspace_bytes() bytes, 256-byte aligned, owned by the caller and
 * valid until tea_finalize(). `cuda_stream` (cudaStream_t, may be NULL = legacy
 * default) is the caller's stream: the library orders its own stream after it
 * on entry and makes it wait for the library on exit. Collective over ranks.  */
tea_status tea_init(tea_ctx **out, const tea_mesh *mesh, const double *density,
                    const double *energy, double dt, const tea_dist *dist,
                    const tea_opts *opts, void *d_workspace, size_t ws_bytes,
                    void *cuda_stream);

/* One implicit timestep: solve A u^{n+1} = u^n with initial guess u^n, stop when
 * ||r||_2 < eps * ||r_0||_2 (reading R5) or after max_iters iterations (CG
 * iterations + CPPCG presteps + outer iterations). inner_steps = s >= 1
 * Chebyshev matvecs per preconditioner application (CPPCG only, s <= 64).
 * On return u^n <- u^{n+1}. Host-synchronous. Collective over ranks.
 * stats may be NULL.                                                          */
tea_status tea_solve(tea_ctx *ctx, tea_method method, double eps, int max_iters,
                     int inner_steps, tea_stats *stats);

/* Copy this rank's owned cells of u into their places in the HOST global array
 * u_host (nx*ny doubles); other entries are untouched. Host-synchronous.      */
tea_status tea_fetch(tea_ctx *ctx, double *u_host);

/* Replace u (and the right-hand side u^n) by the HOST global array u_host:
 * resume from a checkpoint written by tea_fetch. Host-synchronous.            */
tea_status tea_set_u(tea_ctx *ctx, const double *u_host);

/* Per-kernel-class device time accumulated since the last reset in profile mode (eager
 * launches bracketed by events: every HOST launch is counted, including the no-op launches
 * issued after the solve finished -- tea_trace_read() counts only launches that did work):
 * ms[i], launches[i] and bytes[i] for i < TEA_K_COUNT (any may be NULL). bytes are
 * the ALGORITHMIC HBM bytes of those launches (fp64 streams x 8 B x owned cells, the
 * model of DESIGN.md §4; halos and redundant overlap compute excluded).
 * reset != 0 clears.                                                           */
tea_status tea_kernel_times(tea_ctx *ctx, double *ms, long long *launches, double *bytes,
                            int reset);

/* In-graph kernel timing (tea_opts.trace): up to `cap` slots, one per (kernel class,
 * algorithmic bytes per launch) pair seen since tea_init, summed over this rank's blocks:
 * kid[i] (TEA_K_*), bytes_per_launch[i] (DESIGN.md §4 model), launches[i] (launches that
 * did their work) and ms[i] (their summed device durations). Returns the slot count (or a
 * negative tea_status). reset != 0 zeroes the counters after reading. Host-synchronous. */
int tea_trace_read(tea_ctx *ctx, int cap, int *kid, double *bytes_per_launch,
                   long long *launches, double *ms, int reset);

/* Kernel launches issued by the library since tea_init (all modes; graph
 * replays count their kernel nodes).                                          */
long long tea_launch_count(const tea_ctx *ctx);

/* Free the context, its graphs, streams, events and NCCL communicator (not the
 * workspace). Safe on a failed context; NULL is a no-op.                      */
tea_status tea_finalize(tea_ctx *ctx);

/* Last error message of ctx (or of the last failed tea_init when ctx is NULL). */
const char *tea_last_error(const tea_ctx *ctx);

/* ---- host-only helpers (no GPU needed; used by tests and tooling) ---------- */

/* Cells owned by block b: columns [x0,x1), rows [y0,y1) of the global mesh.  */
tea_status tea_block_extent(const tea_mesh *mesh, int px, int py, int b, int *x0, int *x1,
                            int *y0, int *y1);

/* CPPCG inner-loop schedule for s steps and halo depth d on a block with
 * neighbours: writes up to cap ops as (code, arg) pairs into ops[2*i..2*i+1]
 * and returns the op count (or a negative tea_status). Codes:
 *   1 = exchange r at depth arg (after the outer update)
 *   2 = Chebyshev step i computing z_i on owned cells extended by arg
 *   3 = exchange the pair (z_{i-1}, z_{i-2}) at depth arg
 *   4 = exchange z_s at depth arg (final fix-up when d == 1)
 * A block without neighbours uses the same schedule with every exchange a no-op. */
int tea_cheb_schedule(int s, int d, int *ops, int cap);

/* Rows per CTA tile the fused Chebyshev passes use for a pass of `levels` stencil levels
 * (1..6) over width x height cells, given `ctas_per_sm` resident CTAs per SM (the library
 * derives it from the kernel's registers and shared memory) on `nsm` SMs: the cost model of
 * DESIGN.md §4.4 (a wave costs its busiest SM's CTA count). Returns the rows, or TEA_ERR_ARG. */
int tea_tb_plan(int levels, int width, int height, int ctas_per_sm, int nsm);

/* Cross-process halo messages of `rank` for one exchange at halo depth `depth` (corners
 * when `corners` != 0, `nfields` fields per box), in the order tea_solve posts them inside
 * one NCCL group: all sends, then all receives, each sorted by (sending block, receiving
 * block, direction from the sender) -- the canonical order both ranks of a pair share (NCCL
 * matches a pair's point-to-point calls in posting order). Writes up to cap
 * 6-tuples (op 0 send / 1 recv, peer rank, sending block, receiving block, direction
 * 0..7 = W, E, S, N, SW, SE, NW, NE, length in doubles) into out[6*i..6*i+5] and returns
 * the message count (when it exceeds cap nothing is written), or a negative tea_status. */
int tea_halo_order(const tea_mesh *mesh, int px, int py, int nranks, int rank, int depth,
                   int corners, int nfields, long long *out, int cap);

#ifdef __cplusplus
}
#endif
#endif /* TEA_H */
