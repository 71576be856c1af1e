// tea_capi.cu -- host driver and C ABI of the B200 TeaLeaf CG / CPPCG library.
//
// Context, block decomposition, workspace layout in HBM, halo plans
// (matrix powers), the CG / CPPCG control flow (Sec. III), CUDA-graph
// capture with a device-side WHILE loop, NCCL plumbing, and the extern "C" entry
// points declared in include/tea.h. All arithmetic on fields runs in the kernels
// of tea_kernels.cu; this file only sequences them.
#include "tea.h"
#include "tea_internal.h"

#include <nccl.h>
#include <nvtx3/nvToolsExt.h>

#include <algorithm>
#include <chrono>
#include <cmath>
#include <cstdlib>
#include <thread>
#include <cstdarg>
#include <cstdio>
#include <cstring>
#include <map>
#include <memory>
#include <string>
#include <vector>

using namespace tea;

#ifndef TEA_CPPCG_UPD
#define TEA_CPPCG_UPD 0  // 1: CPPCG fused passes do u += alpha p in the last pass instead of the
                         // SpMV (measured slower: SpMV 165 -> 137 us but last pass 151 -> 199 us,
                         // profiles/r02_upd_ab.txt)
#endif

namespace {

constexpr int kNDir = 8;
// direction d: 0 W(-x) 1 E(+x) 2 S(-y) 3 N(+y) 4 SW 5 SE 6 NW 7 NE
constexpr int kDX[kNDir] = {-1, 1, 0, 0, -1, 1, -1, 1};
constexpr int kDY[kNDir] = {0, 0, -1, 1, -1, -1, 1, 1};
constexpr int kOpp[kNDir] = {1, 0, 3, 2, 7, 6, 5, 4};

inline size_t round_up(size_t x, size_t a) { return (x + a - 1) / a * a; }

// exchange kinds
// X_ZD1: z_s at depth d + 1 (CPPCG1F on blocks, exchanged while its one reduction is in flight)
enum { X_R1 = 0, X_RD, X_Z2, X_Z1, X_U1, X_ZD1, X_COUNT };

struct XPlan {
    int nf = 0, depth = 0;
    int nsend = 0, nrecv = 0;  // boxes
    int *d_send = nullptr, *d_recv = nullptr;
    size_t soff[kNDir] = {}, slen[kNDir] = {}, roff[kNDir] = {}, rlen[kNDir] = {};
};

struct BlockLayout {
    int bi, bj, gx0, gx1, gy0, gy1, bx, by;
    int nz;          // planes (1: 2D)
    long long ps;    // plane stride (doubles), rows * pitch
    int H, X0, pitch, rows, planes;
    size_t field_bytes, scalars_off, partials_off, partials_cap, boxes_off, xdesc_off, halo_off,
        halo_cap, total;
    bool has_nbr;
};

void split(int n, int p, int i, int *a, int *b) {
    int base = n / p, rem = n % p;
    *a = i * base + std::min(i, rem);
    *b = *a + base + (i < rem ? 1 : 0);
}

BlockLayout layout_block(const tea_mesh &m, int px, int py, int d, int b) {
    BlockLayout L{};
    L.bi = b % px;
    L.bj = b / px;
    split(m.nx, px, L.bi, &L.gx0, &L.gx1);
    split(m.ny, py, L.bj, &L.gy0, &L.gy1);
    L.bx = L.gx1 - L.gx0;
    L.by = L.gy1 - L.gy0;
    // halo margins: the fused passes read up to M (<= 5) rows and MR (<= 6) columns beyond
    // their output region, which reaches d cells into the halo on extended bounds
    L.H = d + kTbMaxSteps + 2;
    L.X0 = (int)round_up(d + 8, 16);
    L.pitch = (int)round_up(L.X0 + L.bx + d + 8, 32);
    L.rows = L.by + 2 * L.H;
    L.nz = m.nz > 1 ? m.nz : 1;
    L.ps = (long long)L.rows * L.pitch;
    L.planes = L.nz > 1 ? L.nz + 2 * L.H : 1;
    L.field_bytes = round_up((size_t)L.planes * L.ps * sizeof(double), 256);
    size_t off = L.field_bytes * F_COUNT;
    L.scalars_off = off;
    off += round_up(sizeof(Scalars), 256);
    // two values per CTA of the largest grid any reducing launch can use: 2D stencil and
    // pointwise tiles down to one row (tile_rows = 1) on the extended region; 3D stencil
    // tiles down to one plane, 3D pointwise tiles one row x one plane
    L.partials_cap = 2 * (size_t)std::max(max_ctas(L.bx + 2 * d + 2, L.by + 2 * d + 2),
                                          L.nz > 1 ? max_ctas3(L.bx, L.by, L.nz) : 0);
    L.partials_cap = std::max(L.partials_cap, (size_t)6 * 1024);  // k_persist: 2 x 3 x CTAs
    L.partials_off = off;
    off += round_up(L.partials_cap * sizeof(double), 256);
    L.has_nbr = (px * py > 1);
    L.boxes_off = off;
    off += L.has_nbr ? 16384 : 0;
    // direct-exchange descriptors of every block of the process (used in block 0's copy)
    L.xdesc_off = off;
    off += L.has_nbr ? round_up((size_t)X_COUNT * px * py * 16 * sizeof(XCopy), 256) : 0;
    L.halo_off = off;
    // per field and depth d: two faces in x, two in y, four corners
    size_t per_field = 2 * (size_t)d * (L.bx + L.by) + 4 * (size_t)d * d;
    L.halo_cap = L.has_nbr ? 2 * per_field : 0;  // up to 2 fields per exchange
    off += L.has_nbr ? 2 * round_up(L.halo_cap * sizeof(double), 256) : 0;
    L.total = round_up(off, 256);
    return L;
}

struct BlockCtx {
    BlockLayout L;
    int id, rank;
    double *f[F_COUNT];  // orig pointers (cell (0,0))
    Scalars *S;
    double *partials;
    int nbr[kNDir];
    double *sendbuf = nullptr, *recvbuf = nullptr;
    XPlan xp[X_COUNT];
    Region owned() const { return Region{0, L.bx, 0, L.by}; }
    Region ext(int e) const {
        return Region{nbr[0] >= 0 ? -e : 0, L.bx + (nbr[1] >= 0 ? e : 0), nbr[2] >= 0 ? -e : 0,
                      L.by + (nbr[3] >= 0 ? e : 0)};
    }
};

struct PendingEv {
    int kid;
    cudaEvent_t a, b;
};

}  // namespace

struct tea_ctx {
    tea_mesh mesh{};
    tea_opts opts{};
    double dt = 0, rx = 0, ry = 0;
    int px = 1, py = 1, d = 1, rank = 0, nranks = 1;
    std::vector<BlockCtx> blocks;
    cudaStream_t user_stream = nullptr, stream = nullptr;
    cudaEvent_t ev_in = nullptr, ev_t0 = nullptr, ev_t1 = nullptr;
    // halo/compute overlap (tea_opts.overlap): exchange stream and its fork/join events
    cudaStream_t xstream = nullptr;
    cudaEvent_t ev_fork = nullptr, ev_join = nullptr;
    Scalars *hS = nullptr;  // pinned host mirror (head only)
    ncclComm_t comm = nullptr;
    // halos exchanged on the second stream use their own communicator (split from comm): an
    // exchange there may run concurrently with an allreduce on the compute stream, and two
    // concurrent NCCL operations must not share one communicator's connections
    ncclComm_t xcomm = nullptr;
    // TEA_NCCL_SELF=1 (diagnostic, one process, several blocks): halos and dot products go
    // through a 1-rank NCCL communicator -- grouped ncclSend/ncclRecv to self in the canonical
    // order, ncclAllReduce, the split exchange communicator on the second stream, chunked graphs
    // and the polled host waits -- the multi-process code path, on one GPU (NCCL refuses two
    // ranks on one device). Results are bitwise those of the device-copy transport.
    bool nccl_self = false;
    std::string err;
    bool failed = false;
    long long launches = 0;
    // profile
    bool profiling = false;
    std::vector<PendingEv> pending;
    std::vector<cudaEvent_t> evpool;
    size_t evnext = 0;
    double kms[TEA_K_COUNT] = {};
    long long kcount[TEA_K_COUNT] = {};
    double kbytes[TEA_K_COUNT] = {};
    // graphs: key -> exec
    std::map<long long, cudaGraphExec_t> graphs;
    std::map<long long, int> graph_kernels;
    // capture state
    cudaGraphConditionalHandle cond = 0;
    // direct in-process halo exchange (all blocks local): descriptors per exchange kind
    XCopy *xdesc[16] = {};
    int nxdesc[16] = {};
    // in-graph kernel timing (tea_opts.trace): slot i times launches of (kid, bytes)
    std::vector<std::pair<int, double>> tslots;
    int cur_tslot = -1;
    int ty_override = 0;
    int coef_slot = -1;  // constant-memory coefficient slot of the fused passes
};

static std::string g_init_error;

namespace {

struct TeaError {
    tea_status st;
    std::string msg;
};

[[noreturn]] void fail(tea_status st, const char *fmt, ...) {
    char buf[512];
    va_list ap;
    va_start(ap, fmt);
    vsnprintf(buf, sizeof buf, fmt, ap);
    va_end(ap);
    throw TeaError{st, buf};
}

#define CK(call)                                                                        \
    do {                                                                                \
        cudaError_t e_ = (call);                                                        \
        if (e_ != cudaSuccess)                                                          \
            fail(TEA_ERR_CUDA, "%s:%d %s: %s", __FILE__, __LINE__, #call,               \
                 cudaGetErrorString(e_));                                               \
    } while (0)
#define NK(call)                                                                        \
    do {                                                                                \
        ncclResult_t r_ = (call);                                                       \
        if (r_ != ncclSuccess)                                                          \
            fail(TEA_ERR_NCCL, "%s:%d %s: %s", __FILE__, __LINE__, #call,               \
                 ncclGetErrorString(r_));                                               \
    } while (0)

// Host wait for the library stream. Multi-process runs poll instead of blocking: a peer that
// died or an NCCL error would otherwise hang the rank forever (SURVEY §5 failure detection).
// ncclCommGetAsyncError is checked every poll; after TEA_NCCL_TIMEOUT_S seconds (default
// 600) without completion, or on an NCCL error, the communicator is aborted and the call
// fails with TEA_ERR_NCCL.
void wait_stream(tea_ctx *c) {
    if (!c->comm) {
        CK(cudaStreamSynchronize(c->stream));
        return;
    }
    static const double timeout_s = [] {
        const char *e = std::getenv("TEA_NCCL_TIMEOUT_S");
        const double v = e ? std::atof(e) : 0.0;
        return v > 0.0 ? v : 600.0;
    }();
    const auto t0 = std::chrono::steady_clock::now();
    for (long long n = 0;; ++n) {
        const cudaError_t q = cudaStreamQuery(c->stream);
        if (q == cudaSuccess) return;
        if (q != cudaErrorNotReady) CK(q);
        ncclResult_t ar = ncclSuccess;
        NK(ncclCommGetAsyncError(c->comm, &ar));
        if (ar == ncclSuccess && c->xcomm) NK(ncclCommGetAsyncError(c->xcomm, &ar));
        const double dt =
            std::chrono::duration<double>(std::chrono::steady_clock::now() - t0).count();
        if (ar != ncclSuccess && ar != ncclInProgress) {
            if (c->xcomm) ncclCommAbort(c->xcomm);
            c->xcomm = nullptr;
            ncclCommAbort(c->comm);
            c->comm = nullptr;
            fail(TEA_ERR_NCCL, "NCCL async error: %s", ncclGetErrorString(ar));
        }
        if (dt > timeout_s) {
            if (c->xcomm) ncclCommAbort(c->xcomm);
            c->xcomm = nullptr;
            ncclCommAbort(c->comm);
            c->comm = nullptr;
            fail(TEA_ERR_NCCL, "no completion after %.0f s (TEA_NCCL_TIMEOUT_S): a peer rank "
                 "is gone or stalled; communicator aborted", dt);
        }
        if (n > 64) std::this_thread::sleep_for(std::chrono::microseconds(n > 4096 ? 200 : 20));
    }
}

// NVTX phase ranges (nvtx3, header only: no-ops unless a tool such as nsys is attached)
struct Nvtx {
    explicit Nvtx(const char *name) { nvtxRangePushA(name); }
    ~Nvtx() { nvtxRangePop(); }
};

KArgs kargs(tea_ctx *c, const BlockCtx &b, bool set_cond = false) {
    KArgs a;
    a.pitch = b.L.pitch;
    a.S = b.S;
    a.partials = b.partials;
    a.cond = c->cond;
    a.set_cond = set_cond ? 1 : 0;
    a.kz = b.f[F_KZ];
    a.ps = b.L.ps;
    a.nz = b.L.nz;
    a.coef_slot = c->coef_slot;
    // 2D blocks: faces formed on the fly from g (held in the otherwise unused Kz field)
    a.g = (b.L.nz == 1 && c->opts.kform >= 0) ? b.f[F_KZ] : nullptr;
    a.hrx = 0.5 * c->rx;
    a.hry = 0.5 * c->ry;
    a.tslot = c->cur_tslot;
    return a;
}

// kernel classes whose kernels carry the trace_begin / trace_end hooks
bool traced_kid(int kid) {
    switch (kid) {
        case TEA_K_RESIDUAL: case TEA_K_SPMV: case TEA_K_UPDATE: case TEA_K_CHEB_FIRST:
        case TEA_K_CHEB_STEP: case TEA_K_CHEB_LAST: case TEA_K_TB_FIRST: case TEA_K_TB_MID:
        case TEA_K_TB_LAST: case TEA_K_BJ: case TEA_K_CG1: case TEA_K_CG1W: case TEA_K_STAT:
            return true;
        default:
            return false;
    }
}
int trace_slot(tea_ctx *c, int kid, double bytes) {
    if (!c->opts.trace || !traced_kid(kid)) return -1;
    for (size_t i = 0; i < c->tslots.size(); ++i)
        if (c->tslots[i].first == kid && c->tslots[i].second == bytes) return (int)i;
    if ((int)c->tslots.size() >= kTraceSlots) return -1;  // full: this pair goes untimed
    c->tslots.emplace_back(kid, bytes);
    return (int)c->tslots.size() - 1;
}

// Issue one kernel launch (profiled with an event pair when profiling). `bytes` =
// the launch's algorithmic HBM bytes, accumulated per kernel class.
template <class F>
void K(tea_ctx *c, int kid, double bytes, F &&f) {
    c->cur_tslot = trace_slot(c, kid, bytes);
    struct Reset {
        int &v;
        ~Reset() { v = -1; }
    } reset_{c->cur_tslot};
    if (c->profiling) {
        if (c->evnext + 2 > c->evpool.size()) {
            for (int i = 0; i < 256; ++i) {
                cudaEvent_t e;
                CK(cudaEventCreate(&e));
                c->evpool.push_back(e);
            }
        }
        cudaEvent_t a = c->evpool[c->evnext++], b = c->evpool[c->evnext++];
        CK(cudaEventRecord(a, c->stream));
        f();
        CK(cudaGetLastError());
        CK(cudaEventRecord(b, c->stream));
        c->pending.push_back({kid, a, b});
        c->kbytes[kid] += bytes;
    } else {
        f();
        CK(cudaGetLastError());
    }
    c->launches++;
}

void resolve_profile(tea_ctx *c) {
    if (!c->profiling) return;
    wait_stream(c);
    for (auto &p : c->pending) {
        float ms = 0.f;
        CK(cudaEventElapsedTime(&ms, p.a, p.b));
        c->kms[p.kid] += ms;
        c->kcount[p.kid] += 1;
    }
    c->pending.clear();
    c->evnext = 0;
}

Launch plan(tea_ctx *c, const Region &R) {
    return plan_stencil(R, c->opts.tile_rows > 0 ? c->opts.tile_rows : c->ty_override, 1184);
}
// stencil kernels: 2D march over rows, or the 3D march over planes
// every reducing launch writes NV <= 2 partials per CTA into the block's scratch
const Launch &checked(const BlockCtx &b, const Launch &L) {
    const size_t ctas = (size_t)L.grid.x * L.grid.y * L.grid.z;
    if (2 * ctas > b.L.partials_cap)
        fail(TEA_ERR_STATE, "launch of %zu CTAs exceeds the reduction scratch (%zu partials)",
             ctas, b.L.partials_cap);
    return L;
}
Launch plan_st(tea_ctx *c, const BlockCtx &b, const Region &R) {
    if (b.L.nz > 1) return checked(b, plan_stencil3(R, b.L.nz, c->opts.tile_rows));
    return checked(b, plan(c, R));
}
// the SpMV: large 2D blocks (where the default tile is the 32-row cap) get wave-fitted tiles
Launch plan_spmv(tea_ctx *c, const BlockCtx &b, const Region &R) {
    Launch L = plan_st(c, b, R);
    if (b.L.nz > 1 && c->opts.tile_rows <= 0) {
        // 3D: one wave at the SpMV's 4 CTAs/SM (TEA_SPMV3_MINB), so each warp marches as many
        // planes as fit -- fewer (tz + 2) / tz re-read planes (256^3: tz 32 -> 128, SpMV
        // 4776 -> 4965 GB/s, profiles/r01k_tz3.txt)
        const int cols = (int)(L.grid.x * L.grid.y);
        const int gz = std::max(1, 592 / std::max(cols, 1));
        return checked(b, plan_stencil3(R, b.L.nz, std::max(4, (b.L.nz + gz - 1) / gz)));
    }
    if (b.L.nz > 1 || c->opts.tile_rows > 0 || c->ty_override > 0) return L;
    // blocks >= 2M cells get whole waves too (2048 x 1024, the 8-GPU 4096^2 block: the
    // default 8-row tiles were 1.4 waves of 740 slots); smaller ones keep plan_stencil's
    // latency-tuned short tiles (1024^2: 8 rows, the measured optimum)
    const double cells = (double)(R.j1 - R.j0) * (R.k1 - R.k0);
    if (L.ty < 32 && cells < 2.0e6) return L;
    const int ty = spmv_wave_rows(R.j1 - L.jstart, R.k1 - R.k0);
    // one reduction partial per CTA must fit the block's scratch (fewer CTAs: always true)
    return checked(b, plan_stencil(R, ty, 0));
}
// pointwise kernels: the 2D tiling of one plane, planes on grid.z
Launch plan_pw(tea_ctx *c, const BlockCtx &b, const Region &R) {
    // 3D: the planes already multiply the CTA count, so the small-block rule of
    // plan_stencil (shorter tiles until >= 2 tiles per SM, a 2D latency fix) must not
    // apply: it cut 256^3 tiles to one row (CG 67 -> 85 ms per timestep). 8-row tiles.
    const int tr = c->opts.tile_rows > 0 ? c->opts.tile_rows : c->ty_override;
    Launch L = b.L.nz > 1 ? plan_stencil(R, tr > 0 ? tr : 8, 1184) : plan(c, R);
    L.grid.z = b.L.nz;
    return checked(b, L);
}

// ------------------------------------------------------------------ reductions
// Combine the block-local sums of slots [first, first+n) (0 pw, 1 gam, 2 rr) into
// the global sums on every local block and across ranks.
void reduce(tea_ctx *c, int first, int n) {
    Nvtx nv_("tea reduce");
    const int nb = (int)c->blocks.size();
    if (nb > 1) {
        std::vector<Scalars *> L;
        for (auto &b : c->blocks) L.push_back(b.S);
        K(c, TEA_K_SCALAR, 0.0, [&] { launch_combine(L.data(), nb, n, first, c->stream); });
    }
    if (c->nranks > 1 || c->nccl_self) {
        double *p = &c->blocks[0].S->red_pw + first;
        K(c, TEA_K_SCALAR, 0.0,
          [&] { launch_mask_done(c->blocks[0].S, first, n, c->rank != 0, c->stream); });
        NK(ncclAllReduce(p, p, n, ncclDouble, ncclSum, c->comm, c->stream));
    }
}

// ------------------------------------------------------------------ halo exchange
// One cross-process halo message: global ids of the sending and receiving block, the
// direction seen from the sender, its length (doubles), the peer rank and the local buffer.
struct HaloMsg {
    int src, dst, dir;
    double *buf;
    size_t len;
    int peer;
    bool operator<(const HaloMsg &o) const {
        return src != o.src ? src < o.src : (dst != o.dst ? dst < o.dst : dir < o.dir);
    }
};
// NCCL matches the sends and receives between two ranks in posting order: with several
// blocks per rank one pair of ranks can carry several messages (a face and a corner to two
// blocks of the same rank, possibly of equal size), so both sides post them in ONE canonical
// order -- (sending block, receiving block, direction seen from the sender). Shared by the
// exchange and the host-only tea_halo_order (tests/test_dist_gloo.py replays it over gloo).
void halo_post_order(std::vector<HaloMsg> &sends, std::vector<HaloMsg> &recvs) {
    std::sort(sends.begin(), sends.end());
    std::sort(recvs.begin(), recvs.end());
}

void exchange(tea_ctx *c, int kind, const std::vector<int> &fids_per_block_field,
              cudaStream_t xs = nullptr) {
    // fids: field ids (same for every block), 1 or 2 entries; xs: the stream to run on
    // (default: the compute stream)
    const cudaStream_t st = xs ? xs : c->stream;
    const int nb = (int)c->blocks.size();
    if (c->px * c->py == 1) return;
    Nvtx nv_("tea halo exchange");
    const int nf = (int)fids_per_block_field.size();
    for (auto &b : c->blocks) {
        const XPlan &x = b.xp[kind];
        if (x.nsend == 0) continue;
        const double *F[4];
        for (int i = 0; i < nf; ++i) F[i] = b.f[fids_per_block_field[i]];
        K(c, TEA_K_PACK, 0.0, [&] {
            launch_pack(F, nf, b.L.pitch, x.d_send, x.nsend, b.sendbuf, st);
        });
    }
    // transport
    bool remote0 = false;
    for (auto &b : c->blocks)
        for (int d = 0; d < kNDir; ++d)
            if (b.nbr[d] >= 0 && b.nbr[d] / (c->px * c->py / c->nranks) != c->rank) remote0 = true;
    if (!remote0 && c->nxdesc[kind] > 0) {
        // every neighbour is in this process: one direct-copy launch, no pack / copy / unpack
        XFields F{};
        for (size_t i = 0; i < c->blocks.size() && i < (size_t)kXMaxBlocks; ++i) {
            for (int j = 0; j < nf && j < 2; ++j) F.f[i][j] = c->blocks[i].f[fids_per_block_field[j]];
            F.pitch[i] = c->blocks[i].L.pitch;
        }
        K(c, TEA_K_PACK, 0.0, [&] { launch_xcopy(c->xdesc[kind], c->nxdesc[kind], F, st); });
        return;
    }
    // transport
    bool remote = false;
    for (auto &b : c->blocks)
        for (int d = 0; d < kNDir; ++d)
            if (b.nbr[d] >= 0) {
                int nbid = b.nbr[d];
                int nrank = nbid / (c->px * c->py / c->nranks);
                if (nrank != c->rank || c->nccl_self) remote = true;
            }
    const int bpr = c->px * c->py / c->nranks;
    const ncclComm_t hcomm = (xs && c->xcomm) ? c->xcomm : c->comm;
    std::vector<HaloMsg> sends, recvs;
    for (size_t i = 0; i < c->blocks.size(); ++i) {
        auto &b = c->blocks[i];
        const int gid = c->rank * bpr + (int)i;
        const XPlan &x = b.xp[kind];
        for (int d = 0; d < kNDir; ++d) {
            int nbid = b.nbr[d];
            if (nbid < 0) continue;
            int nrank = nbid / bpr;
            if (nrank == c->rank && !c->nccl_self) {
                BlockCtx &nbk = c->blocks[nbid - c->rank * bpr];
                const XPlan &y = nbk.xp[kind];
                int od = kOpp[d];
                if (x.slen[d] != y.rlen[od])
                    fail(TEA_ERR_STATE, "halo size mismatch %zu vs %zu", x.slen[d], y.rlen[od]);
                CK(cudaMemcpyAsync(nbk.recvbuf + y.roff[od], b.sendbuf + x.soff[d],
                                   x.slen[d] * sizeof(double), cudaMemcpyDeviceToDevice,
                                   st));
            } else {
                sends.push_back({gid, nbid, d, b.sendbuf + x.soff[d], x.slen[d], nrank});
                recvs.push_back({nbid, gid, kOpp[d], b.recvbuf + x.roff[d], x.rlen[d], nrank});
            }
        }
    }
    if (remote) {
        halo_post_order(sends, recvs);
        NK(ncclGroupStart());
        for (const HaloMsg &m : sends) NK(ncclSend(m.buf, m.len, ncclDouble, m.peer, hcomm, st));
        for (const HaloMsg &m : recvs) NK(ncclRecv(m.buf, m.len, ncclDouble, m.peer, hcomm, st));
        NK(ncclGroupEnd());
    }
    for (auto &b : c->blocks) {
        const XPlan &x = b.xp[kind];
        if (x.nrecv == 0) continue;
        double *F[4];
        for (int i = 0; i < nf; ++i) F[i] = b.f[fids_per_block_field[i]];
        K(c, TEA_K_UNPACK, 0.0, [&] {
            launch_unpack(F, nf, b.L.pitch, x.d_recv, x.nrecv, b.recvbuf, st);
        });
    }
    (void)nb;
}

// The reduction that ends an iteration and the depth-1 halo exchange of the field the next
// stencil pass reads (CG: r with [r.r]; block Jacobi: z with [r.z, r.r]; Jacobi / Chebyshev:
// u with [r.r]) depend on the same kernel and not on each other: with the overlap on (auto
// across processes) the exchange runs on the second stream (its own communicator) while the
// allreduce is in flight on the compute stream ("the r halo exchange is issued
// together with the rr allreduce"); joined before the next iteration.
void reduce_exchange(tea_ctx *c, int first, int n, int kind, const std::vector<int> &fields) {
    const bool want = c->opts.overlap > 0 || (c->opts.overlap == 0 && (c->nranks > 1 || c->nccl_self));
    if (c->px * c->py > 1 && c->xstream && want && !c->profiling) {
        CK(cudaEventRecord(c->ev_fork, c->stream));
        CK(cudaStreamWaitEvent(c->xstream, c->ev_fork, 0));
        exchange(c, kind, fields, c->xstream);
        CK(cudaEventRecord(c->ev_join, c->xstream));
        reduce(c, first, n);
        CK(cudaStreamWaitEvent(c->stream, c->ev_join, 0));
        return;
    }
    reduce(c, first, n);
    exchange(c, kind, fields);
}

// Boxes of owned cells sent to direction d, and halo cells received from it.
void send_box(const BlockLayout &L, int d, int dep, int *j0, int *j1, int *k0, int *k1) {
    *j0 = 0;
    *j1 = L.bx;
    *k0 = 0;
    *k1 = L.by;
    if (kDX[d] < 0) *j1 = dep;
    if (kDX[d] > 0) *j0 = L.bx - dep;
    if (kDY[d] < 0) *k1 = dep;
    if (kDY[d] > 0) *k0 = L.by - dep;
}
void recv_box(const BlockLayout &L, int d, int dep, int *j0, int *j1, int *k0, int *k1) {
    *j0 = 0;
    *j1 = L.bx;
    *k0 = 0;
    *k1 = L.by;
    if (kDX[d] < 0) { *j0 = -dep; *j1 = 0; }
    if (kDX[d] > 0) { *j0 = L.bx; *j1 = L.bx + dep; }
    if (kDY[d] < 0) { *k0 = -dep; *k1 = 0; }
    if (kDY[d] > 0) { *k0 = L.by; *k1 = L.by + dep; }
}

void build_xplans(tea_ctx *c, BlockCtx &b, int *d_boxes_base) {
    struct K2 {
        int nf, dep;
        bool corners;
    } kinds[X_COUNT] = {{1, 1, false}, {1, c->d, c->d > 1}, {2, c->d, c->d > 1},
                        {1, 1, false}, {1, 1, false}, {1, c->d + 1, true}};
    std::vector<int> host;
    int *dptr = d_boxes_base;
    for (int kd = 0; kd < X_COUNT; ++kd) {
        XPlan &x = b.xp[kd];
        x.nf = kinds[kd].nf;
        x.depth = kinds[kd].dep;
        std::vector<int> sb, rb;
        size_t so = 0, ro = 0;
        for (int d = 0; d < kNDir; ++d) {
            x.soff[d] = so;
            x.roff[d] = ro;
            x.slen[d] = x.rlen[d] = 0;
            if (b.nbr[d] < 0) continue;
            if (d >= 4 && !kinds[kd].corners) continue;
            for (int f = 0; f < x.nf; ++f) {
                int j0, j1, k0, k1;
                send_box(b.L, d, x.depth, &j0, &j1, &k0, &k1);
                sb.insert(sb.end(), {f, j0, j1, k0, k1});
                so += (size_t)(j1 - j0) * (k1 - k0);
                recv_box(b.L, d, x.depth, &j0, &j1, &k0, &k1);
                rb.insert(rb.end(), {f, j0, j1, k0, k1});
                ro += (size_t)(j1 - j0) * (k1 - k0);
            }
            x.slen[d] = so - x.soff[d];
            x.rlen[d] = ro - x.roff[d];
        }
        if (so > b.L.halo_cap || ro > b.L.halo_cap) fail(TEA_ERR_STATE, "halo buffer too small");
        x.nsend = (int)sb.size() / 5;
        x.nrecv = (int)rb.size() / 5;
        x.d_send = dptr;
        CK(cudaMemcpyAsync(dptr, sb.data(), sb.size() * sizeof(int), cudaMemcpyHostToDevice,
                           c->stream));
        dptr += 16 * 5 * 2;
        x.d_recv = dptr;
        CK(cudaMemcpyAsync(dptr, rb.data(), rb.size() * sizeof(int), cudaMemcpyHostToDevice,
                           c->stream));
        dptr += 16 * 5 * 2;
        CK(cudaStreamSynchronize(c->stream));
    }
}

// Descriptors of the direct in-process exchange (k_xcopy): for every block, neighbour direction
// and field of each exchange kind, the send box of the block and the matching receive box of
// the neighbour (same shapes as the packed path's).
void build_xcopy(tea_ctx *c) {
    struct K2 {
        int nf, dep;
        bool corners;
    } kinds[X_COUNT] = {{1, 1, false}, {1, c->d, c->d > 1}, {2, c->d, c->d > 1},
                        {1, 1, false}, {1, 1, false}, {1, c->d + 1, true}};
    const BlockCtx &b0 = c->blocks[0];
    XCopy *base = (XCopy *)((char *)b0.S - b0.L.scalars_off + b0.L.xdesc_off);
    const size_t per_kind = (size_t)c->px * c->py * 16;
    for (int kd = 0; kd < X_COUNT; ++kd) {
        std::vector<XCopy> v;
        for (size_t i = 0; i < c->blocks.size(); ++i) {
            const BlockCtx &b = c->blocks[i];
            for (int d = 0; d < kNDir; ++d) {
                if (b.nbr[d] < 0 || (d >= 4 && !kinds[kd].corners)) continue;
                const int nl = b.nbr[d] - c->rank * (int)c->blocks.size();
                const BlockCtx &nb = c->blocks[nl];
                int sj0, sj1, sk0, sk1, dj0, dj1, dk0, dk1;
                send_box(b.L, d, kinds[kd].dep, &sj0, &sj1, &sk0, &sk1);
                recv_box(nb.L, kOpp[d], kinds[kd].dep, &dj0, &dj1, &dk0, &dk1);
                if (sj1 - sj0 != dj1 - dj0 || sk1 - sk0 != dk1 - dk0)
                    fail(TEA_ERR_STATE, "direct exchange box mismatch");
                for (int f = 0; f < kinds[kd].nf; ++f)
                    v.push_back(XCopy{(int)i, nl, f, sj0, sk0, dj0, dk0, sj1 - sj0, sk1 - sk0});
            }
        }
        if (v.size() > per_kind) fail(TEA_ERR_STATE, "direct exchange table too small");
        c->xdesc[kd] = base + kd * per_kind;
        c->nxdesc[kd] = (int)v.size();
        if (!v.empty())
            CK(cudaMemcpyAsync(c->xdesc[kd], v.data(), v.size() * sizeof(XCopy),
                               cudaMemcpyHostToDevice, c->stream));
    }
}

// ------------------------------------------------------------------ Chebyshev schedule
struct ChebOpS {
    int code, arg;
};
std::vector<ChebOpS> cheb_schedule(int s, int d) {
    std::vector<ChebOpS> ops;
    if (s < 1 || d < 1) return ops;
    // final segment: up to d-1 steps ending at extension 1; other segments up to d
    // steps ending at extension 0 (each needs its operands valid to its length).
    int mlast = std::min(s, d - 1);
    int rest = s - mlast;
    std::vector<int> segs;
    if (rest > 0) {
        int nfull = (rest + d - 1) / d;
        int first = rest - (nfull - 1) * d;
        segs.push_back(first);
        for (int i = 1; i < nfull; ++i) segs.push_back(d);
    }
    if (mlast > 0) segs.push_back(mlast);
    int step = 0;
    for (size_t g = 0; g < segs.size(); ++g) {
        bool final_seg = (g + 1 == segs.size()) && mlast > 0;
        int m = segs[g];
        int depth = final_seg ? m + 1 : m;
        ops.push_back({g == 0 ? 1 : 3, depth});
        for (int i = 0; i < m; ++i) {
            ++step;
            int e = final_seg ? (m - i) : (m - 1 - i);
            ops.push_back({2, e});
        }
    }
    if (mlast == 0) ops.push_back({4, 1});
    // r is read pointwise by every step (and by the stencil of step 1): exchange it
    // once, deep enough for all of them.
    int rdep = 1, i = 0;
    for (auto &o : ops)
        if (o.code == 2) {
            ++i;
            rdep = std::max(rdep, i == 1 ? o.arg + 1 : o.arg);
        }
    // d >= 2: at least depth 2 so the corners come along (extended regions are
    // rectangles; their corner cells read r pointwise)
    ops[0].arg = d > 1 ? std::min(d, std::max(rdep, 2)) : 1;
    (void)step;
    return ops;
}

// ------------------------------------------------------------------ phase bodies
int zbuf(int i) { return F_Z0 + ((i - 1) % 3); }  // per-step path: z_i lives in Z[(i-1)%3]

// start of a field's allocation (orig points at cell (0,0,0))
double *field_base(const BlockCtx &b, int f) {
    return b.f[f] - (b.L.nz > 1 ? (size_t)b.L.H * b.L.ps : 0) - (size_t)b.L.H * b.L.pitch - b.L.X0;
}

// algorithmic bytes of a launch: streams x 8 B x owned cells
double sbytes(const BlockCtx &b, int streams) {
    return 8.0 * streams * (double)b.L.bx * (double)b.L.by * (double)b.L.nz;
}
// face-coefficient streams of a 2D stencil launch: g alone (tea_opts.kform) or Kx + Ky
int kstreams(const tea_ctx *c, const BlockCtx &b) {
    return (b.L.nz == 1 && c->opts.kform >= 0) ? 1 : 2;
}

void body_cg(tea_ctx *c, int par, bool last_sets_cond) {
    for (auto &b : c->blocks) {
        Region R = b.owned();
        Launch L = plan_spmv(c, b, R);
        K(c, TEA_K_SPMV, sbytes(b, 6 + kstreams(c, b)), [&] {
            launch_spmv(kargs(c, b), L, R, b.f[F_R0], b.f[F_P0 + par], b.f[F_P1 - par],
                        b.f[F_W], b.f[F_U], b.f[F_KX], b.f[F_KY], c->stream);
        });
    }
    reduce(c, 0, 1);
    for (auto &b : c->blocks) {
        Region R = b.owned();
        Launch L = plan_pw(c, b, R);
        K(c, TEA_K_UPDATE, sbytes(b, 3), [&] {
            launch_update(kargs(c, b, last_sets_cond), L, R, b.f[F_W], b.f[F_R0], c->stream);
        });
    }
    reduce_exchange(c, 1, 2, X_R1, {F_R0});
}

// Chebyshev chain z = B(A) r, one kernel per step (blocks with neighbours; or
// tb_steps == 1). fused: the first step also does r_out = r_in - alpha w (single
// block only). Returns the field holding z_s.
int cheb_chain(tea_ctx *c, int s, bool restart, bool fused, int rin, int rout, bool sets_cond,
               bool reduce_dots = true) {
    auto ops = cheb_schedule(s, c->d);
    int r = fused ? rout : rin;
    int step = 0;
    for (auto &op : ops) {
        if (op.code == 1) {  // X_RD is depth d >= arg (a superset of what is read)
            if (!fused) exchange(c, op.arg == 1 ? X_R1 : X_RD, {r});
        } else if (op.code == 3) {
            // pair (z_{i-1}, z_{i-2}) before step i = step+1; for i == 2 only z_1 matters
            exchange(c, X_Z2, {zbuf(step), step >= 2 ? zbuf(step - 1) : zbuf(step)});
        } else if (op.code == 4) {
            exchange(c, X_Z1, {zbuf(s)});
        } else {
            ++step;
            const int mode = step == 1 ? 0 : (step == 2 ? 1 : 2);
            const bool last = step == s;
            for (auto &b : c->blocks) {
                Region R = b.ext(op.arg);
                Region D = b.owned();
                Launch L = plan_st(c, b, R);
                const bool fu = fused && step == 1;
                const double *z1 = step >= 2 ? b.f[zbuf(step - 1)] : nullptr;
                const double *z2 = step >= 3 ? b.f[zbuf(step - 2)] : nullptr;
                int kid = step == 1 ? TEA_K_CHEB_FIRST : (last ? TEA_K_CHEB_LAST : TEA_K_CHEB_STEP);
                const int streams =
                    (mode == 0 ? (fu ? 4 : 2) : (mode == 1 ? 3 : 4)) + kstreams(c, b);
                K(c, kid, sbytes(b, streams), [&] {
                    launch_cheb(kargs(c, b, last && sets_cond), L, R, D, mode, step, last, fu,
                                restart, b.f[fu ? rin : r], b.f[F_W], b.f[rout], z1, z2,
                                b.f[zbuf(step)], b.f[F_KX], b.f[F_KY], c->stream);
                });
            }
            if (last && reduce_dots) reduce(c, 1, 2);
        }
    }
    return zbuf(s);
}

// Split s steps into passes of at most Mmax, balanced (e.g. 10 -> 4,3,3).
std::vector<int> tb_passes(int s, int mmax) {
    std::vector<int> v;
    const int P = (s + mmax - 1) / mmax;
    for (int p = 0; p < P; ++p) v.push_back(s / P + (p < s % P ? 1 : 0));
    return v;
}

int tb_steps(const tea_ctx *c) {
    int m = c->opts.tb_steps;
    if (m == 0) {
        // measured (profiles/r01g_tmem_cpa.txt, TMEM/cp.async passes): 5 steps per pass
        // beat one kernel per step from 640^2 up (50 vs 59 us per outer; 1024^2 72 vs 86,
        // 4096^2 ~500 vs 1520); smaller CPPCG blocks run the persistent solver.
        const double cells = (double)c->blocks[0].L.bx * c->blocks[0].L.by;
        m = cells >= 4.0e5 ? kTbMaxSteps : 1;
    }
    return std::min(m, kTbMaxSteps);
}

bool single_block(tea_ctx *c) { return c->px * c->py == 1; }
bool is3d(const tea_ctx *c) { return c->blocks[0].L.nz > 1; }

// Extra work of a temporally blocked chain (single-reduction CPPCG in fused form, CPPCG1F):
// pre = the first pass starts with the outer update p = z_s + beta p, u += alpha p,
// r' = r - alpha A p (reads z_s, p_in, r, u; writes p_out, u, r'); post = the last pass ends
// with q = A z_s and z_s . q (a third value in its grid reduction).
struct ChainX {
    bool pre = false, post = false;
    bool even = false;  // CPPCG1F on one block: the pass split of chain_passes(.., true)
    int zs = -1, pin = -1, pout = -1;
    // CPPCG with neighbour blocks, update fused into the first pass: exchange (r_old, w) at
    // depth d -- it needs no alpha, so it is issued before (and with overlap: concurrently
    // with) the p.w reduction, which this chain then performs
    bool xw = false;
    // CPPCG1F with neighbour blocks: r is already valid on ext(d) (no exchange before the
    // passes); after the last pass z_s is exchanged at depth d + 1 while the chain's one
    // reduction [z.q, r.z, r.r] is in flight
    bool noexch = false, xz = false;
    // CPPCG with the fused passes (faces from g): the last pass does u += alpha p with the
    // direction the SpMV just wrote (field pnew); the SpMV then skips its lazy u update
    bool upd = false;
    int pnew = -1;
};

// Passes of a chain. CPPCG1F on one block (pre and post): an even number of passes >= 2, so
// the first pass's output pair never aliases the z_s it reads (the last pass's pair).
std::vector<int> chain_passes(const tea_ctx *c, int s, bool f1) {
    if (!f1) return tb_passes(s, tb_steps(c));
    const int mmax = std::min(tb_steps(c), kTbMaxSteps);
    int P = std::max(2, (s + mmax - 1) / mmax);
    if (P % 2) ++P;
    std::vector<int> v;
    for (int p = 0; p < P; ++p) v.push_back(s / P + (p < s % P ? 1 : 0));
    return v;
}

// Temporally blocked chain: passes of M steps, each ONE kernel per block
// (tea_cheb_tb.cu). z pairs ping-pong: pass p writes (z_{last-1}, z_last) into
// pair p%2 = (Z0,Z1) or (Z2,Z3). Returns the field holding z_s.
// With neighbour blocks (matrix powers, P:L423-495 -- on chip): r is exchanged ONCE at
// depth d >= s + 1 (corners included); pass p then runs on bounds extended by
// 1 + (steps after it), so the last pass leaves z_s valid on the 1-cell ring the next
// SpMV reads; no z exchange. (One block: every extension is empty.)
int cheb_chain_tb(tea_ctx *c, int s, bool restart, bool fused, int rin, int rout,
                  bool sets_cond, bool reduce_dots = true, const ChainX &x = ChainX()) {
    const bool f1 = x.pre;  // CPPCG1F's one-block fused outer update
    const auto passes = chain_passes(c, s, x.even);
    const int pairA[2] = {F_Z0, F_Z2}, pairB[2] = {F_Z1, F_Z3};
    const bool blocks = !single_block(c);
    // Overlap: the depth-d exchange of r runs on the exchange stream while
    // the first pass computes, on the compute stream, every output cell whose inputs
    // (M rows / columns around it) are owned cells; the frame of the extended region
    // follows the exchange. The first pass must not be the last (its dot products are one
    // grid reduction); profiling keeps every launch on the compute stream.
    const bool want = c->opts.overlap > 0 || (c->opts.overlap == 0 && (c->nranks > 1 || c->nccl_self));
    const bool ovl = blocks && !x.noexch && c->xstream && want && !c->profiling &&
                     passes.size() > 1;
    if (blocks && !x.noexch) {
        // depth d >= s + 1, with corners: r, or (r_old, w) for the fused update
        const int kind = x.xw ? X_Z2 : X_RD;
        const std::vector<int> fields = x.xw ? std::vector<int>{rin, F_W} : std::vector<int>{rin};
        if (ovl) {
            CK(cudaEventRecord(c->ev_fork, c->stream));
            CK(cudaStreamWaitEvent(c->xstream, c->ev_fork, 0));
            exchange(c, kind, fields, c->xstream);
            CK(cudaEventRecord(c->ev_join, c->xstream));
        } else {
            exchange(c, kind, fields);
        }
    }
    if (x.xw) reduce(c, 0, 1);  // p.w -> alpha, while the exchange is in flight
    int step0 = 1, after = s;
    const int r = (fused || f1) ? rout : rin;
    for (size_t p = 0; p < passes.size(); ++p) {
        const int M = passes[p];
        after -= M;
        const bool first = p == 0, last = p + 1 == passes.size();
        const bool fu = fused && first;
        const bool pre = x.pre && first, post = x.post && last;
        // (post with odd M: z.(A z) from faces, no extra level -- tea_cheb_tb.cu POSTF)
        const int levels = M + (pre ? 1 : 0) + ((post && (M + (pre ? 1 : 0)) % 2 == 0) ? 1 : 0);
        const int o = p % 2, in = (p + 1) % 2;
        // the regions this pass is launched on, per block: the whole (extended) region, or
        // for the overlapped first pass the halo-free interior now and the frame after the
        // exchange has landed
        std::vector<std::vector<Region>> regs(c->blocks.size());
        std::vector<std::vector<Region>> frame(c->blocks.size());
        for (size_t i = 0; i < c->blocks.size(); ++i) {
            const BlockCtx &b = c->blocks[i];
            const Region R = blocks ? b.ext(1 + after) : b.owned();
            if (!(ovl && first)) {
                regs[i].push_back(R);
                continue;
            }
            const Region O = b.owned();
            Region I{b.nbr[0] >= 0 ? O.j0 + M : R.j0, b.nbr[1] >= 0 ? O.j1 - M : R.j1,
                     b.nbr[2] >= 0 ? O.k0 + M : R.k0, b.nbr[3] >= 0 ? O.k1 - M : R.k1};
            if (I.j0 >= I.j1 || I.k0 >= I.k1) {
                frame[i].push_back(R);  // block too small for an interior: all after
                continue;
            }
            regs[i].push_back(I);
            auto add = [&](Region q) {
                if (q.j0 < q.j1 && q.k0 < q.k1) frame[i].push_back(q);
            };
            add(Region{R.j0, R.j1, R.k0, I.k0});  // bottom band (full width)
            add(Region{R.j0, R.j1, I.k1, R.k1});  // top band
            add(Region{R.j0, I.j0, I.k0, I.k1});  // west strip
            add(Region{I.j1, R.j1, I.k0, I.k1});  // east strip
        }
        for (int phase = 0; phase < 2; ++phase) {
          if (phase == 1) {
              if (!(ovl && first)) break;
              CK(cudaStreamWaitEvent(c->stream, c->ev_join, 0));
          }
          for (size_t i = 0; i < c->blocks.size(); ++i)
          for (const Region &R : (phase == 0 ? regs[i] : frame[i])) {
            auto &b = c->blocks[i];
            const Region D = b.owned();
            const int jlim = b.L.pitch - b.L.X0;
            int ty = c->opts.tb_rows > 0 ? c->opts.tb_rows : 0;
            // tall tiles keep the 2-level-row pipeline fill small; whole waves (tb_auto_rows)
            if (ty <= 0) ty = tb_auto_rows(levels, R.j1 - R.j0, R.k1 - R.k0);
            // the reduction partials (2 or 3 per CTA) must fit the block's scratch
            const size_t nv = post ? 3 : 2;
            while (ty < R.k1 - R.k0 &&
                   nv * (size_t)tb_ctas(levels, R.j1 - R.j0, R.k1 - R.k0, ty) > b.L.partials_cap)
                ty *= 2;
            // algorithmic streams: reads, then writes
            int streams;
            const bool upd = x.upd && last;
            if (pre)
                streams = 4 + kstreams(c, b) + 3 + (last ? 1 : 2);  // z_s, p, r, u, g -> p, u, r', z..
            else
                streams = (first ? (fu ? 2 : 1) : 3) + kstreams(c, b) + (fu ? 1 : 0) +
                          (last ? 1 : 2) + (upd ? 3 : 0);  // writes: r', z_last(, z_{last-1}); p, u -> u
            const int kid = last ? TEA_K_TB_LAST : (first ? TEA_K_TB_FIRST : TEA_K_TB_MID);
            TbArgs f;
            f.rin = b.f[first && (fu || pre) ? rin : r];
            f.win = b.f[F_W];
            f.rout = b.f[rout];
            f.zin1 = pre ? b.f[x.zs] : (first ? nullptr : b.f[pairB[in]]);
            f.zin2 = first ? nullptr : b.f[pairA[in]];
            f.zoutA = b.f[pairA[o]];
            f.zoutB = b.f[pairB[o]];
            f.kx = b.f[F_KX];
            f.ky = b.f[F_KY];
            if (pre) {
                f.pin = b.f[x.pin];
                f.pout = b.f[x.pout];
                f.uio = b.f[F_U];
            }
            if (upd) {
                f.pin = b.f[x.pnew];
                f.uio = b.f[F_U];
            }
            K(c, kid, sbytes(b, streams), [&] {
                launch_cheb_tb(kargs(c, b, last && sets_cond), R, D, M, ty, jlim, step0, first,
                               fu, last, restart, pre, post, upd, f, c->stream);
            });
          }
        }
        step0 += M;
    }
    const int zs_out = pairB[(passes.size() - 1) % 2];
    if (x.xz && blocks) {
        // the next outer update runs on ext(d) and needs z_s on ext(d + 1): exchange it while
        // the single reduction is in flight ("the communications can be
        // overlapped")
        const bool ovx = c->xstream && want && !c->profiling;
        if (ovx) {
            CK(cudaEventRecord(c->ev_fork, c->stream));
            CK(cudaStreamWaitEvent(c->xstream, c->ev_fork, 0));
            exchange(c, X_ZD1, {zs_out}, c->xstream);
            CK(cudaEventRecord(c->ev_join, c->xstream));
            if (reduce_dots) reduce(c, 0, 3);
            CK(cudaStreamWaitEvent(c->stream, c->ev_join, 0));
        } else {
            exchange(c, X_ZD1, {zs_out});
            if (reduce_dots) reduce(c, 0, 3);
        }
        return zs_out;
    }
    if (reduce_dots) reduce(c, x.post ? 0 : 1, x.post ? 3 : 2);
    return zs_out;
}


// fused passes: 2D; with neighbour blocks only when the halo is deep enough for the whole
// chain at once (d >= s + 1, the paper's deep-halo regime)
bool use_tb(tea_ctx *c, int s) {
    if (is3d(c) || tb_steps(c) <= 1 || c->coef_slot < 0) return false;
    // the passes address a field with 32-bit offsets
    if ((double)c->blocks[0].L.rows * c->blocks[0].L.pitch >= 2147483648.0) return false;
    return single_block(c) || c->d >= s + 1;
}
// CPPCG1F: the pre / post levels form faces from g (kform >= 0) and need >= 2 passes
bool use_tb1f(tea_ctx *c, int s) {
    return use_tb(c, s) && c->opts.kform >= 0 && (!single_block(c) || s >= 2);
}

// reduce_dots = false: the caller folds the chain's [r.z, r.r] into its own single
// reduction (single-reduction CPPCG)
int chain(tea_ctx *c, int s, bool restart, bool fused, int rin, int rout, bool sets_cond,
          bool reduce_dots = true) {
    if (use_tb(c, s))
        return cheb_chain_tb(c, s, restart, fused, rin, rout, sets_cond, reduce_dots);
    return cheb_chain(c, s, restart, fused, rin, rout, sets_cond, reduce_dots);
}

// field holding z_s after a chain (same for every chain of a context and s)
int zs_field(tea_ctx *c, int s) {
    if (use_tb(c, s)) {
        const int P = (int)tb_passes(s, tb_steps(c)).size();
        return (P - 1) % 2 == 0 ? F_Z1 : F_Z3;
    }
    return zbuf(s);
}
// ... of CPPCG1F's chains: one block fused -> an even pass count -> Z3
int zs_field1f(tea_ctx *c, int s) {
    if (use_tb1f(c, s)) {
        const int P = (int)chain_passes(c, s, single_block(c)).size();
        return (P - 1) % 2 == 0 ? F_Z1 : F_Z3;
    }
    return zbuf(s);
}

void body_pcg(tea_ctx *c, int s, int par, bool sets_cond) {
    const bool fused = single_block(c);
    const int zs = zs_field(c, s);
    // with the fused passes and faces from g the last pass updates u (the SpMV's lazy update
    // moved where HBM bandwidth is idle: SpMV 7 -> 5 streams, last pass 5 -> 8)
    const bool upd = TEA_CPPCG_UPD && use_tb(c, s) && c->opts.kform >= 0;
    for (auto &b : c->blocks) {
        Region R = b.owned();
        Launch L = plan_spmv(c, b, R);
        K(c, TEA_K_SPMV, sbytes(b, (upd ? 4 : 6) + kstreams(c, b)), [&] {
            launch_spmv(kargs(c, b), L, R, b.f[zs], b.f[F_P0 + par], b.f[F_P1 - par],
                        b.f[F_W], b.f[F_U], b.f[F_KX], b.f[F_KY], c->stream, !upd);
        });
    }
    if (!fused && use_tb(c, s)) {
        // blocks with the fused passes: r -= alpha w in the first pass on the extended
        // bounds, from (r_old, w) exchanged at depth d -- no separate update kernel (its 3
        // streams), and the exchange overlaps the p.w reduction
        ChainX x;
        x.xw = true;
        x.upd = upd;
        x.pnew = F_P1 - par;
        cheb_chain_tb(c, s, false, true, F_R0 + par, F_R1 - par, sets_cond, true, x);
        return;
    }
    reduce(c, 0, 1);
    if (fused && use_tb(c, s)) {
        ChainX x;
        x.upd = upd;
        x.pnew = F_P1 - par;
        cheb_chain_tb(c, s, false, true, F_R0 + par, F_R1 - par, sets_cond, true, x);
    } else if (fused) {
        chain(c, s, false, true, F_R0 + par, F_R1 - par, sets_cond);
    } else {
        for (auto &b : c->blocks) {
            Region R = b.owned();
            Launch L = plan_pw(c, b, R);
            K(c, TEA_K_UPDATE, sbytes(b, 3), [&] {
                launch_update_nodot(kargs(c, b), L, R, b.f[F_W], b.f[F_R0], c->stream);
            });
        }
        chain(c, s, false, false, F_R0, F_R0, sets_cond);
    }
}

// Block-Jacobi PCG outer iteration (Sec. IV.C.1): spmv on z; fused update + strip solves.
void body_bj(tea_ctx *c, int par, bool sets_cond) {
    for (auto &b : c->blocks) {
        Region R = b.owned();
        Launch L = plan_spmv(c, b, R);
        K(c, TEA_K_SPMV, sbytes(b, 6 + kstreams(c, b)), [&] {
            launch_spmv(kargs(c, b), L, R, b.f[F_Z0], b.f[F_P0 + par], b.f[F_P1 - par],
                        b.f[F_W], b.f[F_U], b.f[F_KX], b.f[F_KY], c->stream);
        });
    }
    reduce(c, 0, 1);
    for (auto &b : c->blocks) {
        // reads r, w, Ky, c', 1/den; writes r, z
        K(c, TEA_K_BJ, sbytes(b, 7), [&] {
            launch_bj(kargs(c, b), b.owned(), true, sets_cond, b.f[F_W], b.f[F_R0], b.f[F_Z0],
                      b.f[F_KY], b.f[F_BJC], b.f[F_BJD], c->stream);
        });
    }
    reduce_exchange(c, 1, 2, X_Z1, {F_Z0});
}

// Single-reduction CG iteration (Chronopoulos-Gear): one fused kernel on a
// single block (r, w, s ping-pong: Z0/Z1 hold w, Z2/Z3 hold s); update -> halo -> A r
// with blocks. Either way ONE reduction [del, gam, rr] per iteration.
void body_cg1(tea_ctx *c, int par, bool sets_cond) {
    if (single_block(c)) {
        BlockCtx &b = c->blocks[0];
        Region R = b.owned();
        Launch L = plan_st(c, b, R);
        K(c, TEA_K_CG1, sbytes(b, 10 + kstreams(c, b)), [&] {
            launch_cg1(kargs(c, b, sets_cond), L, R, b.f[F_R0 + par], b.f[F_Z0 + par],
                       b.f[F_Z2 + par], b.f[F_R1 - par], b.f[F_Z1 - par], b.f[F_Z3 - par],
                       b.f[F_P0], b.f[F_U], b.f[F_KX], b.f[F_KY], c->stream);
        });
        return;
    }
    for (auto &b : c->blocks) {
        Region R = b.owned();
        Launch L = plan_pw(c, b, R);
        K(c, TEA_K_UPDATE, sbytes(b, 9), [&] {
            launch_cg1_update(kargs(c, b), L, R, b.f[F_Z0], b.f[F_Z2], b.f[F_P0], b.f[F_U],
                              b.f[F_R0], c->stream);
        });
    }
    exchange(c, X_R1, {F_R0});
    for (auto &b : c->blocks) {
        Region R = b.owned();
        Launch L = plan_st(c, b, R);
        K(c, TEA_K_CG1W, sbytes(b, 2 + kstreams(c, b)), [&] {
            launch_cg1_w(kargs(c, b, sets_cond), L, R, b.f[F_R0], b.f[F_Z0], b.f[F_KX],
                         b.f[F_KY], c->stream);
        });
    }
    reduce(c, 0, 3);
}

// Single-reduction CPPCG outer iteration (Chronopoulos-Gear PCG with M^-1 = B(A); oracle
// ORA_CPPCG1): pointwise update (alpha, beta from the last reduction; p = z + b p,
// s = q + b s, u += a p, r -= a s) -> Chebyshev chain z = B(A) r with r.z, r.r (no
// reduction of its own) -> q = A z with z.q -> ONE reduction of [z.q, r.z, r.r].
// Fields: z in zs_field, q in W, s in R1, p in P0 (no ping-pong: the update is pointwise).
void body_pcg1(tea_ctx *c, int s, int /*par*/, bool sets_cond) {
    const int zs = zs_field(c, s);
    for (auto &b : c->blocks) {
        Region R = b.owned();
        Launch L = plan_pw(c, b, R);
        K(c, TEA_K_UPDATE, sbytes(b, 10), [&] {
            launch_cg1_update(kargs(c, b), L, R, b.f[F_W], b.f[F_R1], b.f[F_P0], b.f[F_U],
                              b.f[F_R0], c->stream, b.f[zs]);
        });
    }
    chain(c, s, false, false, F_R0, F_R0, false, false);
    for (auto &b : c->blocks) {
        Region R = b.owned();
        Launch L = plan_st(c, b, R);
        K(c, TEA_K_CG1W, sbytes(b, 2 + kstreams(c, b)), [&] {
            launch_cg1_w(kargs(c, b, sets_cond), L, R, b.f[zs], b.f[F_W], b.f[F_KX], b.f[F_KY],
                         c->stream, true);
        });
    }
    reduce(c, 0, 3);
}

// Single-reduction CPPCG in fused form (CPPCG1F; oracle ORA_CPPCG1F, reading R23): ONE
// reduction of [z.q, r.z, r.r] per outer iteration, like CPPCG1, with A p applied instead of
// carried. One block with the fused passes: TWO kernels per outer iteration -- the first pass
// does the outer update (p = z_s + beta p, u += alpha p, r' = r - alpha A p) and the first
// Chebyshev steps, the last pass the last steps and q = A z_s with the three dots (15 streams:
// 5 reads + 5 writes, then 4 + 1; CPPCG: 3 kernels, 18 streams). Blocks / one kernel per
// step: the update as one stencil pass (k_cg1f_pre), the chain (with the post level on the
// fused path, else q = A z_s by k_cg1_w), then the reduction.
// Fields: z_s in zs_field1f, p ping-pong P0/P1 by par; r ping-pong R0/R1 by par on the one-block
// fused path, in place (R0) otherwise.
void body_pcg1f(tea_ctx *c, int s, int par, bool sets_cond) {
    const int zs = zs_field1f(c, s);
    if (single_block(c) && use_tb1f(c, s)) {
        ChainX x;
        x.pre = x.post = x.even = true;
        x.zs = zs;
        x.pin = F_P0 + par;
        x.pout = F_P1 - par;
        cheb_chain_tb(c, s, false, false, F_R0 + par, F_R1 - par, sets_cond, true, x);
        return;
    }
    const bool tb = use_tb1f(c, s);
    for (auto &b : c->blocks) {
        // fused passes across blocks: the update runs on ext(d) (z_s arrived at depth d + 1
        // with the last reduction; p is kept valid on ext(d + 1) by this kernel's ring), so r
        // needs no exchange at all; else on the owned cells, r exchanged by the chain
        Region R = tb ? b.ext(c->d) : b.owned();
        Launch L = plan_spmv(c, b, R);
        K(c, TEA_K_UPDATE, sbytes(b, 7 + kstreams(c, b)), [&] {  // z, p, r, u -> p, r, u
            launch_cg1f_pre(kargs(c, b), L, R, b.owned(), b.f[zs], b.f[F_P0 + par],
                            b.f[F_P1 - par], b.f[F_R0], b.f[F_U], b.f[F_KX], b.f[F_KY],
                            c->stream);
        });
    }
    if (tb) {
        ChainX x;
        x.post = true;
        x.noexch = true;
        x.xz = true;
        cheb_chain_tb(c, s, false, false, F_R0, F_R0, sets_cond, true, x);
        return;
    }
    chain(c, s, false, false, F_R0, F_R0, false, false);
    for (auto &b : c->blocks) {
        Region R = b.owned();
        Launch L = plan_st(c, b, R);
        K(c, TEA_K_CG1W, sbytes(b, 2 + kstreams(c, b)), [&] {
            launch_cg1_w(kargs(c, b, sets_cond), L, R, b.f[zs], b.f[F_W], b.f[F_KX], b.f[F_KY],
                         c->stream, true);
        });
    }
    reduce(c, 0, 3);
}

// Stand-alone Jacobi / Chebyshev iteration: u ping-pongs between U and Z0 (par),
// the new iterate overwrites u_{k-1} in place; halo of the new iterate exchanged.
void body_stat(tea_ctx *c, bool cheb, int par, bool sets_cond) {
    const int in = par ? F_Z0 : F_U, out = par ? F_U : F_Z0;
    for (auto &b : c->blocks) {
        Region R = b.owned();
        Launch L = plan_st(c, b, R);
        K(c, TEA_K_STAT, sbytes(b, (cheb ? 4 : 3) + kstreams(c, b)), [&] {
            launch_stat(kargs(c, b, sets_cond), L, R, cheb, b.f[in], b.f[F_U0], b.f[out],
                        b.f[F_KX], b.f[F_KY], c->stream);
        });
    }
    reduce_exchange(c, 2, 1, X_U1, {out});
}

void read_state(tea_ctx *c) {
    CK(cudaMemcpyAsync(c->hS, c->blocks[0].S, offsetof(Scalars, cheb_a),
                       cudaMemcpyDeviceToHost, c->stream));
    wait_stream(c);
    resolve_profile(c);
}

// Run a phase loop until the device reports done. `body(par, sets_cond)` issues
// one iteration; bodies come in pairs (p / r ping-pong parity).
template <class B>
void run_loop(tea_ctx *c, long long key, int iters_hint, B body) {
    const int mode = c->profiling ? 2 : c->opts.loop_mode;
    if (mode == 2) {
        const int chunk = c->opts.check_interval > 0 ? c->opts.check_interval : 16;
        for (;;) {
            for (int i = 0; i < (chunk + 1) / 2; ++i) {
                body(0, false);
                body(1, false);
            }
            read_state(c);
            if (c->hS->done) return;
        }
    }
    if (mode == 1) {
        const int chunk = c->opts.check_interval > 0 ? c->opts.check_interval : 32;
        long long k = key * 1000003LL + 17 + chunk;
        auto it = c->graphs.find(k);
        if (it == c->graphs.end()) {
            long long l0 = c->launches;
            cudaGraph_t g;
            CK(cudaStreamBeginCapture(c->stream, cudaStreamCaptureModeThreadLocal));
            for (int i = 0; i < (chunk + 1) / 2; ++i) {
                body(0, false);
                body(1, false);
            }
            CK(cudaStreamEndCapture(c->stream, &g));
            cudaGraphExec_t ge;
            CK(cudaGraphInstantiate(&ge, g, 0));
            CK(cudaGraphDestroy(g));
            c->graph_kernels[k] = (int)(c->launches - l0);
            c->launches = l0;
            it = c->graphs.emplace(k, ge).first;
        }
        for (;;) {
            CK(cudaGraphLaunch(it->second, c->stream));
            c->launches += c->graph_kernels[k];
            read_state(c);
            if (c->hS->done) return;
        }
    }
    // mode 0: one graph with a WHILE conditional node around a 2-iteration body
    auto it = c->graphs.find(key);
    if (it == c->graphs.end()) {
        long long l0 = c->launches;
        cudaGraph_t g, bodyg;
        CK(cudaGraphCreate(&g, 0));
        cudaGraphConditionalHandle h;
        CK(cudaGraphConditionalHandleCreate(&h, g, 1, cudaGraphCondAssignDefault));
        cudaGraphNodeParams np = {};
        np.type = cudaGraphNodeTypeConditional;
        np.conditional.handle = h;
        np.conditional.type = cudaGraphCondTypeWhile;
        np.conditional.size = 1;
        cudaGraphNode_t node;
        CK(cudaGraphAddNode(&node, g, nullptr, 0, &np));
        bodyg = np.conditional.phGraph_out[0];
        CK(cudaStreamBeginCaptureToGraph(c->stream, bodyg, nullptr, nullptr, 0,
                                         cudaStreamCaptureModeThreadLocal));
        c->cond = h;
        body(0, true);
        body(1, true);
        c->cond = 0;
        cudaGraph_t captured;
        CK(cudaStreamEndCapture(c->stream, &captured));
        cudaGraphExec_t ge;
        CK(cudaGraphInstantiate(&ge, g, 0));
        CK(cudaGraphDestroy(g));
        c->graph_kernels[key] = (int)(c->launches - l0);
        c->launches = l0;
        it = c->graphs.emplace(key, ge).first;
    }
    const int it0 = c->hS->it;
    CK(cudaGraphLaunch(it->second, c->stream));
    read_state(c);
    const int bodies = (c->hS->it - it0) / 2 + 1;
    c->launches += (long long)bodies * c->graph_kernels[key];
    (void)iters_hint;
}

tea_status map_status(int ds, bool maxed) {
    switch (ds) {
        case DS_CONVERGED: return TEA_OK;
        case DS_LIMIT: return maxed ? TEA_NOT_CONVERGED : TEA_OK;
        case DS_BREAKDOWN:
        case DS_EIGFAIL: return TEA_ERR_BREAKDOWN;
        default: return TEA_ERR_STATE;
    }
}

// Whole solve in one cooperative launch (k_persist): one 2D block in one process, CG or
// CPPCG, device-loop mode, no per-kernel profiling. Auto (persist = 0): where it measured
// faster than the graph path (profiles/r01f_persist.txt): CG up to 1024^2 cells, CPPCG up
// to 512^2 (beyond, the per-phase barrier no longer hides behind the tile work).
bool use_persist(const tea_ctx *c, tea_method method) {
    if (c->opts.persist < 0) return false;
    if (method != TEA_CG && method != TEA_CPPCG) return false;
    if (c->px * c->py != 1 || c->nranks != 1 || is3d(c) || c->profiling) return false;
    if (c->opts.loop_mode != 0) return false;
    if (c->opts.persist == 1) return true;
    const double cells = (double)c->blocks[0].L.bx * c->blocks[0].L.by;
    return cells <= (method == TEA_CG ? TEA_PERSIST_AUTO_CG : TEA_PERSIST_AUTO_CPPCG);
}

void solve_persist(tea_ctx *c, int s, bool two_phase) {
    BlockCtx &b = c->blocks[0];
    PersistArgs P{};
    P.a = kargs(c, b);
    P.R = b.owned();
    Launch L = plan_st(c, b, P.R);
    if (c->opts.tile_rows <= 0) {
        // one tile per resident CTA: the phase time is the slowest CTA's tile chain, so
        // the tallest tiles that still fit the co-resident grid in ONE round
        const int cap = std::min(persist_ctas(1 << 30), (int)(b.L.partials_cap / 6));
        const int gx = (int)L.grid.x, height = P.R.k1 - P.R.k0;
        const int gy = std::max(1, cap / gx);
        const int ty = std::max(1, (height + gy - 1) / gy);
        L = plan_stencil(P.R, ty, 0);
    }
    P.jstart = L.jstart;
    P.ty = L.ty;
    P.gx = (int)L.grid.x;
    P.ntiles = (int)(L.grid.x * L.grid.y);
    P.s = s;
    P.two_phase = two_phase ? 1 : 0;
    P.kx = b.f[F_KX];
    P.ky = b.f[F_KY];
    P.u0 = b.f[F_U0];
    P.u = b.f[F_U];
    P.w = b.f[F_W];
    P.r[0] = b.f[F_R0];
    P.r[1] = b.f[F_R1];
    P.p[0] = b.f[F_P0];
    P.p[1] = b.f[F_P1];
    for (int i = 0; i < 3; ++i) P.z[i] = b.f[F_Z0 + i];
    P.part = b.partials;
    const int ctas = std::min(persist_ctas(P.ntiles), (int)(b.L.partials_cap / 6));
    K(c, TEA_K_PERSIST, 0.0, [&] { CK(launch_persist(P, ctas, c->stream)); });
    read_state(c);
}

tea_status solve_impl(tea_ctx *c, tea_method method, double eps, int max_iters, int s,
                      tea_stats *st) {
    if (c->failed) fail(TEA_ERR_STATE, "context already failed: %s", c->err.c_str());
    if (method < TEA_CG || method > TEA_CPPCG1F) fail(TEA_ERR_ARG, "bad method %d", (int)method);
    if (method == TEA_BJCG && is3d(c)) fail(TEA_ERR_ARG, "block Jacobi is 2D only");
    if (max_iters < 0) fail(TEA_ERR_ARG, "max_iters < 0");
    const bool pcg = method == TEA_CPPCG || method == TEA_CPPCG1 || method == TEA_CPPCG1F;
    if (pcg && (s < 1 || s > kMaxS))
        fail(TEA_ERR_ARG, "inner_steps must be in [1,%d]", kMaxS);
    const int pre = c->opts.presteps;
    if ((pcg || method == TEA_CHEBY) && (pre < 1 || pre > kMaxPre))
        fail(TEA_ERR_ARG, "presteps must be in [1,%d]", kMaxPre);
    c->profiling = c->opts.profile != 0;

    CK(cudaEventRecord(c->ev_in, c->user_stream));
    CK(cudaStreamWaitEvent(c->stream, c->ev_in, 0));
    CK(cudaEventRecord(c->ev_t0, c->stream));

    const bool two_phase = pcg || method == TEA_CHEBY;
    const int lim1 = two_phase ? std::min(pre, max_iters) : max_iters;
    for (auto &b : c->blocks)
        K(c, TEA_K_SCALAR, 0.0, [&] {
            launch_scalars(kargs(c, b), SC_BEGIN, eps, lim1, max_iters, c->opts.eig_margin_lo,
                           c->opts.eig_margin_hi, c->stream);
        });
    Nvtx nv_solve("tea_solve");
    const bool persist = use_persist(c, method);
    int ds = DS_RUNNING;
    bool phase2 = false;
    if (persist) {
        solve_persist(c, s, two_phase);
        ds = c->hS->status;
        phase2 = two_phase && c->hS->presteps > 0;
    } else {
    exchange(c, X_U1, {F_U});
    for (auto &b : c->blocks) {
        Region R = b.owned();
        Launch L = plan_st(c, b, R);
        K(c, TEA_K_RESIDUAL, sbytes(b, 3 + kstreams(c, b)), [&] {
            launch_residual(kargs(c, b), L, R, b.f[F_U], b.f[F_KX], b.f[F_KY], b.f[F_U0],
                            b.f[F_R0], c->stream);
        });
    }
    reduce(c, 1, 2);
    if (method == TEA_BJCG) {  // z = M^{-1} r, r.z, r.r (no update)
        // Thomas coefficients of the strips (they depend on A only) into the two fields
        // block Jacobi never uses (F_BJC = Z2, F_BJD = Z3): ~0.1 ms at 4096^2, no HBM kept
        // for them across solves of other methods
        for (auto &b : c->blocks)
            K(c, TEA_K_INIT, 0.0, [&] {
                launch_bj_setup(kargs(c, b), b.owned(), b.f[F_KX], b.f[F_KY], b.f[F_BJC],
                                b.f[F_BJD], c->stream);
            });
        for (auto &b : c->blocks)
            K(c, TEA_K_BJ, sbytes(b, 5), [&] {
                launch_bj(kargs(c, b), b.owned(), false, false, b.f[F_W], b.f[F_R0], b.f[F_Z0],
                          b.f[F_KY], b.f[F_BJC], b.f[F_BJD], c->stream);
            });
        reduce(c, 1, 2);
    }
    if (method == TEA_CG1) {  // w = A r, gam = r.r, del = w.r
        exchange(c, X_R1, {F_R0});
        for (auto &b : c->blocks) {
            Region R = b.owned();
            Launch L = plan_st(c, b, R);
            K(c, TEA_K_CG1W, sbytes(b, 2 + kstreams(c, b)), [&] {
                launch_cg1_w(kargs(c, b), L, R, b.f[F_R0], b.f[F_Z0], b.f[F_KX], b.f[F_KY],
                             c->stream);
            });
        }
        reduce(c, 0, 3);
    }
    for (auto &b : c->blocks)
        K(c, TEA_K_SCALAR, 0.0, [&] {
            launch_scalars(kargs(c, b), SC_R0, 0, 0, 0, 0, 0, c->stream);
        });
    if (method == TEA_BJCG)
        exchange(c, X_Z1, {F_Z0});
    else
        exchange(c, X_R1, {F_R0});
    read_state(c);

    // ---- phase 1: CG (or the CPPCG presteps), or block-Jacobi PCG
    if (!c->hS->done) {
        Nvtx nv_("tea phase 1 (CG / presteps)");
        if (method == TEA_BJCG)
            run_loop(c, 3, lim1, [&](int par, bool sc) { body_bj(c, par, sc); });
        else if (method == TEA_CG1)
            run_loop(c, 4, lim1, [&](int par, bool sc) { body_cg1(c, par, sc); });
        else if (method == TEA_JACOBI)
            run_loop(c, 5, lim1, [&](int par, bool sc) { body_stat(c, false, par, sc); });
        else
            run_loop(c, 1, lim1, [&](int par, bool sc) { body_cg(c, par, sc); });
    }
    ds = c->hS->status;
    if (method == TEA_JACOBI) {  // the final iterate is in Z0 after an odd count
        if (c->hS->it % 2 == 1)
            for (auto &b : c->blocks)
                CK(cudaMemcpyAsync(field_base(b, F_U), field_base(b, F_Z0), b.L.field_bytes,
                                   cudaMemcpyDeviceToDevice, c->stream));
    }
    phase2 = two_phase && ds == DS_LIMIT && c->hS->it < max_iters;
    if (phase2 && method == TEA_CHEBY) {
        for (auto &b : c->blocks)
            K(c, TEA_K_EIG, 0.0, [&] { launch_eig_setup(kargs(c, b), 1, c->stream); });
        read_state(c);
        const int pre0 = c->hS->it;
        if (!c->hS->done)
            run_loop(c, 6, max_iters, [&](int par, bool sc) { body_stat(c, true, par, sc); });
        if ((c->hS->it - pre0) % 2 == 1)
            for (auto &b : c->blocks)
                CK(cudaMemcpyAsync(field_base(b, F_U), field_base(b, F_Z0), b.L.field_bytes,
                                   cudaMemcpyDeviceToDevice, c->stream));
        ds = c->hS->status;
    } else if (phase2) {
        Nvtx nv_("tea phase 2 (eigen-estimate, restart, PCG)");
        // ---- eigen-estimate, coefficients, restart z = B(A) r, p = z
        for (auto &b : c->blocks)
            K(c, TEA_K_EIG, 0.0, [&] { launch_eig_setup(kargs(c, b), s, c->stream); });
        // the fused passes read the coefficients from constant memory (every block's copy
        // is identical: they derive from globally reduced scalars)
        if (use_tb(c, s)) CK(tb_coef_upload(c->coef_slot, c->blocks[0].S, c->stream));
        if (method == TEA_CPPCG1F) {
            // z = B(A) r, q = A z, [z.q, r.z, r.r] in one reduction (b_0 = 0)
            if (use_tb1f(c, s)) {
                ChainX x;
                x.post = true;
                x.even = single_block(c);
                x.xz = !single_block(c);  // blocks: z_s to depth d + 1 for the first update
                cheb_chain_tb(c, s, true, false, F_R0, F_R0, false, true, x);
            } else {
                chain(c, s, true, false, F_R0, F_R0, false, false);
                const int zs = zs_field1f(c, s);
                for (auto &b : c->blocks) {
                    Region R = b.owned();
                    Launch L = plan_st(c, b, R);
                    K(c, TEA_K_CG1W, sbytes(b, 2 + kstreams(c, b)), [&] {
                        launch_cg1_w(kargs(c, b), L, R, b.f[zs], b.f[F_W], b.f[F_KX], b.f[F_KY],
                                     c->stream, true);
                    });
                }
                reduce(c, 0, 3);
            }
        } else if (method == TEA_CPPCG1) {
            // z = B(A) r, q = A z, [z.q, r.z, r.r] in one reduction; p = s = 0 (b_0 = 0)
            chain(c, s, true, false, F_R0, F_R0, false, false);
            const int zs = zs_field(c, s);
            for (auto &b : c->blocks) {
                Region R = b.owned();
                Launch L = plan_st(c, b, R);
                K(c, TEA_K_CG1W, sbytes(b, 2 + kstreams(c, b)), [&] {
                    launch_cg1_w(kargs(c, b), L, R, b.f[zs], b.f[F_W], b.f[F_KX], b.f[F_KY],
                                 c->stream, true);
                });
            }
            reduce(c, 0, 3);
        } else {
            chain(c, s, true, false, F_R0, F_R0, false);
        }
        read_state(c);
        if (!c->hS->done) {
            if (method == TEA_CPPCG1)
                run_loop(c, 7 + 16LL * s, max_iters,
                         [&](int par, bool sc) { body_pcg1(c, s, par, sc); });
            else if (method == TEA_CPPCG1F)
                run_loop(c, 8 + 16LL * s, max_iters,
                         [&](int par, bool sc) { body_pcg1f(c, s, par, sc); });
            else
                run_loop(c, 2 + 16LL * s, max_iters,
                         [&](int par, bool sc) { body_pcg(c, s, par, sc); });
        }
        ds = c->hS->status;
    }
    }  // !persist
    CK(cudaEventRecord(c->ev_t1, c->stream));
    CK(cudaEventRecord(c->ev_in, c->stream));
    CK(cudaStreamWaitEvent(c->user_stream, c->ev_in, 0));
    wait_stream(c);
    float ms = 0.f;
    CK(cudaEventElapsedTime(&ms, c->ev_t0, c->ev_t1));
    const Scalars &h = *c->hS;
    const bool maxed = h.it >= max_iters;
    tea_status rs = map_status(ds, maxed);
    if (st) {
        st->iterations = h.it;
        st->presteps = phase2 ? h.presteps : 0;
        st->outer = phase2 ? h.outer : 0;
        st->inner_matvecs = phase2 && pcg ? s * (h.outer + 1) : 0;
        st->matvecs = 1 + h.it + st->inner_matvecs + (method == TEA_CG1 ? 1 : 0) +
                      (phase2 && method == TEA_CPPCG1 ? 1 : 0) +
                      (phase2 && method == TEA_CPPCG1F ? 1 + h.outer : 0);
        st->status = rs;
        st->r0 = h.r0;
        st->rnorm = std::sqrt(h.red_rr);
        st->eig_min = phase2 ? h.eig_min : 0.0;
        st->eig_max = phase2 ? h.eig_max : 0.0;
        st->ritz_min = phase2 ? h.ritz_min : 0.0;
        st->ritz_max = phase2 ? h.ritz_max : 0.0;
        st->seconds = ms * 1e-3;
    }
    if (rs < 0) fail(rs, "solver breakdown (device status %d) at iteration %d", ds, h.it);
    return rs;
}

}  // namespace

// ====================================================================== C ABI
extern "C" {

const char *tea_version(void) { return "tea-b200 0.1 (sm_100a, fp64)"; }
int tea_abi_version(void) { return TEA_ABI_VERSION; }

tea_status tea_get_nccl_id(void *id128) {
    if (!id128) return TEA_ERR_ARG;
    ncclUniqueId id;
    if (ncclGetUniqueId(&id) != ncclSuccess) return TEA_ERR_NCCL;
    static_assert(sizeof(id) == 128, "ncclUniqueId size");
    std::memcpy(id128, &id, sizeof id);
    return TEA_OK;
}

static tea_status check_decomp(const tea_mesh *m, const tea_dist *dist, int *px, int *py,
                               int *d, int *rank, int *nranks, std::string *why) {
    if (!m || m->nx < 1 || m->ny < 1 || !(m->xmax > m->xmin) || !(m->ymax > m->ymin)) {
        *why = "bad mesh";
        return TEA_ERR_ARG;
    }
    *px = dist ? dist->px : 1;
    *py = dist ? dist->py : 1;
    *d = dist ? dist->halo_depth : 1;
    *rank = dist ? dist->rank : 0;
    *nranks = dist ? dist->nranks : 1;
    if (*px < 1 || *py < 1 || *nranks < 1 || *rank < 0 || *rank >= *nranks) {
        *why = "bad px/py/rank/nranks";
        return TEA_ERR_ARG;
    }
    if ((*px * *py) % *nranks != 0) {
        *why = "px*py must be a multiple of nranks";
        return TEA_ERR_ARG;
    }
    if (*nranks > 1 && *px * *py != *nranks) {
        *why = "multi-process runs need exactly one block per rank (px*py == nranks)";
        return TEA_ERR_ARG;
    }
    if (m->nz > 1 && (*px * *py != 1 || *nranks != 1)) {
        *why = "3D meshes run on a single block (px = py = nranks = 1)";
        return TEA_ERR_ARG;
    }
    if (m->nz > 1 && !(m->zmax > m->zmin)) {
        *why = "bad z extent";
        return TEA_ERR_ARG;
    }
    if (*px * *py > 64) {
        *why = "at most 64 blocks";
        return TEA_ERR_ARG;
    }
    if (*d < 1 || *d > 16) {
        *why = "halo_depth must be in [1,16]";
        return TEA_ERR_ARG;
    }
    const int minw = std::min(m->nx / *px, m->ny / *py);
    if (*px * *py > 1 && minw < *d + 1) {
        *why = "blocks must be at least halo_depth+1 cells wide";
        return TEA_ERR_ARG;
    }
    return TEA_OK;
}

tea_status tea_workspace_bytes(const tea_mesh *mesh, const tea_dist *dist, size_t *bytes) {
    int px, py, d, rank, nranks;
    std::string why;
    if (!bytes) return TEA_ERR_ARG;
    tea_status s = check_decomp(mesh, dist, &px, &py, &d, &rank, &nranks, &why);
    if (s != TEA_OK) {
        g_init_error = why;
        return s;
    }
    const int bpr = px * py / nranks;
    size_t tot = 0;
    for (int b = rank * bpr; b < (rank + 1) * bpr; ++b) tot += layout_block(*mesh, px, py, d, b).total;
    *bytes = tot;
    return TEA_OK;
}

tea_status tea_init(tea_ctx **out, const tea_mesh *mesh, const double *density,
                    const double *energy, double dt, const tea_dist *dist, const tea_opts *opts,
                    void *d_workspace, size_t ws_bytes, void *cuda_stream) {
    if (!out) return TEA_ERR_ARG;
    *out = nullptr;
    std::unique_ptr<tea_ctx> c(new tea_ctx());
    try {
        int px, py, d, rank, nranks;
        std::string why;
        tea_status s = check_decomp(mesh, dist, &px, &py, &d, &rank, &nranks, &why);
        if (s != TEA_OK) fail(s, "%s", why.c_str());
        if (!density || !energy || !d_workspace) fail(TEA_ERR_ARG, "null pointer argument");
        if (!(dt >= 0.0) || !std::isfinite(dt)) fail(TEA_ERR_ARG, "bad dt");
        if (((uintptr_t)d_workspace) % 256) fail(TEA_ERR_ARG, "workspace must be 256-B aligned");
        size_t need = 0;
        tea_workspace_bytes(mesh, dist, &need);
        if (ws_bytes < need) fail(TEA_ERR_ARG, "workspace too small: %zu < %zu", ws_bytes, need);
        c->mesh = *mesh;
        c->px = px;
        c->py = py;
        c->d = d;
        c->rank = rank;
        c->nranks = nranks;
        c->dt = dt;
        const double dx = (mesh->xmax - mesh->xmin) / mesh->nx;
        const double dy = (mesh->ymax - mesh->ymin) / mesh->ny;
        c->rx = dt / (dx * dx);
        c->ry = dt / (dy * dy);
        tea_opts o{};
        o.presteps = 30;
        o.eig_margin_lo = 0.95;
        o.eig_margin_hi = 1.05;
        if (opts) {
            o = *opts;
            if (o.presteps == 0) o.presteps = 30;
            if (o.eig_margin_lo == 0.0) o.eig_margin_lo = 0.95;
            if (o.eig_margin_hi == 0.0) o.eig_margin_hi = 1.05;
        }
        if (o.loop_mode < 0 || o.loop_mode > 2) fail(TEA_ERR_ARG, "bad loop_mode");
        if (o.persist < -1 || o.persist > 1) fail(TEA_ERR_ARG, "bad persist");
        if (o.overlap < -1 || o.overlap > 1) fail(TEA_ERR_ARG, "bad overlap");
        if (o.kform < -1 || o.kform > 1) fail(TEA_ERR_ARG, "bad kform");
        if (o.trace < 0 || o.trace > 1) fail(TEA_ERR_ARG, "bad trace");
        const char *nse = std::getenv("TEA_NCCL_SELF");
        c->nccl_self = nranks == 1 && px * py > 1 && nse && std::atoi(nse) == 1;
        // NCCL kernels inside a WHILE-conditional graph body are not a supported
        // capture target: multi-process runs use chunked graphs (same kernels).
        const char *nsw = std::getenv("TEA_NCCL_SELF_WHILE");  // diagnostic: keep the WHILE graph
        if ((nranks > 1 || (c->nccl_self && !(nsw && std::atoi(nsw) == 1))) && o.loop_mode == 0)
            o.loop_mode = 1;
        c->opts = o;
        // every cell this rank stages (its blocks plus the margin; all of a 3D mesh): a
        // density <= 0 would silently become an insulating internal boundary
        {
            const int bpr0 = px * py / nranks, m0 = d + 1;
            const long long nzc = mesh->nz > 1 ? mesh->nz : 1;
            for (int bi = rank * bpr0; bi < (rank + 1) * bpr0; ++bi) {
                const BlockLayout L0 = layout_block(*mesh, px, py, d, bi);
                const int x0 = nzc > 1 ? 0 : std::max(0, L0.gx0 - m0);
                const int x1 = nzc > 1 ? mesh->nx : std::min(mesh->nx, L0.gx1 + m0);
                const int y0 = nzc > 1 ? 0 : std::max(0, L0.gy0 - m0);
                const int y1 = nzc > 1 ? mesh->ny : std::min(mesh->ny, L0.gy1 + m0);
                for (long long l = 0; l < nzc; ++l)
                    for (int k = y0; k < y1; ++k) {
                        const size_t row = ((size_t)l * mesh->ny + k) * mesh->nx;
                        for (int j = x0; j < x1; ++j) {
                            const double rh = density[row + j], en = energy[row + j];
                            if (!(rh > 0.0) || !std::isfinite(rh))
                                fail(TEA_ERR_ARG, "density must be finite and > 0 (cell %d,%d,%lld)",
                                     j, k, l);
                            if (!std::isfinite(en))
                                fail(TEA_ERR_ARG, "energy must be finite (cell %d,%d,%lld)", j, k, l);
                        }
                    }
            }
        }

        c->user_stream = (cudaStream_t)cuda_stream;
        CK(cudaStreamCreateWithFlags(&c->stream, cudaStreamNonBlocking));
        CK(cudaEventCreateWithFlags(&c->ev_in, cudaEventDisableTiming));
        CK(cudaEventCreate(&c->ev_t0));
        CK(cudaEventCreate(&c->ev_t1));
        if (px * py > 1) {
            CK(cudaStreamCreateWithFlags(&c->xstream, cudaStreamNonBlocking));
            CK(cudaEventCreateWithFlags(&c->ev_fork, cudaEventDisableTiming));
            CK(cudaEventCreateWithFlags(&c->ev_join, cudaEventDisableTiming));
        }
        CK(cudaMallocHost((void **)&c->hS, sizeof(Scalars)));
        std::memset(c->hS, 0, sizeof(Scalars));
        CK(cudaEventRecord(c->ev_in, c->user_stream));
        CK(cudaStreamWaitEvent(c->stream, c->ev_in, 0));

        if (nranks > 1) {
            if (!dist->nccl_id) fail(TEA_ERR_ARG, "nccl_id required when nranks > 1");
            ncclUniqueId id;
            std::memcpy(&id, dist->nccl_id, sizeof id);
            NK(ncclCommInitRank(&c->comm, nranks, id, rank));
            if (px * py > 1) NK(ncclCommSplit(c->comm, 0, rank, &c->xcomm, nullptr));
        } else if (c->nccl_self) {
            ncclUniqueId id;
            NK(ncclGetUniqueId(&id));
            NK(ncclCommInitRank(&c->comm, 1, id, 0));
            NK(ncclCommSplit(c->comm, 0, 0, &c->xcomm, nullptr));
        }

        const int bpr = px * py / nranks;
        char *ws = (char *)d_workspace;
        c->blocks.resize(bpr);
        for (int i = 0; i < bpr; ++i) {
            BlockCtx &b = c->blocks[i];
            b.id = rank * bpr + i;
            b.rank = rank;
            b.L = layout_block(*mesh, px, py, d, b.id);
            const BlockLayout &L = b.L;
            for (int f = 0; f < F_COUNT; ++f)
                b.f[f] = (double *)(ws + f * L.field_bytes) + (L.nz > 1 ? (size_t)L.H * L.ps : 0) +
                         (size_t)L.H * L.pitch + L.X0;
            b.S = (Scalars *)(ws + L.scalars_off);
            b.partials = (double *)(ws + L.partials_off);
            for (int dd = 0; dd < kNDir; ++dd) {
                int nbi = L.bi + kDX[dd], nbj = L.bj + kDY[dd];
                b.nbr[dd] = (nbi >= 0 && nbi < px && nbj >= 0 && nbj < py) ? nbj * px + nbi : -1;
            }
            CK(cudaMemsetAsync(ws, 0, L.total, c->stream));
            if (L.has_nbr) {
                b.sendbuf = (double *)(ws + L.halo_off);
                b.recvbuf = (double *)(ws + L.halo_off + round_up(L.halo_cap * sizeof(double), 256));
                build_xplans(c.get(), b, (int *)(ws + L.boxes_off));
            }
            if (L.nz > 1) {  // 3D, single block: stage plane by plane, zero margins
                const size_t hp = (size_t)mesh->nx * sizeof(double);
                const size_t plane = (size_t)mesh->nx * mesh->ny;
                for (int l = 0; l < L.nz; ++l) {
                    CK(cudaMemcpy2DAsync(b.f[F_W] + l * L.ps, L.pitch * sizeof(double),
                                         density + l * plane, hp, hp, mesh->ny,
                                         cudaMemcpyHostToDevice, c->stream));
                    CK(cudaMemcpy2DAsync(b.f[F_Z0] + l * L.ps, L.pitch * sizeof(double),
                                         energy + l * plane, hp, hp, mesh->ny,
                                         cudaMemcpyHostToDevice, c->stream));
                }
                const double dz = (mesh->zmax - mesh->zmin) / mesh->nz;
                K(c.get(), TEA_K_INIT, 0.0, [&] {
                    launch_init_fields3(kargs(c.get(), b), b.f[F_W], b.f[F_Z0], b.f[F_U0],
                                        b.f[F_U], b.f[F_KX], b.f[F_KY], b.f[F_KZ], L.bx, L.by,
                                        L.nz, c->rx, c->ry, dt / (dz * dz), o.mean_mode,
                                        c->stream);
                });
                CK(cudaMemsetAsync(ws + F_W * L.field_bytes, 0, L.field_bytes, c->stream));
                CK(cudaMemsetAsync(ws + F_Z0 * L.field_bytes, 0, L.field_bytes, c->stream));
                ws += L.total;
                continue;
            }
            // stage rho -> W, e -> Z0 over the block plus margin m (clipped to the mesh)
            const int m = d + 1;
            const int gx0 = std::max(0, L.gx0 - m), gx1 = std::min(mesh->nx, L.gx1 + m);
            const int gy0 = std::max(0, L.gy0 - m), gy1 = std::min(mesh->ny, L.gy1 + m);
            const size_t hp = (size_t)mesh->nx * sizeof(double);
            double *dW = b.f[F_W] + (size_t)(gy0 - L.gy0) * L.pitch + (gx0 - L.gx0);
            double *dZ = b.f[F_Z0] + (size_t)(gy0 - L.gy0) * L.pitch + (gx0 - L.gx0);
            CK(cudaMemcpy2DAsync(dW, L.pitch * sizeof(double), density + (size_t)gy0 * mesh->nx + gx0,
                                 hp, (gx1 - gx0) * sizeof(double), gy1 - gy0,
                                 cudaMemcpyHostToDevice, c->stream));
            CK(cudaMemcpy2DAsync(dZ, L.pitch * sizeof(double), energy + (size_t)gy0 * mesh->nx + gx0,
                                 hp, (gx1 - gx0) * sizeof(double), gy1 - gy0,
                                 cudaMemcpyHostToDevice, c->stream));
            Region owned{0, L.bx, 0, L.by};
            Region all{-d, L.bx + d + 1, -d, L.by + d + 1};
            Region kxr{-d, L.bx + d + 1, -d, L.by + d};
            Region kyr{-d, L.bx + d, -d, L.by + d + 1};
            // g on every cell a face of kxr / kyr touches; the stored
            // faces are formed from the same g by the same expression as the kernels'
            Region gall{-d - 1, L.bx + d + 1, -d - 1, L.by + d + 1};
            K(c.get(), TEA_K_INIT, 0.0, [&] {
                launch_init_fields(kargs(c.get(), b), b.f[F_W], b.f[F_Z0], b.f[F_U0], b.f[F_U],
                                   b.f[F_KX], b.f[F_KY], b.f[F_KZ], owned, all, kxr, kyr, gall,
                                   0.5 * c->rx, 0.5 * c->ry, o.mean_mode, c->stream);
            });
            // the staging fields are solver fields with zero halos: clear them again
            CK(cudaMemsetAsync(ws + F_W * L.field_bytes, 0, L.field_bytes, c->stream));
            CK(cudaMemsetAsync(ws + F_Z0 * L.field_bytes, 0, L.field_bytes, c->stream));
            ws += L.total;
        }
        if (nranks == 1 && px * py > 1 && bpr <= kXMaxBlocks && !c->nccl_self)
            build_xcopy(c.get());
        CK(cudaStreamSynchronize(c->stream));
        c->coef_slot = tb_slot_acquire();
        *out = c.release();
        return TEA_OK;
    } catch (const TeaError &e) {
        g_init_error = e.msg;
        if (c->stream) cudaStreamSynchronize(c->stream);
        tea_finalize(c.release());
        return e.st;
    }
}

tea_status tea_solve(tea_ctx *ctx, tea_method method, double eps, int max_iters, int inner_steps,
                     tea_stats *stats) {
    if (!ctx) return TEA_ERR_ARG;
    try {
        return solve_impl(ctx, method, eps, max_iters, inner_steps, stats);
    } catch (const TeaError &e) {
        ctx->err = e.msg;
        if (e.st != TEA_ERR_ARG) ctx->failed = true;
        if (stats) stats->status = e.st;
        return e.st;
    }
}

tea_status tea_fetch(tea_ctx *ctx, double *u_host) {
    if (!ctx || !u_host) return TEA_ERR_ARG;
    try {
        if (ctx->failed) fail(TEA_ERR_STATE, "context failed: %s", ctx->err.c_str());
        for (auto &b : ctx->blocks) {
            const BlockLayout &L = b.L;
            const size_t plane = (size_t)ctx->mesh.nx * ctx->mesh.ny;
            for (int l = 0; l < L.nz; ++l)
                CK(cudaMemcpy2DAsync(u_host + l * plane + (size_t)L.gy0 * ctx->mesh.nx + L.gx0,
                                     ctx->mesh.nx * sizeof(double), b.f[F_U] + l * L.ps,
                                     L.pitch * sizeof(double), L.bx * sizeof(double), L.by,
                                     cudaMemcpyDeviceToHost, ctx->stream));
        }
        CK(cudaStreamSynchronize(ctx->stream));
        return TEA_OK;
    } catch (const TeaError &e) {
        ctx->err = e.msg;
        return e.st;
    }
}

tea_status tea_set_u(tea_ctx *ctx, const double *u_host) {
    if (!ctx || !u_host) return TEA_ERR_ARG;
    try {
        if (ctx->failed) fail(TEA_ERR_STATE, "context failed: %s", ctx->err.c_str());
        for (auto &b : ctx->blocks) {
            const BlockLayout &L = b.L;
            const size_t plane = (size_t)ctx->mesh.nx * ctx->mesh.ny;
            for (int l = 0; l < L.nz; ++l)
                CK(cudaMemcpy2DAsync(b.f[F_U] + l * L.ps, L.pitch * sizeof(double),
                                     u_host + l * plane + (size_t)L.gy0 * ctx->mesh.nx + L.gx0,
                                     ctx->mesh.nx * sizeof(double), L.bx * sizeof(double), L.by,
                                     cudaMemcpyHostToDevice, ctx->stream));
        }
        CK(cudaStreamSynchronize(ctx->stream));
        return TEA_OK;
    } catch (const TeaError &e) {
        ctx->err = e.msg;
        return e.st;
    }
}

tea_status tea_kernel_times(tea_ctx *ctx, double *ms, long long *launches, double *bytes,
                            int reset) {
    if (!ctx) return TEA_ERR_ARG;
    for (int i = 0; i < TEA_K_COUNT; ++i) {
        if (ms) ms[i] = ctx->kms[i];
        if (launches) launches[i] = ctx->kcount[i];
        if (bytes) bytes[i] = ctx->kbytes[i];
    }
    if (reset) {
        std::memset(ctx->kms, 0, sizeof ctx->kms);
        std::memset(ctx->kcount, 0, sizeof ctx->kcount);
        std::memset(ctx->kbytes, 0, sizeof ctx->kbytes);
    }
    return TEA_OK;
}

int tea_trace_read(tea_ctx *ctx, int cap, int *kid, double *bytes_per_launch,
                   long long *launches, double *ms, int reset) {
    if (!ctx || cap < 0) return TEA_ERR_ARG;
    try {
        if (ctx->failed) fail(TEA_ERR_STATE, "context failed: %s", ctx->err.c_str());
        const int n = (int)ctx->tslots.size();
        std::vector<unsigned long long> ns(n, 0ull), cnt(n, 0ull);
        std::vector<unsigned long long> h(2 * kTraceSlots);
        CK(cudaStreamSynchronize(ctx->stream));
        for (auto &b : ctx->blocks) {
            CK(cudaMemcpy(h.data(), b.S->trace_ns, sizeof(unsigned long long) * kTraceSlots,
                          cudaMemcpyDeviceToHost));
            CK(cudaMemcpy(h.data() + kTraceSlots, b.S->trace_n,
                          sizeof(unsigned long long) * kTraceSlots, cudaMemcpyDeviceToHost));
            for (int i = 0; i < n; ++i) {
                ns[i] += h[i];
                cnt[i] += h[kTraceSlots + i];
            }
            if (reset) {
                CK(cudaMemset(b.S->trace_ns, 0, sizeof(unsigned long long) * kTraceSlots));
                CK(cudaMemset(b.S->trace_n, 0, sizeof(unsigned long long) * kTraceSlots));
            }
        }
        for (int i = 0; i < n && i < cap; ++i) {
            if (kid) kid[i] = ctx->tslots[i].first;
            if (bytes_per_launch) bytes_per_launch[i] = ctx->tslots[i].second;
            if (launches) launches[i] = (long long)cnt[i];
            if (ms) ms[i] = 1e-6 * (double)ns[i];
        }
        return n;
    } catch (const TeaError &e) {
        ctx->err = e.msg;
        return e.st;
    }
}

long long tea_launch_count(const tea_ctx *ctx) { return ctx ? ctx->launches : 0; }

tea_status tea_finalize(tea_ctx *ctx) {
    if (!ctx) return TEA_OK;
    if (ctx->stream) cudaStreamSynchronize(ctx->stream);
    for (auto &g : ctx->graphs) cudaGraphExecDestroy(g.second);
    for (auto e : ctx->evpool) cudaEventDestroy(e);
    if (ctx->ev_in) cudaEventDestroy(ctx->ev_in);
    if (ctx->ev_t0) cudaEventDestroy(ctx->ev_t0);
    if (ctx->ev_t1) cudaEventDestroy(ctx->ev_t1);
    if (ctx->ev_fork) cudaEventDestroy(ctx->ev_fork);
    if (ctx->ev_join) cudaEventDestroy(ctx->ev_join);
    if (ctx->xstream) cudaStreamDestroy(ctx->xstream);
    if (ctx->hS) cudaFreeHost(ctx->hS);
    // a failed context may hold NCCL operations that were captured but never launched (a
    // failed graph instantiation) or a peer that is gone: ncclCommDestroy can then wait
    // forever, so it is aborted instead (TEA_NCCL_SELF_WHILE diagnostic, round 2)
    if (ctx->xcomm) (ctx->failed ? ncclCommAbort : ncclCommDestroy)(ctx->xcomm);
    if (ctx->comm) (ctx->failed ? ncclCommAbort : ncclCommDestroy)(ctx->comm);
    if (ctx->stream) cudaStreamDestroy(ctx->stream);
    tb_slot_release(ctx->coef_slot);
    delete ctx;
    return TEA_OK;
}

const char *tea_last_error(const tea_ctx *ctx) {
    return ctx ? ctx->err.c_str() : g_init_error.c_str();
}

tea_status tea_block_extent(const tea_mesh *mesh, int px, int py, int b, int *x0, int *x1,
                            int *y0, int *y1) {
    if (!mesh || px < 1 || py < 1 || b < 0 || b >= px * py) return TEA_ERR_ARG;
    split(mesh->nx, px, b % px, x0, x1);
    split(mesh->ny, py, b / px, y0, y1);
    return TEA_OK;
}

int tea_halo_order(const tea_mesh *mesh, int px, int py, int nranks, int rank, int depth,
                   int corners, int nfields, long long *out, int cap) {
    if (!mesh || px < 1 || py < 1 || nranks < 1 || (px * py) % nranks || rank < 0 ||
        rank >= nranks || depth < 1 || nfields < 1 || (!out && cap > 0))
        return TEA_ERR_ARG;
    const int bpr = px * py / nranks;
    std::vector<HaloMsg> sends, recvs;
    for (int i = 0; i < bpr; ++i) {
        const int gid = rank * bpr + i, bi = gid % px, bj = gid / px;
        int x0, x1, y0, y1;
        split(mesh->nx, px, bi, &x0, &x1);
        split(mesh->ny, py, bj, &y0, &y1);
        const int bx = x1 - x0, by = y1 - y0;
        for (int d = 0; d < kNDir; ++d) {
            const int ni = bi + kDX[d], nj = bj + kDY[d];
            if (ni < 0 || ni >= px || nj < 0 || nj >= py) continue;
            if (d >= 4 && !corners) continue;
            const int nbid = nj * px + ni, nrank = nbid / bpr;
            if (nrank == rank) continue;
            // the send box of build_xplans (send_box): depth columns / rows / both
            const size_t len = (size_t)nfields * (kDX[d] ? depth : bx) * (kDY[d] ? depth : by);
            sends.push_back({gid, nbid, d, nullptr, len, nrank});
            recvs.push_back({nbid, gid, kOpp[d], nullptr, len, nrank});
        }
    }
    halo_post_order(sends, recvs);
    const int n = (int)(sends.size() + recvs.size());
    if (n > cap) return n;  // the count only
    int k = 0;
    for (int op = 0; op < 2; ++op)
        for (const HaloMsg &m : op ? recvs : sends) {
            long long *o = out + 6 * k++;
            o[0] = op;
            o[1] = m.peer;
            o[2] = m.src;
            o[3] = m.dst;
            o[4] = m.dir;
            o[5] = (long long)m.len;
        }
    return n;
}

int tea_tb_plan(int levels, int width, int height, int ctas_per_sm, int nsm) {
    if (levels < 1 || levels > 6 || width < 1 || height < 1 || ctas_per_sm < 1 || nsm < 1)
        return TEA_ERR_ARG;
    return tb_plan_rows(levels, width, height, ctas_per_sm, nsm);
}

int tea_cheb_schedule(int s, int d, int *ops, int cap) {
    if (s < 1 || s > kMaxS || d < 1 || d > 16) return TEA_ERR_ARG;
    auto v = cheb_schedule(s, d);
    if ((int)v.size() > cap || !ops) return TEA_ERR_ARG;
    for (size_t i = 0; i < v.size(); ++i) {
        ops[2 * i] = v[i].code;
        ops[2 * i + 1] = v[i].arg;
    }
    return (int)v.size();
}

}  // extern "C"
