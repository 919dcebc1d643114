// sepconv_api.cpp -- the C ABI of include/sepconv.h: plans, validation, variant
// resolution and kernel launches.  Tuning is in sepconv_tune.cpp, the
// host-resident pipeline in sepconv_host.cpp, row bands + NCCL in sepconv_band.cpp.
#include <cuda.h>
#include <cuda_runtime.h>

#include <algorithm>
#include <array>
#include <cmath>
#include <cstdio>
#include <cstdlib>
#include <cstring>
#include <mutex>
#include <new>
#include <string>
#include <vector>

#include "sepconv_internal.h"

namespace sepconv {

std::atomic<uint64_t> g_launches{0};
static thread_local std::string t_last_error;

sepconv_status_t fail(sepconv_status_t st, const char *fmt, ...) {
    char msg[512];
    va_list ap;
    va_start(ap, fmt);
    vsnprintf(msg, sizeof msg, fmt, ap);
    va_end(ap);
    t_last_error = msg;
    return st;
}

sepconv_status_t cuda_fail(cudaError_t e, const char *what) {
    return fail(e == cudaErrorMemoryAllocation ? SEPCONV_E_NOMEM : SEPCONV_E_CUDA, "%s: %s (%s)", what,
                cudaGetErrorString(e), cudaGetErrorName(e));
}

static void clear_error() { t_last_error.clear(); }

// ---- device / driver helpers ---------------------------------------------------------------
typedef CUresult (*EncodeTiledFn)(CUtensorMap *, CUtensorMapDataType, cuuint32_t, void *, const cuuint64_t *,
                                  const cuuint64_t *, const cuuint32_t *, const cuuint32_t *, CUtensorMapInterleave,
                                  CUtensorMapSwizzle, CUtensorMapL2promotion, CUtensorMapFloatOOBfill);

static EncodeTiledFn encode_fn() {
    static EncodeTiledFn fn = nullptr;
    static std::once_flag once;
    std::call_once(once, [] {
        void *p = nullptr;
        cudaDriverEntryPointQueryResult q;
        if (cudaGetDriverEntryPoint("cuTensorMapEncodeTiled", &p, cudaEnableDefault, &q) == cudaSuccess &&
            q == cudaDriverEntryPointSuccess)
            fn = reinterpret_cast<EncodeTiledFn>(p);
    });
    return fn;
}

sepconv_status_t encode_tmap_f32_3d(CUtensorMap *map, const float *base, const uint64_t dims[3],
                                    const uint64_t strides_bytes[2], const uint32_t box[3]) {
    EncodeTiledFn enc = encode_fn();
    if (!enc) return fail(SEPCONV_E_CUDA, "cuTensorMapEncodeTiled unavailable from the driver");
    cuuint64_t d[3] = {dims[0], dims[1], dims[2]};
    cuuint64_t st[2] = {strides_bytes[0], strides_bytes[1]};
    cuuint32_t bx[3] = {box[0], box[1], box[2]};
    cuuint32_t estr[3] = {1, 1, 1};
    CUresult r = enc(map, CU_TENSOR_MAP_DATA_TYPE_FLOAT32, 3, const_cast<float *>(base), d, st, bx, estr,
                     CU_TENSOR_MAP_INTERLEAVE_NONE, CU_TENSOR_MAP_SWIZZLE_NONE, CU_TENSOR_MAP_L2_PROMOTION_L2_256B,
                     CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
    if (r != CUDA_SUCCESS) return fail(SEPCONV_E_CUDA, "cuTensorMapEncodeTiled failed (CUresult %d)", (int)r);
    return SEPCONV_OK;
}

static sepconv_status_t query_device(int device, DeviceInfo *out) {
    int count = 0;
    cudaError_t e = cudaGetDeviceCount(&count);
    if (e != cudaSuccess || count == 0)
        return fail(SEPCONV_E_UNSUPPORTED, "no CUDA device (%s)", cudaGetErrorString(e));
    if (device < 0) SC_CUDA(cudaGetDevice(&device));
    if (device >= count) return fail(SEPCONV_E_INVALID, "device %d out of range (%d devices)", device, count);
    cudaDeviceProp prop;
    SC_CUDA(cudaGetDeviceProperties(&prop, device));
    if (prop.major != 10)
        return fail(SEPCONV_E_UNSUPPORTED, "device %d is sm_%d%d; this library is built for sm_100a (B200)", device,
                    prop.major, prop.minor);
    out->device = device;
    out->sms = prop.multiProcessorCount;
    out->major = prop.major;
    out->minor = prop.minor;
    out->l2 = static_cast<size_t>(prop.l2CacheSize);
    out->smem_optin = prop.sharedMemPerBlockOptin;
    out->name = prop.name;
    return SEPCONV_OK;
}

struct DeviceGuard {
    int prev = -1;
    bool ok = true;
    explicit DeviceGuard(int dev) {
        cudaGetDevice(&prev);
        if (prev != dev) ok = cudaSetDevice(dev) == cudaSuccess;
    }
    ~DeviceGuard() {
        if (prev >= 0) cudaSetDevice(prev);
    }
};

// ---- validation ---------------------------------------------------------------------------------
sepconv_status_t check_kernel(const float *kernel, int K) {
    if (!kernel) return fail(SEPCONV_E_INVALID, "kernel is NULL (expected a host pointer to %d floats)", K);
    return SEPCONV_OK;
}

static bool aligned(const void *p, size_t a) { return (reinterpret_cast<uintptr_t>(p) % a) == 0; }

Geometry plan_geometry(sepconv_plan_t plan) {
    Geometry g;
    g.K = plan->k;
    g.nimg = static_cast<int>(plan->n);
    g.in_rows = static_cast<int>(plan->h);
    g.in_cols = static_cast<int>(plan->w);
    g.ld_in = plan->ld_in;
    g.in_img = plan->h * plan->ld_in;
    g.out_cols = static_cast<int>(plan->wo);
    g.ld_out = plan->ld_out;
    g.out_img = plan->ho * plan->ld_out;
    g.row_begin = 0;
    g.rows = static_cast<int>(plan->ho);
    return g;
}

static long long extent_floats(long long nimg, long long img, long long rows, long long ld, long long cols) {
    return (nimg - 1) * img + (rows - 1) * ld + cols;
}

// ---- launching ------------------------------------------------------------------------------------
static int map_index(bool tma, bool vec16) { return tma ? MAP_TMA : (vec16 ? MAP_DIRECT_VEC : MAP_DIRECT); }  // conv2d

static sepconv_status_t prepare_func(const KernelInfo &ki, int dev, const DeviceInfo &di, int *blocks_per_sm) {
    // attribute setting is cheap but not free: cache per (function, device)
    static std::mutex mu;
    static std::map<std::pair<const void *, int>, int> occ_cache;
    std::lock_guard<std::mutex> lock(mu);
    auto key = std::make_pair(ki.func, dev);
    auto it = occ_cache.find(key);
    if (it != occ_cache.end()) {
        *blocks_per_sm = it->second;
        return SEPCONV_OK;
    }
    if (ki.smem > di.smem_optin)
        return fail(SEPCONV_E_UNSUPPORTED, "kernel needs %zu B shared memory, device allows %zu", ki.smem,
                    di.smem_optin);
    SC_CUDA(cudaFuncSetAttribute(ki.func, cudaFuncAttributeMaxDynamicSharedMemorySize, static_cast<int>(ki.smem)));
    int occ = 0;
    SC_CUDA(cudaOccupancyMaxActiveBlocksPerMultiprocessor(&occ, ki.func, ki.threads, ki.smem));
    if (occ < 1) return fail(SEPCONV_E_UNSUPPORTED, "kernel cannot be resident (occupancy 0)");
    occ_cache[key] = occ;
    *blocks_per_sm = occ;
    return SEPCONV_OK;
}

static sepconv_status_t make_tmap(sepconv_plan_t plan, CUtensorMap *map, const float *base, int cols, int rows,
                                  int nimg, long long ld, long long img, int box_w, int box_h) {
    EncodeTiledFn enc = encode_fn();
    if (!enc) return fail(SEPCONV_E_CUDA, "cuTensorMapEncodeTiled unavailable from the driver");
    const std::array<long long, 8> key{static_cast<long long>(reinterpret_cast<uintptr_t>(base)), cols, rows, nimg,
                                       ld, img, box_w, box_h};
    auto it = plan->tmaps.maps.find(key);
    if (it != plan->tmaps.maps.end()) {
        *map = it->second;
        return SEPCONV_OK;
    }
    cuuint64_t dims[3] = {static_cast<cuuint64_t>(cols), static_cast<cuuint64_t>(rows), static_cast<cuuint64_t>(nimg)};
    cuuint64_t strides[2] = {static_cast<cuuint64_t>(ld) * 4, static_cast<cuuint64_t>(img) * 4};
    cuuint32_t box[3] = {static_cast<cuuint32_t>(box_w), static_cast<cuuint32_t>(box_h), 1};
    cuuint32_t estr[3] = {1, 1, 1};
    CUresult r = enc(map, CU_TENSOR_MAP_DATA_TYPE_FLOAT32, 3, const_cast<float *>(base), dims, strides, box, estr,
                     CU_TENSOR_MAP_INTERLEAVE_NONE, CU_TENSOR_MAP_SWIZZLE_NONE, CU_TENSOR_MAP_L2_PROMOTION_L2_256B,
                     CU_TENSOR_MAP_FLOAT_OOB_FILL_NONE);
    if (r != CUDA_SUCCESS) return fail(SEPCONV_E_CUDA, "cuTensorMapEncodeTiled failed (CUresult %d)", (int)r);
    if (plan->tmaps.maps.size() > 64) plan->tmaps.maps.clear();
    plan->tmaps.maps[key] = *map;
    return SEPCONV_OK;
}

static bool tma_ok(const float *base, long long ld, long long img) {
    return aligned(base, 16) && (ld % 4) == 0 && (img % 4) == 0;
}

// Work schedule (SegmentIter in sepconv_kernels.cuh).  Preferred: `parts` row partitions
// per (image, strip), handed out strip-fastest and strided over the grid, so the CTAs in
// flight walk a few row windows together (2 MB pages and DRAM rows stay hot; neighbouring
// strips read their shared halo columns at the same time) -- measured +8% at K=3..13 on
// 16384^2 over a contiguous split.  The part count and grid are chosen to maximise
//   (useful rows / (useful + warm-up rows)) x (items / (rounds x slots)),
// i.e. the K-1 warm-up rows every segment pays against the idle slots of the last round
// (64 x 4096^2: 4 strips x 64 images x 9 parts = 2304 items = 16 rounds of 144 CTAs).
// Tiny problems (fewer rows than a part needs) fall back to the exactly balanced
// contiguous split (parts = 0).
//
// When the strips do not divide the slots (16 CTA strips on 148 SMs at 16384^2: 144 CTAs,
// 4 SMs idle -- 2.7% of the FP32 pipes the K >= 15 kernels are bound by), the window
// schedule (parts = -q) keeps every slot busy: q windows of P rows one segment per CTA,
// and the e = slots - q*S leftover CTAs share the short last window, m = ceil(S/e)
// segments each; P solves P + o = m*(rows - q*P + o) (o = per-segment overhead in rows).
// $SEPCONV_SCHED = "nowin" disables it, "win" forces it where eligible (tests, A/B runs).
static Sched schedule_uncached(long long slots, int nimg, int nstrips, int rows, int K, bool no_win, bool force_win) {
    const long long strips = static_cast<long long>(nimg) * nstrips;
    // segments may be short: the score below already charges each one its K-1 warm-up rows,
    // and on small images (2048^2: 2 CTA strips) a floor of 4(K-1) rows left 86 of 148 SMs
    // idle at K=17 -- fill beats warm-up there
    const long long min_rows = 8;
    const long long max_parts = std::max<long long>(1, rows / min_rows);
    const double o = (K - 1) + 16.0;                           // warm-up + pipeline fill, rows
    double best = -1.0;
    long long best_p = 0, best_g = 0;
    Sched win{0, 0, 0, 0};
    double win_score = -1.0;
    if (!no_win && strips < slots && slots % strips != 0) {
        const long long q = slots / strips, e = slots - q * strips;
        const long long m = (strips + e - 1) / e;
        long long P = static_cast<long long>(std::ceil((m * static_cast<double>(rows) + (m - 1) * o) / (m * q + 1)));
        P = std::min<long long>(P, rows / q);
        const long long L = rows - q * P;
        if (P >= min_rows) {
            const double makespan = std::max(P + o, L > 0 ? m * (L + o) : 0.0);
            win_score = static_cast<double>(rows) * strips / (static_cast<double>(slots) * makespan);
            win = Sched{static_cast<int>(q * strips + (L > 0 ? e : 0)), static_cast<int>(-q), static_cast<int>(P),
                        static_cast<int>(L > 0 ? e : 0)};
        }
    }
    for (long long p = 1; p <= std::min<long long>(max_parts, 4096); ++p) {
        const long long items = strips * p;
        // grids to try: every slot, and the largest multiple of the strip count that fits
        const long long g_opts[2] = {std::min(slots, items), strips <= slots ? (slots / strips) * strips : 0};
        for (long long g : g_opts) {
            if (g <= 0) continue;
            const long long rounds = (items + g - 1) / g;
            const double fill = static_cast<double>(items) / static_cast<double>(rounds * slots);
            const double seg_rows = static_cast<double>(rows) / p;
            // K-1 warm-up rows + ~16 rows' worth of pipeline fill per segment
            const double useful = seg_rows / (seg_rows + (K - 1) + 16);
            const double score = fill * useful;
            if (score > best + 1e-9) {
                best = score;
                best_p = p;
                best_g = g;
            }
        }
    }
    // contiguous split: every slot busy, ~2 segments per CTA, but the CTAs in flight are
    // spread over the whole image (measured -8% at 16384^2): a locality factor of 0.92
    const long long total = strips * rows;
    const long long g_contig = std::min<long long>(slots, std::max<long long>(1, total / min_rows));
    const double contig_rows = static_cast<double>(total) / g_contig;
    const double contig_score = 0.92 * (contig_rows / (contig_rows + 2.0 * (K - 1 + 16))) *
                                (static_cast<double>(g_contig) / slots);
    // the same model for the strided schedule: rounds x (segment rows + o)
    if (win_score > 0 && (force_win || (win_score > best && win_score > contig_score))) return win;
    if (best_p > 0 && best >= contig_score) return Sched{static_cast<int>(best_g), static_cast<int>(best_p), 0, 0};
    return Sched{static_cast<int>(std::max<long long>(g_contig, 1)), 0, 0, 0};
}

// The search above walks up to 2 x 4096 part counts (~10 us of host time at 16384^2): memoised
// per (slots, images, strips, rows, K, mode), so a steady-state sepconv_run only looks it up.
static int sched_mode() {
    const char *mode = std::getenv("SEPCONV_SCHED");          // read per launch: tests flip it
    if (!mode) return 0;
    return std::strcmp(mode, "nowin") == 0 ? 1 : (std::strcmp(mode, "win") == 0 ? 2 : 0);
}

static Sched schedule(const DeviceInfo &di, int occ, int nimg, int nstrips, int rows, int K) {
    const int mode = sched_mode();
    const bool no_win = mode == 1;
    const bool force_win = mode == 2;
    const long long slots = static_cast<long long>(di.sms) * occ;
    static std::mutex mu;
    static std::map<std::array<long long, 6>, Sched> memo;
    const std::array<long long, 6> key{slots, nimg, nstrips, rows, K, no_win ? 1 : (force_win ? 2 : 0)};
    {
        std::lock_guard<std::mutex> lock(mu);
        auto it = memo.find(key);
        if (it != memo.end()) return it->second;
    }
    const Sched sc = schedule_uncached(slots, nimg, nstrips, rows, K, no_win, force_win);
    std::lock_guard<std::mutex> lock(mu);
    if (memo.size() > 4096) memo.clear();
    memo[key] = sc;
    return sc;
}

// A tuner-mutated schedule (sepconv_choice_t.sched_parts / sched_grid) replaces the model's:
// `parts` strided row partitions per (image, strip) over `grid` CTAs, both clamped to what the
// geometry and the resident slots allow.  Any (parts, grid) is a valid SegmentIter schedule.
static constexpr int kMaxClaims = 1 << 16;

static Sched apply_override(const Sched &model, long long slots, int nimg, int nstrips, int rows, int parts,
                            int grid, int steal = 0, int warps = 1, int stage_rows = 1, int K = 1) {
    if (parts <= 0) return model;
    const long long p = std::max(1, std::min(parts, rows));
    const long long items = static_cast<long long>(nimg) * nstrips * p;
    long long g = grid > 0 ? grid : slots;
    g = std::max<long long>(1, std::min(std::min(g, slots), items));
    Sched sc{static_cast<int>(g), static_cast<int>(p), 0, 0};
    // work stealing: one claim word per (segment, warp), stage counts in 16 bits
    const long long max_stages = ((rows + p - 1) / p + K - 1) / stage_rows + 2;
    if (steal > 0 && steal < 100 && items * warps <= kMaxClaims && max_stages < 65535) sc.steal = steal;
    return sc;
}

// the kernels that carry the work-stealing code (sepconv_kernels.cuh: fused TMA, free-running
// warps, at most 8 per CTA)
static bool steal_ok(int op, bool tma, int map, int K, int warps) {
    return op == OP_SEP && tma && warps <= 8 && !stream_geom(K, OP_SEP, map).lock;
}

static sepconv_status_t ensure_claims(sepconv_plan_t plan) {
    if (plan->claims) return SEPCONV_OK;
    SC_CUDA(cudaMalloc(&plan->claims, kMaxClaims * sizeof(unsigned long long)));
    SC_CUDA(cudaMemset(plan->claims, 0, kMaxClaims * sizeof(unsigned long long)));
    SC_CUDA(cudaDeviceSynchronize());          // zeroed before any stream's first stealing launch
    return SEPCONV_OK;
}

// One streaming pass (ROWS, COLS or SEP) over geometry g.
static sepconv_status_t launch_stream_op(sepconv_plan_t plan, int op, const Geometry &g, const float *in,
                                         long long ld_in, long long in_img, int in_cols, float *out,
                                         long long ld_out, long long out_img, int out_cols, int rows_total,
                                         const float *kernel, bool want_tma, int cfg, int store_path,
                                         cudaStream_t st, int ov_parts = 0, int ov_grid = 0, int ov_steal = 0,
                                         Sched *query = nullptr, long long *query_slots = nullptr,
                                         sepconv_plan_s::Replay *record = nullptr) {
    const int K = g.K;
    const bool tma = want_tma && tma_ok(in, ld_in, in_img);
    const bool vec = aligned(in, 16) && (ld_in % 4) == 0 && (in_img % 4) == 0;
    // variant: 0 direct, 1 direct 16-byte, 2.. TMA configurations (stream_geom)
    const int ntma = stream_variants(op) - 2;
    const int map = tma ? 2 + std::min(std::max(cfg, 0), ntma - 1) : (vec ? 1 : 0);
    const int store8 = (aligned(out, 16) && (ld_out % 4) == 0 && (out_img % 4) == 0) ? 2
                       : (aligned(out, 8) && (ld_out % 2) == 0 && (out_img % 2) == 0) ? 1 : 0;
    // store mode 3 (8-byte rows, even-width right-edge warps on the fast path, K >= 13 fused
    // TMA only): on images up to 8192 columns the edge warp's second loop copy costs 4-19%, on
    // wider ones the extra per-row predicates cost more than it (profiles/r02x_edge8_ab.txt)
    const int smode = (op == OP_SEP && tma && store_path == 2) ? 4
                      : (store8 == 2 && store_path == 0) ? 2
                      : (op == OP_SEP && tma && K >= 13 && (out_cols % 2) == 0 && out_cols <= 8192) ? 3 : 1;
    KernelInfo ki = stream_info(op, map, K, smode);
    int occ = 0;
    sepconv_status_t s = prepare_func(ki, plan->dev.device, plan->dev, &occ);
    if (s != SEPCONV_OK) return s;
    if (ki.cps > 0) occ = std::min(occ, ki.cps);

    StreamParams p;
    std::memset(&p, 0, sizeof p);
    p.in = in;
    p.out = out;
    p.in_img_stride = in_img;
    p.out_img_stride = out_img;
    p.ld_in = ld_in;
    p.ld_out = ld_out;
    p.in_rows = g.in_rows;
    p.in_cols = in_cols;
    p.out_cols = out_cols;
    p.row_begin = g.row_begin;
    p.rows = rows_total;
    p.nimg = g.nimg;
    const int cta_cols = (ki.threads / 32) * kWarpCols;
    p.nstrips = (out_cols + cta_cols - 1) / cta_cols;
    p.total = static_cast<long long>(g.nimg) * p.nstrips * rows_total;
    p.store8 = store8;
    for (int i = 0; i < K; ++i) {
        p.k[i] = kernel[i];
        p.k2[i] = make_float2(kernel[i], kernel[i]);
    }
    if (tma && !query) {
        s = make_tmap(plan, &p.tmap, in, in_cols, g.in_rows, g.nimg, ld_in, in_img, stream_bw(K, op), ki.stage_rows);
        if (s != SEPCONV_OK) return s;
    }
    const long long slots = static_cast<long long>(plan->dev.sms) * occ;
    const Sched sc = apply_override(schedule(plan->dev, occ, g.nimg, p.nstrips, rows_total, K), slots, g.nimg,
                                    p.nstrips, rows_total, ov_parts, ov_grid,
                                    steal_ok(op, tma, map, K, ki.threads / 32) ? ov_steal : 0, ki.threads / 32,
                                    std::max(1, ki.stage_rows), K);
    if (query) {                                               // candidate_sched: report, do not launch
        *query = sc;
        if (query_slots) *query_slots = slots;
        return SEPCONV_OK;
    }
    if (p.total <= 0) return SEPCONV_OK;
    p.parts = sc.parts;
    p.win_rows = sc.win_rows;
    p.extra = sc.extra;
    if (sc.steal > 0) {
        s = ensure_claims(plan);
        if (s != SEPCONV_OK) return s;
        p.steal = sc.steal;
        p.claims = plan->claims;
        p.epoch = ++plan->epoch;
        if (p.epoch == 0) p.epoch = ++plan->epoch;             // 0 is the words' initial value
    }
    cudaError_t e = stream_launch(op, map, K, smode, p, sc.grid, st);
    if (e != cudaSuccess) return cuda_fail(e, "stream kernel launch");
    g_launches.fetch_add(1, std::memory_order_relaxed);
    if (record) {
        record->op = op;
        record->map = map;
        record->smode = smode;
        record->grid = sc.grid;
        record->p = p;
        record->valid = true;
    }
    return SEPCONV_OK;
}

static sepconv_status_t launch_2d(sepconv_plan_t plan, const Geometry &g, const float *in, float *out,
                                  const float *kernel, bool want_tma, cudaStream_t st, int ov_parts = 0,
                                  int ov_grid = 0, Sched *query = nullptr, long long *query_slots = nullptr) {
    const int K = g.K;
    const bool tma = want_tma && tma_ok(in, g.ld_in, g.in_img);
    const bool vec = aligned(in, 16) && (g.ld_in % 4) == 0 && (g.in_img % 4) == 0;
    const int map = map_index(tma, vec);
    KernelInfo ki = conv2d_info(map, K);
    int occ = 0;
    sepconv_status_t s = prepare_func(ki, plan->dev.device, plan->dev, &occ);
    if (s != SEPCONV_OK) return s;
    Conv2DParams p;
    std::memset(&p, 0, sizeof p);
    p.in = in;
    p.out = out;
    p.in_img_stride = g.in_img;
    p.out_img_stride = g.out_img;
    p.ld_in = g.ld_in;
    p.ld_out = g.ld_out;
    p.in_rows = g.in_rows;
    p.in_cols = g.in_cols;
    p.out_cols = g.out_cols;
    p.row_begin = g.row_begin;
    p.rows = g.rows;
    p.nimg = g.nimg;
    const int cta_cols = kNW * kWarpCols;
    p.nstrips = (g.out_cols + cta_cols - 1) / cta_cols;
    p.total = static_cast<long long>(g.nimg) * p.nstrips * g.rows;
    p.store8 = (aligned(out, 8) && (g.ld_out % 2) == 0 && (g.out_img % 2) == 0) ? 1 : 0;   // conv2d: store() only
    // w_ji = fl(k_i * k_j): the outer-product weights of Convolve2D, rounded once
    for (int j = 0; j < K; ++j)
        for (int i = 0; i < K; ++i) p.w[j * K + i] = kernel[i] * kernel[j];
    if (tma && !query) {
        s = make_tmap(plan, &p.tmap, in, g.in_cols, g.in_rows, g.nimg, g.ld_in, g.in_img, box_width(K, true),
                      Conv2DCfg<1>::SR);
        if (s != SEPCONV_OK) return s;
    }
    const long long slots = static_cast<long long>(plan->dev.sms) * occ;
    const Sched sc = apply_override(schedule(plan->dev, occ, g.nimg, p.nstrips, g.rows, K), slots, g.nimg, p.nstrips,
                                    g.rows, ov_parts, ov_grid);
    if (query) {
        *query = sc;
        if (query_slots) *query_slots = slots;
        return SEPCONV_OK;
    }
    if (p.total <= 0) return SEPCONV_OK;
    p.parts = sc.parts;
    p.win_rows = sc.win_rows;
    p.extra = sc.extra;
    cudaError_t e = conv2d_launch(map, K, p, sc.grid, st);
    if (e != cudaSuccess) return cuda_fail(e, "conv2d kernel launch");
    g_launches.fetch_add(1, std::memory_order_relaxed);
    return SEPCONV_OK;
}

sepconv_status_t ensure_buf(sepconv_plan_t plan) {
    if (plan->buf) return SEPCONV_OK;
    plan->ld_buf = (plan->wo + 3) & ~3LL;
    plan->buf_floats = static_cast<size_t>(plan->n * plan->h * plan->ld_buf);
    cudaError_t e = cudaMalloc(&plan->buf, plan->buf_floats * sizeof(float));
    if (e != cudaSuccess) {
        plan->buf = nullptr;
        return cuda_fail(e, "cudaMalloc(unfused separable buffer)");
    }
    return SEPCONV_OK;
}

sepconv_status_t launch_candidate(sepconv_plan_t plan, const Geometry &g, const float *in, float *out,
                                  const float *kernel, const Candidate &c, float *buf, long long ld_buf,
                                  cudaStream_t st) {
    const bool tma = c.mapping == SEPCONV_MAP_TMA;
    // a schedule override was tuned for the plan's whole geometry; bands and host-pipeline
    // chunks (other row counts) use the model
    const bool whole = g.row_begin == 0 && g.rows == plan->ho && g.nimg == plan->n;
    const int ovp = whole ? c.sched_parts : 0, ovg = whole ? c.sched_grid : 0, ovs = whole ? c.sched_steal : 0;
    if (c.algo == SEPCONV_2D) return launch_2d(plan, g, in, out, kernel, tma, st, ovp, ovg);
    if (c.fused)
        return launch_stream_op(plan, OP_SEP, g, in, g.ld_in, g.in_img, g.in_cols, out, g.ld_out, g.out_img,
                                g.out_cols, g.rows, kernel, tma, c.config, c.store, st, ovp, ovg, ovs);
    // Choice 2 as the paper writes it: ConvolveRows into buffer, then ConvolveColumns.
    // The buffer holds the rows this launch's output rows need: [row_begin, row_begin + rows + K - 1).
    if (!buf) return fail(SEPCONV_E_INVALID, "unfused separable needs a workspace");
    const int brows = g.rows + g.K - 1;
    Geometry gr = g;
    gr.row_begin = 0;
    const long long buf_img = static_cast<long long>(brows) * ld_buf;
    // ROWS: input rows [row_begin, row_begin+brows) -> buf rows [0, brows)
    gr.in_rows = g.in_rows;
    {
        Geometry gg = g;
        gg.rows = brows;
        // shift the input pointer so buf row 0 = input row row_begin
        const float *in0 = in + static_cast<long long>(g.row_begin) * g.ld_in;
        gg.in_rows = g.in_rows - g.row_begin;
        gg.row_begin = 0;
        sepconv_status_t s = launch_stream_op(plan, OP_ROWS, gg, in0, g.ld_in, g.in_img, g.in_cols, buf, ld_buf,
                                              buf_img, g.out_cols, brows, kernel, tma, 0, 0, st);
        if (s != SEPCONV_OK) return s;
    }
    {
        Geometry gc = g;
        gc.in_rows = brows;
        gc.row_begin = 0;
        float *out0 = out + static_cast<long long>(g.row_begin) * g.ld_out;
        return launch_stream_op(plan, OP_COLS, gc, buf, ld_buf, buf_img, g.out_cols, out0, g.ld_out, g.out_img,
                                g.out_cols, g.rows, kernel, tma, 0, 0, st);
    }
}

sepconv_status_t candidate_sched(sepconv_plan_t plan, const Geometry &g, const Candidate &c, Sched *sc,
                                 long long *slots) {
    // the same pointers' alignment as the tuner's buffers (cudaMalloc: 256-byte aligned)
    const float *in = reinterpret_cast<const float *>(uintptr_t{256});
    float *out = reinterpret_cast<float *>(uintptr_t{512});
    const bool tma = c.mapping == SEPCONV_MAP_TMA;
    std::vector<float> k(g.K, 0.f);
    if (c.algo == SEPCONV_2D)
        return launch_2d(plan, g, in, out, k.data(), tma, nullptr, c.sched_parts, c.sched_grid, sc, slots);
    if (!c.fused) return fail(SEPCONV_E_INVALID, "candidate_sched: the unfused pair has two schedules");
    return launch_stream_op(plan, OP_SEP, g, in, g.ld_in, g.in_img, g.in_cols, out, g.ld_out, g.out_img, g.out_cols,
                            g.rows, k.data(), tma, c.config, c.store, nullptr, c.sched_parts, c.sched_grid,
                            c.sched_steal, sc, slots);
}

Candidate from_choice(const sepconv_choice_t &c) {
    Candidate r{static_cast<int>(c.algo), c.mapping, c.algo == SEPCONV_SEPARABLE ? c.fused : 0, c.config,
                c.store_path};
    r.sched_parts = c.sched_parts;
    r.sched_grid = c.sched_grid;
    r.sched_steal = c.sched_steal;
    return r;
}

sepconv_choice_t to_choice(const Candidate &c, int K, int source) {
    sepconv_choice_t o;
    std::memset(&o, 0, sizeof o);
    o.algo = static_cast<sepconv_variant_t>(c.algo);
    o.mapping = c.mapping;
    o.fused = c.fused;
    o.config = c.config;
    o.store_path = c.store;
    o.warps = candidate_warps(K, c);
    o.ctas_per_sm = (c.algo == SEPCONV_SEPARABLE && c.fused && c.mapping == SEPCONV_MAP_TMA)
                        ? std::max(1, stream_info(OP_SEP, 2 + c.config, K, 1).cps)
                        : 1;
    o.sched_parts = c.sched_parts;
    o.sched_grid = c.sched_grid;
    o.sched_steal = c.sched_steal;
    o.source = source;
    return o;
}

// Static default before tuning (R16): fused separable with TMA for K >= 2
// (one HBM pass, 2K FMA/px), 2D with TMA for K = 1.
static Candidate default_candidate(int K, sepconv_variant_t v) {
    if (v == SEPCONV_2D || (v == SEPCONV_AUTO && K == 1)) return {SEPCONV_2D, SEPCONV_MAP_TMA, 0, 0, 0};
    return {SEPCONV_SEPARABLE, SEPCONV_MAP_TMA, 1, 0, 0};
}

int candidate_warps(int K, const Candidate &c) {
    if (c.algo == SEPCONV_SEPARABLE && c.fused && c.mapping == SEPCONV_MAP_TMA)
        return stream_info(OP_SEP, 2 + c.config, K, 1).threads / 32;
    return kNW;
}

Candidate resolve(sepconv_plan_t plan, sepconv_variant_t v) {
    const int idx = v == SEPCONV_2D ? 0 : v == SEPCONV_SEPARABLE ? 1 : 2;
    if (plan->tuned) return from_choice(plan->best[idx]);
    return default_candidate(plan->k, v);
}

}  // namespace sepconv

using namespace sepconv;

// ==== C ABI ===========================================================================================
extern "C" {

const char *sepconv_version(void) { return "sepconv-b200 0.1 (sm_100a)"; }

const char *sepconv_status_str(sepconv_status_t s) {
    switch (s) {
        case SEPCONV_OK: return "ok";
        case SEPCONV_E_INVALID: return "invalid argument";
        case SEPCONV_E_ALIGN: return "misaligned pointer";
        case SEPCONV_E_ALIAS: return "input and output overlap";
        case SEPCONV_E_UNSUPPORTED: return "unsupported";
        case SEPCONV_E_NOMEM: return "out of memory";
        case SEPCONV_E_CUDA: return "CUDA error";
        case SEPCONV_E_NCCL: return "NCCL error";
    }
    return "unknown status";
}

const char *sepconv_last_error(void) { return t_last_error.c_str(); }

uint64_t sepconv_launch_count(void) { return g_launches.load(); }

// The clean L2 flush of DESIGN.md R25, shared by the tuner's timing and bench.py: library-owned
// scratch of 2 x L2 written, then a second 2 x L2 read, per device (allocated on first use).
// Not counted by sepconv_launch_count (it is measurement hygiene, not SeparableConvolution).
sepconv_status_t sepconv_l2_flush(sepconv_stream_t stream) {
    clear_error();
    int dev = -1;
    SC_CUDA(cudaGetDevice(&dev));
    struct Scratch {
        float *w = nullptr, *r = nullptr, *sink = nullptr;
        size_t n = 0;
    };
    static std::mutex mu;
    static std::map<int, Scratch> all;
    Scratch sc;
    {
        std::lock_guard<std::mutex> lock(mu);
        auto it = all.find(dev);
        if (it == all.end()) {
            int l2 = 0;
            SC_CUDA(cudaDeviceGetAttribute(&l2, cudaDevAttrL2CacheSize, dev));
            Scratch n;
            n.n = static_cast<size_t>(l2) / 2;                // floats in 2 x L2 bytes
            SC_CUDA(cudaMalloc(&n.w, n.n * 4));
            SC_CUDA(cudaMalloc(&n.r, n.n * 4));
            SC_CUDA(cudaMalloc(&n.sink, 16));
            SC_CUDA(cudaMemset(n.r, 0, n.n * 4));
            SC_CUDA(cudaDeviceSynchronize());
            it = all.emplace(dev, n).first;
        }
        sc = it->second;
    }
    cudaStream_t st = static_cast<cudaStream_t>(stream);
    SC_CUDA(launch_l2_flush(sc.w, static_cast<long long>(sc.n), st));
    SC_CUDA(launch_l2_clean(sc.r, static_cast<long long>(sc.n), sc.sink, st));
    return SEPCONV_OK;
}

static sepconv_status_t validate_desc(const sepconv_plan_desc_t *d) {
    if (!d) return fail(SEPCONV_E_INVALID, "descriptor is NULL");
    if (d->k > SEPCONV_MAX_K) return fail(SEPCONV_E_UNSUPPORTED, "K=%d exceeds SEPCONV_MAX_K=%d", d->k, SEPCONV_MAX_K);
    if (d->k < 1) return fail(SEPCONV_E_INVALID, "K=%d must be >= 1", d->k);
    if (d->n < 1) return fail(SEPCONV_E_INVALID, "n=%lld must be >= 1", (long long)d->n);
    if (d->h < d->k || d->w < d->k)
        return fail(SEPCONV_E_INVALID, "image %lldx%lld smaller than kernel width %d (output would be empty)",
                    (long long)d->h, (long long)d->w, d->k);
    if (d->h > (1LL << 30) || d->w > (1LL << 30) || d->n > (1LL << 30))
        return fail(SEPCONV_E_INVALID, "dimension too large");
    const int64_t ld_in = d->ld_in ? d->ld_in : d->w;
    const int64_t ld_out = d->ld_out ? d->ld_out : d->w - d->k + 1;
    if (ld_in < d->w) return fail(SEPCONV_E_INVALID, "ld_in=%lld < w=%lld", (long long)ld_in, (long long)d->w);
    if (ld_out < d->w - d->k + 1)
        return fail(SEPCONV_E_INVALID, "ld_out=%lld < w-k+1=%lld", (long long)ld_out, (long long)(d->w - d->k + 1));
    if (d->ld_in < 0 || d->ld_out < 0) return fail(SEPCONV_E_INVALID, "negative pitch");
    return SEPCONV_OK;
}

sepconv_status_t sepconv_plan_ex(const sepconv_plan_desc_t *desc, sepconv_plan_t *plan) {
    clear_error();
    if (!plan) return fail(SEPCONV_E_INVALID, "plan out-pointer is NULL");
    *plan = nullptr;
    sepconv_status_t s = validate_desc(desc);
    if (s != SEPCONV_OK) return s;
    DeviceInfo di;
    s = query_device(desc->device, &di);
    if (s != SEPCONV_OK) return s;
    sepconv_plan_s *p = new (std::nothrow) sepconv_plan_s();
    if (!p) return fail(SEPCONV_E_NOMEM, "host allocation of the plan failed");
    p->dev = di;
    p->n = desc->n;
    p->h = desc->h;
    p->w = desc->w;
    p->k = desc->k;
    p->ld_in = desc->ld_in ? desc->ld_in : desc->w;
    p->ho = desc->h - desc->k + 1;
    p->wo = desc->w - desc->k + 1;
    p->ld_out = desc->ld_out ? desc->ld_out : p->wo;
    DeviceGuard guard(di.device);
    cudaError_t e = cudaEventCreateWithFlags(&p->last_work, cudaEventDisableTiming);
    if (e != cudaSuccess) {
        delete p;
        return cuda_fail(e, "cudaEventCreate");
    }
    sepconv_seed_from_cache(p);
    *plan = p;
    return SEPCONV_OK;
}

sepconv_status_t sepconv_plan(int64_t H, int64_t W, int K, sepconv_plan_t *plan) {
    sepconv_plan_desc_t d;
    std::memset(&d, 0, sizeof d);
    d.n = 1;
    d.h = H;
    d.w = W;
    d.k = K;
    d.device = -1;
    return sepconv_plan_ex(&d, plan);
}

void sepconv_destroy(sepconv_plan_t plan) {
    if (!plan) return;
    DeviceGuard guard(plan->dev.device);
    if (plan->last_work) cudaEventSynchronize(plan->last_work);
    cudaDeviceSynchronize();
    sepconv_comm_destroy_internal(plan);
    if (plan->buf) cudaFree(plan->buf);
    for (int i = 0; i < 2; ++i) {
        if (plan->hin[i]) cudaFree(plan->hin[i]);
        if (plan->hout[i]) cudaFree(plan->hout[i]);
        if (plan->hbuf[i]) cudaFree(plan->hbuf[i]);
    }
    for (auto &s : plan->hstream)
        if (s) cudaStreamDestroy(s);
    for (auto &row : plan->hev)
        for (auto &ev : row)
            if (ev) cudaEventDestroy(ev);
    if (plan->last_work) cudaEventDestroy(plan->last_work);
    for (auto &e : plan->tev)
        if (e) cudaEventDestroy(e);
    if (plan->claims) cudaFree(plan->claims);
    delete plan;
}

sepconv_status_t sepconv_out_shape(sepconv_plan_t plan, int64_t *Ho, int64_t *Wo) {
    clear_error();
    if (!plan || !Ho || !Wo) return fail(SEPCONV_E_INVALID, "NULL argument");
    *Ho = plan->ho;
    *Wo = plan->wo;
    return SEPCONV_OK;
}

static sepconv_status_t check_io(sepconv_plan_t plan, const float *in, const float *out) {
    if (!in || !out) return fail(SEPCONV_E_INVALID, "in/out must be non-NULL device pointers");
    if (!aligned(in, 4) || !aligned(out, 4)) return fail(SEPCONV_E_ALIGN, "in/out must be 4-byte aligned");
    const long long ein = extent_floats(plan->n, plan->h * plan->ld_in, plan->h, plan->ld_in, plan->w);
    const long long eout = extent_floats(plan->n, plan->ho * plan->ld_out, plan->ho, plan->ld_out, plan->wo);
    const uintptr_t a0 = reinterpret_cast<uintptr_t>(in), a1 = a0 + ein * 4;
    const uintptr_t b0 = reinterpret_cast<uintptr_t>(out), b1 = b0 + eout * 4;
    if (a0 < b1 && b0 < a1) return fail(SEPCONV_E_ALIAS, "input and output ranges overlap (in-place is not supported)");
    return SEPCONV_OK;
}

static sepconv_status_t check_choice(const sepconv_choice_t *c) {
    if (!c) return fail(SEPCONV_E_INVALID, "choice is NULL");
    if (c->algo != SEPCONV_2D && c->algo != SEPCONV_SEPARABLE)
        return fail(SEPCONV_E_INVALID, "choice.algo must be SEPCONV_2D or SEPCONV_SEPARABLE");
    if (c->mapping != SEPCONV_MAP_DIRECT && c->mapping != SEPCONV_MAP_TMA)
        return fail(SEPCONV_E_INVALID, "choice.mapping must be DIRECT or TMA");
    if (c->config < 0 || c->config >= kSepTmaConfigs)
        return fail(SEPCONV_E_INVALID, "choice.config must be in [0, %d)", kSepTmaConfigs);
    if (c->store_path < 0 || c->store_path > 2) return fail(SEPCONV_E_INVALID, "choice.store_path must be 0, 1 or 2");
    if (c->sched_parts < 0 || c->sched_grid < 0)
        return fail(SEPCONV_E_INVALID, "choice.sched_parts / sched_grid must be >= 0");
    if (c->sched_steal < 0 || c->sched_steal > 99) return fail(SEPCONV_E_INVALID, "choice.sched_steal must be in [0, 99]");
    return SEPCONV_OK;
}

static sepconv_status_t run_resolved(sepconv_plan_t plan, const float *in, const float *kernel, float *out,
                                     const Candidate &c, cudaStream_t st) {
    sepconv_status_t s = check_io(plan, in, out);
    if (s != SEPCONV_OK) return s;
    s = check_kernel(kernel, plan->k);
    if (s != SEPCONV_OK) return s;
    DeviceGuard guard(plan->dev.device);
    if (c.algo == SEPCONV_SEPARABLE && !c.fused) {
        s = ensure_buf(plan);
        if (s != SEPCONV_OK) return s;
    }
    Geometry g = plan_geometry(plan);
    // (no per-call event: sepconv_destroy synchronises the device before freeing anything)
    if (!(c.algo == SEPCONV_SEPARABLE && c.fused))
        // the unfused buffer for a whole-image launch is [n][h][ld_buf] (rows = ho + K - 1 = h)
        return launch_candidate(plan, g, in, out, kernel, c, plan->buf, plan->ld_buf, st);
    // fused separable: replay the last launch's parameter block when nothing but the weights can
    // have changed (same pointers, candidate and schedule mode); else build it and record it
    sepconv_plan_s::Replay &r = plan->replay;
    const int mode = sched_mode();
    if (r.valid && r.in == in && r.out == out && r.algo == c.algo && r.mapping == c.mapping && r.fused == c.fused &&
        r.config == c.config && r.store == c.store && r.sched_parts == c.sched_parts &&
        r.sched_grid == c.sched_grid && r.sched_steal == c.sched_steal && r.sched_mode == mode) {
        for (int i = 0; i < plan->k; ++i) {
            r.p.k[i] = kernel[i];
            r.p.k2[i] = make_float2(kernel[i], kernel[i]);
        }
        if (r.p.steal > 0) {                                   // a fresh claim epoch per launch
            r.p.epoch = ++plan->epoch;
            if (r.p.epoch == 0) r.p.epoch = ++plan->epoch;
        }
        if (r.p.total <= 0) return SEPCONV_OK;
        cudaError_t e = stream_launch(r.op, r.map, plan->k, r.smode, r.p, r.grid, st);
        if (e != cudaSuccess) return cuda_fail(e, "stream kernel launch");
        g_launches.fetch_add(1, std::memory_order_relaxed);
        return SEPCONV_OK;
    }
    r.valid = false;
    s = launch_stream_op(plan, OP_SEP, g, in, g.ld_in, g.in_img, g.in_cols, out, g.ld_out, g.out_img, g.out_cols,
                         g.rows, kernel, c.mapping == SEPCONV_MAP_TMA, c.config, c.store, st, c.sched_parts,
                         c.sched_grid, c.sched_steal, nullptr, nullptr, &r);
    if (s == SEPCONV_OK && r.valid) {
        r.in = in;
        r.out = out;
        r.algo = c.algo;
        r.mapping = c.mapping;
        r.fused = c.fused;
        r.config = c.config;
        r.store = c.store;
        r.sched_parts = c.sched_parts;
        r.sched_grid = c.sched_grid;
        r.sched_steal = c.sched_steal;
        r.sched_mode = mode;
    }
    return s;
}

sepconv_status_t sepconv_run(sepconv_plan_t plan, const float *in, const float *kernel, float *out,
                             sepconv_variant_t variant, sepconv_stream_t stream) {
    clear_error();
    if (!plan) return fail(SEPCONV_E_INVALID, "plan is NULL");
    if (variant != SEPCONV_2D && variant != SEPCONV_SEPARABLE && variant != SEPCONV_AUTO)
        return fail(SEPCONV_E_INVALID, "variant %d is not 2D / SEPARABLE / AUTO", (int)variant);
    return run_resolved(plan, in, kernel, out, resolve(plan, variant), static_cast<cudaStream_t>(stream));
}

sepconv_status_t sepconv_run_choice(sepconv_plan_t plan, const float *in, const float *kernel, float *out,
                                    const sepconv_choice_t *choice, sepconv_stream_t stream) {
    clear_error();
    if (!plan) return fail(SEPCONV_E_INVALID, "plan is NULL");
    sepconv_status_t s = check_choice(choice);
    if (s != SEPCONV_OK) return s;
    return run_resolved(plan, in, kernel, out, from_choice(*choice), static_cast<cudaStream_t>(stream));
}

sepconv_status_t sepconv_get_choice(sepconv_plan_t plan, sepconv_variant_t variant, sepconv_choice_t *choice) {
    clear_error();
    if (!plan || !choice) return fail(SEPCONV_E_INVALID, "NULL argument");
    if (variant != SEPCONV_2D && variant != SEPCONV_SEPARABLE && variant != SEPCONV_AUTO)
        return fail(SEPCONV_E_INVALID, "bad variant");
    const int idx = variant == SEPCONV_2D ? 0 : variant == SEPCONV_SEPARABLE ? 1 : 2;
    if (plan->tuned) *choice = plan->best[idx];
    else *choice = to_choice(resolve(plan, variant), plan->k, SEPCONV_SRC_DEFAULT);
    return SEPCONV_OK;
}

sepconv_status_t sepconv_set_choice(sepconv_plan_t plan, sepconv_variant_t variant, const sepconv_choice_t *choice) {
    clear_error();
    if (!plan) return fail(SEPCONV_E_INVALID, "plan is NULL");
    if (variant != SEPCONV_2D && variant != SEPCONV_SEPARABLE && variant != SEPCONV_AUTO)
        return fail(SEPCONV_E_INVALID, "bad variant");
    sepconv_status_t s = check_choice(choice);
    if (s != SEPCONV_OK) return s;
    if (variant != SEPCONV_AUTO && choice->algo != static_cast<int>(variant))
        return fail(SEPCONV_E_INVALID, "choice.algo does not belong to the variant it is set for");
    if (!plan->tuned) {                                        // the others keep their resolution
        for (int v = 0; v < 3; ++v) {
            const sepconv_variant_t vv = v == 0 ? SEPCONV_2D : v == 1 ? SEPCONV_SEPARABLE : SEPCONV_AUTO;
            plan->best[v] = to_choice(resolve(plan, vv), plan->k, SEPCONV_SRC_DEFAULT);
        }
        plan->tuned = true;
    }
    const int idx = variant == SEPCONV_2D ? 0 : variant == SEPCONV_SEPARABLE ? 1 : 2;
    sepconv_choice_t c = to_choice(from_choice(*choice), plan->k, SEPCONV_SRC_EXPLICIT);
    c.median_us = choice->median_us;
    plan->best[idx] = c;
    return SEPCONV_OK;
}

}  // extern "C"
