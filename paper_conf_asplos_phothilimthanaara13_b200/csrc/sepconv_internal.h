// sepconv_internal.h -- plan object and helpers shared by the host-side C++ files.
#pragma once
#include <cuda.h>
#include <cuda_runtime.h>

#include <array>
#include <atomic>
#include <cstdarg>
#include <cstdint>
#include <map>
#include <string>
#include <utility>

#include "../../include/sepconv.h"
#include "sepconv_launch.h"

namespace sepconv {

// ---- errors --------------------------------------------------------------------------
sepconv_status_t fail(sepconv_status_t st, const char *fmt, ...);
sepconv_status_t cuda_fail(cudaError_t e, const char *what);
// cuTensorMapEncodeTiled for a float32 3-D tensor (dims innermost first, byte strides of dims 1
// and 2), no swizzle, zero fill out of bounds; the driver entry point is resolved once
sepconv_status_t encode_tmap_f32_3d(CUtensorMap *map, const float *base, const uint64_t dims[3],
                                    const uint64_t strides_bytes[2], const uint32_t box[3]);
extern std::atomic<uint64_t> g_launches;

#define SC_CUDA(call)                                              \
    do {                                                           \
        cudaError_t _e = (call);                                   \
        if (_e != cudaSuccess) return ::sepconv::cuda_fail(_e, #call); \
    } while (0)

// ---- geometry of one launch sequence -----------------------------------------------------
// A set of nimg images of in_rows x in_cols (pitch ld_in, image stride in_img),
// producing output rows [row_begin, row_begin + rows) of each image's
// (in_rows-K+1) x (in_cols-K+1) valid region (pitch ld_out, stride out_img).
struct Geometry {
    int K;
    int nimg;
    int in_rows, in_cols;
    long long ld_in, in_img;
    int out_cols;
    long long ld_out, out_img;
    int row_begin, rows;
};

struct Candidate {
    int algo;      // SEPCONV_2D / SEPCONV_SEPARABLE
    int mapping;   // SEPCONV_MAP_DIRECT / SEPCONV_MAP_TMA
    int fused;     // separable only
    int config;    // fused + TMA: stage configuration 0..kSepTmaConfigs-1 (stream_geom)
    int store;     // 0: 16-byte store path when every output row allows it, 1: always the 8-byte path
    int sched_parts = 0;   // work-schedule override (sepconv_choice_t.sched_parts): 0 = model
    int sched_grid = 0;    // CTAs of the override (0 = every resident slot)
    int sched_steal = 0;   // work stealing between warps: minimum stages a victim must have left (0 = off)
};

// The work schedule a launch uses (SegmentIter, sepconv_kernels.cuh): grid CTAs; parts > 0
// strided row partitions, 0 contiguous, -q the window schedule (win_rows, extra).
struct Sched {
    int grid, parts, win_rows, extra;
    int steal = 0;         // work-stealing threshold (strided schedule; 0 = off)
};

struct TensorMapCache {
    // key: every field the encoded map depends on -- (base, cols, rows, images, ld, image
    // stride, box width, box height) -- compared exactly, so two geometries on one base (band
    // interior / tail, the unfused ROWS pass's shifted pointer) never share a map
    std::map<std::array<long long, 8>, CUtensorMap> maps;
};

struct DeviceInfo {
    int device = -1;
    int sms = 0;
    int major = 0, minor = 0;
    size_t l2 = 0;
    size_t smem_optin = 0;
    std::string name;
};

}  // namespace sepconv

struct sepconv_plan_s {
    sepconv::DeviceInfo dev;
    int64_t n = 1, h = 0, w = 0;
    int k = 0;
    int64_t ld_in = 0, ld_out = 0, ho = 0, wo = 0;

    // unfused-separable workspace: the paper's `buffer` [H][W-K+1]
    float *buf = nullptr;
    int64_t ld_buf = 0;
    size_t buf_floats = 0;

    // tuned choices: [0] 2D, [1] SEPARABLE, [2] AUTO; best[i].source says where each came
    // from (tuned on this shape, or SELECT over a size selector)
    bool tuned = false;
    sepconv_choice_t best[3] = {};

    sepconv::TensorMapCache tmaps;

    // replay record of the last whole-plan single-kernel streaming launch (sepconv_run's fast
    // path): the same pointers, candidate and schedule mode reuse its parameter block, grid and
    // kernel, refreshing only the weights
    struct Replay {
        bool valid = false;
        const float *in = nullptr;
        float *out = nullptr;
        int algo = -1, mapping = -1, fused = -1, config = -1, store = -1, sched_parts = 0, sched_grid = 0,
            sched_steal = 0;
        int sched_mode = 0;                 // $SEPCONV_SCHED at record time
        int op = 0, map = 0, smode = 0, grid = 0;
        sepconv::StreamParams p;
    } replay;
    cudaEvent_t last_work = nullptr;

    // work stealing (sched_steal): a launch counter tags the claim words of each launch
    unsigned epoch = 0;
    unsigned long long *claims = nullptr;   // kMaxClaims words, zeroed at allocation

    // NCCL (row bands)
    void *comm = nullptr;
    bool band_external = false;   // sepconv_comm_init(id = NULL): the caller supplies the halo rows
    int nranks = 1, rank = 0;
    cudaStream_t comm_stream = nullptr;
    cudaEvent_t ev_in = nullptr, ev_halo = nullptr;
    // band timeline (sepconv_band_trace): timing events t0, interior start/end, exchange
    // start/end (comm stream), tail start/end of the last sepconv_run_band
    bool trace = false;
    cudaEvent_t tev[7] = {};

    // host-resident pipeline
    cudaStream_t hstream[3] = {nullptr, nullptr, nullptr};
    cudaEvent_t hev[4][2] = {};
    float *hin[2] = {nullptr, nullptr};
    float *hout[2] = {nullptr, nullptr};
    float *hbuf[2] = {nullptr, nullptr};
    int64_t hchunk_rows = 0;
};

namespace sepconv {
// core launcher shared by run / run_host / run_band / tune
sepconv_status_t launch_candidate(sepconv_plan_t plan, const Geometry &g, const float *in, float *out,
                                  const float *kernel, const Candidate &c, float *buf, long long ld_buf,
                                  cudaStream_t st);
Candidate resolve(sepconv_plan_t plan, sepconv_variant_t v);
// the schedule launch_candidate would give c on geometry g (model or override) and the
// resident-slot count it was sized for; single-kernel candidates only (fused, 2D)
sepconv_status_t candidate_sched(sepconv_plan_t plan, const Geometry &g, const Candidate &c, Sched *sc,
                                 long long *slots);
Candidate from_choice(const sepconv_choice_t &c);
sepconv_choice_t to_choice(const Candidate &c, int K, int source);
int candidate_warps(int K, const Candidate &c);
sepconv_status_t check_kernel(const float *kernel, int K);
Geometry plan_geometry(sepconv_plan_t plan);
sepconv_status_t ensure_buf(sepconv_plan_t plan);
}  // namespace sepconv

void sepconv_comm_destroy_internal(sepconv_plan_t plan);   // sepconv_band.cpp

// ---- NCCL, loaded at run time (sepconv_band.cpp); shared by the row-band paths ----------
namespace sepconv {
typedef int nccl_result_t;                 // the subset of the NCCL ABI we use (stable since 2.7)
typedef void *nccl_comm_t;
struct nccl_unique_id_t {
    char internal[SEPCONV_NCCL_ID_BYTES];
};
constexpr int kNcclFloat32 = 7;
struct NcclApi {
    bool ok = false;
    std::string why;
    nccl_result_t (*GetUniqueId)(nccl_unique_id_t *) = nullptr;
    nccl_result_t (*CommInitRank)(nccl_comm_t *, int, nccl_unique_id_t, int) = nullptr;
    nccl_result_t (*CommDestroy)(nccl_comm_t) = nullptr;
    nccl_result_t (*Send)(const void *, size_t, int, int, nccl_comm_t, cudaStream_t) = nullptr;
    nccl_result_t (*Recv)(void *, size_t, int, int, nccl_comm_t, cudaStream_t) = nullptr;
    nccl_result_t (*GroupStart)() = nullptr;
    nccl_result_t (*GroupEnd)() = nullptr;
    const char *(*GetErrorString)(nccl_result_t) = nullptr;
};
NcclApi &nccl();
sepconv_status_t nccl_fail(nccl_result_t r, const char *what);
sepconv_status_t comm_acquire(const unsigned char *id, int nranks, int rank, int device, void **out);
void comm_release(void *comm);
}  // namespace sepconv
void sepconv_seed_from_cache(sepconv_plan_t plan);         // sepconv_tune.cpp
