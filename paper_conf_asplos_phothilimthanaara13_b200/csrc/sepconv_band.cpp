// sepconv_band.cpp -- row-band partition of one image across G GPUs (one process per
// GPU) with the one-sided (K-1)-row input halo exchanged by NCCL send/recv.
//
// The paper splits one output matrix into a first and second part across devices
// and has every task write a sub-region of one big buffer;
// here that split is G row bands.  Windows extend to +y, so
// band g needs K-1 input rows owned by band g+1 and nothing from band g-1.
//
// NCCL is loaded at run time with dlopen: the libnccl.so.2 already in the process
// (PyTorch's) when there is one, so the process never holds two NCCLs; else
// $SEPCONV_NCCL_LIB.  The C ABI therefore does not depend on NCCL at link time.
#include <cuda_runtime.h>
#include <dlfcn.h>

#include <cstdlib>
#include <cstring>
#include <map>
#include <mutex>
#include <string>

#include <nvtx3/nvToolsExt.h>

#include "sepconv_internal.h"

using namespace sepconv;

namespace sepconv {

NcclApi &nccl() {
    static NcclApi api;
    static std::once_flag once;
    std::call_once(once, [] {
        void *h = dlopen("libnccl.so.2", RTLD_NOW | RTLD_NOLOAD);
        if (!h) {
            const char *env = std::getenv("SEPCONV_NCCL_LIB");
            h = dlopen(env ? env : "libnccl.so.2", RTLD_NOW | RTLD_GLOBAL);
        }
        if (!h) {
            api.why = std::string("cannot load libnccl.so.2: ") + dlerror();
            return;
        }
#define SC_SYM(field, name)                                                   \
    api.field = reinterpret_cast<decltype(api.field)>(dlsym(h, name));        \
    if (!api.field) {                                                         \
        api.why = std::string("libnccl.so.2 lacks ") + name;                  \
        return;                                                               \
    }
        SC_SYM(GetUniqueId, "ncclGetUniqueId");
        SC_SYM(CommInitRank, "ncclCommInitRank");
        SC_SYM(CommDestroy, "ncclCommDestroy");
        SC_SYM(Send, "ncclSend");
        SC_SYM(Recv, "ncclRecv");
        SC_SYM(GroupStart, "ncclGroupStart");
        SC_SYM(GroupEnd, "ncclGroupEnd");
        SC_SYM(GetErrorString, "ncclGetErrorString");
#undef SC_SYM
        api.ok = true;
    });
    return api;
}

}  // namespace sepconv

namespace {

// Communicators are shared by every plan of the process that is initialised with the same
// unique id, rank and size (e.g. one plan per kernel width over the same row bands): the
// first sepconv_comm_init creates it collectively, later ones take a reference.
struct SharedComm {
    nccl_comm_t comm = nullptr;
    int nranks = 0, rank = 0, refs = 0, device = -1;
};
std::mutex g_comm_mu;
std::map<std::string, SharedComm> g_comms;

void release_comm(void *comm) {
    std::lock_guard<std::mutex> lock(g_comm_mu);
    for (auto it = g_comms.begin(); it != g_comms.end(); ++it) {
        if (it->second.comm == comm) {
            if (--it->second.refs == 0) {
                if (nccl().ok) nccl().CommDestroy(it->second.comm);
                g_comms.erase(it);
            }
            return;
        }
    }
}

}  // namespace

namespace sepconv {
sepconv_status_t nccl_fail(nccl_result_t r, const char *what) {
    NcclApi &a = nccl();
    return fail(SEPCONV_E_NCCL, "%s: %s", what, a.GetErrorString ? a.GetErrorString(r) : "error");
}

// A communicator for (id, nranks, rank) on `device`, created collectively on first use and
// reference-counted; release with comm_release.
sepconv_status_t comm_acquire(const unsigned char *id, int nranks, int rank, int device, void **out) {
    NcclApi &a = nccl();
    if (!a.ok) return fail(SEPCONV_E_NCCL, "%s", a.why.c_str());
    const std::string key(reinterpret_cast<const char *>(id), SEPCONV_NCCL_ID_BYTES);
    std::lock_guard<std::mutex> lock(g_comm_mu);
    auto it = g_comms.find(key);
    if (it != g_comms.end()) {
        if (it->second.nranks != nranks || it->second.rank != rank || it->second.device != device)
            return fail(SEPCONV_E_INVALID, "NCCL id already used with a different rank, size or device");
        ++it->second.refs;
        *out = it->second.comm;
        return SEPCONV_OK;
    }
    nccl_unique_id_t u;
    std::memcpy(u.internal, id, SEPCONV_NCCL_ID_BYTES);
    nccl_comm_t comm = nullptr;
    int prev = -1;
    cudaGetDevice(&prev);
    cudaSetDevice(device);
    nccl_result_t r = a.CommInitRank(&comm, nranks, u, rank);
    if (prev >= 0) cudaSetDevice(prev);
    if (r != 0) return nccl_fail(r, "ncclCommInitRank");
    SharedComm sc;
    sc.comm = comm;
    sc.nranks = nranks;
    sc.rank = rank;
    sc.refs = 1;
    sc.device = device;
    g_comms[key] = sc;
    *out = comm;
    return SEPCONV_OK;
}

void comm_release(void *comm) { release_comm(comm); }
}  // namespace sepconv

void sepconv_comm_destroy_internal(sepconv_plan_t plan) {
    if (plan->comm) release_comm(plan->comm);
    plan->comm = nullptr;
    if (plan->comm_stream) cudaStreamDestroy(plan->comm_stream);
    if (plan->ev_in) cudaEventDestroy(plan->ev_in);
    if (plan->ev_halo) cudaEventDestroy(plan->ev_halo);
    plan->comm_stream = nullptr;
    plan->ev_in = plan->ev_halo = nullptr;
    plan->band_external = false;
}

// NVTX range on the host timeline (visible to nsys / ncu --nvtx); popped once
struct NvtxScope {
    bool open = true;
    explicit NvtxScope(const char *name) { nvtxRangePushA(name); }
    void end() {
        if (open) nvtxRangePop();
        open = false;
    }
    ~NvtxScope() { end(); }
};

extern "C" {

sepconv_status_t sepconv_band(int64_t H, int K, int G, int g, int64_t *out_row0, int64_t *out_rows,
                              int64_t *in_rows_owned, int64_t *in_rows_alloc) {
    if (K < 1 || K > SEPCONV_MAX_K) return fail(K > SEPCONV_MAX_K ? SEPCONV_E_UNSUPPORTED : SEPCONV_E_INVALID,
                                                "K=%d out of range", K);
    if (H < K) return fail(SEPCONV_E_INVALID, "H=%lld < K=%d", (long long)H, K);
    if (G < 1 || g < 0 || g >= G) return fail(SEPCONV_E_INVALID, "band %d of %d", g, G);
    const int64_t ho = H - K + 1;
    if (G > 1 && ho / G < K - 1)
        return fail(SEPCONV_E_INVALID, "bands of %lld rows are thinner than the K-1=%d halo",
                    (long long)(ho / G), K - 1);
    if (G > ho) return fail(SEPCONV_E_INVALID, "more bands (%d) than output rows (%lld)", G, (long long)ho);
    const int64_t r0 = ho * g / G, r1 = ho * (g + 1) / G;
    if (out_row0) *out_row0 = r0;
    if (out_rows) *out_rows = r1 - r0;
    if (in_rows_alloc) *in_rows_alloc = r1 - r0 + K - 1;
    if (in_rows_owned) *in_rows_owned = (g == G - 1) ? (r1 - r0 + K - 1) : (r1 - r0);
    return SEPCONV_OK;
}

sepconv_status_t sepconv_nccl_unique_id(unsigned char id[SEPCONV_NCCL_ID_BYTES]) {
    if (!id) return fail(SEPCONV_E_INVALID, "id is NULL");
    NcclApi &a = nccl();
    if (!a.ok) return fail(SEPCONV_E_NCCL, "%s", a.why.c_str());
    nccl_unique_id_t u;
    nccl_result_t r = a.GetUniqueId(&u);
    if (r != 0) return nccl_fail(r, "ncclGetUniqueId");
    std::memcpy(id, u.internal, SEPCONV_NCCL_ID_BYTES);
    return SEPCONV_OK;
}

sepconv_status_t sepconv_comm_init(sepconv_plan_t plan, const unsigned char id[SEPCONV_NCCL_ID_BYTES], int nranks,
                                   int rank) {
    if (!plan) return fail(SEPCONV_E_INVALID, "NULL plan");
    if (nranks < 1 || rank < 0 || rank >= nranks) return fail(SEPCONV_E_INVALID, "rank %d of %d", rank, nranks);
    if (plan->n != 1) return fail(SEPCONV_E_INVALID, "row bands split a single image (plan has n=%lld)", (long long)plan->n);
    int prev = -1;
    cudaGetDevice(&prev);
    SC_CUDA(cudaSetDevice(plan->dev.device));
    sepconv_comm_destroy_internal(plan);
    SC_CUDA(cudaStreamCreateWithFlags(&plan->comm_stream, cudaStreamNonBlocking));
    SC_CUDA(cudaEventCreateWithFlags(&plan->ev_in, cudaEventDisableTiming));
    SC_CUDA(cudaEventCreateWithFlags(&plan->ev_halo, cudaEventDisableTiming));
    plan->nranks = nranks;
    plan->rank = rank;
    if (!id) {                        // external-halo mode: the caller moves the halo rows
        plan->band_external = true;
        if (prev >= 0) cudaSetDevice(prev);
        return SEPCONV_OK;
    }
    plan->band_external = false;
    sepconv_status_t st = comm_acquire(id, nranks, rank, plan->dev.device, &plan->comm);
    if (prev >= 0) cudaSetDevice(prev);
    return st;
}

sepconv_status_t sepconv_run_band(sepconv_plan_t plan, float *in_band, const float *kernel, float *out_band,
                                  sepconv_variant_t variant, sepconv_stream_t stream) {
    if (!plan) return fail(SEPCONV_E_INVALID, "plan is NULL");
    if (!plan->comm && !plan->band_external)
        return fail(SEPCONV_E_INVALID, "sepconv_comm_init has not been called on this plan");
    if (!in_band || !out_band) return fail(SEPCONV_E_INVALID, "NULL band pointer");
    if (variant != SEPCONV_2D && variant != SEPCONV_SEPARABLE && variant != SEPCONV_AUTO)
        return fail(SEPCONV_E_INVALID, "bad variant");
    sepconv_status_t s = check_kernel(kernel, plan->k);
    if (s != SEPCONV_OK) return s;
    NcclApi &a = nccl();
    const int K = plan->k;
    const bool last = plan->rank == plan->nranks - 1;
    const int halo = K - 1;
    const int64_t ho = plan->ho;   // this band's output rows (plan h = in_rows_alloc)
    if (!last && ho < halo) return fail(SEPCONV_E_INVALID, "band thinner than the halo");

    int prev = -1;
    cudaGetDevice(&prev);
    if (prev != plan->dev.device) SC_CUDA(cudaSetDevice(plan->dev.device));
    cudaStream_t st = static_cast<cudaStream_t>(stream);
    const Candidate c = resolve(plan, variant);
    if (c.algo == SEPCONV_SEPARABLE && !c.fused) {
        s = ensure_buf(plan);
        if (s != SEPCONV_OK) return s;
    }

    // timeline events (sepconv_band_trace): [0] start, [1,2] interior, [3,4] exchange, [5,6] tail
    cudaEvent_t *tv = plan->trace ? plan->tev : nullptr;
    NvtxScope whole("sepconv_run_band");
    if (tv) SC_CUDA(cudaEventRecord(tv[0], st));

    // 1. the exchange (comm stream, after the caller's writes to in_band on `st`)
    SC_CUDA(cudaEventRecord(plan->ev_in, st));
    SC_CUDA(cudaStreamWaitEvent(plan->comm_stream, plan->ev_in, 0));
    if (tv) SC_CUDA(cudaEventRecord(tv[3], plan->comm_stream));
    NvtxScope xchg("halo exchange (NCCL send/recv)");
    if (halo > 0 && plan->nranks > 1 && !plan->band_external) {
        const size_t cnt = static_cast<size_t>(halo) * plan->ld_in;
        nccl_comm_t comm = static_cast<nccl_comm_t>(plan->comm);
        nccl_result_t r = a.GroupStart();
        if (r == 0 && plan->rank > 0)        // my first K-1 rows complete band rank-1
            r = a.Send(in_band, cnt, kNcclFloat32, plan->rank - 1, comm, plan->comm_stream);
        if (r == 0 && !last)                 // rank+1's first K-1 rows complete my band
            r = a.Recv(in_band + ho * plan->ld_in, cnt, kNcclFloat32, plan->rank + 1, comm, plan->comm_stream);
        nccl_result_t r2 = a.GroupEnd();
        if (r != 0) return nccl_fail(r, "ncclSend/ncclRecv");
        if (r2 != 0) return nccl_fail(r2, "ncclGroupEnd");
    }
    if (tv) SC_CUDA(cudaEventRecord(tv[4], plan->comm_stream));
    SC_CUDA(cudaEventRecord(plan->ev_halo, plan->comm_stream));
    xchg.end();

    // 2. interior rows: need only owned input rows, overlap the exchange
    Geometry g = plan_geometry(plan);
    const int64_t interior = last ? ho : ho - halo;
    NvtxScope inner("interior rows");
    if (tv) SC_CUDA(cudaEventRecord(tv[1], st));
    if (interior > 0) {
        Geometry gi = g;
        gi.row_begin = 0;
        gi.rows = static_cast<int>(interior);
        s = launch_candidate(plan, gi, in_band, out_band, kernel, c, plan->buf, plan->ld_buf, st);
        if (s != SEPCONV_OK) return s;
    }
    if (tv) SC_CUDA(cudaEventRecord(tv[2], st));
    inner.end();
    // 3. tail rows after the halo has landed (and, on every rank, after our send
    //    has read in_band, so the caller may reuse it in stream order)
    NvtxScope tail("tail rows (after the halo)");
    SC_CUDA(cudaStreamWaitEvent(st, plan->ev_halo, 0));
    if (tv) SC_CUDA(cudaEventRecord(tv[5], st));
    if (!last && halo > 0) {
        Geometry gt = g;
        gt.row_begin = static_cast<int>(interior);
        gt.rows = halo;
        s = launch_candidate(plan, gt, in_band, out_band, kernel, c, plan->buf, plan->ld_buf, st);
        if (s != SEPCONV_OK) return s;
    }
    if (tv) SC_CUDA(cudaEventRecord(tv[6], st));
    SC_CUDA(cudaEventRecord(plan->last_work, st));
    if (prev >= 0 && prev != plan->dev.device) cudaSetDevice(prev);
    return SEPCONV_OK;
}

sepconv_status_t sepconv_band_trace(sepconv_plan_t plan, int enable) {
    if (!plan) return fail(SEPCONV_E_INVALID, "plan is NULL");
    int prev = -1;
    cudaGetDevice(&prev);
    SC_CUDA(cudaSetDevice(plan->dev.device));
    if (enable && !plan->tev[0])
        for (auto &e : plan->tev) SC_CUDA(cudaEventCreate(&e));
    plan->trace = enable != 0;
    if (prev >= 0) cudaSetDevice(prev);
    return SEPCONV_OK;
}

sepconv_status_t sepconv_band_timeline(sepconv_plan_t plan, float ms[6]) {
    if (!plan || !ms) return fail(SEPCONV_E_INVALID, "NULL argument");
    if (!plan->trace || !plan->tev[0]) return fail(SEPCONV_E_INVALID, "sepconv_band_trace is not enabled on this plan");
    SC_CUDA(cudaEventSynchronize(plan->tev[6]));
    for (int i = 0; i < 6; ++i) SC_CUDA(cudaEventElapsedTime(&ms[i], plan->tev[0], plan->tev[i + 1]));
    return SEPCONV_OK;
}

}  // extern "C"
