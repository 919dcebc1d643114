// sepconv_host.cpp -- host-resident end-to-end path.
//
// The paper's GPU task chain is prepare / copy-in / execute / copy-out
// and its reported times include the transfers.  Here
// the image is cut into row bands; band b's copy-in (H2D), kernel and copy-out
// (D2H) run on three plan-owned streams with two device slots, so the copy-in of
// band b+1 and the copy-out of band b-1 overlap the kernel of band b.  Each band
// carries its own K-1 halo rows (one-sided), so bands are independent.
#include <cuda_runtime.h>

#include <algorithm>
#include <cstring>

#include "sepconv_internal.h"

using namespace sepconv;

namespace {

constexpr size_t kChunkBytes = 16ull << 20;   // target input bytes per band (small: the pipeline fill/drain
                                              // of one band each way costs ~2 x 16 MB / 55 GB/s per call)

sepconv_status_t ensure_host_pipeline(sepconv_plan_t p, const Candidate &c) {
    if (!p->hstream[0]) {
        for (auto &s : p->hstream) SC_CUDA(cudaStreamCreateWithFlags(&s, cudaStreamNonBlocking));
        for (auto &row : p->hev)
            for (auto &ev : row) SC_CUDA(cudaEventCreateWithFlags(&ev, cudaEventDisableTiming));
    }
    if (!p->hchunk_rows) {
        int64_t r = static_cast<int64_t>(kChunkBytes / (static_cast<size_t>(p->ld_in) * 4));
        r = std::max<int64_t>(r, 4 * p->k);
        r = std::min<int64_t>(r, p->ho);
        p->hchunk_rows = std::max<int64_t>(r, 1);
        for (int i = 0; i < 2; ++i) {
            SC_CUDA(cudaMalloc(&p->hin[i], static_cast<size_t>((p->hchunk_rows + p->k - 1) * p->ld_in) * 4));
            SC_CUDA(cudaMalloc(&p->hout[i], static_cast<size_t>(p->hchunk_rows * p->ld_out) * 4));
        }
    }
    if (c.algo == SEPCONV_SEPARABLE && !c.fused && !p->hbuf[0]) {
        const int64_t ldb = (p->wo + 3) & ~3LL;
        for (int i = 0; i < 2; ++i)
            SC_CUDA(cudaMalloc(&p->hbuf[i], static_cast<size_t>((p->hchunk_rows + p->k - 1) * ldb) * 4));
    }
    return SEPCONV_OK;
}

}  // namespace

extern "C" sepconv_status_t sepconv_run_host(sepconv_plan_t plan, const float *in_host, const float *kernel,
                                             float *out_host, sepconv_variant_t variant, sepconv_stream_t stream) {
    if (!plan) return fail(SEPCONV_E_INVALID, "plan is NULL");
    if (!in_host || !out_host) return fail(SEPCONV_E_INVALID, "in_host/out_host must be non-NULL host pointers");
    if (variant != SEPCONV_2D && variant != SEPCONV_SEPARABLE && variant != SEPCONV_AUTO)
        return fail(SEPCONV_E_INVALID, "bad variant");
    sepconv_status_t s = check_kernel(kernel, plan->k);
    if (s != SEPCONV_OK) return s;
    {
        const uintptr_t a0 = reinterpret_cast<uintptr_t>(in_host);
        const uintptr_t a1 = a0 + static_cast<uintptr_t>(plan->n * plan->h * plan->ld_in) * 4;
        const uintptr_t b0 = reinterpret_cast<uintptr_t>(out_host);
        const uintptr_t b1 = b0 + static_cast<uintptr_t>(plan->n * plan->ho * plan->ld_out) * 4;
        if (a0 < b1 && b0 < a1) return fail(SEPCONV_E_ALIAS, "host input and output overlap");
    }
    int prev = -1;
    cudaGetDevice(&prev);
    if (prev != plan->dev.device) SC_CUDA(cudaSetDevice(plan->dev.device));
    struct Restore {
        int d, cur;
        ~Restore() {
            if (d >= 0 && d != cur) cudaSetDevice(d);
        }
    } restore{prev, plan->dev.device};

    const Candidate c = resolve(plan, variant);
    s = ensure_host_pipeline(plan, c);
    if (s != SEPCONV_OK) return s;
    cudaStream_t sh = plan->hstream[0], sc = plan->hstream[1], sd = plan->hstream[2];
    cudaEvent_t(&ev)[4][2] = plan->hev;   // [0] copy-in done, [1] kernel done, [2] copy-out done, [3] entry
    SC_CUDA(cudaEventRecord(ev[3][0], static_cast<cudaStream_t>(stream)));
    SC_CUDA(cudaStreamWaitEvent(sh, ev[3][0], 0));

    const int64_t R = plan->hchunk_rows, K = plan->k;
    const int64_t ldb = (plan->wo + 3) & ~3LL;
    long long i = 0;
    for (int64_t n = 0; n < plan->n; ++n) {
        for (int64_t r0 = 0; r0 < plan->ho; r0 += R, ++i) {
            const int slot = static_cast<int>(i & 1);
            const int64_t rr = std::min<int64_t>(R, plan->ho - r0);
            const int64_t rin = rr + K - 1;
            // copy-in: input rows [r0, r0 + rr + K - 1) of image n.  The first K-1 of
            // them are the previous band's last K-1 rows, already on the device in the other slot
            // (its copy-in precedes this one on sh): a device-to-device copy, so PCIe carries every
            // input row once (the H2D direction bounds the pipeline)
            if (i >= 2) SC_CUDA(cudaStreamWaitEvent(sh, ev[1][slot], 0));
            const int64_t carry = (r0 > 0) ? K - 1 : 0;
            if (carry > 0)
                SC_CUDA(cudaMemcpy2DAsync(plan->hin[slot], plan->ld_in * 4,
                                          plan->hin[slot ^ 1] + R * plan->ld_in, plan->ld_in * 4, plan->w * 4,
                                          carry, cudaMemcpyDeviceToDevice, sh));
            SC_CUDA(cudaMemcpy2DAsync(plan->hin[slot] + carry * plan->ld_in, plan->ld_in * 4,
                                      in_host + (n * plan->h + r0 + carry) * plan->ld_in, plan->ld_in * 4,
                                      plan->w * 4, rin - carry, cudaMemcpyHostToDevice, sh));
            SC_CUDA(cudaEventRecord(ev[0][slot], sh));
            // execute
            SC_CUDA(cudaStreamWaitEvent(sc, ev[0][slot], 0));
            if (i >= 2) SC_CUDA(cudaStreamWaitEvent(sc, ev[2][slot], 0));
            Geometry g;
            g.K = static_cast<int>(K);
            g.nimg = 1;
            g.in_rows = static_cast<int>(rin);
            g.in_cols = static_cast<int>(plan->w);
            g.ld_in = plan->ld_in;
            g.in_img = rin * plan->ld_in;
            g.out_cols = static_cast<int>(plan->wo);
            g.ld_out = plan->ld_out;
            g.out_img = rr * plan->ld_out;
            g.row_begin = 0;
            g.rows = static_cast<int>(rr);
            s = launch_candidate(plan, g, plan->hin[slot], plan->hout[slot], kernel, c, plan->hbuf[slot], ldb, sc);
            if (s != SEPCONV_OK) return s;
            SC_CUDA(cudaEventRecord(ev[1][slot], sc));
            // copy-out
            SC_CUDA(cudaStreamWaitEvent(sd, ev[1][slot], 0));
            SC_CUDA(cudaMemcpy2DAsync(out_host + (n * plan->ho + r0) * plan->ld_out, plan->ld_out * 4,
                                      plan->hout[slot], plan->ld_out * 4, plan->wo * 4, rr, cudaMemcpyDeviceToHost,
                                      sd));
            SC_CUDA(cudaEventRecord(ev[2][slot], sd));
        }
    }
    SC_CUDA(cudaStreamSynchronize(sd));
    SC_CUDA(cudaStreamSynchronize(sc));
    SC_CUDA(cudaStreamSynchronize(sh));
    return SEPCONV_OK;
}
