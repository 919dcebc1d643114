// kernel_stubs.cpp -- stand-ins for the kernel translation units (inst_*.cu, sepconv_2d.cu) in
// the sanitizer build of the C ABI's host code (tests/test_sanitize_cpu.py): the host logic
// (validation, band arithmetic, SELECT, cache parsing, plan lifecycle) is instrumented without
// compiling ~2 minutes of kernels.  The abi driver never launches a SeparableConvolution
// kernel, so these are never called; if one were, it returns an error rather than a kernel.
#include "sepconv_launch.h"

namespace sepconv {
namespace {
KernelInfo no_info() { return KernelInfo{nullptr, 0, 32, 1, 1}; }
cudaError_t no_launch(const StreamParams &, int, cudaStream_t) { return cudaErrorNotSupported; }
StreamEntry kStub[kMaxK];
const StreamEntry *stub_table() {
    for (auto &e : kStub) {
        e.info[0] = e.info[1] = e.info[2] = e.info[3] = no_info;
        e.launch[0] = e.launch[1] = e.launch[2] = e.launch[3] = no_launch;
    }
    return kStub;
}
}  // namespace
#define SEPCONV_STUB(name) \
    const StreamEntry *name() { return stub_table(); }
SEPCONV_STUB(stream_table_rows_v0)
SEPCONV_STUB(stream_table_rows_v1)
SEPCONV_STUB(stream_table_rows_v2)
SEPCONV_STUB(stream_table_cols_v0)
SEPCONV_STUB(stream_table_cols_v1)
SEPCONV_STUB(stream_table_cols_v2)
SEPCONV_STUB(stream_table_sep_v0)
SEPCONV_STUB(stream_table_sep_v1)
SEPCONV_STUB(stream_table_sep_v2)
SEPCONV_STUB(stream_table_sep_v3)
SEPCONV_STUB(stream_table_sep_v4)
SEPCONV_STUB(stream_table_sep_v5)
SEPCONV_STUB(stream_table_sep_v6)
SEPCONV_STUB(stream_table_sep_v7)
KernelInfo conv2d_info(int, int) { return no_info(); }
cudaError_t conv2d_launch(int, int, const Conv2DParams &, int, cudaStream_t) { return cudaErrorNotSupported; }
}  // namespace sepconv
