// abi_driver.cpp -- the C ABI's host logic under AddressSanitizer + UndefinedBehaviorSanitizer
// (tests/test_sanitize_cpu.py links it against the instrumented host objects of
// libsepconv.so, with kernel_stubs.cpp in place of the kernel translation units).
//   * argument validation of every entry point that can fail before touching a device
//     (include/sepconv.h, sor.h, bs.h), NULL-safety, status strings;
//   * sepconv_band / sor_band over a sweep of shapes, with their partition invariants;
//   * sepconv_select over random (also malformed) selectors;
//   * with a GPU: plan creation against fuzzed tuning-cache files (truncated, garbled and
//     well-formed lines for this device's keys) -- the cache parser is the one piece of the
//     library that reads untrusted text.
// Any sanitizer report aborts (-fno-sanitize-recover=all); the exit status is 0 otherwise.
#include <cuda_runtime.h>

#include <cstdint>
#include <cstdio>
#include <cstdlib>
#include <cstring>
#include <random>
#include <string>

#include "bs.h"
#include "sepconv.h"
#include "sor.h"

static int failures = 0;
#define EXPECT(c)                                                                          \
    do {                                                                                   \
        if (!(c)) {                                                                        \
            std::fprintf(stderr, "%s:%d: expectation failed: %s\n", __FILE__, __LINE__, #c); \
            ++failures;                                                                    \
        }                                                                                  \
    } while (0)

static void validation() {
    for (int s = -8; s <= 1; ++s) EXPECT(sepconv_status_str(static_cast<sepconv_status_t>(s)) != nullptr);
    EXPECT(std::strlen(sepconv_version()) > 0);
    sepconv_destroy(nullptr);
    sor_destroy(nullptr);
    sepconv_plan_t p = nullptr;
    EXPECT(sepconv_plan_ex(nullptr, &p) == SEPCONV_E_INVALID);
    EXPECT(sepconv_plan(64, 64, 3, nullptr) == SEPCONV_E_INVALID);
    struct Bad {
        int64_t n, h, w;
        int k;
        int64_t ld_in, ld_out;
        sepconv_status_t want;
    } bad[] = {{1, 64, 64, 0, 0, 0, SEPCONV_E_INVALID},   {1, 64, 64, 18, 0, 0, SEPCONV_E_UNSUPPORTED},
               {0, 64, 64, 3, 0, 0, SEPCONV_E_INVALID},   {1, 2, 64, 3, 0, 0, SEPCONV_E_INVALID},
               {1, 64, 2, 3, 0, 0, SEPCONV_E_INVALID},    {1, 64, 64, 3, 63, 0, SEPCONV_E_INVALID},
               {1, 64, 64, 3, 0, 61, SEPCONV_E_INVALID},  {1, 64, 64, 3, -1, 0, SEPCONV_E_INVALID},
               {1, 1LL << 31, 64, 3, 0, 0, SEPCONV_E_INVALID}};
    for (const Bad &b : bad) {
        sepconv_plan_desc_t d{b.n, b.h, b.w, b.k, b.ld_in, b.ld_out, -1};
        p = reinterpret_cast<sepconv_plan_t>(0x1);
        EXPECT(sepconv_plan_ex(&d, &p) == b.want);
        EXPECT(p == nullptr);
        EXPECT(std::strlen(sepconv_last_error()) > 0);
    }
    int64_t a, b, c, e;
    EXPECT(sepconv_run(nullptr, nullptr, nullptr, nullptr, SEPCONV_AUTO, nullptr) == SEPCONV_E_INVALID);
    EXPECT(sepconv_out_shape(nullptr, &a, &b) == SEPCONV_E_INVALID);
    EXPECT(sepconv_tune(nullptr, nullptr, nullptr) == SEPCONV_E_INVALID);
    EXPECT(sepconv_get_choice(nullptr, SEPCONV_AUTO, nullptr) == SEPCONV_E_INVALID);
    EXPECT(sepconv_num_candidates(nullptr) == 0);
    EXPECT(sepconv_run_band(nullptr, nullptr, nullptr, nullptr, SEPCONV_AUTO, nullptr) != SEPCONV_OK);
    EXPECT(sepconv_nccl_unique_id(nullptr) == SEPCONV_E_INVALID);
    EXPECT(sepconv_tune_selector(0, -1, nullptr, 0, nullptr, nullptr) != SEPCONV_OK);
    const int64_t down[2] = {512, 256};
    EXPECT(sepconv_tune_selector(5, -1, down, 2, nullptr, nullptr) == SEPCONV_E_INVALID);
    EXPECT(sepconv_tune_selector(5, -1, down, 13, nullptr, nullptr) == SEPCONV_E_INVALID);
    EXPECT(sepconv_band(100, 3, 0, 0, &a, &b, &c, &e) == SEPCONV_E_INVALID);
    EXPECT(sepconv_band(100, 3, 4, 4, &a, &b, &c, &e) == SEPCONV_E_INVALID);
    EXPECT(sepconv_band(100, 30, 8, 0, &a, &b, &c, &e) == SEPCONV_E_UNSUPPORTED);
    sor_plan_t sp = nullptr;
    EXPECT(sor_plan(0, 5, &sp) == SEPCONV_E_INVALID);
    EXPECT(sor_plan(5, -1, &sp) == SEPCONV_E_INVALID);
    EXPECT(sor_iterate(nullptr, 1.5f, 3, SOR_AUTO, nullptr) == SEPCONV_E_INVALID);
    EXPECT(sor_band(100, 0, 0, 2, &a, &b, &c, &e) == SEPCONV_E_INVALID);
    EXPECT(sor_band(100, 2, 0, 3, &a, &b, &c, &e) == SEPCONV_E_INVALID);
    float f[8] = {1, 1, 1, 1, 1, 1, 1, 1}, g[8];
    EXPECT(bs_price(f, f, f, 8, 0.02f, -1.f, g, g, nullptr) == SEPCONV_E_INVALID);
    EXPECT(bs_price(f, f, f, -1, 0.02f, 0.3f, g, g, nullptr) == SEPCONV_E_INVALID);
}

static void bands() {
    for (int64_t H = 1; H <= 160; H += 7)
        for (int K = 1; K <= 17; K += 4)
            for (int G = 1; G <= 9; ++G) {
                int64_t next = 0, total = 0;
                bool ok = true;
                for (int g = 0; g < G; ++g) {
                    int64_t r0 = -1, rows = -1, owned = -1, alloc = -1;
                    sepconv_status_t s = sepconv_band(H, K, G, g, &r0, &rows, &owned, &alloc);
                    if (s != SEPCONV_OK) {
                        ok = false;
                        break;
                    }
                    EXPECT(r0 == next && rows >= 1 && alloc == rows + K - 1 && owned <= alloc);
                    next = r0 + rows;
                    total += rows;
                }
                if (ok) EXPECT(total == H - K + 1);
            }
    for (int64_t n = 1; n <= 80; n += 3)
        for (int G = 1; G <= 6; ++G)
            for (int halo = 2; halo <= 8; halo += 2)
                for (int g = 0; g < G; ++g) {
                    int64_t r0 = -1, rows = -1, a0 = -1, arows = -1;
                    if (sor_band(n, G, g, halo, &r0, &rows, &a0, &arows) == SEPCONV_OK) {
                        EXPECT(r0 % 2 == 0 && rows >= 1 && a0 <= r0 && a0 + arows >= r0 + rows && a0 >= 0 &&
                               a0 + arows <= n);
                    }
                }
}

static void selectors() {
    std::mt19937_64 rng(12345);
    for (int it = 0; it < 20000; ++it) {
        sepconv_selector_t s;
        std::memset(&s, 0, sizeof s);
        s.k = 1 + static_cast<int>(rng() % 17);
        s.m = static_cast<int>(rng() % 15) - 1;                     // -1 .. 13: also malformed
        int64_t c = 0;
        const int valid_m = s.m >= 1 && s.m <= SEPCONV_SELECTOR_LEVELS;
        for (int i = 0; i < SEPCONV_SELECTOR_LEVELS - 1; ++i) {
            c += (rng() % 4 == 0) ? -static_cast<int64_t>(rng() % 100) : static_cast<int64_t>(rng() % 100000);
            s.cutoffs[i] = c;
        }
        for (int i = 0; i < SEPCONV_SELECTOR_LEVELS; ++i) s.algos[i].config = i;
        sepconv_choice_t out;
        const int64_t size = static_cast<int64_t>(rng() % 2000000);
        const sepconv_status_t st = sepconv_select(&s, size, &out);
        bool increasing = valid_m && (s.m == 1 || s.cutoffs[0] > 0);
        for (int i = 1; valid_m && i + 1 < s.m; ++i) increasing = increasing && s.cutoffs[i] > s.cutoffs[i - 1];
        EXPECT((st == SEPCONV_OK) == increasing);
        if (st == SEPCONV_OK) {
            const int i = out.config;
            EXPECT(i >= 0 && i < s.m);
            EXPECT(i == 0 || size >= s.cutoffs[i - 1]);
            EXPECT(i == s.m - 1 || size < s.cutoffs[i]);
        }
    }
    EXPECT(sepconv_select(nullptr, 1, nullptr) == SEPCONV_E_INVALID);
}

static std::string garble(std::mt19937_64 &rng, const std::string &line) {
    std::string s = line;
    switch (rng() % 5) {
        case 0: s.resize(rng() % (s.size() + 1)); break;                       // truncated
        case 1:
            for (int i = 0; i < 4 && !s.empty(); ++i) s[rng() % s.size()] = static_cast<char>(rng() % 256);
            break;
        case 2: s.insert(rng() % (s.size() + 1), std::string(rng() % 300, '9')); break;   // huge numbers
        case 3: s += std::string(rng() % 5000, '['); break;
        default: break;                                                         // well formed
    }
    return s;
}

static void cache_fuzz() {
    int dev = 0;
    cudaDeviceProp prop;
    if (cudaGetDevice(&dev) != cudaSuccess || cudaGetDeviceProperties(&prop, dev) != cudaSuccess) {
        std::printf("no device: cache fuzzing skipped\n");
        return;
    }
    const char *path = "sanitize_cache.jsonl";
    const std::string gpu = std::string(prop.name) + "|" + std::to_string(prop.multiProcessorCount);
    const std::string good_plan = "{\"key\":\"" + gpu +
                                  "|1x300x200|k5|ld200,196\",\"2d\":[0,1,0,0,0,8,1,3.5,0,0],\"sep\":"
                                  "[1,1,1,2,0,8,1,2.5,7,100],\"auto\":[1,1,1,2,0,8,1,2.5,7,100,85]}";
    const std::string good_sel = "{\"key\":\"sel:" + gpu +
                                 "|k5\",\"k\":5,\"m\":3,\"cutoffs\":[10000,90000],\"algos\":[[0,1,0,0,0,8,1,0,0,0],"
                                 "[1,1,1,1,0,8,1,0,0,0],[1,1,1,3,1,16,1,0,0,0]]}";
    std::mt19937_64 rng(777);
    setenv("SEPCONV_TUNE_CACHE", path, 1);
    for (int it = 0; it < 300; ++it) {
        FILE *f = std::fopen(path, "w");
        for (int l = 0; l < 6; ++l) std::fprintf(f, "%s\n", garble(rng, (l & 1) ? good_plan : good_sel).c_str());
        std::fclose(f);
        for (int64_t side : {300, 100, 250}) {
            sepconv_plan_desc_t d{1, side, side == 300 ? 200 : side, 5, 0, 0, -1};
            sepconv_plan_t p = nullptr;
            if (sepconv_plan_ex(&d, &p) != SEPCONV_OK) continue;
            sepconv_choice_t c;
            EXPECT(sepconv_get_choice(p, SEPCONV_AUTO, &c) == SEPCONV_OK);
            EXPECT(c.config >= 0 && c.config < 8 && c.sched_parts >= 0 && c.sched_grid >= 0);
            EXPECT(c.sched_steal >= 0 && c.sched_steal <= 99);
            sepconv_destroy(p);
        }
    }
    {   // the well-formed file: exact entry and SELECT both resolve
        FILE *f = std::fopen(path, "w");
        std::fprintf(f, "%s\n%s\n", good_plan.c_str(), good_sel.c_str());
        std::fclose(f);
        sepconv_plan_desc_t d{1, 300, 200, 5, 0, 0, -1};
        sepconv_plan_t p = nullptr;
        if (sepconv_plan_ex(&d, &p) == SEPCONV_OK) {
            sepconv_choice_t c;
            sepconv_get_choice(p, SEPCONV_AUTO, &c);
            EXPECT(c.source == SEPCONV_SRC_TUNED && c.config == 2 && c.sched_parts == 7 && c.sched_grid == 100 &&
                   c.sched_steal == 85);
            sepconv_choice_t sc;
            sepconv_get_choice(p, SEPCONV_SEPARABLE, &sc);
            EXPECT(sc.sched_parts == 7 && sc.sched_steal == 0);          // the 10-field form: no stealing
            sepconv_destroy(p);
        }
        sepconv_plan_desc_t d2{1, 250, 250, 5, 0, 0, -1};            // 62500 px: level 2 of 3
        if (sepconv_plan_ex(&d2, &p) == SEPCONV_OK) {
            sepconv_choice_t c;
            sepconv_get_choice(p, SEPCONV_AUTO, &c);
            EXPECT(c.source == SEPCONV_SRC_SELECTOR && c.config == 1);
            sepconv_destroy(p);
        }
    }
    std::remove(path);
    unsetenv("SEPCONV_TUNE_CACHE");
    std::printf("cache fuzzing done on %s\n", prop.name);
}

int main() {
    validation();
    bands();
    selectors();
    cache_fuzz();
    if (failures) {
        std::fprintf(stderr, "abi_driver: %d expectation(s) failed\n", failures);
        return 1;
    }
    std::printf("abi sanitize ok\n");
    return 0;
}
