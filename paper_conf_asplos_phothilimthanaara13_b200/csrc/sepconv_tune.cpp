// sepconv_tune.cpp -- the empirical tuner (the paper's autotuner, reduced to
// an exhaustive search: the B200 space is a handful of candidates per plan, so
// timing every one is exact where the paper needed evolutionary search).
//
// For each eligible candidate: warm up, then `reps` timed runs with CUDA events on a
// private stream, the L2 flushed before each run when the working set would fit in L2
// (the same hygiene as bench.py), median.  The fastest overall becomes AUTO's choice,
// the fastest of each algorithm becomes 2D's / SEPARABLE's.  Ties within 1% prefer
// fewer passes, then the lower candidate index (R17).
#include <cuda_runtime.h>
#include <fcntl.h>
#include <sys/file.h>
#include <unistd.h>

#include <algorithm>
#include <cmath>
#include <cstdio>
#include <cstdlib>
#include <cstring>
#include <fstream>
#include <sstream>
#include <string>
#include <thread>
#include <vector>

#include "sepconv_internal.h"

using namespace sepconv;

namespace {

std::vector<Candidate> candidates(sepconv_plan_t p) {
    // fixed order: this is also the tie-break order
    std::vector<Candidate> cs;
    for (int cfg = 0; cfg < kSepTmaConfigs; ++cfg) cs.push_back({SEPCONV_SEPARABLE, SEPCONV_MAP_TMA, 1, cfg, 0});
    // with 16-byte aligned output rows the 8-byte store path is a distinct candidate
    // (it paces the warps differently; measured faster at K=13 on 16384^2)
    const bool rows16 = (p->ld_out % 4) == 0;
    if (rows16)
        for (int cfg = 0; cfg < kSepTmaConfigs; ++cfg) cs.push_back({SEPCONV_SEPARABLE, SEPCONV_MAP_TMA, 1, cfg, 1});
    cs.push_back({SEPCONV_SEPARABLE, SEPCONV_MAP_DIRECT, 1, 0, 0});
    cs.push_back({SEPCONV_2D, SEPCONV_MAP_TMA, 0, 0, 0});
    cs.push_back({SEPCONV_2D, SEPCONV_MAP_DIRECT, 0, 0, 0});
    cs.push_back({SEPCONV_SEPARABLE, SEPCONV_MAP_TMA, 0, 0, 0});
    cs.push_back({SEPCONV_SEPARABLE, SEPCONV_MAP_DIRECT, 0, 0, 0});
    return cs;
}

int passes(const Candidate &c) { return (c.algo == SEPCONV_SEPARABLE && !c.fused) ? 2 : 1; }

std::string cache_key(sepconv_plan_t p) {
    std::ostringstream os;
    os << p->dev.name << "|" << p->dev.sms << "|" << p->n << "x" << p->h << "x" << p->w << "|k" << p->k << "|ld"
       << p->ld_in << "," << p->ld_out;
    return os.str();
}

std::string choice_json(const sepconv_choice_t &c) {
    char b[160];
    snprintf(b, sizeof b, "[%d,%d,%d,%d,%d,%d,%d,%.9g]", (int)c.algo, c.mapping, c.fused, c.config, c.store_path,
             c.warps, c.ctas_per_sm, c.median_us);
    return b;
}

bool parse_choice(const std::string &line, const char *field, sepconv_choice_t *c) {
    std::string f = std::string("\"") + field + "\":[";
    size_t pos = line.find(f);
    if (pos == std::string::npos) return false;
    int algo, map, fused, config, store, warps, ctas;
    float us;
    if (sscanf(line.c_str() + pos + f.size(), "%d,%d,%d,%d,%d,%d,%d,%f", &algo, &map, &fused, &config, &store, &warps,
               &ctas, &us) != 8)
        return false;
    if (store < 0 || store > 1) return false;
    if (config < 0 || config >= kSepTmaConfigs) return false;
    if ((algo != SEPCONV_2D && algo != SEPCONV_SEPARABLE) || (map != 0 && map != 1)) return false;
    c->algo = static_cast<sepconv_variant_t>(algo);
    c->mapping = map;
    c->fused = fused;
    c->config = config;
    c->store_path = store;
    c->warps = warps;
    c->ctas_per_sm = ctas;
    c->median_us = us;
    return true;
}

bool load_cache(const std::string &path, const std::string &key, sepconv_choice_t best[3]) {
    std::ifstream f(path);
    if (!f) return false;
    std::string line, want = "\"key\":\"" + key + "\"";
    bool found = false;
    while (std::getline(f, line)) {
        if (line.find(want) == std::string::npos) continue;
        sepconv_choice_t b[3];
        if (parse_choice(line, "2d", &b[0]) && parse_choice(line, "sep", &b[1]) && parse_choice(line, "auto", &b[2])) {
            std::memcpy(best, b, sizeof b);
            found = true;   // the last matching line wins
        }
    }
    return found;
}

// Read-modify-write of the JSON-lines cache under an exclusive flock on "<path>.lock", through a
// temp file unique to this process and thread, then an atomic rename: several ranks or
// processes sharing one cache (multi-GPU bench runs) neither truncate each other's temp file
// nor lose each other's entries.
struct CacheLock {
    int fd = -1;
    explicit CacheLock(const std::string &path) {
        fd = ::open((path + ".lock").c_str(), O_RDWR | O_CREAT | O_CLOEXEC, 0644);
        if (fd >= 0) ::flock(fd, LOCK_EX);
    }
    ~CacheLock() {
        if (fd >= 0) {
            ::flock(fd, LOCK_UN);
            ::close(fd);
        }
    }
};

void store_cache(const std::string &path, const std::string &key, const std::string &entry) {
    CacheLock lock(path);
    std::vector<std::string> keep;
    {
        std::ifstream f(path);
        std::string line, want = "\"key\":\"" + key + "\"";
        while (f && std::getline(f, line))
            if (!line.empty() && line.find(want) == std::string::npos) keep.push_back(line);
    }
    std::ostringstream tn;
    tn << path << ".tmp." << ::getpid() << "." << std::hash<std::thread::id>{}(std::this_thread::get_id());
    const std::string tmp = tn.str();
    {
        std::ofstream o(tmp, std::ios::trunc);
        if (!o) return;
        for (auto &l : keep) o << l << "\n";
        o << entry << "\n";
        if (!o.good()) {
            o.close();
            std::remove(tmp.c_str());
            return;
        }
    }
    if (std::rename(tmp.c_str(), path.c_str()) != 0) std::remove(tmp.c_str());
}

void store_choices(const std::string &path, const std::string &key, const sepconv_choice_t best[3]) {
    store_cache(path, key, "{\"key\":\"" + key + "\",\"2d\":" + choice_json(best[0]) + ",\"sep\":" +
                               choice_json(best[1]) + ",\"auto\":" + choice_json(best[2]) + "}");
}

// The paper's selector picks a rule by input-size cutoffs (SELECT).  Here: a
// plan of an untuned shape adopts the cached choice of the nearest tuned size (same GPU,
// SM count, K and image count; sizes compared in log2 of the pixel count, within 2x).
bool select_nearest(const std::string &path, sepconv_plan_t p, sepconv_choice_t best[3]) {
    std::ifstream f(path);
    if (!f) return false;
    std::ostringstream pre;
    pre << p->dev.name << "|" << p->dev.sms << "|";
    const std::string want_pre = "\"key\":\"" + pre.str();
    const double my = std::log2(static_cast<double>(p->h) * static_cast<double>(p->w));
    double best_d = 1.0 + 1e-9;
    bool found = false;
    std::string line;
    while (std::getline(f, line)) {
        const size_t at = line.find(want_pre);
        if (at == std::string::npos) continue;
        long long n = 0, h = 0, w = 0;
        int k = 0;
        if (sscanf(line.c_str() + at + want_pre.size(), "%lldx%lldx%lld|k%d", &n, &h, &w, &k) != 4) continue;
        if (k != p->k || n != p->n) continue;
        const double d = std::fabs(std::log2(static_cast<double>(h) * static_cast<double>(w)) - my);
        sepconv_choice_t b[3];
        if (d < best_d && parse_choice(line, "2d", &b[0]) && parse_choice(line, "sep", &b[1]) &&
            parse_choice(line, "auto", &b[2])) {
            best_d = d;
            std::memcpy(best, b, sizeof b);
            found = true;
        }
    }
    return found;
}

}  // namespace

// Called by sepconv_plan_ex: an exact cache hit makes the plan tuned; otherwise the nearest
// tuned size class (NEXT-2 of SURVEY 8(f)) seeds AUTO / 2D / SEPARABLE until sepconv_tune.
void sepconv_seed_from_cache(sepconv_plan_t plan) {
    const char *env = std::getenv("SEPCONV_TUNE_CACHE");
    if (!env || !*env) return;
    if (load_cache(env, cache_key(plan), plan->best) || select_nearest(env, plan, plan->best)) plan->tuned = true;
}

extern "C" {

int sepconv_num_candidates(sepconv_plan_t plan) {
    if (!plan) return 0;
    return static_cast<int>(candidates(plan).size());
}

sepconv_status_t sepconv_get_candidate(sepconv_plan_t plan, int index, sepconv_choice_t *choice) {
    if (!plan || !choice) return fail(SEPCONV_E_INVALID, "NULL argument");
    auto cs = candidates(plan);
    if (index < 0 || index >= static_cast<int>(cs.size())) return fail(SEPCONV_E_INVALID, "candidate index out of range");
    std::memset(choice, 0, sizeof *choice);
    choice->algo = static_cast<sepconv_variant_t>(cs[index].algo);
    choice->mapping = cs[index].mapping;
    choice->fused = cs[index].fused;
    choice->config = cs[index].config;
    choice->store_path = cs[index].store;
    choice->warps = candidate_warps(plan->k, cs[index]);
    choice->ctas_per_sm = 1;
    return SEPCONV_OK;
}

sepconv_status_t sepconv_tune(sepconv_plan_t plan, const sepconv_tune_opts_t *opts, sepconv_choice_t *chosen) {
    if (!plan) return fail(SEPCONV_E_INVALID, "plan is NULL");
    const int reps = (opts && opts->reps > 0) ? opts->reps : 20;
    const int flags = opts ? opts->flags : 0;
    std::string path;
    if (opts && opts->cache_path) path = opts->cache_path;
    else if (const char *env = std::getenv("SEPCONV_TUNE_CACHE")) path = env;
    const std::string key = cache_key(plan);

    if (!path.empty() && !(flags & SEPCONV_TUNE_FORCE) && load_cache(path, key, plan->best)) {
        plan->tuned = true;
        if (chosen) *chosen = plan->best[2];
        return SEPCONV_OK;
    }

    int prev = -1;
    cudaGetDevice(&prev);
    cudaSetDevice(plan->dev.device);
    struct Restore {
        int d;
        ~Restore() {
            if (d >= 0) cudaSetDevice(d);
        }
    } restore{prev};

    const size_t in_floats = static_cast<size_t>(plan->n * plan->h * plan->ld_in);
    const size_t out_floats = static_cast<size_t>(plan->n * plan->ho * plan->ld_out);
    float *din = nullptr, *dout = nullptr, *flush = nullptr;
    cudaStream_t st = nullptr;
    cudaEvent_t e0 = nullptr, e1 = nullptr;
    sepconv_status_t status = SEPCONV_OK;
    const size_t flush_floats = plan->dev.l2 / 2;   // 2x L2 bytes
    const bool need_flush = !(flags & SEPCONV_TUNE_NO_L2_FLUSH) &&
                            (in_floats + out_floats) * 4 < 2 * plan->dev.l2;
    std::vector<float> kern(plan->k);
    for (int i = 0; i < plan->k; ++i) {   // normalised binomial (the benchmark kernel)
        double c = 1;
        for (int j = 0; j < i; ++j) c = c * (plan->k - 1 - j) / (j + 1);
        kern[i] = static_cast<float>(c / std::pow(2.0, plan->k - 1));
    }
    auto cs = candidates(plan);
    std::vector<float> med(cs.size(), -1.f);

    do {
        cudaError_t e;
        if ((e = cudaMalloc(&din, in_floats * 4)) != cudaSuccess) { status = cuda_fail(e, "tune: cudaMalloc(in)"); break; }
        if ((e = cudaMalloc(&dout, out_floats * 4)) != cudaSuccess) { status = cuda_fail(e, "tune: cudaMalloc(out)"); break; }
        if (need_flush && (e = cudaMalloc(&flush, flush_floats * 4)) != cudaSuccess) {
            status = cuda_fail(e, "tune: cudaMalloc(flush)");
            break;
        }
        if ((e = cudaStreamCreateWithFlags(&st, cudaStreamNonBlocking)) != cudaSuccess) { status = cuda_fail(e, "tune: stream"); break; }
        cudaEventCreate(&e0);
        cudaEventCreate(&e1);
        launch_fill_pattern(din, static_cast<long long>(in_floats), 1234u, st);
        Geometry g = plan_geometry(plan);
        for (size_t ci = 0; ci < cs.size() && status == SEPCONV_OK; ++ci) {
            const Candidate &c = cs[ci];
            if (c.algo == SEPCONV_SEPARABLE && !c.fused) {
                status = ensure_buf(plan);
                if (status != SEPCONV_OK) break;
            }
            std::vector<float> t;
            for (int r = 0; r < reps + 2; ++r) {
                if (need_flush) launch_l2_flush(flush, static_cast<long long>(flush_floats), st);
                cudaEventRecord(e0, st);
                status = launch_candidate(plan, g, din, dout, kern.data(), c, plan->buf, plan->ld_buf, st);
                if (status != SEPCONV_OK) break;
                cudaEventRecord(e1, st);
                if ((e = cudaEventSynchronize(e1)) != cudaSuccess) { status = cuda_fail(e, "tune: run"); break; }
                float ms = 0;
                cudaEventElapsedTime(&ms, e0, e1);
                if (r >= 2) t.push_back(ms * 1000.f);
            }
            if (status != SEPCONV_OK) break;
            std::sort(t.begin(), t.end());
            med[ci] = t[t.size() / 2];
        }
    } while (0);

    if (st) cudaStreamSynchronize(st);
    if (din) cudaFree(din);
    if (dout) cudaFree(dout);
    if (flush) cudaFree(flush);
    if (e0) cudaEventDestroy(e0);
    if (e1) cudaEventDestroy(e1);
    if (st) cudaStreamDestroy(st);
    if (status != SEPCONV_OK) return status;

    auto better = [&](size_t a, size_t b) {   // is candidate a better than incumbent b?
        if (med[a] < 0) return false;
        if (med[b] < 0) return true;
        if (med[a] < med[b] * 0.99f) return true;
        if (med[b] < med[a] * 0.99f) return false;
        if (passes(cs[a]) != passes(cs[b])) return passes(cs[a]) < passes(cs[b]);
        return false;   // keep the lower index
    };
    size_t bi[3] = {SIZE_MAX, SIZE_MAX, SIZE_MAX};
    for (size_t i = 0; i < cs.size(); ++i) {
        const int slot = cs[i].algo == SEPCONV_2D ? 0 : 1;
        if (bi[slot] == SIZE_MAX || better(i, bi[slot])) bi[slot] = i;
        if (bi[2] == SIZE_MAX || better(i, bi[2])) bi[2] = i;
    }
    for (int s = 0; s < 3; ++s) {
        const Candidate &c = cs[bi[s]];
        sepconv_choice_t &o = plan->best[s];
        std::memset(&o, 0, sizeof o);
        o.algo = static_cast<sepconv_variant_t>(c.algo);
        o.mapping = c.mapping;
        o.fused = c.fused;
        o.config = c.config;
        o.store_path = c.store;
        o.warps = candidate_warps(plan->k, c);
        o.ctas_per_sm = 1;
        o.median_us = med[bi[s]];
    }
    plan->tuned = true;
    if (!path.empty()) store_choices(path, key, plan->best);
    if (chosen) *chosen = plan->best[2];
    return SEPCONV_OK;
}

}  // extern "C"
