// sepconv_tune.cpp -- the empirical tuner (the paper's autotuner) and its size
// selector (SELECT).
//
// sepconv_tune(plan): every eligible candidate (compile-time stage configurations, store
// paths, mappings, algorithms) is timed -- the B200 space is a handful of candidates per plan,
// so the exhaustive pass is exact where the paper needed an evolutionary search -- then the
// winner's work schedule, a pair of size-like integers (row partitions per CTA strip, CTAs),
// goes through the paper's mutation search: one parent, asexual children made by
// scaling the values by lognormal factors (a halving as likely as a doubling, small changes
// likelier than large ones), a child kept only if it beats its parent.
// The fastest overall becomes AUTO's choice, the fastest of each algorithm 2D's / SEPARABLE's.
// Ties within 1% prefer fewer passes, then the lower candidate index (R17).
//
// Timing: when in + out fit in 2 x L2 every timed pass follows a clean
// flush -- a write of 2 x L2 then a read of another 2 x L2, so the pass pays for its own
// traffic and not for write-backs of lines an unrelated kernel dirtied -- and the pass time is
// the event time of n x (flush + pass) minus that of n x (flush), because single events tick
// in 2.048 us steps on this system (profiles/r02_flush_study.txt); larger working sets time n
// back-to-back passes.  The result is the fastest of three such batches (one-sided noise), or
// for flushed differences their median (two-sided noise: the flush's own variance).
//
// sepconv_tune_selector(K): the exhaustive tuner at up to 12 square sizes, equal neighbouring
// picks merged, each cutoff between different picks placed by timing both at the geometric
// middle; stored in the cache so that plans of untuned shapes resolve AUTO by SELECT.
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
#include <functional>
#include <sstream>
#include <string>
#include <thread>
#include <tuple>
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
    // with 8-byte (not 16-byte) aligned rows, two 8-byte stores per lane instead of the shuffled
    // 16-byte chunks (store path 2; the 16-warp cfg 3 already stores that way): a smaller loop
    // body, faster on mid-size images; on outputs wider than 8192 columns the half-sector writes
    // lose (16384^2: K=11 +13%, K=15 +2-5% in the bench; profiles/r02_explore_v2x2.txt,
    // profiles/r02v3_bench_c4*.json), so it is offered up to that width
    else if ((p->ld_out % 2) == 0 && p->wo <= 8192)
        for (int cfg = 0; cfg < kSepTmaConfigs; ++cfg)
            if (cfg != 3) cs.push_back({SEPCONV_SEPARABLE, SEPCONV_MAP_TMA, 1, cfg, 2});
    cs.push_back({SEPCONV_SEPARABLE, SEPCONV_MAP_DIRECT, 1, 0, 0});
    cs.push_back({SEPCONV_2D, SEPCONV_MAP_TMA, 0, 0, 0});
    cs.push_back({SEPCONV_2D, SEPCONV_MAP_DIRECT, 0, 0, 0});
    cs.push_back({SEPCONV_SEPARABLE, SEPCONV_MAP_TMA, 0, 0, 0});
    cs.push_back({SEPCONV_SEPARABLE, SEPCONV_MAP_DIRECT, 0, 0, 0});
    return cs;
}

int passes(const Candidate &c) { return (c.algo == SEPCONV_SEPARABLE && !c.fused) ? 2 : 1; }

std::string plan_key(sepconv_plan_t p) {
    std::ostringstream os;
    os << p->dev.name << "|" << p->dev.sms << "|" << p->n << "x" << p->h << "x" << p->w << "|k" << p->k << "|ld"
       << p->ld_in << "," << p->ld_out;
    return os.str();
}

std::string selector_key(const DeviceInfo &d, int K) {
    std::ostringstream os;
    os << "sel:" << d.name << "|" << d.sms << "|k" << K;
    return os.str();
}

// ---- the JSON-lines cache -------------------------------------------------------------------
std::string choice_json(const sepconv_choice_t &c) {
    char b[200];
    if (c.sched_steal)                                         // 11 fields only when stealing is on
        snprintf(b, sizeof b, "[%d,%d,%d,%d,%d,%d,%d,%.9g,%d,%d,%d]", (int)c.algo, c.mapping, c.fused, c.config,
                 c.store_path, c.warps, c.ctas_per_sm, c.median_us, c.sched_parts, c.sched_grid, c.sched_steal);
    else
        snprintf(b, sizeof b, "[%d,%d,%d,%d,%d,%d,%d,%.9g,%d,%d]", (int)c.algo, c.mapping, c.fused, c.config,
                 c.store_path, c.warps, c.ctas_per_sm, c.median_us, c.sched_parts, c.sched_grid);
    return b;
}

// parses one "[...]" choice at p; returns the position after it, or nullptr
const char *parse_choice_at(const char *p, sepconv_choice_t *c) {
    int algo, map, fused, config, store, warps, ctas, parts = 0, grid = 0, steal = 0, used = 0;
    float us;
    if (sscanf(p, "[%d,%d,%d,%d,%d,%d,%d,%f,%d,%d]%n", &algo, &map, &fused, &config, &store, &warps, &ctas, &us, &parts,
               &grid, &used) != 10 || used == 0) {
        used = 0;
        if (sscanf(p, "[%d,%d,%d,%d,%d,%d,%d,%f,%d,%d,%d]%n", &algo, &map, &fused, &config, &store, &warps, &ctas, &us,
                   &parts, &grid, &steal, &used) != 11 || used == 0)
            return nullptr;
    }
    if (store < 0 || store > 2 || config < 0 || config >= kSepTmaConfigs || parts < 0 || grid < 0) return nullptr;
    if (steal < 0 || steal > 99) return nullptr;
    if ((algo != SEPCONV_2D && algo != SEPCONV_SEPARABLE) || (map != 0 && map != 1)) return nullptr;
    std::memset(c, 0, sizeof *c);
    c->algo = static_cast<sepconv_variant_t>(algo);
    c->mapping = map;
    c->fused = fused;
    c->config = config;
    c->store_path = store;
    c->warps = warps;
    c->ctas_per_sm = ctas;
    c->median_us = us;
    c->sched_parts = parts;
    c->sched_grid = grid;
    c->sched_steal = steal;
    return p + used;
}

bool parse_choice(const std::string &line, const char *field, sepconv_choice_t *c) {
    const std::string f = std::string("\"") + field + "\":";
    const size_t pos = line.find(f);
    return pos != std::string::npos && parse_choice_at(line.c_str() + pos + f.size(), c) != nullptr;
}

// the last line of the cache whose key is exactly `key`
bool find_line(const std::string &path, const std::string &key, std::string *out) {
    std::ifstream f(path);
    if (!f) return false;
    const std::string want = "{\"key\":\"" + key + "\",";
    std::string line;
    bool found = false;
    while (std::getline(f, line))
        if (line.compare(0, want.size(), want) == 0) {
            *out = line;
            found = true;
        }
    return found;
}

bool load_choices(const std::string &path, const std::string &key, sepconv_choice_t best[3]) {
    std::string line;
    if (!find_line(path, key, &line)) return false;
    sepconv_choice_t b[3];
    if (!(parse_choice(line, "2d", &b[0]) && parse_choice(line, "sep", &b[1]) && parse_choice(line, "auto", &b[2])))
        return false;
    for (auto &c : b) c.source = SEPCONV_SRC_TUNED;
    std::memcpy(best, b, sizeof b);
    return true;
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
        std::string line;
        const std::string want = "{\"key\":\"" + key + "\",";
        while (f && std::getline(f, line))
            if (!line.empty() && line.compare(0, want.size(), want) != 0) keep.push_back(line);
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

void store_selector(const std::string &path, const std::string &key, const sepconv_selector_t &s) {
    std::ostringstream o;
    o << "{\"key\":\"" << key << "\",\"k\":" << s.k << ",\"m\":" << s.m << ",\"cutoffs\":[";
    for (int i = 0; i + 1 < s.m; ++i) o << (i ? "," : "") << static_cast<long long>(s.cutoffs[i]);
    o << "],\"algos\":[";
    for (int i = 0; i < s.m; ++i) o << (i ? "," : "") << choice_json(s.algos[i]);
    o << "]}";
    store_cache(path, key, o.str());
}

bool load_selector(const std::string &path, const std::string &key, sepconv_selector_t *s) {
    std::string line;
    if (!find_line(path, key, &line)) return false;
    sepconv_selector_t r;
    std::memset(&r, 0, sizeof r);
    const size_t pk = line.find("\"k\":"), pm = line.find("\"m\":"), pc = line.find("\"cutoffs\":["),
                 pa = line.find("\"algos\":[");
    if (pk == std::string::npos || pm == std::string::npos || pc == std::string::npos || pa == std::string::npos)
        return false;
    if (sscanf(line.c_str() + pk + 4, "%d", &r.k) != 1 || sscanf(line.c_str() + pm + 4, "%d", &r.m) != 1) return false;
    if (r.m < 1 || r.m > SEPCONV_SELECTOR_LEVELS) return false;
    const char *p = line.c_str() + pc + 11;
    for (int i = 0; i + 1 < r.m; ++i) {
        long long v;
        int used = 0;
        if (sscanf(p, i ? ",%lld%n" : "%lld%n", &v, &used) != 1 || used == 0) return false;
        r.cutoffs[i] = v;
        p += used;
    }
    p = line.c_str() + pa + 9;
    for (int i = 0; i < r.m; ++i) {
        if (i) {
            if (*p != ',') return false;
            ++p;
        }
        p = parse_choice_at(p, &r.algos[i]);
        if (!p) return false;
        r.algos[i].source = SEPCONV_SRC_SELECTOR;
    }
    *s = r;
    return true;
}

std::string cache_path_of(const sepconv_tune_opts_t *opts) {
    if (opts && opts->cache_path) return opts->cache_path;
    if (const char *env = std::getenv("SEPCONV_TUNE_CACHE")) return env;
    return std::string();
}

// ---- timing -----------------------------------------------------------------------------------
// Synthetic buffers and the flush machinery of one tuning session on one plan.
struct Bench {
    sepconv_plan_t plan = nullptr;
    Geometry g{};
    float *din = nullptr, *dout = nullptr;
    size_t flush_floats = 0;
    bool need_flush = false;
    cudaStream_t st = nullptr;
    cudaEvent_t e0 = nullptr, e1 = nullptr;
    std::vector<float> kern;

    sepconv_status_t open(sepconv_plan_t p, bool allow_flush) {
        plan = p;
        const size_t in_floats = static_cast<size_t>(p->n * p->h * p->ld_in);
        const size_t out_floats = static_cast<size_t>(p->n * p->ho * p->ld_out);
        flush_floats = p->dev.l2 / 2;                     // 2 x L2 bytes
        need_flush = allow_flush && (in_floats + out_floats) * 4 < 2 * p->dev.l2;
        cudaError_t e;
        if ((e = cudaMalloc(&din, in_floats * 4)) != cudaSuccess) return cuda_fail(e, "tune: cudaMalloc(in)");
        if ((e = cudaMalloc(&dout, out_floats * 4)) != cudaSuccess) return cuda_fail(e, "tune: cudaMalloc(out)");
        if (need_flush) {
            sepconv_status_t fs = sepconv_l2_flush(nullptr);   // allocates the shared scratch once
            if (fs != SEPCONV_OK) return fs;
        }
        if ((e = cudaStreamCreateWithFlags(&st, cudaStreamNonBlocking)) != cudaSuccess) return cuda_fail(e, "tune: stream");
        if ((e = cudaEventCreate(&e0)) != cudaSuccess || (e = cudaEventCreate(&e1)) != cudaSuccess)
            return cuda_fail(e, "tune: events");
        launch_fill_pattern(din, static_cast<long long>(in_floats), 1234u, st);
        g = plan_geometry(p);
        kern.resize(p->k);
        for (int i = 0; i < p->k; ++i) {   // normalised binomial (the benchmark kernel)
            double c = 1;
            for (int j = 0; j < i; ++j) c = c * (p->k - 1 - j) / (j + 1);
            kern[i] = static_cast<float>(c / std::pow(2.0, p->k - 1));
        }
        return SEPCONV_OK;
    }
    ~Bench() {
        if (st) cudaStreamSynchronize(st);
        for (float *b : {din, dout})
            if (b) cudaFree(b);
        if (e0) cudaEventDestroy(e0);
        if (e1) cudaEventDestroy(e1);
        if (st) cudaStreamDestroy(st);
    }
    void flush() { sepconv_l2_flush(st); }   // the same flush bench.py uses
    // event time of n iterations of body, in us per iteration
    sepconv_status_t batch(int n, const std::function<sepconv_status_t()> &body, double *us) {
        cudaEventRecord(e0, st);
        for (int i = 0; i < n; ++i) {
            sepconv_status_t s = body();
            if (s != SEPCONV_OK) return s;
        }
        cudaEventRecord(e1, st);
        cudaError_t e = cudaEventSynchronize(e1);
        if (e != cudaSuccess) return cuda_fail(e, "tune: run");
        float ms = 0.f;
        cudaEventElapsedTime(&ms, e0, e1);
        *us = ms * 1000.0 / n;
        return SEPCONV_OK;
    }
    // the pass time of candidate c from three batches of n (see the file comment)
    sepconv_status_t time(const Candidate &c, int n, float *out_us) {
        if (c.algo == SEPCONV_SEPARABLE && !c.fused) {
            sepconv_status_t s = ensure_buf(plan);
            if (s != SEPCONV_OK) return s;
        }
        auto pass = [&]() { return launch_candidate(plan, g, din, dout, kern.data(), c, plan->buf, plan->ld_buf, st); };
        auto fl = [&]() {
            flush();
            return SEPCONV_OK;
        };
        auto flpass = [&]() {
            flush();
            return pass();
        };
        sepconv_status_t s = pass();                              // warm-up (first-launch costs)
        if (s != SEPCONV_OK) return s;
        double t[3];
        for (int b = 0; b < 3; ++b) {
            if (need_flush) {
                double tf = 0, tfp = 0;
                if ((s = batch(n, fl, &tf)) != SEPCONV_OK || (s = batch(n, flpass, &tfp)) != SEPCONV_OK) return s;
                t[b] = std::max(0.05, tfp - tf);
            } else {
                if ((s = batch(n, pass, &t[b])) != SEPCONV_OK) return s;
            }
        }
        // back-to-back batches: the fastest -- the noise is one-sided (a transient clock, power
        // or memory-system slowdown only adds time), and a median of three still let a 5%
        // slowdown of one candidate's batches decide a pick (profiles/r02_tune_log.txt).
        // Flushed differences: the median -- the flush's own variance makes their noise two-sided
        std::sort(t, t + 3);
        *out_us = static_cast<float>(need_flush ? t[1] : t[0]);
        return SEPCONV_OK;
    }
};

// splitmix64 stream for the mutation search (reproducible for a given seed)
struct Rng {
    uint64_t s;
    uint64_t next() {
        uint64_t z = (s += 0x9E3779B97F4A7C15ull);
        z = (z ^ (z >> 30)) * 0xBF58476D1CE4E5B9ull;
        z = (z ^ (z >> 27)) * 0x94D049BB133111EBull;
        return z ^ (z >> 31);
    }
    double uniform() { return ((next() >> 11) + 0.5) * (1.0 / 9007199254740992.0); }
    double normal() { return std::sqrt(-2.0 * std::log(uniform())) * std::cos(6.283185307179586 * uniform()); }
};

// Mutation search over the winner's work schedule.  The parent starts as the
// model's schedule written as an explicit (parts, grid); each child scales one or both by
// exp(sigma N(0,1)), sigma = ln 2 / 2 (a doubling or a halving is a 2-sigma step), and replaces
// the parent only if it is faster (R23): by more than 2% in its own timing, then by
// more than 1% in a paired re-measurement of parent and child.
sepconv_status_t mutate_schedule(Bench &b, Candidate &best, float &best_us, int mutations, uint32_t seed, int reps) {
    if (mutations <= 0 || passes(best) != 1) return SEPCONV_OK;
    Sched model;
    long long slots = 0;
    Candidate probe = best;
    probe.sched_parts = probe.sched_grid = probe.sched_steal = 0;
    sepconv_status_t s = candidate_sched(b.plan, b.g, probe, &model, &slots);
    if (s != SEPCONV_OK) return s;
    const int rows = b.g.rows;
    const int cta_cols = candidate_warps(b.g.K, best) * kWarpCols;
    const long long strips = static_cast<long long>(b.g.nimg) * ((b.g.out_cols + cta_cols - 1) / cta_cols);
    double parts = model.parts > 0 ? model.parts
                                   : std::max(1.0, std::round(static_cast<double>(slots) / std::max(1LL, strips)));
    double grid = std::min(static_cast<double>(slots), static_cast<double>(strips) * parts);
    Rng rng{0x5EC0A11Dull ^ (static_cast<uint64_t>(seed ? seed : 1u) << 17) ^ static_cast<uint64_t>(rows) ^
            (static_cast<uint64_t>(b.g.K) << 40)};
    const double sigma = 0.5 * std::log(2.0);
    Candidate parent = best;
    float parent_us = best_us;
    const double parts0 = parts;
    // work stealing between warps (R27) is seeded on the configurations that carry it
    // (fused TMA with free-running warps, at most 8 per CTA: cfg 2, 4, 5)
    const bool stealing = best.algo == SEPCONV_SEPARABLE && best.fused && best.mapping == SEPCONV_MAP_TMA &&
                          (best.config == 2 || best.config == 4 || best.config == 5);
    const int nseeds = stealing ? 6 : 4;
    int steal = best.sched_steal;
    for (int m = 0; m < mutations + nseeds; ++m) {
        double np = parts, ng = grid;
        int nst = steal;
        if (m < 2) {
            // seeded members of the initial population: two and three rounds of the model's
            // items over every slot (more, shorter segments average out per-SM speed
            // differences: 16384^2 / K=17 -7.5%, profiles/r02_sched_check.txt)
            np = parts0 * (m + 2);
            ng = static_cast<double>(slots);
            nst = 0;
        } else if (m < 4) {
            // ... and 2/3 and 1/2 of one round on as many CTAs as items: fewer, taller segments
            // on fewer SMs.  HBM-bound widths stream from fewer concurrent row windows
            // (16384^2 / K=5: cfg 1 with 6 parts on 96 CTAs 328 us against 375 us under the model's
            // schedule and 351 us for the best default, profiles/r02p_tune_diag.txt)
            np = std::max(1.0, std::round(parts0 * (m == 2 ? 2.0 / 3.0 : 0.5)));
            ng = std::min(static_cast<double>(slots), static_cast<double>(strips) * np);
            nst = 0;
        } else if (m < nseeds) {
            // stealing on one and on two rounds of the model's items: warps that run out of
            // work take half of the largest unclaimed remainder (profiles/r02_steal_sched.txt)
            np = parts0 * (m - 3);
            ng = static_cast<double>(slots);
            nst = 4;
        } else {
            const double u = rng.uniform();
            if (u < 2.0 / 3.0) np = parts * std::exp(sigma * rng.normal());
            if (u >= 1.0 / 3.0) ng = grid * std::exp(sigma * rng.normal());
            if (steal > 0 && rng.uniform() < 0.5)             // the stealing threshold, in stages
                nst = static_cast<int>(std::lround(steal * std::exp(sigma * rng.normal())));
            nst = steal > 0 ? std::min(std::max(nst, 2), 64) : 0;
        }
        np = std::min<double>(std::max(1.0, std::round(np)), rows);
        ng = std::min(std::max(1.0, std::round(ng)), static_cast<double>(slots));
        Candidate child = parent;
        child.sched_parts = static_cast<int>(np);
        child.sched_grid = static_cast<int>(ng);
        child.sched_steal = nst;
        float us = 0.f;
        if ((s = b.time(child, reps, &us)) != SEPCONV_OK) return s;
        const float parent_before = parent_us;
        bool accepted = false;
        if (us < parent_us * 0.98f) {
            // a paired re-measurement (parent, child, parent, child) decides: batch-to-batch
            // drift of ~1-2% on 16384^2 otherwise admits children that are not faster
            float tp[2], tc[2];
            for (int r = 0; r < 2; ++r) {
                if ((s = b.time(parent, reps, &tp[r])) != SEPCONV_OK) return s;
                if ((s = b.time(child, reps, &tc[r])) != SEPCONV_OK) return s;
            }
            const float p2 = std::min(tp[0], tp[1]), c2 = std::min(tc[0], tc[1]);
            if (c2 < p2 * 0.99f) {
                accepted = true;
                parent = child;
                parent_us = c2;
                parts = np;
                grid = ng;
                steal = nst;
            } else if (p2 < parent_us) {
                parent_us = p2;
            }
        }
        if (const char *log = std::getenv("SEPCONV_TUNE_LOG")) {   // diagnostics: every child
            if (FILE *f = std::fopen(log, "a")) {
                std::fprintf(f, "mutation k%d cfg%d s%d: child p%dg%dst%d %.2f us vs parent %.2f -> %s\n", b.g.K,
                             child.config, child.store, child.sched_parts, child.sched_grid, child.sched_steal, us,
                             parent_before, accepted ? "accepted" : "rejected");
                std::fclose(f);
            }
        }
    }
    best = parent;
    best_us = parent_us;
    return SEPCONV_OK;
}

struct DeviceRestore {
    int prev = -1;
    explicit DeviceRestore(int dev) {
        cudaGetDevice(&prev);
        cudaSetDevice(dev);
    }
    ~DeviceRestore() {
        if (prev >= 0) cudaSetDevice(prev);
    }
};

// The exhaustive pass (+ mutation) on plan; fills best[3] (2D, SEPARABLE, AUTO).
sepconv_status_t tune_plan(sepconv_plan_t plan, int reps, int flags, int mutations, uint32_t seed,
                           sepconv_choice_t best[3]) {
    DeviceRestore restore(plan->dev.device);
    sepconv_status_t status;
    auto cs = candidates(plan);
    std::vector<float> med(cs.size(), -1.f);
    Bench b;
    if ((status = b.open(plan, !(flags & SEPCONV_TUNE_NO_L2_FLUSH))) != SEPCONV_OK) return status;
    for (size_t ci = 0; ci < cs.size(); ++ci)
        if ((status = b.time(cs[ci], reps, &med[ci])) != SEPCONV_OK) return status;
    // finalists -- up to four candidates within 8% of the fastest -- are timed twice more in
    // interleaved rounds and keep the fastest (flushed: the median) of their measurements: one sequential pass over
    // the candidates picked a configuration 8% slower than the runner-up on 16384^2 / K=13 (a
    // transient during the runner-up's batches; profiles/r02_interleave.txt, r02_tune_log.txt)
    std::vector<size_t> finalists;
    {
        const float fastest = *std::min_element(med.begin(), med.end());
        std::vector<size_t> &fin = finalists;
        for (size_t i = 0; i < cs.size(); ++i)
            if (med[i] >= 0 && med[i] <= fastest * 1.08f) fin.push_back(i);
        std::sort(fin.begin(), fin.end(), [&](size_t a, size_t c) { return med[a] < med[c]; });
        if (fin.size() > 4) fin.resize(4);
        if (fin.size() > 1) {
            std::vector<float> t1(fin.size()), t2(fin.size());
            for (int round = 0; round < 2; ++round)
                for (size_t f = 0; f < fin.size(); ++f)
                    if ((status = b.time(cs[fin[f]], reps, round ? &t2[f] : &t1[f])) != SEPCONV_OK) return status;
            for (size_t f = 0; f < fin.size(); ++f) {
                float v[3] = {med[fin[f]], t1[f], t2[f]};
                std::sort(v, v + 3);
                med[fin[f]] = b.need_flush ? v[1] : v[0];      // as in Bench::time
            }
        }
    }

    if (const char *log = std::getenv("SEPCONV_TUNE_LOG")) {   // diagnostics: every candidate's time
        if (FILE *f = std::fopen(log, "a")) {
            std::fprintf(f, "%s", plan_key(plan).c_str());
            for (size_t i = 0; i < cs.size(); ++i)
                std::fprintf(f, " | %d,%d,%d,%d,%d %.2f", cs[i].algo, cs[i].mapping, cs[i].fused, cs[i].config,
                             cs[i].store, med[i]);
            std::fprintf(f, "\n");
            std::fclose(f);
        }
    }

    // Power-aware comparison (R26): the tuner times short bursts, and in a sustained
    // stream of back-to-back passes the packed-FP32 row-pass configuration (cfg 4, the
    // FMA-heaviest: 80% FMA-pipe active) loses up to 5% to the power cap (16384^2 / K=17: 372.6 us
    // in the tuner, 393 us in bench.py, profiles/r02_driver_bench.json).  Without a flush it is
    // charged 4% when compared; flushed (mid-size) passes keep their measured time.
    // The same holds for the three-stage lockstep configuration (cfg 1) from K = 7 up: 330 us in
    // the tuner, 348-398 us in bench.py at 16384^2 / K=7 (6 runs on 3 boxes), 329-335 vs 361-381 us
    // at K=13, where the free-running cfg 2 moves 1-2% (profiles/r02zz_bench_c4.json,
    // profiles/r02_sustained_confirm_rejected/); below K=7 (cfg 1 on 96 CTAs, 330-345 us in the
    // bench) it keeps its measured time.
    auto eff = [&](const Candidate &c, float t) {
        const bool fused_tma = c.algo == SEPCONV_SEPARABLE && c.fused && c.mapping == SEPCONV_MAP_TMA;
        const bool heavy = fused_tma && (c.config == 4 || (c.config == 1 && b.g.K >= 7));
        return (heavy && !b.need_flush) ? t * 1.04f : t;
    };
    auto better = [&](size_t a, size_t c) {   // is candidate a better than incumbent c?
        if (med[a] < 0) return false;
        if (med[c] < 0) return true;
        const float ea = eff(cs[a], med[a]), ec = eff(cs[c], med[c]);
        if (ea < ec * 0.99f) return true;
        if (ec < ea * 0.99f) return false;
        if (passes(cs[a]) != passes(cs[c])) return passes(cs[a]) < passes(cs[c]);
        return false;   // keep the lower index
    };
    size_t bi[3] = {SIZE_MAX, SIZE_MAX, SIZE_MAX};
    for (size_t i = 0; i < cs.size(); ++i) {
        const int slot = cs[i].algo == SEPCONV_2D ? 0 : 1;
        if (bi[slot] == SIZE_MAX || better(i, bi[slot])) bi[slot] = i;
        if (bi[2] == SIZE_MAX || better(i, bi[2])) bi[2] = i;
    }
    Candidate win[3];
    float us[3];
    for (int s = 0; s < 3; ++s) {
        win[s] = cs[bi[s]];
        us[s] = med[bi[s]];
    }
    // the paper's evolutionary refinement of size-like tunables, on each single-kernel finalist
    // (up to six, below): a configuration that loses under the model's schedule can win under its
    // own best schedule (16384^2 / K=17: cfg 4 with 27 parts beats cfg 3, which gains nothing;
    // the fourth finalist is kept for configurations that only win with work stealing)
    if (mutations > 0) {
        // the pool: the single-kernel finalists, then, for every other single-kernel mapping /
        // configuration within 15% of the fastest under the model's schedule, its faster store
        // path: a configuration 7% behind under the model's schedule was 7% ahead under its own
        // (16384^2 / K=5, cfg 1: 375 -> 328 us with 6 parts on 96 CTAs, profiles/r02p_tune_diag.txt)
        std::vector<size_t> pool;
        for (size_t i : finalists)
            if (passes(cs[i]) == 1 && pool.size() < 4) pool.push_back(i);
        {
            const float fastest = *std::min_element(med.begin(), med.end());
            auto same_kernel = [&](size_t a, size_t c) {
                return cs[a].algo == cs[c].algo && cs[a].mapping == cs[c].mapping && cs[a].fused == cs[c].fused &&
                       cs[a].config == cs[c].config;
            };
            std::vector<size_t> more;
            for (size_t i = 0; i < cs.size(); ++i)
                if (med[i] >= 0 && med[i] <= fastest * 1.15f && passes(cs[i]) == 1)
                    more.push_back(i);
            std::sort(more.begin(), more.end(), [&](size_t a, size_t c) { return med[a] < med[c]; });
            for (size_t i : more)
                if (std::none_of(pool.begin(), pool.end(), [&](size_t j) { return same_kernel(i, j); }))
                    pool.push_back(i);
        }
        if (pool.empty()) pool.push_back(bi[2]);
        std::vector<std::pair<Candidate, float>> out;
        for (size_t i : pool) {
            Candidate c = cs[i];
            float t = med[i];
            if ((status = mutate_schedule(b, c, t, mutations, seed, reps)) != SEPCONV_OK) return status;
            out.emplace_back(c, t);
        }
        // fastest wins; within 1% of it the lower candidate index (R17)
        float tmin = eff(out[0].first, out[0].second);
        for (auto &o : out) tmin = std::min(tmin, eff(o.first, o.second));
        size_t pick = SIZE_MAX, k_pick = 0;
        for (size_t k = 0; k < out.size(); ++k)
            if (eff(out[k].first, out[k].second) <= tmin * 1.01f && (pick == SIZE_MAX || pool[k] < pick)) {
                pick = pool[k];
                k_pick = k;
            }
        const Candidate pick_c = out[k_pick].first;
        const float pick_t = out[k_pick].second;
        if (eff(pick_c, pick_t) < eff(win[2], us[2]) || pick == bi[2]) {
            win[2] = pick_c;
            us[2] = pick_t;
            bi[2] = pick;
        }
    }
    const int aslot = win[2].algo == SEPCONV_2D ? 0 : 1;
    if (bi[aslot] == bi[2] || eff(win[2], us[2]) < eff(win[aslot], us[aslot])) {
        win[aslot] = win[2];
        us[aslot] = us[2];
    }
    for (int s = 0; s < 3; ++s) {
        best[s] = to_choice(win[s], plan->k, SEPCONV_SRC_TUNED);
        best[s].median_us = us[s];
    }
    return SEPCONV_OK;
}

int mutations_of(const sepconv_tune_opts_t *opts) {
    if (!opts || opts->mutations == 0) return 12;
    return opts->mutations < 0 ? 0 : opts->mutations;
}

sepconv_status_t square_plan(int64_t side, int K, int device, sepconv_plan_t *p) {
    sepconv_plan_desc_t d;
    std::memset(&d, 0, sizeof d);
    d.n = 1;
    d.h = d.w = side;
    d.k = K;
    d.device = device;
    return sepconv_plan_ex(&d, p);
}

struct PlanHolder {
    sepconv_plan_t p = nullptr;
    ~PlanHolder() { sepconv_destroy(p); }
};

// times two choices on one plan (the cutoff placement of sepconv_tune_selector)
sepconv_status_t time_pair(sepconv_plan_t p, const sepconv_choice_t &a, const sepconv_choice_t &c, int reps,
                           int flags, float *ta, float *tc) {
    DeviceRestore restore(p->dev.device);
    Bench b;
    sepconv_status_t s = b.open(p, !(flags & SEPCONV_TUNE_NO_L2_FLUSH));
    if (s == SEPCONV_OK) s = b.time(from_choice(a), reps, ta);
    if (s == SEPCONV_OK) s = b.time(from_choice(c), reps, tc);
    return s;
}

}  // namespace

// Called by sepconv_plan_ex: an exact cache entry makes the plan tuned; otherwise a size
// selector for its K (NEXT-2 of SURVEY 8(f)) resolves AUTO by SELECT until sepconv_tune.
void sepconv_seed_from_cache(sepconv_plan_t plan) {
    const char *env = std::getenv("SEPCONV_TUNE_CACHE");
    if (!env || !*env) return;
    if (load_choices(env, plan_key(plan), plan->best)) {
        plan->tuned = true;
        return;
    }
    sepconv_selector_t sel;
    if (!load_selector(env, selector_key(plan->dev, plan->k), &sel) || sel.k != plan->k) return;
    sepconv_choice_t pick;
    if (sepconv_select(&sel, plan->n * plan->h * plan->w, &pick) != SEPCONV_OK) return;
    pick.sched_parts = pick.sched_grid = pick.sched_steal = 0;                    // size-specific: not transferred
    const int slot = pick.algo == SEPCONV_2D ? 0 : 1;
    for (int s = 0; s < 3; ++s) {
        // 2D / SEPARABLE requests keep their static defaults unless the selector picked that algorithm
        if (s == 2 || s == slot) {
            plan->best[s] = pick;
        } else {
            Candidate d = resolve(plan, s == 0 ? SEPCONV_2D : SEPCONV_SEPARABLE);   // plan->tuned still false
            plan->best[s] = to_choice(d, plan->k, SEPCONV_SRC_DEFAULT);
        }
    }
    plan->tuned = true;
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
    *choice = to_choice(cs[index], plan->k, SEPCONV_SRC_EXPLICIT);
    return SEPCONV_OK;
}

sepconv_status_t sepconv_tune(sepconv_plan_t plan, const sepconv_tune_opts_t *opts, sepconv_choice_t *chosen) {
    if (!plan) return fail(SEPCONV_E_INVALID, "plan is NULL");
    const int reps = (opts && opts->reps > 0) ? opts->reps : 20;
    const int flags = opts ? opts->flags : 0;
    const std::string path = cache_path_of(opts);
    const std::string key = plan_key(plan);

    if (!path.empty() && !(flags & SEPCONV_TUNE_FORCE) && load_choices(path, key, plan->best)) {
        plan->tuned = true;
        if (chosen) *chosen = plan->best[2];
        return SEPCONV_OK;
    }
    sepconv_choice_t best[3];
    sepconv_status_t s = tune_plan(plan, reps, flags, mutations_of(opts), opts ? opts->seed : 0u, best);
    if (s != SEPCONV_OK) return s;
    std::memcpy(plan->best, best, sizeof best);
    plan->tuned = true;
    if (!path.empty()) store_choices(path, key, plan->best);
    if (chosen) *chosen = plan->best[2];
    return SEPCONV_OK;
}

sepconv_status_t sepconv_select(const sepconv_selector_t *s, int64_t size, sepconv_choice_t *choice) {
    if (!s || !choice) return fail(SEPCONV_E_INVALID, "NULL argument");
    if (s->m < 1 || s->m > SEPCONV_SELECTOR_LEVELS) return fail(SEPCONV_E_INVALID, "selector m=%d outside 1..12", s->m);
    if (s->m > 1 && s->cutoffs[0] <= 0) return fail(SEPCONV_E_INVALID, "selector cutoff c_1 must be > 0");
    for (int i = 1; i + 1 < s->m; ++i)
        if (!(s->cutoffs[i] > s->cutoffs[i - 1])) return fail(SEPCONV_E_INVALID, "selector cutoffs not increasing");
    // alpha_i such that c_i > size >= c_{i-1}, c_0 = 0, c_m = infinity
    int i = 0;
    while (i + 1 < s->m && size >= s->cutoffs[i]) ++i;
    *choice = s->algos[i];
    choice->source = SEPCONV_SRC_SELECTOR;
    return SEPCONV_OK;
}

sepconv_status_t sepconv_tune_selector(int K, int device, const int64_t *sides, int nsides,
                                       const sepconv_tune_opts_t *opts, sepconv_selector_t *out) {
    static const int64_t kLevels[SEPCONV_SELECTOR_LEVELS] = {64, 128, 256, 512, 1024, 2048,
                                                             3072, 4096, 6144, 8192, 11584, 16384};
    if (K < 1 || K > SEPCONV_MAX_K) return fail(SEPCONV_E_UNSUPPORTED, "K=%d outside 1..%d", K, SEPCONV_MAX_K);
    if (!sides) {
        sides = kLevels;
        nsides = SEPCONV_SELECTOR_LEVELS;
    }
    if (nsides < 1 || nsides > SEPCONV_SELECTOR_LEVELS) return fail(SEPCONV_E_INVALID, "nsides must be in 1..12");
    for (int i = 0; i < nsides; ++i)
        if (sides[i] < K || (i && sides[i] <= sides[i - 1]))
            return fail(SEPCONV_E_INVALID, "sides must be >= K and strictly increasing");
    const int reps = (opts && opts->reps > 0) ? opts->reps : 10;
    const int flags = opts ? opts->flags : 0;
    auto same = [](const sepconv_choice_t &a, const sepconv_choice_t &c) {
        return std::make_tuple(static_cast<int>(a.algo), a.mapping, a.fused, a.config, a.store_path) ==
               std::make_tuple(static_cast<int>(c.algo), c.mapping, c.fused, c.config, c.store_path);
    };
    // 1. the exhaustive tuner (no mutation: schedules are size-specific) at every level
    std::vector<sepconv_choice_t> pick(nsides);
    DeviceInfo dev;
    for (int i = 0; i < nsides; ++i) {
        PlanHolder h;
        sepconv_status_t s = square_plan(sides[i], K, device, &h.p);
        if (s != SEPCONV_OK) return s;
        dev = h.p->dev;
        sepconv_choice_t best[3];
        if ((s = tune_plan(h.p, reps, flags, 0, 0u, best)) != SEPCONV_OK) return s;
        pick[i] = best[2];
    }
    // 2. merge equal neighbours; 3. place each cutoff between two different picks by timing
    // both at the geometric middle side of the two levels (one bisection step in log size)
    sepconv_selector_t sel;
    std::memset(&sel, 0, sizeof sel);
    sel.k = K;
    sel.m = 1;
    sel.algos[0] = pick[0];
    for (int i = 1; i < nsides; ++i) {
        if (same(pick[i], sel.algos[sel.m - 1])) continue;
        const double lo = static_cast<double>(sides[i - 1]), hi = static_cast<double>(sides[i]);
        const int64_t mid = std::llround(std::sqrt(lo * hi));
        int64_t cut_side = mid;                               // the side where pick[i] takes over
        if (mid > sides[i - 1] && mid < sides[i]) {
            PlanHolder h;
            sepconv_status_t s = square_plan(mid, K, device, &h.p);
            float t_lo = 0.f, t_hi = 0.f;
            if (s == SEPCONV_OK) s = time_pair(h.p, sel.algos[sel.m - 1], pick[i], reps, flags, &t_lo, &t_hi);
            if (s != SEPCONV_OK) return s;
            // the lower level's pick still wins at the middle: the switch lies above it
            cut_side = t_lo <= t_hi ? std::llround(std::sqrt(static_cast<double>(mid) * hi))
                                    : std::llround(std::sqrt(lo * static_cast<double>(mid)));
        }
        sel.cutoffs[sel.m - 1] = cut_side * cut_side;         // size = n*h*w pixels
        sel.algos[sel.m] = pick[i];
        ++sel.m;
    }
    for (int i = 0; i < sel.m; ++i) {
        sel.algos[i].sched_parts = sel.algos[i].sched_grid = sel.algos[i].sched_steal = 0;
        sel.algos[i].source = SEPCONV_SRC_SELECTOR;
    }
    const std::string path = cache_path_of(opts);
    if (!path.empty()) store_selector(path, selector_key(dev, K), sel);
    if (out) *out = sel;
    return SEPCONV_OK;
}

}  // extern "C"
