// sg_plan.cpp -- the mapping flow of Fig. 3.1:
//   annotated graph -> partitioning (Algorithm 1, aided by the PEE)
//   -> PDG -> ILP multi-GPU mapping over the GPU topology -> code generation.
#include "sg_plan.h"

#include <algorithm>
#include <chrono>
#include <cstdio>
#include <cstdlib>
#include <cmath>
#include <functional>
#include <numeric>
#include <set>
#include <tuple>

#include "sg_codegen.h"

namespace sg {

// ============================================================ PEE (B200)
// Section 3.3 of the paper predicts a partition's kernel time from per-node
// work and the kernel parameters the code generator will choose ("the PEE
// includes the same optimization done by the GPU code generator",
// PAPER.md:579-581).  Here: the code generator's own mode decision
// (register_mode_eligible) and its algorithmic work counts, priced with B200
// throughputs:
//   Tcomp = flops/(FP32 peak * eff) + int ops/INT peak + fp64 work + shared-memory bytes/SMEM bw
//   Tdt   = boundary-stream bytes / HBM bandwidth
//   T     = max(Tcomp, Tdt) + per-level barrier and per-fragment launch costs
// (the max() of Eq. III.8 survives: compute and data movement overlap).
namespace {
constexpr double kClk = 1.9e9;
constexpr double kSM = 148;
constexpr double kFp32 = kSM * 128 * 2 * kClk;    // flop/s
constexpr double kInt = kSM * 64 * kClk;          // int min/max per s
constexpr double kFp64 = 37e12;                   // flop/s
constexpr double kSmem = kSM * 128 * kClk;        // bytes/s
constexpr double kHbm = 6.5536e12;                // bytes/s (MEASURED_PEAKS.json copy)
constexpr double kLaunch = 8.5e-6;                // s per kernel launch incl. ramp / tail (fitted)
constexpr double kFragIters = 1 << 20;            // iterations per fragment assumed when planning (the
                                                  // runtime's default at the bench sizes: n / (8 G))
constexpr double kLoopFiring = 25e-9;             // s per sequential loop firing
constexpr long long kIlpNodeBudget = 4000000;     // branch-and-bound nodes per mapping (deterministic)
constexpr int kFusedMaxInEdges = 8;               // staged: more boundary inputs -> general path expected
constexpr double kFrameParRef = 1.0;               // par_eff the fitted e_frame corresponds to
constexpr double kSplitMargin = 0.05;             // a cut must beat one partition by more than the PEE's noise

// Model constants, fitted by least squares on log time to the partition corpus measured on the B200
// (scripts/pee_calibrate.py -> profiles/pee_corpus_r02.json, 707 partitions; scripts/pee_fit.py), the way
// the paper fits its C1, C2.  One set serves both estimates: at plan time the kernel
// shape (register variant, fused or general staged path, tile) is inferred from the work; after code
// generation the generated kernel's own shape is used (pee_refine).
struct PeeModel {
    double e_reg;      // register mode: fraction of the fp32 peak
    double c_row;      // register rows: ns per (items of one iteration)^2 (one thread holds the row)
    double c_demand;   // demand-ordered wide single-component rows: ns per items^2
    double e_staged;   // staged fused kernels: fraction of the fp32 peak
    double e_frame;    // frame FIRs
    double e_general;  // staged general path (fused path declined): fraction of the fp32 peak
    double c_edge;     // fused: ns per boundary edge per tile
    double c_level;    // ns per compute level per tile
    double e_gen_hbm;  // general path: fraction of the HBM bandwidth its boundary streams reach
    double c_gen_edge; // general path: ns per boundary edge per tile
    double c_gather;   // views only (gather kernels): ns per output item and (boundary input + 1)
};
// fitted on the round-2 corpus (profiles/pee_corpus_r02.json); the general-path constants on the corpus of
// the code generator before gather kernels existed, where that path ran (a 2-D DCT split: 58.8 ns/block)
// e_frame re-centred (geometric mean of measured / estimated) on the frame-FIR partitions of the corpus of the
// sliding-window kernels, which report their parallel efficiency (e_frame x par_eff; profiles/pee_corpus_r02b.json,
// validated again on r02c); c_demand on the bench times of the rolled four-run demand kernels (DCT 16x16
// 0.873 ns/block over a 512-item row, MatMul 16 1.51 ns over 768 items: c = t / row^2, geometric mean)
constexpr PeeModel kModel{0.8, 2.782e-6, 2.9e-6, 1.0, 0.595, 0.0034, 0.7779, 8.674, 0.5677, 5.783, 5.649e-4};

struct KernelShape {  // the code generator's decisions the model needs
    bool demand = false, inplace = false, fused = true, gather = false;
    double tile = 1;
    double par_eff = 1;  // frame-FIR levels: the code generator's simulated parallel efficiency
};

double model_ns(const PartitionWork& w, int mode, bool bitslice, double bitslice_ops, const KernelShape& k,
                const PeeModel& m) {
    const double hbm = (w.in_bytes + w.out_bytes) / kHbm * 1e9;
    if (bitslice) return std::max(bitslice_ops / kInt * 1e9, hbm);
    if (mode == 4) return std::max(kLoopFiring * w.loop_firings * 1e9, hbm);
    if (mode == 1) {
        const double row2 = w.row_items * w.row_items;
        if (k.demand) return std::max(hbm, m.c_demand * row2);
        const double tc = (w.flops / (kFp32 * m.e_reg) + w.intops / kInt + w.dfma * 80.0 / kFp64) * 1e9;
        return std::max({tc, hbm, k.inplace ? 0.0 : m.c_row * row2});
    }
    if (k.gather) return std::max(hbm, m.c_gather * (w.out_bytes / 4.0) * (w.in_edges + 1));
    const double e = k.fused ? (w.frame ? m.e_frame * k.par_eff : m.e_staged) : m.e_general;
    const double W = std::max(1.0, k.tile);
    const double recompute = 1.0 + w.halo_firings / (W * std::max(1.0, w.firings));
    const double tc = (w.flops / (kFp32 * e) + w.intops / kInt + w.dfma * 80.0 / kFp64) * recompute * 1e9 +
                      kLoopFiring * w.loop_firings * 1e9;
    const double edges = w.in_edges + w.out_edges;
    if (!k.fused) return std::max(tc, hbm / m.e_gen_hbm) + m.c_gen_edge * edges / W + m.c_level * (w.levels + 1) / W;
    return std::max(tc, hbm) + m.c_edge * edges / W + m.c_level * (w.levels + 1) / W;
}
}  // namespace

PeeEstimate pee_estimate(const Flat& f, const std::vector<int>& nodes) {
    PeeEstimate est;
    bool loop = false;
    for (int v : nodes) loop = loop || f.nodes[v].type == N_LOOP;
    est.mode = loop && nodes.size() == 1 ? 4 : (register_mode_eligible(f, nodes, nullptr) ? 1 : 2);
    est.bitslice = est.mode == 1 && bitslice_eligible(f, nodes, nullptr);
    est.work = partition_work(f, nodes, est.mode == 1 && !est.bitslice);
    const PartitionWork& w = est.work;
    if (est.bitslice) {
        // bitslice mode: one LOP3 covers 32 iterations; an S-box is a ~44-gate circuit, a word <-> bits
        // conversion a share of a 32x32 transpose (~5 ops per bit)
        for (int v : nodes) {
            const Node& n = f.nodes[v];
            if (n.type != N_FILTER) continue;
            switch (n.kind) {
            case SG_K_XOR: case SG_K_XOR_CONST: est.bitslice_ops += (double)n.rep * n.iv[0] / 32.0; break;
            case SG_K_SBOX: est.bitslice_ops += (double)n.rep * 44.0 / 32.0; break;
            case SG_K_INTO_BITS: case SG_K_BITS_TO_INT: est.bitslice_ops += (double)n.rep * 5.0; break;
            default: break;
            }
        }
    }
    // the kernel shape the code generator will pick, inferred: register rows of one wide dependence
    // component are demand-ordered (>= 384 items, sg_codegen.cpp), several components run in place;
    // staged tiles hold ~150k live firings' worth of iterations (frame FIRs: one frame)
    KernelShape k;
    k.demand = est.mode == 1 && w.row_items >= 384 && w.components == 1;
    k.inplace = est.mode == 1 && w.components > 1;
    k.tile = w.frame ? 1.0 : std::min(4096.0, std::max(1.0, 150000.0 / std::max(1.0, w.firings)));
    // staged partitions: views only -> the gather kernel (HBM-bound like the fused path); with compute,
    // the fused path declines for merges of many boundary streams (runtime index readers: the general
    // path) -- observed over the corpus
    const bool compute = (w.flops + w.intops + w.dfma + w.loop_firings) > 0;
    k.gather = est.mode == 2 && !compute;
    est.fused = k.fused = est.mode != 2 || !compute || w.in_edges <= kFusedMaxInEdges;
    if (!k.fused) {  // the general path's tile: every buffer of the tile in ~100 KB of shared memory
        double W = 1;
        while (W < 1024 && 2 * W * 8.0 * std::max(1.0, w.row_items) <= 100.0 * 1024) W *= 2;
        k.tile = W;
    }
    est.t = model_ns(w, est.mode, est.bitslice, est.bitslice_ops, k, kModel);
    est.t_dt = (w.in_bytes + w.out_bytes) / kHbm * 1e9;
    est.t_comp = est.t;
    return est;
}

double pee_refine(const PeeEstimate& est, const KernelInfo& ki) {
    KernelShape k;
    k.demand = ki.mode == 1 && ki.reg_variant == 2;
    k.inplace = ki.mode == 1 && ki.reg_variant == 1;
    k.fused = ki.mode != 2 || ki.fused;
    k.gather = ki.mode == 5;
    k.tile = std::max(1, ki.tile);
    k.par_eff = ki.fused ? std::max(0.05, ki.par_eff / kFrameParRef) : 1.0;
    return model_ns(est.work, est.mode, est.bitslice, est.bitslice_ops, k, kModel);
}

double launch_ns_per_iter(int64_t frag) { return kLaunch / (double)(frag > 0 ? frag : (int64_t)kFragIters) * 1e9; }

double paper_model(const std::vector<double>& t, const std::vector<double>& fr, int S, int W, int F, double D,
                   double C1, double C2, double* tcomp, double* tdt, double* tdb) {
    double tc = 0;  // Eq. III.9: Tcomp = sum_i t_i / min(f_i, S)
    for (size_t i = 0; i < t.size(); i++) tc += t[i] / std::min(fr[i], (double)S);
    double td = C1 * D / F;                 // Eq. III.10
    double tb = C2 * D / (F + (double)W * S);  // Eq. III.11 (all threads swap WS and DB)
    double texec = std::max(tc, td) + tb;   // Eq. III.8
    if (tcomp) *tcomp = tc;
    if (tdt) *tdt = td;
    if (tdb) *tdb = tb;
    return texec / W;                       // Eq. III.12
}

// ===================================================== partition structure
// "A partition is convex if there is no path between two internal nodes that
// goes through an external node" (footnote).
bool is_convex(const Flat& f, const std::vector<char>& in) {
    const int N = (int)f.nodes.size();
    std::vector<char> seen(N, 0);
    std::vector<int> st;
    for (int v = 0; v < N; v++) {
        if (!in[v]) continue;
        for (int e : f.nodes[v].out) {
            int w = f.edges[e].dst;
            if (w >= 0 && !in[w] && !seen[w]) { seen[w] = 1; st.push_back(w); }
        }
    }
    while (!st.empty()) {
        int u = st.back();
        st.pop_back();
        for (int e : f.nodes[u].out) {
            int w = f.edges[e].dst;
            if (w < 0) continue;
            if (in[w]) return false;
            if (!seen[w]) { seen[w] = 1; st.push_back(w); }
        }
    }
    return true;
}

namespace {
struct PartState {
    const Flat& f;
    double cap;
    int64_t frag = 0;
    std::vector<int> owner;                    // node -> partition id (-1 none)
    std::vector<std::vector<int>> members;     // partition id -> nodes (empty = dead)
    std::vector<double> T;
    std::vector<char> io;                      // IO-bound flag
    PartState(const Flat& fl, double c, int64_t fr) : f(fl), cap(c), frag(fr), owner(fl.nodes.size(), -1) {}

    mutable std::map<std::vector<int>, PeeEstimate> memo;
    double cost(const std::vector<int>& nodes, bool* io_bound = nullptr) const {
        std::vector<int> key(nodes);
        std::sort(key.begin(), key.end());
        auto it = memo.find(key);
        if (it == memo.end()) it = memo.emplace(key, pee_estimate(f, key)).first;
        if (io_bound) *io_bound = it->second.io_bound();
        return it->second.t + launch_ns_per_iter(frag);  // merging saves a kernel launch per fragment
    }
    int make(const std::vector<int>& nodes) {
        int id = (int)members.size();
        members.push_back(nodes);
        bool iob = false;
        T.push_back(cost(nodes, &iob));
        io.push_back(iob);
        for (int v : nodes) owner[v] = id;
        return id;
    }
    bool connected(const std::vector<int>& a, const std::vector<int>& b) const {
        std::vector<char> inb(f.nodes.size(), 0);
        for (int v : b) inb[v] = 1;
        for (int v : a) {
            for (int e : f.nodes[v].out) if (f.edges[e].dst >= 0 && inb[f.edges[e].dst]) return true;
            for (int e : f.nodes[v].in) if (f.edges[e].src >= 0 && inb[f.edges[e].src]) return true;
        }
        return false;
    }
    // Try-Merge: connected, convex, and T(merged) < T(a) + T(b).
    bool try_merge_sets(const std::vector<std::vector<int>>& sets, const std::vector<double>& Ts,
                        std::vector<int>& merged, double& tm) const {
        merged.clear();
        for (auto& s : sets) merged.insert(merged.end(), s.begin(), s.end());
        std::sort(merged.begin(), merged.end());
        std::vector<char> in(f.nodes.size(), 0);
        for (int v : merged) in[v] = 1;
        if (!is_convex(f, in)) return false;
        tm = cost(merged);
        double sum = std::accumulate(Ts.begin(), Ts.end(), 0.0);
        if (!(tm < sum)) return false;
        if (cap > 0 && tm > cap) return false;
        return true;
    }
    bool try_merge(int a, int b) {
        if (a == b || members[a].empty() || members[b].empty()) return false;
        if (!connected(members[a], members[b])) return false;
        std::vector<int> m;
        double tm;
        if (!try_merge_sets({members[a], members[b]}, {T[a], T[b]}, m, tm)) return false;
        for (int v : members[b]) owner[v] = a;
        members[a] = m;
        members[b].clear();
        T[a] = tm;
        bool iob = false;
        cost(m, &iob);
        io[a] = iob;
        return true;
    }
    std::vector<int> neighbours(int p) const {
        std::set<int> s;
        for (int v : members[p]) {
            for (int e : f.nodes[v].out) { int w = f.edges[e].dst; if (w >= 0 && owner[w] >= 0 && owner[w] != p) s.insert(owner[w]); }
            for (int e : f.nodes[v].in) { int w = f.edges[e].src; if (w >= 0 && owner[w] >= 0 && owner[w] != p) s.insert(owner[w]); }
        }
        return std::vector<int>(s.begin(), s.end());
    }
    std::vector<int> live() const {
        std::vector<int> r;
        for (int i = 0; i < (int)members.size(); i++) if (!members[i].empty()) r.push_back(i);
        return r;
    }
};

}  // namespace

std::vector<std::vector<int>> algorithm1(const Flat& f, double cap, int64_t iters_per_fragment) {
    PartState S(f, cap, iters_per_fragment);
    // ---- Phase 1: inside innermost pipelines (Alg. 1 lines 2-10), recorded by Flat::build
    for (auto& pipe : f.pipes) {
        size_t i = 0;
        while (i < pipe.size()) {
            int p = S.make({pipe[i]});
            size_t j = i + 1;
            while (j < pipe.size()) {            // Try-Merge one neighbour node in pipe with p
                int q = S.make({pipe[j]});
                if (!S.try_merge(p, q)) {        // h <- last failed node
                    S.members[q].clear();
                    S.owner[pipe[j]] = -1;
                    break;
                }
                j++;
            }
            i = j;
        }
    }
    // ---- Phase 2: nodes outside partitions (lines 13-20)
    for (int n = 0; n < (int)f.nodes.size(); n++) {
        if (S.owner[n] >= 0) continue;
        int p = S.make({n});
        bool merged = true;
        while (merged) {
            merged = false;
            std::set<int> cand;
            for (int v : S.members[p]) {
                for (int e : f.nodes[v].out) { int w = f.edges[e].dst; if (w >= 0 && S.owner[w] < 0) cand.insert(w); }
                for (int e : f.nodes[v].in) { int w = f.edges[e].src; if (w >= 0 && S.owner[w] < 0) cand.insert(w); }
            }
            for (int k : cand) {
                if (S.owner[k] >= 0) continue;
                int q = S.make({k});
                if (S.try_merge(p, q)) merged = true;
                else { S.members[q].clear(); S.owner[k] = -1; }
            }
        }
    }
    // ---- Phase 3: IO-bound first, ascending T, three rounds (lines 23-31)
    for (int round = 0; round < 3; round++) {
        bool merged = true;
        while (merged) {
            merged = false;
            std::vector<int> L1, L12 = S.live();
            for (int p : L12) if (S.io[p]) L1.push_back(p);
            std::vector<int>& outer = round == 2 ? L12 : L1;
            std::sort(outer.begin(), outer.end(), [&](int a, int b) { return S.T[a] < S.T[b]; });
            for (int p : outer) {
                std::vector<int> nb = S.neighbours(p);
                std::sort(nb.begin(), nb.end(), [&](int a, int b) { return S.T[a] < S.T[b]; });
                for (int q : nb) {
                    bool ok = round == 0 ? (bool)S.io[q] : true;
                    if (!ok) continue;
                    if (S.try_merge(p, q)) { merged = true; break; }
                }
                if (merged) break;
            }
        }
    }
    // ---- Phase 4 (lines 34-35): (1) two neighbours at once, (2) all nodes at once
    bool merged = true;
    while (merged) {
        merged = false;
        for (int p : S.live()) {
            std::vector<int> nb = S.neighbours(p);
            for (size_t a = 0; a < nb.size() && !merged; a++)
                for (size_t b = a + 1; b < nb.size() && !merged; b++) {
                    int q = nb[a], r = nb[b];
                    std::vector<int> m;
                    double tm;
                    if (S.try_merge_sets({S.members[p], S.members[q], S.members[r]}, {S.T[p], S.T[q], S.T[r]}, m, tm)) {
                        for (int v : S.members[q]) S.owner[v] = p;
                        for (int v : S.members[r]) S.owner[v] = p;
                        S.members[p] = m;
                        S.members[q].clear();
                        S.members[r].clear();
                        S.T[p] = tm;
                        bool iob;
                        S.cost(m, &iob);
                        S.io[p] = iob;
                        merged = true;
                    }
                }
            if (merged) break;
        }
    }
    std::vector<std::vector<int>> parts;
    for (int p : S.live()) parts.push_back(S.members[p]);
    if (cap <= 0 && parts.size() > 1) {  // all nodes at once: never worse than single-partition
        std::vector<int> all(f.nodes.size());
        std::iota(all.begin(), all.end(), 0);
        double sum = 0;
        for (int p : S.live()) sum += S.T[p];
        if (S.cost(all) < sum * (1.0 + kSplitMargin)) parts = {all};
    }
    return parts;
}

// ========================================================= topology
// NVSwitch (B200 HGX): every GPU k has an uplink k->switch and a downlink
// switch->k; traffic i->j loads uplink i and downlink j.  The dtlist rule of
// section 3.2.1 applied to this star.
Topology Topology::nvswitch(int G) {
    Topology t;
    t.G = G;
    t.L = 2 * G;
    t.dt.assign((size_t)t.L * G * G, 0);
    for (int i = 0; i < G; i++)
        for (int j = 0; j < G; j++) {
            if (i == j) continue;
            t.dt[(size_t)i * G * G + (size_t)i * G + j] = 1;          // uplink of i
            t.dt[(size_t)(G + j) * G * G + (size_t)i * G + j] = 1;    // downlink of j
        }
    return t;
}

// Fig. 3.3: Host - SW1 - {SW2: GPU1, GPU2}, {SW3: GPU3, GPU4}.
// Links (each direction separately): GPUk<->its switch, SW2<->SW1, SW3<->SW1.
// "the load of an uplink l is contributed by the data transfer from GPU i to
// GPU j if and only if i is a child of l and j is not"; downlinks mirror it.
Topology Topology::pcie_tree4() {
    Topology t;
    t.G = 4;
    // links: 0-3 GPUk->SW (up), 4-7 SW->GPUk (down), 8 SW2->SW1, 9 SW1->SW2, 10 SW3->SW1, 11 SW1->SW3
    t.L = 12;
    t.dt.assign((size_t)t.L * 16, 0);
    auto sw = [](int g) { return g < 2 ? 0 : 1; };  // 0 = SW2, 1 = SW3
    for (int i = 0; i < 4; i++)
        for (int j = 0; j < 4; j++) {
            if (i == j) continue;
            t.dt[(size_t)i * 16 + i * 4 + j] = 1;        // leaf uplink of i
            t.dt[(size_t)(4 + j) * 16 + i * 4 + j] = 1;  // leaf downlink of j
            if (sw(i) != sw(j)) {                        // crosses SW1
                int up = sw(i) == 0 ? 8 : 10, down = sw(j) == 0 ? 9 : 11;
                t.dt[(size_t)up * 16 + i * 4 + j] = 1;
                t.dt[(size_t)down * 16 + i * 4 + j] = 1;
            }
        }
    return t;
}

// ===================================================== ILP (Eq. III.1-III.7)
double mapping_cost(const std::vector<double>& T, const std::vector<PdgEdge>& pdg, const Topology& topo, double lat,
                    double bw, const std::vector<int>& a) {
    std::vector<double> gl(topo.G, 0.0), ll(topo.L, 0.0);
    for (size_t i = 0; i < T.size(); i++) gl[a[i]] += T[i];                       // III.4
    std::set<std::tuple<int, int, int>> shipped;                                   // duplicated data: once per
    for (auto& e : pdg) {                                                          // III.6-III.7 (src, dst) GPU
        int k = a[e.src], h = a[e.dst];
        if (k == h) continue;
        if (e.data >= 0 && !shipped.insert(std::make_tuple(e.data, k, h)).second) continue;
        for (int l = 0; l < topo.L; l++) if (topo.carries(l, k, h)) ll[l] += e.bytes;
    }
    double tmax = 0;
    for (double x : gl) tmax = std::max(tmax, x);                                  // III.1
    for (int l = 0; l < topo.L; l++) tmax = std::max(tmax, lat + ll[l] / bw);      // III.2-III.3
    return tmax;
}

MapResult map_partitions(const std::vector<double>& T, const std::vector<PdgEdge>& pdg, const Topology& topo,
                         double lat, double bw, int time_limit_ms, int method, long long node_limit) {
    const int P = (int)T.size(), G = topo.G;
    MapResult best;
    best.assign.assign(P, 0);
    if (P == 0) { best.optimal = true; best.tmax = 0; return best; }
    if (method == 1) {  // brute force over G^P
        std::vector<int> a(P, 0);
        best.tmax = mapping_cost(T, pdg, topo, lat, bw, a);
        for (;;) {
            int i = 0;
            while (i < P && ++a[i] == G) a[i++] = 0;
            if (i == P) break;
            double c = mapping_cost(T, pdg, topo, lat, bw, a);
            if (c < best.tmax - 1e-12) { best.tmax = c; best.assign = a; }
        }
        best.optimal = true;
        return best;
    }
    // branch and bound: partitions by decreasing T; LPT incumbent
    // interchangeable partitions (same T, the same PDG edges to the same other partitions, none between
    // them): classes; members are branched consecutively and in non-decreasing GPU order (symmetry
    // breaking: sorting a consecutive run of identical jobs keeps first-use GPU labels valid)
    std::vector<int> cls(P);
    {
        std::vector<std::vector<std::tuple<int, double, int, int>>> sig(P);
        for (auto& e : pdg) {
            if (e.src == e.dst) continue;
            sig[e.src].push_back(std::make_tuple(e.dst, e.bytes, 1, e.data));
            sig[e.dst].push_back(std::make_tuple(e.src, e.bytes, 0, e.data));
        }
        for (auto& v : sig) std::sort(v.begin(), v.end());
        std::map<std::pair<double, std::vector<std::tuple<int, double, int, int>>>, int> ids;
        for (int i = 0; i < P; i++) {
            auto key = std::make_pair(T[i], sig[i]);
            auto it = ids.find(key);
            cls[i] = it == ids.end() ? (ids[key] = i) : it->second;
        }
        for (auto& e : pdg)  // members adjacent to each other are not interchangeable
            if (e.src != e.dst && cls[e.src] == cls[e.dst]) {
                const int c = cls[e.src];
                for (int i = 0; i < P; i++) if (cls[i] == c) cls[i] = i;
            }
    }
    std::vector<int> ord(P);
    std::iota(ord.begin(), ord.end(), 0);
    std::stable_sort(ord.begin(), ord.end(), [&](int x, int y) {
        return T[x] != T[y] ? T[x] > T[y] : cls[x] < cls[y];
    });
    {
        std::vector<int> a(P, 0);
        std::vector<double> gl(G, 0);
        for (int i : ord) {
            int g = (int)(std::min_element(gl.begin(), gl.end()) - gl.begin());
            a[i] = g;
            gl[g] += T[i];
        }
        best.assign = a;
        best.tmax = mapping_cost(T, pdg, topo, lat, bw, a);
        std::vector<int> z(P, 0);
        double cz = mapping_cost(T, pdg, topo, lat, bw, z);
        if (cz < best.tmax) { best.tmax = cz; best.assign = z; }
        // local search on the incumbent (single moves, then pairwise swaps, first improvement) so the
        // branch and bound starts from a tight upper bound
        for (bool improved = true; improved;) {
            improved = false;
            for (int i = 0; i < P && !improved; i++)
                for (int g = 0; g < G && !improved; g++) {
                    if (g == best.assign[i]) continue;
                    std::vector<int> b = best.assign;
                    b[i] = g;
                    double c = mapping_cost(T, pdg, topo, lat, bw, b);
                    if (c < best.tmax * (1 - 1e-12)) { best.tmax = c; best.assign = b; improved = true; }
                }
            for (int i = 0; i < P && !improved; i++)
                for (int j = i + 1; j < P && !improved; j++) {
                    if (best.assign[i] == best.assign[j]) continue;
                    std::vector<int> b = best.assign;
                    std::swap(b[i], b[j]);
                    double c = mapping_cost(T, pdg, topo, lat, bw, b);
                    if (c < best.tmax * (1 - 1e-12)) { best.tmax = c; best.assign = b; improved = true; }
                }
        }
    }
    bool symmetric = true;  // all GPUs interchangeable (true for the NVSwitch star)
    {
        Topology s = Topology::nvswitch(G);
        symmetric = s.L == topo.L && s.dt == topo.dt;
    }
    struct Adj { int other; double bytes; bool out; int data; };
    std::vector<std::vector<Adj>> adj(P);  // edges to earlier-ordered partitions
    std::vector<int> rank(P);
    for (int k = 0; k < P; k++) rank[ord[k]] = k;
    for (auto& e : pdg) {
        if (e.src == e.dst) continue;
        int later = rank[e.src] > rank[e.dst] ? e.src : e.dst;
        int other = later == e.src ? e.dst : e.src;
        adj[later].push_back({other, e.bytes, later == e.src, e.data});
    }
    std::map<std::tuple<int, int, int>, int> shipped;  // (data, src GPU, dst GPU) -> edges carrying it
    std::vector<double> suffix(P + 1, 0.0);
    for (int k = P - 1; k >= 0; k--) suffix[k] = suffix[k + 1] + T[ord[k]];
    std::vector<int> a(P, -1);
    std::vector<double> gl(G, 0.0), ll(topo.L, 0.0);
    auto t0 = std::chrono::steady_clock::now();
    bool timed_out = false;
    long long nodes = 0;
    double total = suffix[0];
    std::function<void(int, int, double)> rec = [&](int k, int used, double cur) {
        if (timed_out) return;
        if (node_limit > 0 && nodes >= node_limit) { timed_out = true; return; }  // deterministic budget
        if ((++nodes & 4095) == 0 && time_limit_ms > 0) {
            auto ms = std::chrono::duration_cast<std::chrono::milliseconds>(std::chrono::steady_clock::now() - t0).count();
            if (ms > time_limit_ms) { timed_out = true; return; }
        }
        double lb = std::max(cur, total / G);
        if (k < P) lb = std::max(lb, T[ord[k]]);
        if (lb >= best.tmax - 1e-12) return;
        if (k == P) {
            best.tmax = cur;
            for (int i = 0; i < P; i++) best.assign[i] = a[i];
            return;
        }
        int i = ord[k];
        int gmax = symmetric ? std::min(G - 1, used) : G - 1;
        const int gmin = k > 0 && cls[ord[k - 1]] == cls[i] ? a[ord[k - 1]] : 0;
        for (int g = gmin; g <= gmax; g++) {
            a[i] = g;
            gl[g] += T[i];
            double c = std::max(cur, gl[g]);
            std::vector<std::pair<int, double>> touched;
            std::vector<std::tuple<int, int, int>> counted;
            for (auto& pr : adj[i]) {
                int j = pr.other;
                double D = pr.bytes;
                int src = pr.out ? g : a[j], dst = pr.out ? a[j] : g;
                if (src == dst) continue;
                if (pr.data >= 0) {
                    auto key = std::make_tuple(pr.data, src, dst);
                    counted.push_back(key);
                    if (shipped[key]++ > 0) continue;  // the same duplicated stream already crosses this pair
                }
                for (int l = 0; l < topo.L; l++)
                    if (topo.carries(l, src, dst)) {
                        ll[l] += D;
                        touched.push_back({l, D});
                        c = std::max(c, lat + ll[l] / bw);
                    }
            }
            rec(k + 1, std::max(used, g + 1), c);
            for (auto& key : counted) shipped[key]--;
            for (auto& t : touched) ll[t.first] -= t.second;
            gl[g] -= T[i];
            a[i] = -1;
        }
    };
    rec(0, 0, lat);
    best.optimal = !timed_out;
    // recompute exactly
    best.tmax = mapping_cost(T, pdg, topo, lat, bw, best.assign);
    return best;
}

// ============================================================ plan assembly
namespace {
// Partitions for a pipeline over Gs GPUs (Algorithm 1's cap depends on Gs).
// cap_mult scales Algorithm 1's G-aware cap (0: no cap).
std::vector<std::vector<int>> make_partitions(const Flat& f, int Gs, const sg_plan_opts& o, double cap_mult = 1.0) {
    const int N = (int)f.nodes.size();
    std::vector<std::vector<int>> parts;
    switch (o.partitioner) {
    case SG_PART_SINGLE: {
        std::vector<int> all(N);
        std::iota(all.begin(), all.end(), 0);
        parts.push_back(all);
        break;
    }
    case SG_PART_PER_FILTER:
        for (int v = 0; v < N; v++) parts.push_back({v});
        break;
    case SG_PART_USER: {
        if (!o.node_partition || o.n_node_partition != N)
            throw Error(SG_E_ARG, "SG_PART_USER needs node_partition[n_nodes] (n_nodes = " + std::to_string(N) + ")");
        std::map<int, std::vector<int>> m;
        for (int v = 0; v < N; v++) m[o.node_partition[v]].push_back(v);
        for (auto& kv : m) parts.push_back(kv.second);
        break;
    }
    case SG_PART_CHAIN: {  // one partition per chain-fission group; nodes before / after join the first / last
        if (f.chain_first.empty()) throw Error(SG_E_ARG, "SG_PART_CHAIN needs a chain-fissioned graph (chain_groups >= 2)");
        const int m = (int)f.chain_first.size();
        parts.assign(m, {});
        for (int v = 0; v < N; v++) {
            int g = 0;
            while (g + 1 < m && v >= f.chain_first[g + 1]) g++;
            parts[g].push_back(v);
        }
        break;
    }
    case SG_PART_ALGORITHM1: {
        double cap = 0;
        if (Gs > 1 && cap_mult > 0) {
            std::vector<int> all(N);
            std::iota(all.begin(), all.end(), 0);
            double sum = 0;
            for (int v = 0; v < N; v++) sum += pee_estimate(f, {v}).t;
            // G-aware cap: similar-sized partitions (goal 4)
            cap = std::max(pee_estimate(f, all).t, sum / 4) / Gs * 1.25 * cap_mult;
        }
        parts = algorithm1(f, cap, o.iters_per_fragment);
        break;
    }
    default: throw Error(SG_E_ARG, "unknown partitioner");
    }
    // a feedback loop runs sequentially: it is a partition of its own.  Splitting a convex
    // partition into {ancestors of the loop}, {loop}, {the rest} keeps every piece convex and the
    // partition graph acyclic (no path leaves the rest and re-enters the ancestors).
    for (bool again = true; again;) {
        again = false;
        for (size_t i = 0; i < parts.size() && !again; i++) {
            if (parts[i].size() < 2) continue;
            for (int v : parts[i]) {
                if (f.nodes[v].type != N_LOOP) continue;
                std::vector<char> anc(N, 0);
                std::vector<int> st{v};
                while (!st.empty()) {
                    int u = st.back();
                    st.pop_back();
                    for (int e : f.nodes[u].in) {
                        int w = f.edges[e].src;
                        if (w >= 0 && !anc[w]) { anc[w] = 1; st.push_back(w); }
                    }
                }
                std::vector<int> a, rest;
                for (int u : parts[i]) {
                    if (u == v) continue;
                    (anc[u] ? a : rest).push_back(u);
                }
                parts[i] = {v};
                if (!a.empty()) parts.push_back(a);
                if (!rest.empty()) parts.push_back(rest);
                again = true;
                break;
            }
        }
    }
    return parts;
}

struct GroupMap {
    std::vector<double> T;
    std::vector<PdgEdge> pdg;
    MapResult m;
};

// PEE times, PDG and the ILP mapping of `parts` onto Gs GPUs.
GroupMap map_group(const Flat& f, const std::vector<std::vector<int>>& parts, int Gs, const sg_plan_opts& o) {
    const int N = (int)f.nodes.size(), P = (int)parts.size();
    std::vector<int> owner(N, -1);
    for (int i = 0; i < P; i++) for (int v : parts[i]) if (v >= 0 && v < N) owner[v] = i;
    GroupMap gm;
    gm.T.resize(P);
    for (int i = 0; i < P; i++) gm.T[i] = pee_estimate(f, parts[i]).t + launch_ns_per_iter(o.iters_per_fragment);
    // PDG: D_ij = sum of the weights of crossing edges (bytes / iteration)
    // edges out of a duplicate splitter carry the splitter's input stream: one data id per splitter
    std::map<std::tuple<int, int, int>, double> D;
    for (auto& e : f.edges) {
        if (e.src < 0 || e.dst < 0) continue;
        int a = owner[e.src], b = owner[e.dst];
        if (a < 0 || b < 0 || a == b) continue;
        const int data = f.nodes[e.src].type == N_SPLIT_DUP ? e.src : -1;
        if (data >= 0) D[std::make_tuple(a, b, data)] = 4.0 * e.per_iter;  // once per destination partition
        else D[std::make_tuple(a, b, -1)] += 4.0 * e.per_iter;
    }
    for (auto& kv : D) {
        PdgEdge pe;
        pe.src = std::get<0>(kv.first);
        pe.dst = std::get<1>(kv.first);
        pe.data = std::get<2>(kv.first);
        pe.bytes = kv.second;
        gm.pdg.push_back(pe);
    }
    gm.m.assign.assign(P, 0);
    if (Gs > 1) {
        Topology topo = Topology::nvswitch(Gs);
        double bw = o.link_gbps > 0 ? o.link_gbps : 770.0;          // bytes per ns
        double lat_us = o.link_latency_us > 0 ? o.link_latency_us : 10.0;
        double lat = lat_us * 1e3 / (o.iters_per_fragment > 0 ? (double)o.iters_per_fragment : kFragIters);  // reading 12
        // default: a deterministic node budget (plans are reproducible, so cubin caches hit); an
        // explicit ilp_time_limit_ms is a wall-clock budget instead
        gm.m = map_partitions(gm.T, gm.pdg, topo, lat, bw, o.ilp_time_limit_ms > 0 ? o.ilp_time_limit_ms : 0, 0,
                              o.ilp_time_limit_ms > 0 ? 0 : kIlpNodeBudget);
    } else {
        gm.m.tmax = std::accumulate(gm.T.begin(), gm.T.end(), 0.0);
        gm.m.optimal = true;
    }
    return gm;
}

// Balanced contiguous groups of branches for chain fission: m groups minimising the largest group
// cost (linear partition by DP over the branches' PEE times).
// head / tail: work outside the split-join that lands on the first / last group (SG_PART_CHAIN puts the
// nodes before the split-join into group 0 and those after it into the last group).
std::vector<int> balanced_groups(const std::vector<double>& c, int m, double head = 0.0, double tail = 0.0) {
    const int n = (int)c.size();
    m = std::min(m, n);
    std::vector<double> pre(n + 1, 0.0);
    for (int i = 0; i < n; i++) pre[i + 1] = pre[i] + c[i];
    const double INF = 1e300;
    // best[k][i]: first i branches in k groups; cut[k][i]: start of the k-th group
    std::vector<std::vector<double>> best(m + 1, std::vector<double>(n + 1, INF));
    std::vector<std::vector<int>> cut(m + 1, std::vector<int>(n + 1, 0));
    best[0][0] = 0;
    for (int k = 1; k <= m; k++)
        for (int i = k; i <= n; i++)
            for (int j = k - 1; j < i; j++) {
                const double extra = (k == 1 ? head : 0.0) + (k == m && i == n ? tail : 0.0);
                double v = std::max(best[k - 1][j], pre[i] - pre[j] + extra);
                if (v < best[k][i] - 1e-12) { best[k][i] = v; cut[k][i] = j; }
            }
    std::vector<int> first(m);
    for (int k = m, i = n; k >= 1; k--) {
        first[k - 1] = cut[k][i];
        i = cut[k][i];
    }
    return first;
}

// The split-join chain fission applies to: eligible (forward and/or accumulate chain), most nodes.
int fission_target(const Flat& f) {
    int best = -1, bestn = 0;
    for (int k = 0; k < (int)f.sjs.size(); k++) {
        if (!chain_fission_eligible(f, k)) continue;
        int n = f.sjs[k].join - f.sjs[k].split;
        if (n > bestn) { bestn = n; best = k; }
    }
    return best;
}

Flat fissioned(const Flat& f, int sj, int m) {
    const SjInfo& si = f.sjs[sj];
    const int nb = (int)si.first.size();
    std::vector<double> cost(nb);
    for (int b = 0; b < nb; b++) {
        std::vector<int> br;
        for (int v = si.first[b]; v < (b + 1 < nb ? si.first[b + 1] : si.join); v++) br.push_back(v);
        cost[b] = br.empty() ? 0.0 : pee_estimate(f, br).t;
    }
    std::vector<int> head, tail;
    for (int v = 0; v < si.split; v++) head.push_back(v);
    for (int v = si.join + 1; v < (int)f.nodes.size(); v++) tail.push_back(v);
    // head / tail priced by their own work only (alone they would be partitions with the split-join's
    // boundary streams, which they are not inside a group)
    auto work_ns = [&](const std::vector<int>& nodes) {
        if (nodes.empty()) return 0.0;
        const PartitionWork w = partition_work(f, nodes);
        return (w.flops / (kFp32 * kModel.e_staged) + w.intops / kInt + w.dfma * 80.0 / kFp64 +
                kLoopFiring * w.loop_firings) * 1e9;
    };
    const double th = work_ns(head), tt = work_ns(tail);
    return chain_fission(f, sj, balanced_groups(cost, m, th, tt));
}

// Graph variants and partitionings the planner compares (pipeline of Gs GPUs): the graph as written
// and, when a split-join is eligible, its chain fission into Gs groups; Algorithm 1
// with the G-aware cap, twice the cap, and no cap.  The ILP objective Tmax decides (ties: the first).
struct Candidate {
    int variant = 0;
    std::vector<std::vector<int>> parts;
    double tmax = 0, maxload = 0;
};
GroupMap map_group(const Flat& f, const std::vector<std::vector<int>>& parts, int Gs, const sg_plan_opts& o);

Candidate best_candidate(const std::vector<Flat>& variants, int Gs, const sg_plan_opts& o, GroupMap* gm_out,
                         std::vector<std::pair<Candidate, GroupMap>>* all = nullptr) {
    Candidate best;
    bool have = false;
    GroupMap bgm;
    for (int vi = 0; vi < (int)variants.size(); vi++) {
        std::vector<double> mults = {1.0};
        if (o.partitioner == SG_PART_ALGORITHM1 && Gs > 1) mults = {1.0, 2.0, 0.0};
        if (o.partitioner == SG_PART_ALGORITHM1 && vi == 0) mults.push_back(-2.0);  // one partition
        if (const char* env = std::getenv("SG_A1_CAPS")) {  // experiments: fixed cap multipliers ("1,2")
            mults.clear();
            for (const char* c = env; *c;) {
                mults.push_back(std::atof(c));
                while (*c && *c != ',') c++;
                if (*c == ',') c++;
            }
        }
        // a fissioned graph's groups are a candidate partitioning of their own (cap < 0 below)
        if (o.partitioner == SG_PART_ALGORITHM1 && !variants[vi].chain_first.empty()) mults.push_back(-1.0);
        std::set<std::vector<std::vector<int>>> seen;
        for (double cm : mults) {
            sg_plan_opts oc = o;
            if (cm == -1.0) oc.partitioner = SG_PART_CHAIN;
            if (cm == -2.0) oc.partitioner = SG_PART_SINGLE;
            auto parts = make_partitions(variants[vi], Gs, oc, cm);
            auto key = parts;
            for (auto& q : key) std::sort(q.begin(), q.end());
            std::sort(key.begin(), key.end());
            if (!seen.insert(key).second) continue;
            GroupMap gm = map_group(variants[vi], parts, Gs, o);
            if (std::getenv("SG_PLAN_DEBUG")) {
                std::fprintf(stderr, "[sg plan] variant %d cap x%.1f: %zu partitions, Tmax %.4f ns (ilp %s) T =", vi, cm,
                             parts.size(), gm.m.tmax, gm.m.optimal ? "optimal" : "budget");
                for (size_t i = 0; i < parts.size() && i < 24; i++) std::fprintf(stderr, " %.3f/%zu", gm.T[i], parts[i].size());
                std::fprintf(stderr, "\n");
            }
            // ties on Tmax (e.g. every candidate bound by the same link): the smaller largest GPU load
            std::vector<double> load(Gs, 0.0);
            for (size_t i = 0; i < parts.size(); i++) load[gm.m.assign[i]] += gm.T[i];
            const double maxload = *std::max_element(load.begin(), load.end());
            // a plan of several partitions is charged the PEE's noise margin against one partition
            const double score = gm.m.tmax * (parts.size() > 1 ? 1.0 + kSplitMargin : 1.0);
            if (all) {
                Candidate c;
                c.variant = vi;
                c.parts = parts;
                c.tmax = score;
                c.maxload = maxload;
                all->push_back({c, gm});
            }
            const bool tie = have && std::fabs(score - best.tmax) <= 1e-9 * std::max(1.0, best.tmax);
            if (!have || score < best.tmax * (1 - 1e-9) || (tie && maxload < best.maxload * (1 - 1e-9))) {
                best.maxload = maxload;
                have = true;
                best.variant = vi;
                best.parts = parts;
                best.tmax = score;
                bgm = gm;
            }
        }
    }
    if (gm_out) *gm_out = bgm;
    if (all)  // best first (the order the planner falls back in when a partition cannot be generated)
        std::stable_sort(all->begin(), all->end(), [](const std::pair<Candidate, GroupMap>& a,
                                                      const std::pair<Candidate, GroupMap>& b) {
            return a.first.tmax != b.first.tmax ? a.first.tmax < b.first.tmax : a.first.maxload < b.first.maxload;
        });
    return best;
}

// Eq. III.1-III.7 objective of a given mapping inside one group of Gs GPUs (same link model as map_group)
double group_tmax(const std::vector<double>& T, const std::vector<PdgEdge>& pdg, const std::vector<int>& a, int Gs,
                  const sg_plan_opts& o) {
    if (Gs <= 1) return std::accumulate(T.begin(), T.end(), 0.0);
    const double bw = o.link_gbps > 0 ? o.link_gbps : 770.0;
    const double lat = (o.link_latency_us > 0 ? o.link_latency_us : 10.0) * 1e3 /
                       (o.iters_per_fragment > 0 ? (double)o.iters_per_fragment : kFragIters);
    return mapping_cost(T, pdg, Topology::nvswitch(Gs), lat, bw, a);
}

// Throughput bound of R replica groups of Gs GPUs each on the NVSwitch star:
// group r runs the group mapping `a` on GPUs r*Gs .. r*Gs+Gs-1 and 1/R of the fragments, so every
// GPU's compute (Eq. III.4) and every link's load (Eq. III.6-III.7) is 1/R of the group's; the
// input GPU's uplink also ships the other groups' input share and the output GPU's downlink
// receives their output share.  Links carry Lat (Eq. III.3) only when they carry bytes, so a
// mapping that moves nothing is not charged a transfer.
double hybrid_cost(const Flat& f, const std::vector<double>& T, const std::vector<PdgEdge>& pdg,
                   const std::vector<int>& a, int in_gpu, int out_gpu, int Gs, int R, const sg_plan_opts& o) {
    const int G = Gs * R;
    const double bw = o.link_gbps > 0 ? o.link_gbps : 770.0;
    const double lat = (o.link_latency_us > 0 ? o.link_latency_us : 10.0) * 1e3 /
                       (o.iters_per_fragment > 0 ? (double)o.iters_per_fragment : kFragIters);
    std::vector<double> comp(Gs, 0.0), up(G, 0.0), down(G, 0.0);
    for (size_t i = 0; i < T.size(); i++) comp[a[i]] += T[i];
    for (int r = 0; r < R; r++) {
        std::set<std::tuple<int, int, int>> shipped;
        for (auto& e : pdg) {
            int k = a[e.src], h = a[e.dst];
            if (k == h) continue;
            if (e.data >= 0 && !shipped.insert(std::make_tuple(e.data, k, h)).second) continue;
            up[r * Gs + k] += e.bytes / R;
            down[r * Gs + h] += e.bytes / R;
        }
        if (r == 0) continue;
        const double bi = 4.0 * (double)f.in_per_iter / R, bo = 4.0 * (double)f.out_per_iter / R;
        up[in_gpu] += bi;
        down[r * Gs + in_gpu] += bi;
        up[r * Gs + out_gpu] += bo;
        down[out_gpu] += bo;
    }
    double t = 0;
    for (double c : comp) t = std::max(t, c / R);
    for (int g = 0; g < G; g++) {
        if (up[g] > 0) t = std::max(t, lat + up[g] / bw);
        if (down[g] > 0) t = std::max(t, lat + down[g] / bw);
    }
    return t;
}

int io_gpu(const Flat& f, const std::vector<std::vector<int>>& parts, const std::vector<int>& a, int node) {
    for (size_t i = 0; i < parts.size(); i++)
        for (int v : parts[i]) if (v == node) return a[i];
    return 0;
}
}  // namespace

namespace {
void assemble_plan(Plan& p, std::vector<std::vector<int>> parts, const GroupMap& gm, int G, int R, int Gs,
                   const sg_plan_opts& o);
}

void build_plan(Plan& p, const sg_graph& g, int G, const sg_plan_opts& o) {
    if (o.transport < SG_TRANSPORT_AUTO || o.transport > SG_TRANSPORT_HOST)
        throw Error(SG_E_ARG, "transport must be SG_TRANSPORT_AUTO, _P2P or _HOST");
    if (o.chain_groups < -1 || o.chain_groups == 1) throw Error(SG_E_ARG, "chain_groups must be -1, 0 or >= 2");
    Flat f0 = Flat::build(g);
    p.G = G;
    p.opts = o;
    // graph variants: as written, and the order-preserving chain fission of the
    // largest eligible split-join -- forced with chain_groups >= 2, considered by the planner for
    // Algorithm 1 on more than one GPU (per replica group)
    const int fsj = o.chain_groups == -1 ? -1 : fission_target(f0);
    if (o.chain_groups >= 2 && fsj < 0) throw Error(SG_E_PLAN, "chain_groups: no eligible split-join (SURVEY.md 8(e))");
    auto variants_for = [&](int Gs) {
        std::vector<Flat> v;
        if (o.chain_groups >= 2) { v.push_back(fissioned(f0, fsj, o.chain_groups)); return v; }
        v.push_back(f0);
        if (fsj >= 0 && Gs > 1 && o.partitioner == SG_PART_ALGORITHM1) v.push_back(fissioned(f0, fsj, Gs));
        return v;
    };
    p.flat = f0;
    const Flat& f = p.flat;
    // ---- replica groups (hybrid replica x pipeline; R = 1 is the paper's mapping)
    int R = 1;
    bool has_loop = false;
    for (auto& n : f.nodes) has_loop |= n.type == N_LOOP;
    if (has_loop && o.replicas > 1)
        throw Error(SG_E_UNSUPPORTED, "replicas > 1: a feedback loop carries state from one fragment to the next");
    if (o.replicas > 1) {
        if (G % o.replicas) throw Error(SG_E_ARG, "replicas must divide n_gpus");
        R = o.replicas;
    } else if (o.replicas < 0 && G > 1 && !has_loop) {
        double best = 0;
        for (int r = 1; r <= G; r++) {
            if (G % r) continue;
            auto vars = variants_for(G / r);
            GroupMap gm;
            Candidate cd = best_candidate(vars, G / r, o, &gm);
            const Flat& fv = vars[cd.variant];
            auto& pr = cd.parts;
            double c = hybrid_cost(fv, gm.T, gm.pdg, gm.m.assign, io_gpu(fv, pr, gm.m.assign, fv.edges[fv.in_edge].dst),
                                   io_gpu(fv, pr, gm.m.assign, fv.edges[fv.out_edge].src), G / r, r, o);
            if (r == 1 || c < best * 0.999) { best = c; R = r; }
        }
    } else if (o.replicas < -1) {
        throw Error(SG_E_ARG, "replicas must be -1 (auto), 0/1 (pipeline) or a divisor of n_gpus");
    }
    const int Gs = G / R;
    p.R = R;
    p.Gs = Gs;
    // ---- graph variant + partitions (Algorithm 1 candidates compared by the ILP objective); a candidate
    // with a partition the code generator cannot fit (SG_E_SIZE: shared memory) yields to the next one
    auto vars = variants_for(Gs);
    std::vector<std::pair<Candidate, GroupMap>> cands;
    best_candidate(vars, Gs, o, nullptr, &cands);
    // After code generation the estimate is refined with the kernels' own decisions; a plan whose refined
    // Tmax exceeds its planning score by more than half also has the one-partition candidate (and the next
    // few) generated, and the smallest refined Tmax wins -- the planner never keeps a cut the generated code
    // shows to be slower than what it had to compare with.
    auto attempt = [&](size_t ci) -> bool {
        try {
            p.flat = vars[cands[ci].first.variant];
            p.chain_fission = o.chain_groups >= 2 || cands[ci].first.variant == 1;
            assemble_plan(p, cands[ci].first.parts, cands[ci].second, G, R, Gs, o);
            return true;
        } catch (const Error& e) {
            if (e.code != SG_E_SIZE) throw;
            return false;
        }
    };
    // One GPU: a fused kernel whose frame-FIR level cannot fill the CTA (the code generator's simulated
    // parallel efficiency, KernelInfo::split_level) is also tried as two partitions cut at that level
    // boundary (convex: levels rise along every edge); the refined estimates decide (static discrepancy,
    // the estimate sees the code generator's own decisions).
    auto level_split = [&]() {
        if (o.plan_only || Gs != 1 || p.parts.size() != 1 || o.partitioner != SG_PART_ALGORITHM1 ||
            std::getenv("SG_NO_LEVEL_SPLIT"))
            return;
        const int sl = p.kernels[0].ki.split_level;
        const std::vector<std::pair<int, int>> nlev = p.kernels[0].ki.node_level;
        if (sl <= 1 || nlev.empty()) return;
        std::vector<std::vector<int>> parts(2);
        for (auto& nl : nlev) parts[nl.second >= sl ? 1 : 0].push_back(nl.first);
        if (parts[0].empty() || parts[1].empty()) return;
        const double one = p.est_tmax;
        const std::vector<std::vector<int>> single{p.parts[0].nodes};
        const Flat fsave = p.flat;
        const bool chain = p.chain_fission;
        try {
            GroupMap gm = map_group(p.flat, parts, 1, o);
            assemble_plan(p, parts, gm, G, R, Gs, o);
            if (std::getenv("SG_PLAN_DEBUG"))
                std::fprintf(stderr, "[sg plan] level split before level %d: %.3f ns vs one partition %.3f ns\n",
                             sl, p.est_tmax, one);
            if (p.est_tmax < one * (1.0 - kSplitMargin)) return;
        } catch (const Error& e) {
            if (e.code != SG_E_SIZE) throw;
        }
        p.flat = fsave;
        p.chain_fission = chain;
        GroupMap gm1 = map_group(p.flat, single, 1, o);
        assemble_plan(p, single, gm1, G, R, Gs, o);
    };
    int best_ci = -1;
    double best_ref = 0;
    size_t tried = 0;
    double single_score = 0;  // the one-partition candidate's planning score
    for (auto& c : cands) if (c.first.parts.size() == 1) single_score = c.first.tmax;
    for (size_t ci = 0; ci < cands.size() && tried < 4; ci++) {
        if (!attempt(ci)) continue;
        tried++;
        const bool cut = cands[ci].first.parts.size() > 1;
        if (o.plan_only || (p.est_tmax <= cands[ci].first.tmax * 1.5 &&
                            (!cut || single_score <= 0 || p.est_tmax <= 0.9 * single_score))) {
            level_split();
            return;
        }
        if (best_ci < 0 || p.est_tmax < best_ref) { best_ci = (int)ci; best_ref = p.est_tmax; }
    }
    for (size_t ci = 0; ci < cands.size(); ci++)  // the one-partition candidate, if not yet tried
        if (cands[ci].first.parts.size() == 1 && (int)ci != best_ci && attempt(ci)) {
            if (best_ci < 0 || p.est_tmax < best_ref) { best_ci = (int)ci; best_ref = p.est_tmax; }
            break;
        }
    if (best_ci < 0) throw Error(SG_E_SIZE, "no candidate partitioning fits the code generator's shared memory");
    if (!attempt((size_t)best_ci)) throw Error(SG_E_SIZE, "internal: candidate no longer fits");
    level_split();
}

namespace {
// Partitions -> ordered, mapped, generated plan (the graph variant is p.flat).
void assemble_plan(Plan& p, std::vector<std::vector<int>> parts, const GroupMap& gm, int G, int R, int Gs,
                   const sg_plan_opts& o) {
    const Flat& f = p.flat;
    const int N = (int)f.nodes.size();
    // validate: cover, convex; order topologically
    std::vector<int> owner(N, -1);
    for (size_t i = 0; i < parts.size(); i++) {
        std::sort(parts[i].begin(), parts[i].end());
        std::vector<char> in(N, 0);
        for (int v : parts[i]) {
            if (v < 0 || v >= N || owner[v] >= 0) throw Error(SG_E_PLAN, "partitions must cover each node exactly once");
            owner[v] = (int)i;
            in[v] = 1;
        }
        if (!is_convex(f, in)) throw Error(SG_E_PLAN, "partition " + std::to_string(i) + " is not convex");
    }
    for (int v = 0; v < N; v++) if (owner[v] < 0) throw Error(SG_E_PLAN, "node not covered by any partition");
    const int P = (int)parts.size();
    std::vector<std::set<int>> succ(P);
    std::vector<int> indeg(P, 0);
    for (auto& e : f.edges) {
        if (e.src < 0 || e.dst < 0) continue;
        int a = owner[e.src], b = owner[e.dst];
        if (a != b && succ[a].insert(b).second) indeg[b]++;
    }
    std::vector<int> order;
    std::vector<int> ready;
    for (int i = 0; i < P; i++) if (!indeg[i]) ready.push_back(i);
    while (!ready.empty()) {
        std::sort(ready.begin(), ready.end(), std::greater<int>());
        int x = ready.back();
        ready.pop_back();
        order.push_back(x);
        for (int y : succ[x]) if (--indeg[y] == 0) ready.push_back(y);
    }
    if ((int)order.size() != P) throw Error(SG_E_PLAN, "partition graph is cyclic");
    p.parts.assign(P, Partition());
    p.part_order = order;
    p.part_time.assign(P, 0.0);
    p.part_mode.assign(P, 0);
    std::vector<double> T(P);
    std::vector<PeeEstimate> ests(P);
    for (int i = 0; i < P; i++) {
        p.parts[i].nodes = parts[i];
        PeeEstimate est = ests[i] = pee_estimate(f, parts[i]);
        p.parts[i].t_est = T[i] = est.t;
        p.parts[i].t_comp = est.t_comp;
        p.parts[i].t_dt = est.t_dt;
        p.part_time[i] = est.t;
    }
    // ---- PDG and mapping inside one replica group of Gs GPUs
    p.pdg = gm.pdg;
    p.part_gpu.assign(P, 0);
    for (int i = 0; i < P; i++) p.part_gpu[i] = gm.m.assign[i];
    p.est_tmax = R == 1 ? gm.m.tmax
                        : hybrid_cost(f, gm.T, gm.pdg, gm.m.assign, io_gpu(f, parts, gm.m.assign, f.edges[f.in_edge].dst),
                                      io_gpu(f, parts, gm.m.assign, f.edges[f.out_edge].src), Gs, R, o);
    p.ilp_optimal = gm.m.optimal;
    // ---- rings: a duplicated stream crosses to a GPU once (PDG data ids, reading 15)
    p.ring_rep.assign(f.edges.size(), -1);
    p.ring_lo.assign(f.edges.size(), 0);
    p.ring_extra.assign(f.edges.size(), 0);
    {
        std::map<std::pair<int, int>, int> first;  // (dup splitter, destination GPU) -> representative edge
        for (int e = 0; e < (int)f.edges.size(); e++) {
            const Edge& ed = f.edges[e];
            if (ed.src < 0 || ed.dst < 0) continue;
            const int ps = owner[ed.src], pd = owner[ed.dst];
            if (ps == pd) continue;
            int rep = e;
            const int hg = p.part_gpu[pd];
            if (f.nodes[ed.src].type == N_SPLIT_DUP && p.part_gpu[ps] != hg) {
                auto it = first.find({ed.src, hg});
                if (it == first.end()) first[{ed.src, hg}] = e;
                else rep = it->second;
            }
            p.ring_rep[e] = rep;
            int64_t lo, ex;
            edge_window(f, e, lo, ex);
            if (rep == e) {
                p.ring_lo[e] = lo;
                p.ring_extra[e] = ex;
            } else {  // union [min lo, max(lo + extra)) -- members have the same items per iteration
                const int64_t hi = std::max(p.ring_lo[rep] + p.ring_extra[rep], lo + ex);
                p.ring_lo[rep] = std::min(p.ring_lo[rep], lo);
                p.ring_extra[rep] = hi - p.ring_lo[rep];
            }
        }
    }
    // ---- devices
    p.virtual_gpus = o.virtual_gpus != 0;
    p.devices.assign(G, 0);
    for (int gi = 0; gi < G; gi++) p.devices[gi] = o.devices ? o.devices[gi] : (p.virtual_gpus ? 0 : gi);
    p.input_gpu = p.part_gpu[owner[f.edges[f.in_edge].dst]];
    p.output_gpu = p.part_gpu[owner[f.edges[f.out_edge].src]];
    p.iters_per_fragment = o.iters_per_fragment;
    // ---- code generation + NVRTC (one kernel per partition)
    p.kernels.clear();
    p.kernels.resize(P);
    CodegenOpts co;
    co.mode = o.codegen_mode;
    co.threads = o.threads;
    co.tile = o.tile_iters;
    for (int i = 0; i < P; i++) {
        if (o.plan_only) {  // partitions and mapping only: keep the PEE's mode decision
            p.kernels[i].ki.mode = register_mode_eligible(f, parts[i], nullptr) ? 1 : 2;
            if (parts[i].size() == 1 && f.nodes[parts[i][0]].type == N_LOOP) p.kernels[i].ki.mode = 4;
            p.kernels[i].ki.tile = 1;
            partition_boundary(f, parts[i], p.kernels[i].ki.in_edges, p.kernels[i].ki.out_edges);
            p.part_mode[i] = p.kernels[i].ki.mode;
            p.parts[i].mode = p.kernels[i].ki.mode;
            p.parts[i].gpu = p.part_gpu[i];
            continue;
        }
        p.kernels[i].ki = generate_kernel(f, parts[i], i, co);
        compile_kernel(p.kernels[i], o.verbose);
        p.part_mode[i] = p.kernels[i].ki.mode;
        p.parts[i].mode = p.kernels[i].ki.mode;
        p.parts[i].gpu = p.part_gpu[i];
        p.parts[i].tile = p.kernels[i].ki.tile;
        p.parts[i].threads = p.kernels[i].ki.threads;
        // the PEE with the generated kernel's own decisions (static discrepancy)
        p.parts[i].t_est = p.part_time[i] = pee_refine(ests[i], p.kernels[i].ki);
    }
    if (!o.plan_only) {  // Tmax of this mapping with the refined partition times
        std::vector<double> Tr(P);
        for (int i = 0; i < P; i++) Tr[i] = p.part_time[i] + launch_ns_per_iter(o.iters_per_fragment);
        p.est_tmax = R == 1 ? group_tmax(Tr, gm.pdg, gm.m.assign, Gs, o)
                            : hybrid_cost(f, Tr, gm.pdg, gm.m.assign, io_gpu(f, parts, gm.m.assign, f.edges[f.in_edge].dst),
                                          io_gpu(f, parts, gm.m.assign, f.edges[f.out_edge].src), Gs, R, o);
    }
    // ---- info arrays
    p.reps.resize(N);
    p.ninit.resize(N);
    p.node_type.resize(N);
    p.node_kind.resize(N);
    p.node_part.resize(N);
    for (int v = 0; v < N; v++) {
        p.reps[v] = f.nodes[v].rep;
        p.ninit[v] = f.nodes[v].ninit;
        p.node_type[v] = (int32_t)f.nodes[v].type;
        p.node_kind[v] = f.nodes[v].kind;
        p.node_part[v] = owner[v];
    }
}
}  // namespace

}  // namespace sg
