// sg_pee.cpp -- the work a partition's kernel actually executes, for the B200 PEE.
//
// "The PEE includes the same optimization done by the GPU code generator" (PAPER.md:579-581,
// section 3.3: otherwise the estimate suffers a static discrepancy).  The code generator
// (sg_codegen.cpp) resolves every view (splitter, joiner, IDENTITY, DELAY, DECIMATE, EXPAND,
// PERMUTE, FFT_REORDER) at compile time, computes only the live firings of a filter whose outputs
// are read at a stride (dead-firing elimination), drops FMA terms whose input is an EXPAND zero
// slot (zero-tap pruning), and computes identical firings once (CSE: same kind and parameters, same
// input values).  This file repeats those decisions on the partition's node set, per steady-state
// iteration, without generating code:
//
//  1. Liveness.  Steady-state demand is shift-invariant (iteration k+1 needs firing g + rep_u of u
//     wherever iteration k needs g), so demand is tracked per firing residue (g - ninit_u) mod rep_u:
//     the boundary outputs of one iteration K demand residues of their producers; a live firing of u
//     demands the producers of every non-zero item in its peek window, resolved through the
//     partition's views (a view outside the partition is a boundary input).
//  2. Work.  In topological order, every live firing of a compute node is priced with zero inputs
//     pruned; a node whose parameters and input values (per live residue) equal those of an earlier
//     node is a CSE duplicate and costs nothing.
// The result is the executed work per iteration, the live firings, and the items read / written by
// those firings (the shared-memory traffic of the staged kernels).
#include <algorithm>
#include <cstring>
#include <functional>
#include <map>
#include <set>
#include <unordered_map>
#include <unordered_set>

#include "sg_codegen.h"
#include "sg_plan.h"

namespace sg {

namespace {
int64_t fdiv(int64_t a, int64_t b) {
    int64_t q = a / b, r = a % b;
    return (r != 0 && ((r < 0) != (b < 0))) ? q - 1 : q;
}
int64_t fmodp(int64_t a, int64_t b) { return a - fdiv(a, b) * b; }

inline uint64_t mix(uint64_t h, uint64_t x) {
    h ^= x + 0x9e3779b97f4a7c15ULL + (h << 6) + (h >> 2);
    h *= 0xff51afd7ed558ccdULL;
    return h ^ (h >> 33);
}

struct Item {
    enum K { PHYS, ZERO } k = PHYS;
    int edge = -1;
    int64_t pos = 0;
};

// Integer view resolution inside a node set (the code generator's Resolver on constant positions).
struct IntResolver {
    const Flat& f;
    const std::vector<char>& in;
    bool phys(int e) const {
        const Edge& ed = f.edges[e];
        if (ed.src < 0 || !in[ed.src]) return true;
        const Node& u = f.nodes[ed.src];
        if (u.type == N_FILTER) return !is_view_kind(u.kind);
        return u.type == N_LOOP;
    }
    Item resolve(int e, int64_t pos) const {
        for (int guard = 0; guard < 100000; guard++) {
            if (phys(e)) return {Item::PHYS, e, pos};
            const Edge& ed = f.edges[e];
            const Node& u = f.nodes[ed.src];
            switch (u.type) {
            case N_SPLIT_DUP: e = u.in[0]; continue;
            case N_SPLIT_RR: {
                const int b = ed.sport;
                int64_t w = u.w[b], P = 0;
                for (int i = 0; i < b; i++) P += u.w[i];
                pos = fdiv(pos, w) * u.wsum + P + fmodp(pos, w);
                e = u.in[0];
                continue;
            }
            case N_JOIN: {
                const int64_t S = u.wsum;
                const int64_t q = fdiv(pos, S);
                int64_t o = fmodp(pos, S), P = 0;
                int b = 0;
                while (o >= P + u.w[b]) { P += u.w[b]; b++; }
                pos = q * u.w[b] + (o - P);
                e = u.in[b];
                continue;
            }
            case N_FILTER:
                switch (u.kind) {
                case SG_K_IDENTITY: e = u.in[0]; continue;
                case SG_K_DELAY: pos -= u.iv[0]; e = u.in[0]; continue;
                case SG_K_DECIMATE: pos *= u.iv[0]; e = u.in[0]; continue;
                case SG_K_EXPAND:
                    if (fmodp(pos, u.iv[0]) != 0) return {Item::ZERO, -1, 0};
                    pos = fdiv(pos, u.iv[0]);
                    e = u.in[0];
                    continue;
                case SG_K_PERMUTE: {
                    const int64_t n = u.iv[0], m = (int64_t)u.iv.size() - 1;
                    pos = fdiv(pos, m) * n + u.iv[1 + fmodp(pos, m)];
                    e = u.in[0];
                    continue;
                }
                case SG_K_FFT_REORDER: {
                    const int64_t n = u.iv[0], F = 2 * n;
                    const int64_t q = fdiv(pos, F), o = fmodp(pos, F), m = o / 2, r = o % 2;
                    const int64_t sc = m < n / 2 ? 2 * m : 2 * (m - n / 2) + 1;
                    pos = q * F + 2 * sc + r;
                    e = u.in[0];
                    continue;
                }
                default: break;
                }
                break;
            default: break;
            }
            throw Error(SG_E_UNSUPPORTED, "internal: PEE view resolution");
        }
        throw Error(SG_E_UNSUPPORTED, "internal: PEE view chain too long");
    }
};

// fp32 flops / int ops / fp64 work of one firing of compute node v whose peek window has `nz`
// non-zero items out of n.peek (zero taps pruned as the code generator does)
void firing_work(const Flat& f, int v, int64_t nz, double& fl, double& io, double& dd) {
    const Node& n = f.nodes[v];
    fl = io = dd = 0;
    if (n.type == N_LOOP) {
        int64_t a, b, c;
        node_work(f, v, a, b, c);
        fl = (double)a / n.rep;
        io = (double)b / n.rep;
        dd = (double)c / n.rep;
        return;
    }
    switch (n.kind) {
    case SG_K_FIR: fl = 2.0 * (double)std::min<int64_t>(nz, n.iv[0]); break;
    case SG_K_ADD:
        if (f.dtype == SG_F32) fl = (double)nz;
        else io = (double)nz;
        break;
    case SG_K_BEAM_FIR: {  // zero history at the frame start: output t uses min(L, t + 1) taps
        const int64_t L = n.iv[0], dec = n.iv[1], frame = n.iv[2];
        double taps = 0;
        for (int64_t t = 0; t < frame; t += dec) taps += (double)std::min<int64_t>(L, t + 1);
        fl = 8.0 * taps;
        break;
    }
    default: {
        int64_t a, b, c;
        node_work(f, v, a, b, c);
        fl = (double)a / n.rep;
        io = (double)b / n.rep;
        dd = (double)c / n.rep;
    }
    }
}
}  // namespace

PartitionWork partition_work(const Flat& f, const std::vector<int>& nodes, bool components) {
    PartitionWork w;
    const int N = (int)f.nodes.size();
    std::vector<char> in(N, 0);
    for (int v : nodes) in[v] = 1;
    IntResolver R{f, in};
    auto compute = [&](int v) {
        const Node& n = f.nodes[v];
        return in[v] && ((n.type == N_FILTER && !is_view_kind(n.kind)) || n.type == N_LOOP);
    };
    std::vector<int> ins, outs;
    partition_boundary(f, nodes, ins, outs);
    for (int e : ins) w.in_bytes += 4.0 * f.edges[e].per_iter;
    for (int e : outs) w.out_bytes += 4.0 * f.edges[e].per_iter;
    w.in_edges = (int)ins.size();
    w.out_edges = (int)outs.size();
    w.row_items = (w.in_bytes + w.out_bytes) / 4.0;
    // a reference iteration far from the stream start (every firing index positive)
    int64_t K = 1;
    for (int v : nodes) {
        const Node& n = f.nodes[v];
        if (n.rep > 0) K = std::max<int64_t>(K, (std::llabs(n.ninit) + n.halo) / n.rep + 2);
    }
    auto first_firing = [&](int u) { return f.nodes[u].ninit + K * f.nodes[u].rep; };
    // producer firing residue of an item on a physical edge produced inside the partition
    auto producer = [&](const Item& it, int& u, int64_t& g) {
        u = -1;
        if (it.k != Item::PHYS) return;
        const Edge& ed = f.edges[it.edge];
        if (ed.src < 0 || !in[ed.src]) return;
        u = ed.src;
        g = fdiv(it.pos - ed.pre, ed.push);
    };
    // ---- 1. liveness by residue, consumers first (node ids are topological)
    std::vector<std::vector<char>> live(N);
    for (int v : nodes)
        if (compute(v)) live[v].assign((size_t)std::max<int64_t>(1, f.nodes[v].rep), 0);
    auto demand = [&](int u, int64_t g) {
        if (u < 0 || !compute(u)) return;
        const Node& n = f.nodes[u];
        live[u][(size_t)fmodp(g - n.ninit, n.rep)] = 1;
    };
    for (int e : outs) {
        const Edge& ed = f.edges[e];
        const Node& s = f.nodes[ed.src];
        // positions produced by the source node's firings of iteration K (views: the same window)
        const int64_t p0 = ed.pre + (s.ninit + K * s.rep) * ed.push;
        for (int64_t i = 0; i < ed.per_iter; i++) {
            Item it = R.resolve(e, p0 + i);
            int u;
            int64_t g;
            producer(it, u, g);
            demand(u, g);
        }
    }
    std::vector<int> order(nodes.begin(), nodes.end());
    std::sort(order.begin(), order.end());
    for (auto it = order.rbegin(); it != order.rend(); ++it) {
        const int v = *it;
        if (!compute(v)) continue;
        const Node& n = f.nodes[v];
        const int64_t g0 = first_firing(v);
        for (int64_t r = 0; r < n.rep; r++) {
            if (!live[v][(size_t)r]) continue;
            const int64_t g = g0 + r;
            for (int e : n.in) {
                const Edge& ed = f.edges[e];
                for (int64_t i = 0; i < ed.peek; i++) {
                    Item x = R.resolve(e, g * ed.pop + i);
                    int u;
                    int64_t gu;
                    producer(x, u, gu);
                    demand(u, gu);
                }
            }
        }
    }
    // ---- 1b. dependence components of one iteration (register mode picks its kernel variant by them:
    // one wide component -> the demand-ordered kernel): outputs whose cones share an input item
    if (components) {
        std::map<std::pair<int, int64_t>, int> id;
        std::vector<int> uf;
        auto get = [&](int e, int64_t pos) {
            auto it = id.find({e, pos});
            if (it != id.end()) return it->second;
            int k = (int)uf.size();
            uf.push_back(k);
            id[{e, pos}] = k;
            return k;
        };
        std::function<int(int)> find = [&](int x) { return uf[x] == x ? x : uf[x] = find(uf[x]); };
        auto unite = [&](int a, int b) { a = find(a); b = find(b); if (a != b) uf[a] = b; };
        std::vector<int> out_ids;
        for (int e : outs) {
            const Edge& ed = f.edges[e];
            const Node& s0 = f.nodes[ed.src];
            const int64_t p0 = ed.pre + (s0.ninit + K * s0.rep) * ed.push;
            for (int64_t i = 0; i < ed.per_iter; i++) {
                const int me = get(-2 - e, p0 + i);
                out_ids.push_back(me);
                std::set<std::pair<int, int64_t>> seen;
                std::vector<Item> st{R.resolve(e, p0 + i)};
                while (!st.empty()) {
                    Item x = st.back();
                    st.pop_back();
                    if (x.k != Item::PHYS) continue;
                    int u;
                    int64_t g;
                    producer(x, u, g);
                    if (u < 0) { unite(me, get(x.edge, x.pos)); continue; }
                    if (!seen.insert({u, g}).second) continue;
                    for (int ie : f.nodes[u].in) {
                        const Edge& ied = f.edges[ie];
                        for (int64_t q = 0; q < ied.peek; q++) st.push_back(R.resolve(ie, g * ied.pop + q));
                    }
                }
            }
        }
        std::set<int> roots;
        for (int o : out_ids) roots.insert(find(o));
        w.components = (int)roots.size();
    }
    // ---- 2. work per live firing, zero taps pruned, CSE duplicates skipped (producers first)
    std::unordered_map<int, int> cls;           // node -> class representative
    std::unordered_map<uint64_t, int> by_key;   // node key -> representative
    auto value_id = [&](const Item& x) -> uint64_t {
        if (x.k == Item::ZERO) return 0;
        int u;
        int64_t g;
        producer(x, u, g);
        if (u < 0) return mix(mix(1, (uint64_t)x.edge), (uint64_t)x.pos);  // boundary input item
        const Edge& ed = f.edges[x.edge];
        const int64_t j = x.pos - ed.pre - g * ed.push;
        auto c = cls.find(u);
        const int rep = c == cls.end() ? u : c->second;
        return mix(mix(mix(2, (uint64_t)rep), (uint64_t)g), (uint64_t)(j * 64 + ed.sport));
    };
    std::vector<int> level(N, 0);
    for (int v : order) {
        if (!compute(v)) continue;
        const Node& n = f.nodes[v];
        uint64_t key = mix(mix(7, (uint64_t)n.type), (uint64_t)(n.kind + 1000));
        for (int32_t x : n.iv) key = mix(key, (uint64_t)(uint32_t)x);
        for (float x : n.fv) {
            uint32_t b;
            std::memcpy(&b, &x, 4);
            key = mix(key, b);
        }
        key = mix(mix(key, (uint64_t)n.rep), (uint64_t)n.ninit);
        const int64_t g0 = first_firing(v);
        double fl_sum = 0, io_sum = 0, dd_sum = 0, reads = 0, nlive = 0;
        int lvl = 0;
        for (int64_t r = 0; r < n.rep; r++) {
            if (!live[v][(size_t)r]) continue;
            const int64_t g = g0 + r;
            int64_t nz = 0;
            key = mix(key, (uint64_t)r);
            for (int e : n.in) {
                const Edge& ed = f.edges[e];
                for (int64_t i = 0; i < ed.peek; i++) {
                    Item x = R.resolve(e, g * ed.pop + i);
                    key = mix(key, value_id(x));
                    if (x.k == Item::ZERO) continue;
                    nz++;
                    int u;
                    int64_t gu;
                    producer(x, u, gu);
                    if (u >= 0) lvl = std::max(lvl, level[u]);
                }
            }
            double fl, io, dd;
            firing_work(f, v, nz, fl, io, dd);
            fl_sum += fl;
            io_sum += io;
            dd_sum += dd;
            reads += (double)nz;
            nlive += 1;
        }
        level[v] = lvl + 1;
        w.levels = std::max(w.levels, level[v]);
        auto k = by_key.find(key);
        if (k != by_key.end()) { cls[v] = k->second; w.cse_nodes++; continue; }
        by_key[key] = v;
        cls[v] = v;
        w.flops += fl_sum;
        w.intops += io_sum;
        w.dfma += dd_sum;
        w.reads += reads;
        w.firings += nlive;
        w.writes += nlive * (double)n.push;
        if (n.type == N_FILTER && n.kind == SG_K_BEAM_FIR) w.frame = true;
        if (n.type == N_LOOP) w.loop_firings += (double)n.rep * (double)n.loop->sched.size();
        // halo recompute of a tile: peek windows reaching into the previous tile
        w.halo_firings += (double)n.halo * nlive / (double)std::max<int64_t>(1, n.rep);
    }
    return w;
}

}  // namespace sg
