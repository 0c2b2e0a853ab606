// sg_internal.h -- internal data structures of the stream-graph executor.
//
// Layers: graph IR + SDF analysis (sg_graph.cpp), planner
// (sg_plan.cpp: PEE, Algorithm 1, PDG, ILP), code generator (sg_codegen.cpp),
// runtime (sg_runtime.cpp: NVRTC, modules, launches, multi-GPU pipeline),
// C ABI (sg_capi.cpp).
#pragma once

#include <cstdint>
#include <map>
#include <memory>
#include <mutex>
#include <stdexcept>
#include <string>
#include <vector>

#include "../../include/sg.h"

namespace sg {

struct Error : std::runtime_error {
    sg_status code;
    Error(sg_status c, const std::string& m) : std::runtime_error(m), code(c) {}
};

// ------------------------------------------------------------------ builder
enum ElemType { E_FILTER = 0, E_PIPE = 1, E_SJ = 2, E_LOOP = 3 };

struct Elem {
    ElemType type = E_FILTER;
    // filter
    int kind = -1;
    std::vector<int32_t> iv;
    std::vector<float> fv;
    // pipeline
    std::vector<int> kids;
    // split-join
    int split_kind = 0;  // 0 dup, 1 rr
    std::vector<int32_t> split_w, join_w;
    std::vector<int> branches;  // elem ids of branch pipelines (loop: body, loop stream)
    std::vector<bool> branch_done;
    // feedback loop: enqueued items (raw 4-byte words)
    std::vector<uint32_t> enq;
};

}  // namespace sg

struct sg_graph {
    sg_dtype dtype = SG_F32;
    std::vector<sg::Elem> elems;
    int top = 0;
    std::vector<int> open;  // stack of open pipelines (elem ids); bottom = top
    std::vector<std::pair<int, int>> open_branch;  // (sj, branch) matching open[1..]
};

namespace sg {

// --------------------------------------------------------- flattened graph
enum NodeType { N_FILTER = 0, N_SPLIT_DUP = 1, N_SPLIT_RR = 2, N_JOIN = 3, N_LOOP = 4 };

struct Flat;
// A feedback loop, seen from outside as one stateful filter (N_LOOP) whose firing is one steady-state
// iteration of the loop's own SDF graph: pop P = r_J * join_w[0], push Q = r_S * (split port-0 weight).
struct LoopInfo {
    std::shared_ptr<Flat> sub;          // J (node 0), body, S, loop stream; sub->in_edge / out_edge = outer ports
    int J = 0, S = -1, back = -1;       // joiner, splitter, returning edge (loop stream -> J port 1)
    std::vector<uint32_t> enq;          // initial contents of the returning edge
    int64_t P = 0, Q = 0;
    // static schedule of one firing (one steady iteration of the loop graph), found by simulation
    std::vector<int> sched;             // sub node ids in firing order
    std::vector<int64_t> init_level;    // per sub edge: items queued at the stream start
    std::vector<int64_t> cap;           // per sub edge: FIFO capacity (power of two >= max live items)
};

struct Node {
    NodeType type = N_FILTER;
    int kind = -1;
    std::vector<int32_t> iv;
    std::vector<float> fv;
    std::vector<int32_t> w;   // split / join weights
    int64_t wsum = 0;
    std::vector<int> in, out;  // edge ids, by port
    // filter rates (splitters/joiners: per edge, see Edge)
    int64_t pop = 0, push = 0, peek = 0, prework = 0;
    // analysis
    int64_t rep = 0;     // repetition vector entry
    int64_t ninit = 0;   // init-schedule firings (signed: negative = lag)
    int64_t halo = 0;    // extra firings before a range start (same for every start)
    int elem = -1;       // builder element (filters)
    std::shared_ptr<LoopInfo> loop;  // N_LOOP only
};

struct Edge {
    int src = -1, dst = -1;  // node ids (-1: graph input / output)
    int sport = 0, dport = 0;
    int64_t push = 0;  // items the producer pushes per firing onto this edge
    int64_t pop = 0;   // items the consumer pops per firing from this edge
    int64_t peek = 0;  // items the consumer reads per firing (>= pop)
    int64_t pre = 0;   // prework items of the producer on this edge
    int64_t per_iter = 0;  // items per steady-state iteration (= rep_src * push)
};

// A split-join of the hierarchy in the flat graph: splitter, joiner, and the first node of each branch
// (branch b = nodes [first[b], first[b + 1]), the last one ending before the joiner; branches are
// contiguous in construction order).
struct SjInfo {
    int split = -1, join = -1;
    std::vector<int> first;
};

struct Flat {
    sg_dtype dtype = SG_F32;
    std::vector<Node> nodes;  // topological (construction) order
    std::vector<Edge> edges;
    int in_edge = -1, out_edge = -1;
    int64_t in_per_iter = 0, out_per_iter = 0;
    std::vector<std::vector<int>> pipes;  // innermost pipelines (every kid a filter), node ids in order
    std::vector<SjInfo> sjs;              // split-joins, in construction order
    std::vector<int> chain_first;         // chain-fissioned graph: first node id of each group (S_g); group g
                                          // = nodes [chain_first[g], chain_first[g + 1]) (empty if not fissioned)
    // Builds from the hierarchy; throws Error.
    static Flat build(const sg_graph& g);
    void solve_rates();       // balance equations -> rep
    void solve_init();        // init schedule (signed) + halos
    int64_t input_items(int64_t n) const;   // minimal input prefix for n iterations
    int64_t output_items(int64_t n) const;
    bool is_physical(int e) const { return edges[e].src < 0 || nodes[edges[e].src].type == N_FILTER; }
};

// Order-preserving chain fission of split-join `sj`: its branches are cut into the
// contiguous groups starting at branch group_first[0] = 0 < group_first[1] < ...; a duplicate
// splitter becomes a forward chain S_1 -> S_2 -> ... (S_g feeds group g's branches and relays the
// stream to S_{g+1}); a roundrobin(1) joiner feeding ADD(n_branches) becomes an accumulate chain
// acc_g = ADD(acc_{g-1}, y_first(g), ..., y_last(g)) (J_g = roundrobin(1) over acc_{g-1} and group g's
// branches), bit-identical to the sequential ADD (s = 0 + acc_{g-1} = acc_{g-1} exactly).
// chain_fission_eligible: which of the two chains apply (0 none, bit 1 forward, bit 2 accumulate).
int chain_fission_eligible(const Flat& f, int sj);
Flat chain_fission(const Flat& f, int sj, const std::vector<int>& group_first);

// kind metadata
struct KindRates { int64_t peek, pop, push, prework; };
KindRates kind_rates(int kind, const std::vector<int32_t>& iv, const std::vector<float>& fv, sg_dtype dt);
const char* kind_name(int kind);

// ------------------------------------------------------------------ planner
struct Topology {
    int G = 1;
    int L = 0;
    std::vector<uint8_t> dt;  // [L][G][G]: link l carries i->j
    bool carries(int l, int i, int j) const { return dt[(size_t)l * G * G + (size_t)i * G + j] != 0; }
    static Topology nvswitch(int G);
    static Topology pcie_tree4();  // Fig. 3.3
};

// PDG edge: bytes per iteration from partition src to partition dst.  `data` >= 0
// names the stream a duplicate splitter copies (its node id): edges with the same `data` carry the
// same items, so a link carries them once per destination GPU (SURVEY.md 8(c)-4 reading 15).
struct PdgEdge { int src, dst; double bytes; int data = -1; };

struct Partition {
    std::vector<int> nodes;  // node ids (sorted, topological)
    double t_est = 0;        // PEE estimate, ns per iteration
    double t_comp = 0, t_dt = 0;
    int mode = 0;            // 1 register, 2 staged
    int gpu = 0;
    int tile = 0, threads = 0;
};

}  // namespace sg
