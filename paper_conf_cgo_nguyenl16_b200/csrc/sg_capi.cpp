// sg_capi.cpp -- the extern "C" boundary declared in include/sg.h.
// Every entry point catches all C++ exceptions and converts them to sg_status;
// the message is kept in a thread-local buffer for sg_last_error().
#include <cuda_runtime.h>

#include <algorithm>
#include <cstring>
#include <numeric>

#include "sg_plan.h"
#include "sg_runtime.h"

struct sg_plan_s {
    sg::Plan plan;
};

namespace {
thread_local std::string t_err;

sg_status fail(sg_status c, const std::string& m) {
    t_err = m;
    return c;
}

template <class F>
sg_status guard(F&& f) {
    try {
        t_err.clear();
        f();
        return SG_OK;
    } catch (const sg::Error& e) {
        return fail(e.code, e.what());
    } catch (const std::bad_alloc&) {
        return fail(SG_E_NOMEM, "host allocation failed");
    } catch (const std::exception& e) {
        return fail(SG_E_ARG, e.what());
    } catch (...) {
        return fail(SG_E_ARG, "unknown error");
    }
}

sg::Elem& current_pipe(sg_graph* g) { return g->elems[g->open.back()]; }
}  // namespace

extern "C" {

const char* sg_last_error(void) { return t_err.c_str(); }
const char* sg_version(void) { return "sg-b200 0.1 (sm_100a, NVRTC)"; }

sg_status sg_graph_create(sg_dtype dtype, sg_graph** out) {
    if (!out) return fail(SG_E_ARG, "out is NULL");
    if (dtype != SG_F32 && dtype != SG_I32) return fail(SG_E_ARG, "bad dtype");
    return guard([&] {
        auto* g = new sg_graph();
        g->dtype = dtype;
        sg::Elem top;
        top.type = sg::E_PIPE;
        g->elems.push_back(top);
        g->top = 0;
        g->open.push_back(0);
        *out = g;
    });
}

void sg_graph_destroy(sg_graph* g) { delete g; }

sg_status sg_add_filter(sg_graph* g, const sg_filter_desc* d, int32_t* elem_id) {
    if (!g || !d) return fail(SG_E_ARG, "NULL argument");
    if (d->n_i < 0 || d->n_f < 0 || (d->n_i && !d->p_i) || (d->n_f && !d->p_f)) return fail(SG_E_ARG, "bad parameter arrays");
    return guard([&] {
        sg::Elem e;
        e.type = sg::E_FILTER;
        e.kind = (int)d->kind;
        e.iv.assign(d->p_i, d->p_i + d->n_i);
        e.fv.assign(d->p_f, d->p_f + d->n_f);
        sg::kind_rates(e.kind, e.iv, e.fv, g->dtype);  // validates (throws)
        int id = (int)g->elems.size();
        g->elems.push_back(std::move(e));
        current_pipe(g).kids.push_back(id);
        if (elem_id) *elem_id = id;
    });
}

sg_status sg_add_splitjoin(sg_graph* g, sg_split_kind kind, const int32_t* split_w, const int32_t* join_w,
                           int32_t nb, int32_t* sj_id) {
    if (!g) return fail(SG_E_ARG, "NULL graph");
    if (nb < 1) return fail(SG_E_ARG, "split-join needs >= 1 branch");
    if (kind != SG_SPLIT_DUPLICATE && kind != SG_SPLIT_ROUNDROBIN) return fail(SG_E_ARG, "bad split kind");
    return guard([&] {
        sg::Elem e;
        e.type = sg::E_SJ;
        e.split_kind = kind == SG_SPLIT_DUPLICATE ? 0 : 1;
        e.split_w.assign(nb, 1);
        e.join_w.assign(nb, 1);
        if (kind == SG_SPLIT_ROUNDROBIN && split_w) e.split_w.assign(split_w, split_w + nb);
        if (join_w) e.join_w.assign(join_w, join_w + nb);
        for (int b = 0; b < nb; b++)
            if (e.split_w[b] < 1 || e.join_w[b] < 1) throw sg::Error(SG_E_ARG, "weights must be >= 1");
        int id = (int)g->elems.size();
        g->elems.push_back(e);
        for (int b = 0; b < nb; b++) {
            sg::Elem p;
            p.type = sg::E_PIPE;
            g->elems.push_back(p);
            g->elems[id].branches.push_back((int)g->elems.size() - 1);
        }
        g->elems[id].branch_done.assign(nb, false);
        current_pipe(g).kids.push_back(id);
        if (sj_id) *sj_id = id;
    });
}

sg_status sg_add_feedbackloop(sg_graph* g, const int32_t join_w[2], sg_split_kind kind, const int32_t* split_w,
                              int32_t n_enq, const void* enq, int32_t* loop_id) {
    if (!g || !join_w) return fail(SG_E_ARG, "NULL argument");
    if (kind != SG_SPLIT_DUPLICATE && kind != SG_SPLIT_ROUNDROBIN) return fail(SG_E_ARG, "bad split kind");
    if (n_enq < 0 || (n_enq > 0 && !enq)) return fail(SG_E_ARG, "bad enqueue list");
    return guard([&] {
        sg::Elem e;
        e.type = sg::E_LOOP;
        e.split_kind = kind == SG_SPLIT_DUPLICATE ? 0 : 1;
        e.join_w.assign(join_w, join_w + 2);
        e.split_w.assign(2, 1);
        if (kind == SG_SPLIT_ROUNDROBIN && split_w) e.split_w.assign(split_w, split_w + 2);
        if (e.join_w[0] < 0 || e.join_w[1] < 1 || e.split_w[0] < 0 || e.split_w[1] < 1)
            throw sg::Error(SG_E_ARG, "feedback loop weights: join_w = {>=0, >=1}, split_w = {>=0, >=1}");
        if (e.join_w[0] == 0) throw sg::Error(SG_E_UNSUPPORTED, "feedback loop without outer input (join_w[0] = 0)");
        if (kind == SG_SPLIT_ROUNDROBIN && e.split_w[0] == 0) throw sg::Error(SG_E_UNSUPPORTED, "feedback loop without output");
        e.enq.assign((const uint32_t*)enq, (const uint32_t*)enq + n_enq);
        int id = (int)g->elems.size();
        g->elems.push_back(e);
        for (int b = 0; b < 2; b++) {
            sg::Elem p;
            p.type = sg::E_PIPE;
            g->elems.push_back(p);
            g->elems[id].branches.push_back((int)g->elems.size() - 1);
        }
        g->elems[id].branch_done.assign(2, false);
        current_pipe(g).kids.push_back(id);
        if (loop_id) *loop_id = id;
    });
}

sg_status sg_branch_begin(sg_graph* g, int32_t sj, int32_t b) {
    if (!g) return fail(SG_E_ARG, "NULL graph");
    if (sj < 0 || sj >= (int)g->elems.size() || (g->elems[sj].type != sg::E_SJ && g->elems[sj].type != sg::E_LOOP))
        return fail(SG_E_ARG, "not a split-join or feedback-loop id");
    sg::Elem& e = g->elems[sj];
    if (b < 0 || b >= (int)e.branches.size()) return fail(SG_E_ARG, "branch out of range");
    if (e.branch_done[b]) return fail(SG_E_STRUCTURE, "branch already filled");
    // the split-join must belong to the currently open pipeline
    const auto& kids = current_pipe(g).kids;
    if (std::find(kids.begin(), kids.end(), sj) == kids.end())
        return fail(SG_E_STRUCTURE, "split-join is not in the currently open pipeline");
    g->open.push_back(e.branches[b]);
    g->open_branch.push_back({sj, b});
    return SG_OK;
}

sg_status sg_branch_end(sg_graph* g) {
    if (!g) return fail(SG_E_ARG, "NULL graph");
    if (g->open.size() <= 1) return fail(SG_E_STRUCTURE, "no open branch");
    auto sb = g->open_branch.back();
    g->elems[sb.first].branch_done[sb.second] = true;
    g->open.pop_back();
    g->open_branch.pop_back();
    return SG_OK;
}

void sg_plan_opts_default(sg_plan_opts* o) {
    if (!o) return;
    std::memset(o, 0, sizeof(*o));
    o->partitioner = SG_PART_ALGORITHM1;
    o->transport = SG_TRANSPORT_AUTO;
}

sg_status sg_plan(const sg_graph* g, int32_t n_gpus, const sg_plan_opts* opts, sg_plan_t** out) {
    if (!g || !out) return fail(SG_E_ARG, "NULL argument");
    if (n_gpus < 1 || n_gpus > 64) return fail(SG_E_ARG, "n_gpus must be in [1, 64]");
    return guard([&] {
        sg_plan_opts o;
        sg_plan_opts_default(&o);
        if (opts) o = *opts;
        auto* p = new sg_plan_s();
        try {
            sg::build_plan(p->plan, *g, n_gpus, o);
        } catch (...) {
            delete p;
            throw;
        }
        *out = p;
    });
}

int64_t sg_input_items(const sg_plan_t* p, int64_t n) {
    if (!p || n < 0) return -1;
    return p->plan.flat.input_items(n);
}
int64_t sg_output_items(const sg_plan_t* p, int64_t n) {
    if (!p || n < 0) return -1;
    return p->plan.flat.output_items(n);
}

sg_status sg_plan_info(const sg_plan_t* pp, sg_plan_info_t* o) {
    if (!pp || !o) return fail(SG_E_ARG, "NULL argument");
    const sg::Plan& p = pp->plan;
    std::memset(o, 0, sizeof(*o));
    o->n_nodes = (int32_t)p.flat.nodes.size();
    o->n_edges = (int32_t)p.flat.edges.size();
    o->n_partitions = (int32_t)p.parts.size();
    o->n_gpus = p.G;
    o->in_per_iter = p.flat.in_per_iter;
    o->out_per_iter = p.flat.out_per_iter;
    o->reps = p.reps.data();
    o->init_firings = p.ninit.data();
    o->node_type = p.node_type.data();
    o->node_kind = p.node_kind.data();
    o->node_partition = p.node_part.data();
    o->partition_gpu = p.part_gpu.data();
    o->partition_time = p.part_time.data();
    o->partition_mode = p.part_mode.data();
    o->est_tmax = p.est_tmax;
    o->input_device = p.devices[p.input_gpu];
    o->output_device = p.devices[p.output_gpu];
    o->iters_per_fragment = p.iters_per_fragment;
    o->ilp_optimal = p.ilp_optimal ? 1 : 0;
    double written = 0, pruned = 0;
    int64_t intops = 0;
    for (const auto& ck : p.kernels) {
        written += (double)ck.ki.flops_per_iter;
        pruned += ck.ki.flops_exec_per_iter >= 0 ? std::min<double>((double)ck.ki.flops_exec_per_iter,
                                                                    (double)ck.ki.flops_per_iter)
                                                 : (double)ck.ki.flops_per_iter;
        intops += ck.ki.intops_per_iter;
    }
    o->flops_per_iter_written = written;
    o->flops_per_iter_pruned = pruned;
    o->intops_per_iter = intops;
    o->replicas = p.R;
    o->chain_fission = p.chain_fission ? 1 : 0;
    return SG_OK;
}

const char* sg_plan_source(const sg_plan_t* p, int32_t part) {
    if (!p || part < 0 || part >= (int)p->plan.kernels.size()) return nullptr;
    return p->plan.kernels[part].ki.source.c_str();
}

sg_status sg_run(sg_plan_t* p, const void* input, int64_t n, void* output, void* stream) {
    if (!p) return fail(SG_E_ARG, "NULL plan");
    if (n < 0) return fail(SG_E_ARG, "negative n_iters");
    if (n == 0) return SG_OK;
    if (!input || !output) return fail(SG_E_ARG, "NULL buffer");
    return guard([&] { p->plan.run(input, n, output, (cudaStream_t)stream); });
}

sg_status sg_run_host(sg_plan_t* p, const void* hin, int64_t n, void* hout) {
    if (!p) return fail(SG_E_ARG, "NULL plan");
    if (n < 0) return fail(SG_E_ARG, "negative n_iters");
    if (n == 0) return SG_OK;
    if (!hin || !hout) return fail(SG_E_ARG, "NULL buffer");
    return guard([&] { p->plan.run_host(hin, n, hout); });
}

int32_t sg_topology_links(int32_t kind, int32_t G) {
    if (kind == 0 && G >= 1 && G <= 64) return 2 * G;
    if (kind == 1 && G == 4) return 12;
    return -1;
}

sg_status sg_topology_dtlist(int32_t kind, int32_t G, uint8_t* dt) {
    if (!dt || sg_topology_links(kind, G) < 0) return fail(SG_E_ARG, "bad topology kind / size");
    sg::Topology t = kind == 0 ? sg::Topology::nvswitch(G) : sg::Topology::pcie_tree4();
    std::memcpy(dt, t.dt.data(), t.dt.size());
    return SG_OK;
}

sg_status sg_map_ilp(int32_t P, const double* T, int32_t ne, const int32_t* es, const int32_t* ed, const double* eb,
                     int32_t topo_kind, int32_t G, double lat, double bw, int32_t ms, int32_t method, int32_t* assign,
                     double* tmax, int32_t* optimal) {
    if (P < 0 || (P && (!T || !assign)) || ne < 0 || (ne && (!es || !ed || !eb)) || bw <= 0)
        return fail(SG_E_ARG, "bad ILP arguments");
    if (sg_topology_links(topo_kind, G) < 0) return fail(SG_E_ARG, "bad topology");
    return guard([&] {
        std::vector<double> Tv(T, T + P);
        std::vector<sg::PdgEdge> pdg;
        for (int i = 0; i < ne; i++) {
            if (es[i] < 0 || es[i] >= P || ed[i] < 0 || ed[i] >= P) throw sg::Error(SG_E_ARG, "PDG edge out of range");
            pdg.push_back({es[i], ed[i], eb[i]});
        }
        sg::Topology t = topo_kind == 0 ? sg::Topology::nvswitch(G) : sg::Topology::pcie_tree4();
        sg::MapResult m = sg::map_partitions(Tv, pdg, t, lat, bw, ms > 0 ? ms : 10000, method);
        for (int i = 0; i < P; i++) assign[i] = m.assign[i];
        if (tmax) *tmax = m.tmax;
        if (optimal) *optimal = m.optimal ? 1 : 0;
    });
}

double sg_paper_model(int32_t n, const double* t, const double* f, int32_t S, int32_t W, int32_t F, double D,
                      double C1, double C2, double* tcomp, double* tdt, double* tdb) {
    if (n < 0 || (n && (!t || !f)) || S < 1 || W < 1 || F < 1) return -1.0;
    std::vector<double> tv(t, t + n), fv(f, f + n);
    return sg::paper_model(tv, fv, S, W, F, D, C1, C2, tcomp, tdt, tdb);
}

int32_t sg_plan_pdg(const sg_plan_t* p, int32_t cap, int32_t* src, int32_t* dst, double* bytes) {
    if (!p) return -1;
    const auto& e = p->plan.pdg;
    for (int i = 0; i < (int)e.size() && i < cap; i++) {
        if (src) src[i] = e[i].src;
        if (dst) dst[i] = e[i].dst;
        if (bytes) bytes[i] = e[i].bytes;
    }
    return (int32_t)e.size();
}

int32_t sg_pee_features(const sg_plan_t* p, int32_t part, double* out, int32_t cap) {
    if (!p || !out || part < 0 || part >= (int32_t)p->plan.parts.size()) return -1;
    try {
        const sg::Plan& pl = p->plan;
        const auto& nodes = pl.parts[part].nodes;
        sg::PeeEstimate est = sg::pee_estimate(pl.flat, nodes);
        const sg::PartitionWork& w = est.work;
        const sg::KernelInfo& ki = pl.kernels[part].ki;
        const bool gen = !pl.opts.plan_only;
        const double v[29] = {(double)est.mode, w.flops, w.intops, w.dfma, w.reads, w.writes, w.firings, w.in_bytes,
                              w.out_bytes, (double)w.levels, w.halo_firings, w.loop_firings, (double)w.cse_nodes,
                              w.frame ? 1.0 : 0.0, est.bitslice ? 1.0 : 0.0, pl.part_time[part], (double)w.in_edges,
                              (double)w.out_edges, w.row_items,
                              gen ? (ki.fused ? 1.0 : 0.0) : -1.0, gen ? (double)ki.tile : -1.0,
                              gen ? (double)ki.threads : -1.0, gen ? (double)ki.smem : -1.0,
                              gen ? (double)ki.source.size() : -1.0, gen ? (double)ki.reg_variant : -1.0,
                              (double)w.components, est.fused ? 1.0 : 0.0, gen ? (double)ki.mode : -1.0,
                              gen ? ki.par_eff : -1.0};
        int32_t n = std::min<int32_t>(cap, 29);
        for (int32_t i = 0; i < n; i++) out[i] = v[i];
        return n;
    } catch (...) {
        return -1;
    }
}

sg_status sg_comm_unique_id(uint8_t id[128]) {
    if (!id) return fail(SG_E_ARG, "NULL id");
    return guard([&] { sg::nccl_unique_id(id); });
}

sg_status sg_comm_init(sg_plan_t* p, int32_t nranks, int32_t rank, const uint8_t id[128], int32_t device) {
    if (!p || !id) return fail(SG_E_ARG, "NULL argument");
    return guard([&] { p->plan.comm_init(nranks, rank, id, device); });
}

sg_status sg_run_rank(sg_plan_t* p, const void* input, int64_t n, void* output, void* stream) {
    if (!p) return fail(SG_E_ARG, "NULL plan");
    if (n < 0) return fail(SG_E_ARG, "negative n_iters");
    if (n == 0) return SG_OK;
    return guard([&] { p->plan.run_rank(input, n, output, (cudaStream_t)stream); });
}

int64_t sg_rank_schedule(const sg_plan_t* p, int32_t rank, int64_t n, sg_rank_op* ops, int64_t cap) {
    if (!p || n < 0 || rank < 0 || rank >= p->plan.G) return -1;
    try {
        auto v = sg::rank_schedule(p->plan, rank, n, sg::fragment_size(p->plan, std::max<int64_t>(n, 1)));
        for (int64_t i = 0; i < (int64_t)v.size() && i < cap; i++) {
            ops[i].op = v[i].op;
            ops[i].part = v[i].part;
            ops[i].edge = v[i].edge;
            ops[i].peer = v[i].peer;
            ops[i].fragment = v[i].frag;
            ops[i].k_begin = v[i].kb;
            ops[i].k_end = v[i].ke;
            ops[i].items = v[i].items;
        }
        return (int64_t)v.size();
    } catch (...) {
        return -1;
    }
}

sg_status sg_profile_partitions(sg_plan_t* p, int64_t n, int32_t reps, double* ns_per_iter) {
    if (!p || !ns_per_iter) return fail(SG_E_ARG, "NULL argument");
    if (n <= 0 || reps <= 0) return fail(SG_E_ARG, "n_iters and reps must be positive");
    return guard([&] { p->plan.profile_partitions(n, reps, ns_per_iter); });
}

int64_t sg_last_launch_count(const sg_plan_t* p) { return p ? p->plan.last_launches : -1; }

void sg_plan_destroy(sg_plan_t* p) { delete p; }

}  // extern "C"
