// sg_dist.cpp -- one process per GPU: the pipelined multi-GPU execution of
// PAPER.md:552-567 (section 3.2.3, Fig. 3.5) with boundary streams carried by
// NCCL point-to-point over NVLink / NVSwitch.
//
// Every rank builds the same plan (same graph, n_gpus = world size, so the same
// Algorithm-1 partitions, PDG and ILP mapping) and calls sg_run_rank.  A rank
// runs only the partitions the ILP mapped to it, fragment by fragment, on its
// compute stream; cut-edge fragments travel on one comm stream per rank:
//
//     issue order   R(0) | K(0) R(1) S(0) | K(1) R(2) S(1) | ...
//
// R(f) = ncclRecv of every incoming cut edge of fragment f, S(f) = ncclSend of
// every outgoing one, both in global edge-id order (so the k-th message between
// two ranks is the same edge/fragment on both sides: NCCL matches P2P by order),
// K(f) = the rank's partition kernels of fragment f.  Receiving f+1 before
// sending f lets a middle rank's compute of fragment f+1 overlap its transfers;
// double-buffered slots are recycled through CUDA events only.  The rank graph
// is acyclic (partitions are convex and topologically ordered), so every
// blocking P2P op is eventually matched.
#include <dlfcn.h>
#include <nccl.h>

#include <algorithm>
#include <cstring>

#include "sg_plan.h"
#include "sg_runtime.h"

namespace sg {

namespace {
struct Nccl {
    decltype(&ncclGetUniqueId) get_id = nullptr;
    decltype(&ncclCommInitRank) init_rank = nullptr;
    decltype(&ncclSend) send = nullptr;
    decltype(&ncclRecv) recv = nullptr;
    decltype(&ncclGroupStart) gstart = nullptr;
    decltype(&ncclGroupEnd) gend = nullptr;
    decltype(&ncclCommDestroy) destroy = nullptr;
    decltype(&ncclGetErrorString) errstr = nullptr;
    bool ok = false;
};
Nccl& nccl() {
    static Nccl n;
    static std::once_flag once;
    std::call_once(once, [] {
        void* h = dlopen("libnccl.so.2", RTLD_NOW | RTLD_GLOBAL);
        if (!h) {
            if (const char* p = std::getenv("SG_NCCL_LIB")) h = dlopen(p, RTLD_NOW | RTLD_GLOBAL);
        }
        if (!h) {
            const char* guesses[] = {"/opt/prime-rl/.venv/lib/python3.12/site-packages/nvidia/nccl/lib/libnccl.so.2",
                                     "/usr/lib/x86_64-linux-gnu/libnccl.so.2"};
            for (const char* g : guesses)
                if ((h = dlopen(g, RTLD_NOW | RTLD_GLOBAL))) break;
        }
        if (!h) return;
        n.get_id = (decltype(n.get_id))dlsym(h, "ncclGetUniqueId");
        n.init_rank = (decltype(n.init_rank))dlsym(h, "ncclCommInitRank");
        n.send = (decltype(n.send))dlsym(h, "ncclSend");
        n.recv = (decltype(n.recv))dlsym(h, "ncclRecv");
        n.gstart = (decltype(n.gstart))dlsym(h, "ncclGroupStart");
        n.gend = (decltype(n.gend))dlsym(h, "ncclGroupEnd");
        n.destroy = (decltype(n.destroy))dlsym(h, "ncclCommDestroy");
        n.errstr = (decltype(n.errstr))dlsym(h, "ncclGetErrorString");
        n.ok = n.get_id && n.init_rank && n.send && n.recv && n.gstart && n.gend && n.destroy;
    });
    if (!n.ok) throw Error(SG_E_COMM, "NCCL not available (libnccl.so.2 not found; set SG_NCCL_LIB)");
    return n;
}
#define SG_NC(x)                                                                                              \
    do {                                                                                                      \
        ncclResult_t r_ = (x);                                                                                \
        if (r_ != ncclSuccess)                                                                                \
            throw Error(SG_E_COMM, std::string(#x) + ": " + (nccl().errstr ? nccl().errstr(r_) : "nccl error")); \
    } while (0)
#define SG_RT2(x)                                                                                             \
    do {                                                                                                      \
        cudaError_t r_ = (x);                                                                                 \
        if (r_ != cudaSuccess) throw Error(SG_E_CUDA, std::string(#x) + ": " + cudaGetErrorString(r_));       \
    } while (0)
}  // namespace

void nccl_unique_id(uint8_t out[128]) {
    ncclUniqueId id;
    SG_NC(nccl().get_id(&id));
    std::memcpy(out, &id, sizeof id < 128 ? sizeof id : 128);
}

std::vector<RankOp> rank_schedule(const Plan& p, int rank, int64_t n, int64_t F) {
    std::vector<RankOp> ops;
    if (n <= 0) return ops;
    const int64_t nfrag = (n + F - 1) / F;
    // replica groups: rank = group * Gs + local GPU; the group handles fragments f with f % R == group
    const int grp = rank / p.Gs, base = grp * p.Gs;
    rank %= p.Gs;
    std::vector<int> cut;
    for (int e = 0; e < (int)p.flat.edges.size(); e++) {
        const Edge& ed = p.flat.edges[e];
        if (ed.src < 0 || ed.dst < 0) continue;
        int ps = p.node_part[ed.src], pd = p.node_part[ed.dst];
        // one message per shared ring (a duplicated stream crosses to a GPU once): its representative
        if (ps != pd && p.part_gpu[ps] != p.part_gpu[pd] && p.ring_rep[e] == e) cut.push_back(e);
    }
    auto window = [&](int e, int64_t ka, int64_t kb) {
        int64_t lo, ex;
        p.cut_window(e, lo, ex);
        return p.flat.edges[e].per_iter * (kb - ka) + ex;
    };
    auto recvs = [&](int64_t f) {
        int64_t ka = f * F, kb = std::min(n, ka + F);
        for (int e : cut) {
            const Edge& ed = p.flat.edges[e];
            if (p.part_gpu[p.node_part[ed.dst]] == rank)
                ops.push_back({SG_OP_RECV, p.node_part[ed.dst], e, base + p.part_gpu[p.node_part[ed.src]], f, ka, kb,
                               window(e, ka, kb)});
        }
    };
    auto sends = [&](int64_t f) {
        int64_t ka = f * F, kb = std::min(n, ka + F);
        for (int e : cut) {
            const Edge& ed = p.flat.edges[e];
            if (p.part_gpu[p.node_part[ed.src]] == rank)
                ops.push_back({SG_OP_SEND, p.node_part[ed.src], e, base + p.part_gpu[p.node_part[ed.dst]], f, ka, kb,
                               window(e, ka, kb)});
        }
    };
    if (grp < nfrag) recvs(grp);
    for (int64_t f = grp; f < nfrag; f += p.R) {
        int64_t ka = f * F, kb = std::min(n, ka + F);
        for (int q : p.part_order)
            if (p.part_gpu[q] == rank) ops.push_back({SG_OP_LAUNCH, q, -1, base + rank, f, ka, kb, 0});
        if (f + p.R < nfrag) recvs(f + p.R);
        sends(f);
    }
    return ops;
}

int64_t fragment_size(const Plan& p, int64_t n) {
    int64_t F = p.iters_per_fragment;
    if (F <= 0) {
        int64_t wave = 1;
        for (auto& ck : p.kernels) wave = std::max<int64_t>(wave, (int64_t)ck.ki.tile * 148 * 2);
        // one GPU without replicas: partitions run back to back on one stream, so fragments buy no overlap
        // and only cost waves -- one fragment (ring memory permitting); several GPUs:
        // about 8 fragments per GPU so the pipeline fills
        F = (p.G == 1 && p.R == 1) ? n : std::max<int64_t>(wave, (n + 8 * p.G - 1) / (8 * p.G));
        int64_t ring = 0;
        for (auto& e : p.flat.edges)
            if (e.src >= 0 && e.dst >= 0 && p.node_part[e.src] != p.node_part[e.dst]) ring += 4 * e.per_iter;
        if (ring > 0) F = std::min<int64_t>(F, std::max<int64_t>(wave, ((int64_t)1 << 30) / ring));
        // replica groups: every group gets fragments (at least two rounds of R)
        if (p.R > 1) F = std::min<int64_t>(F, std::max<int64_t>(1, (n + 2 * p.R - 1) / (2 * p.R)));
    }
    return std::max<int64_t>(1, std::min(F, n));
}

void Plan::comm_init(int nranks, int rank, const uint8_t id[128], int device) {
    if (nranks != G) throw Error(SG_E_ARG, "world size must equal the plan's n_gpus");
    if (rank < 0 || rank >= nranks) throw Error(SG_E_ARG, "bad rank");
    SG_RT2(cudaSetDevice(device));
    ncclUniqueId uid;
    std::memcpy(&uid, id, sizeof uid);
    ncclComm_t c = nullptr;
    SG_NC(nccl().init_rank(&c, nranks, uid, rank));
    comm = c;
    comm_rank = rank;
    comm_device = device;
}

void Plan::run_rank(const void* in, int64_t n, void* out, cudaStream_t user) {
    if (!comm) throw Error(SG_E_COMM, "sg_comm_init was not called");
    if (n <= 0) return;
    const int me = comm_rank % Gs, dev = comm_device;  // this rank's GPU inside its replica group
    SG_RT2(cudaSetDevice(dev));
    const int64_t F = fragment_size(*this, n);
    const int D = ring_depth;
    if (!dist_ready || dist_F < F) {
        for (auto& kv : dist_slots) for (void* q : kv.second) cudaFree(q);
        for (auto& kv : dist_ev) for (auto ev : kv.second) cudaEventDestroy(ev);
        dist_slots.clear();
        dist_ev.clear();
        if (!dist_compute) SG_RT2(cudaStreamCreateWithFlags(&dist_compute, cudaStreamNonBlocking));
        if (!dist_comm) SG_RT2(cudaStreamCreateWithFlags(&dist_comm, cudaStreamNonBlocking));
        if (!dist_join) SG_RT2(cudaEventCreateWithFlags(&dist_join, cudaEventDisableTiming));
        for (int e = 0; e < (int)flat.edges.size(); e++) {
            const Edge& ed = flat.edges[e];
            if (ed.src < 0 || ed.dst < 0) continue;
            int ps = node_part[ed.src], pd = node_part[ed.dst];
            if (ps == pd || (part_gpu[ps] != me && part_gpu[pd] != me)) continue;
            if (ring_rep[e] != e) continue;  // shares its representative's slots
            int64_t lo, ex;
            cut_window(e, lo, ex);
            for (int s = 0; s < D; s++) {
                void* q = nullptr;
                SG_RT2(cudaMalloc(&q, (size_t)(ed.per_iter * F + ex) * 4));
                dist_slots[e].push_back(q);
            }
            // per slot: 0 data ready for consumer, 1 consumer done, 2 producer done, 3 send done
            for (int s = 0; s < 4 * D; s++) {
                cudaEvent_t ev;
                SG_RT2(cudaEventCreateWithFlags(&ev, cudaEventDisableTiming));
                dist_ev[e].push_back(ev);
            }
        }
        dist_F = F;
        dist_ready = true;
    }
    // slots cycle over this group's fragments (f = group + R * j)
    auto EV = [&](int e, int kind, int64_t f) { return dist_ev[ring_rep[e]][kind * D + (int)((f / R) % D)]; };
    auto SLOT = [&](int e, int64_t f) { return dist_slots[ring_rep[e]][(int)((f / R) % D)]; };
    SG_RT2(cudaEventRecord(dist_join, user));
    SG_RT2(cudaStreamWaitEvent(dist_compute, dist_join, 0));
    SG_RT2(cudaStreamWaitEvent(dist_comm, dist_join, 0));
    const int64_t n_in = flat.input_items(n);
    last_launches = 0;
    std::vector<RankOp> ops = rank_schedule(*this, comm_rank, n, F);
    for (size_t p = 0; p < parts.size(); p++)  // this rank's feedback loops restart from their enqueued items
        if (part_gpu[p] == me && kernels[p].ki.state_words > 0) reset_state(kernels[p], dev, dist_compute);
    size_t i = 0;
    while (i < ops.size()) {
        const RankOp& o = ops[i];
        if (o.op == SG_OP_LAUNCH) {
            CompiledKernel& ck = kernels[o.part];
            IoBinding io;
            for (int e : ck.ki.in_edges) {
                const Edge& ed = flat.edges[e];
                if (ed.src < 0) {
                    if (!in) throw Error(SG_E_ARG, "this rank consumes the graph input: pass it");
                    io.in.push_back(in);
                    io.in_base.push_back(0);
                    io.in_limit.push_back(n_in);
                    continue;
                }
                int64_t lo, ex;
                cut_window(e, lo, ex);
                bool remote = part_gpu[node_part[ed.src]] != me;
                SG_RT2(cudaStreamWaitEvent(dist_compute, EV(e, remote ? 0 : 2, o.frag), 0));
                io.in.push_back(SLOT(e, o.frag));
                io.in_base.push_back(o.kb * ed.per_iter + lo);
                io.in_limit.push_back(ed.per_iter * F + ex);
            }
            for (int e : ck.ki.out_edges) {
                const Edge& ed = flat.edges[e];
                if (ed.dst < 0) {
                    if (!out) throw Error(SG_E_ARG, "this rank produces the graph output: pass it");
                    io.out.push_back(out);
                    io.out_base.push_back(0);
                    continue;
                }
                int64_t lo, ex;
                cut_window(e, lo, ex);
                bool remote = part_gpu[node_part[ed.dst]] != me;
                if (o.frag / R >= D) SG_RT2(cudaStreamWaitEvent(dist_compute, EV(e, remote ? 3 : 1, o.frag), 0));
                io.out.push_back(SLOT(e, o.frag));
                io.out_base.push_back(o.kb * ed.per_iter + lo);
            }
            last_launches += launch_kernel(ck, dev, io, o.kb, o.ke, dist_compute, flat.dtype == SG_F32);
            for (int e : ck.ki.in_edges)
                if (flat.edges[e].src >= 0) SG_RT2(cudaEventRecord(EV(e, 1, o.frag), dist_compute));
            for (int e : ck.ki.out_edges)
                if (flat.edges[e].dst >= 0) SG_RT2(cudaEventRecord(EV(e, 2, o.frag), dist_compute));
            i++;
            continue;
        }
        // a run of consecutive comm ops of the same kind and fragment -> one NCCL group
        size_t j = i;
        while (j < ops.size() && ops[j].op == o.op && ops[j].frag == o.frag) j++;
        for (size_t k = i; k < j; k++) {
            const RankOp& c = ops[k];
            if (c.op == SG_OP_RECV && c.frag / R >= D) SG_RT2(cudaStreamWaitEvent(dist_comm, EV(c.edge, 1, c.frag), 0));
            if (c.op == SG_OP_SEND) SG_RT2(cudaStreamWaitEvent(dist_comm, EV(c.edge, 2, c.frag), 0));
        }
        SG_NC(nccl().gstart());
        for (size_t k = i; k < j; k++) {
            const RankOp& c = ops[k];
            if (c.op == SG_OP_RECV)
                SG_NC(nccl().recv(SLOT(c.edge, c.frag), (size_t)c.items, ncclInt32, c.peer, (ncclComm_t)comm, dist_comm));
            else
                SG_NC(nccl().send(SLOT(c.edge, c.frag), (size_t)c.items, ncclInt32, c.peer, (ncclComm_t)comm, dist_comm));
        }
        SG_NC(nccl().gend());
        for (size_t k = i; k < j; k++) {
            const RankOp& c = ops[k];
            SG_RT2(cudaEventRecord(EV(c.edge, c.op == SG_OP_RECV ? 0 : 3, c.frag), dist_comm));
        }
        i = j;
    }
    SG_RT2(cudaEventRecord(dist_join, dist_compute));
    SG_RT2(cudaStreamWaitEvent(user, dist_join, 0));
    SG_RT2(cudaEventRecord(dist_join, dist_comm));
    SG_RT2(cudaStreamWaitEvent(user, dist_join, 0));
}

void Plan::dist_release() {
    for (auto& kv : dist_slots) for (void* q : kv.second) cudaFree(q);
    for (auto& kv : dist_ev) for (auto ev : kv.second) cudaEventDestroy(ev);
    dist_slots.clear();
    dist_ev.clear();
    if (dist_compute) cudaStreamDestroy(dist_compute);
    if (dist_comm) cudaStreamDestroy(dist_comm);
    if (dist_join) cudaEventDestroy(dist_join);
    dist_compute = dist_comm = nullptr;
    dist_join = nullptr;
    if (comm && nccl().destroy) nccl().destroy((ncclComm_t)comm);
    comm = nullptr;
}

}  // namespace sg
