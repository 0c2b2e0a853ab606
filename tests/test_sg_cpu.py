"""CPU tests of the product library (no GPU): the C ABI loads and exports every
symbol include/sg.h declares; the SDF analysis agrees with the oracle's
independent solver; error codes; the planner (topology dtlist of Fig. 3.3,
ILP exactness against brute force and HiGHS, Algorithm 1 invariants, the
paper's Eq. III.8-III.12); code generation + NVRTC sm_100a compilation of the
benchmark programs and of random graphs.
"""
import os
import re

import numpy as np
import pytest

from workloads import apps
from workloads.spec import Filter, Pipeline, Program, SplitJoin

ROOT = os.path.dirname(os.path.dirname(os.path.abspath(__file__)))


@pytest.fixture(scope="module")
def sg():
    from paper_conf_cgo_nguyenl16_b200 import build, sg as s
    build.build()
    s.lib()
    return s


def test_library_exports_every_declared_symbol(sg):
    hdr = open(os.path.join(ROOT, "include", "sg.h")).read()
    hdr = re.sub(r"/\*.*?\*/", "", hdr, flags=re.S)
    declared = set(re.findall(r"\b(sg_[a-z0-9_]+)\s*\(", hdr))
    assert len(declared) >= 20
    L = sg.lib()
    for name in sorted(declared):
        assert hasattr(L, name), f"libsg.so does not export {name}"
    assert set(sg.EXPORTS) == declared


def test_library_is_sm100a(sg):
    import subprocess
    so = os.path.join(ROOT, "paper_conf_cgo_nguyenl16_b200", "libsg.so")
    out = subprocess.run(["cuobjdump", "--list-elf", so], capture_output=True, text=True).stdout
    assert "sm_100a" in out


# ------------------------------------------------------- SDF analysis vs oracle
@pytest.mark.parametrize("name", list(apps.CONFIGS) + list(apps.EXTRA))
def test_rates_match_oracle(sg, oracle_lib, name):
    prog = {**apps.CONFIGS, **apps.EXTRA}[name]()
    r = oracle_lib.rates(prog)
    with sg.plan(prog, 1, partitioner="single", plan_only=1) as p:
        i = p.info()
        assert i["reps"] == r["reps"]
        assert i["in_per_iter"] == r["in_per_iter"] and i["out_per_iter"] == r["out_per_iter"]
        for n in (1, 2, 5):
            assert p.input_items(n) == oracle_lib.in_items(prog, n)
            assert p.output_items(n) == n * r["out_per_iter"]
        assert p.input_items(0) == 0 and p.output_items(0) == 0


@pytest.mark.parametrize("seed", range(24))
def test_random_graph_rates_and_in_items_match_oracle(sg, oracle_lib, seed):
    prog = apps.random_program(seed, "f32" if seed % 2 else "i32")
    r = oracle_lib.rates(prog)
    with sg.plan(prog, 1, partitioner="single", plan_only=1) as p:
        i = p.info()
        assert i["reps"] == r["reps"]
        for n in (1, 3):
            assert p.input_items(n) == oracle_lib.in_items(prog, n), n
            got = p.output_items(n)
            # output items of n iterations = what the oracle emits on in_items(n) inputs
            x = np.zeros(oracle_lib.in_items(prog, n), np.int32 if prog.dtype == "i32" else np.float32)
            assert oracle_lib.run_items(prog, x, 10 ** 9).size >= got


def test_delay_prework_counts_in_output(sg, oracle_lib):
    prog = Program("d", "f32", Pipeline([Filter("FIR", [3, 1], [1.0, 2.0, 3.0]), Filter("DELAY", [5])]))
    with sg.plan(prog, 1) as p:
        assert p.output_items(4) == 4                       # first 4 stream items: prework zeros
        assert p.input_items(4) == oracle_lib.in_items(prog, 4) == 0
        assert p.output_items(9) == 9
        assert p.input_items(9) == oracle_lib.in_items(prog, 9) == 6


# ------------------------------------------------------------------ errors
def test_inconsistent_rates_rejected(sg):
    bad = Program("bad", "f32", Pipeline([SplitJoin("dup", [Filter("IDENTITY"), Filter("DECIMATE", [2])])]))
    with pytest.raises(sg.SgError) as e:
        sg.plan(bad, 1)
    assert e.value.code == sg.SG_E_RATE


def test_structure_errors(sg):
    g = sg.Graph("f32")
    sj = g.add_splitjoin(True, 2)
    g.branch_begin(sj, 0)
    g.add_filter("IDENTITY")
    g.branch_end()
    with pytest.raises(sg.SgError) as e:          # branch 1 never filled
        sg.Plan(g, 1)
    assert e.value.code == sg.SG_E_STRUCTURE
    with pytest.raises(sg.SgError):
        g.branch_end()                            # nothing open
    empty = sg.Graph("f32")
    with pytest.raises(sg.SgError) as e:
        sg.Plan(empty, 1)
    assert e.value.code == sg.SG_E_STRUCTURE


def test_bad_parameters_rejected(sg):
    g = sg.Graph("f32")
    with pytest.raises(sg.SgError) as e:
        g.add_filter("FIR", [4, 1], [1.0, 2.0])   # 4 taps, 2 coefficients
    assert e.value.code == sg.SG_E_ARG
    gi = sg.Graph("i32")
    with pytest.raises(sg.SgError) as e:
        gi.add_filter("FIR", [1, 1], [1.0])        # float kind on an int graph
    assert e.value.code == sg.SG_E_UNSUPPORTED
    with pytest.raises(sg.SgError):
        sg.plan(apps.bitonic(8), 0)


def test_run_without_gpu_fails_loudly(sg):
    import torch
    if torch.cuda.is_available():
        pytest.skip("GPU present")
    with sg.plan(apps.bitonic(8), 1) as p:
        x = np.zeros(8 * 4, np.int32)
        y = np.zeros(8 * 4, np.int32)
        with pytest.raises(sg.SgError) as e:
            p.run_host(x, 4, y)
        assert e.value.code == sg.SG_E_CUDA
        with pytest.raises(sg.SgError) as e:
            p.profile_partitions(4)
        assert e.value.code == sg.SG_E_CUDA
        with pytest.raises(sg.SgError) as e:
            p.profile_partitions(0)
        assert e.value.code == sg.SG_E_ARG


# ---------------------------------------------------------------- topology
def test_pcie_tree_dtlist_matches_fig_3_3(sg):
    """PAPER.md:468-490 (section 3.2.1, Fig. 3.3): GPU1->GPU2 uses two links,
    GPU2->GPU3 uses four, and link SW2->SW1 carries exactly (1,3),(1,4),(2,3),(2,4)."""
    import json
    gold = json.load(open(os.path.join(ROOT, "tests", "golden", "fig3_3_pcie_tree.json")))
    dt = np.array(sg.topology_dtlist(1, 4))
    assert dt.shape == (12, 4, 4)
    for src, dst, n in gold["links_used"]:
        assert int(dt[:, src - 1, dst - 1].sum()) == n
    up_sw2 = 8  # link index of SW2 -> SW1 in sg_topology_dtlist(1, 4)
    pairs = sorted((i + 1, j + 1) for i in range(4) for j in range(4) if dt[up_sw2, i, j])
    assert pairs == sorted(tuple(p) for p in gold["sw2_to_sw1_pairs"])
    # the uplink rule: uplink l carries i->j iff i is under l and j is not
    for l in range(12):
        assert not any(dt[l, i, i] for i in range(4))


def test_nvswitch_star(sg):
    G = 8
    dt = np.array(sg.topology_dtlist(0, G))
    assert dt.shape == (2 * G, G, G)
    for i in range(G):
        for j in range(G):
            used = set(np.nonzero(dt[:, i, j])[0])
            assert used == (set() if i == j else {i, G + j})


# --------------------------------------------------------------------- ILP
def _rand_instance(seed, P, G):
    rng = np.random.default_rng(seed)
    T = list(rng.uniform(1, 10, P))
    edges = []
    for i in range(P - 1):
        edges.append((i, i + 1, float(rng.uniform(0, 40))))
    for _ in range(P // 2):
        a, b = sorted(rng.choice(P, 2, replace=False))
        edges.append((int(a), int(b), float(rng.uniform(0, 20))))
    return T, edges


@pytest.mark.parametrize("seed", range(12))
@pytest.mark.parametrize("G,topo", [(2, 0), (3, 0), (4, 0), (4, 1)])
def test_ilp_branch_and_bound_equals_brute_force(sg, seed, G, topo):
    P = 6 if G < 4 else 5
    T, edges = _rand_instance(seed, P, G)
    lat, bw = 0.3, 10.0
    a1, t1, opt1 = sg.map_ilp(T, edges, G, topo, lat, bw, method=0)
    a2, t2, opt2 = sg.map_ilp(T, edges, G, topo, lat, bw, method=1)
    assert opt1 and opt2
    assert abs(t1 - t2) <= 1e-9 * max(1, t2)


def _milp_tmax(T, edges, G, dt, lat, bw):
    """The same model, Eq. III.1-III.7 linearised, solved by HiGHS."""
    from scipy.optimize import LinearConstraint, milp, Bounds
    P, E, L = len(T), len(edges), dt.shape[0]
    nv = P * G + E * G * G + 1
    idx_n = lambda i, j: i * G + j
    idx_e = lambda e, k, h: P * G + e * G * G + k * G + h
    it = nv - 1
    c = np.zeros(nv)
    c[it] = 1
    A, lo, hi = [], [], []

    def row():
        return np.zeros(nv)

    for i in range(P):                                   # III.5
        r = row()
        for j in range(G):
            r[idx_n(i, j)] = 1
        A.append(r); lo.append(1); hi.append(1)
    for j in range(G):                                   # III.1 + III.4
        r = row()
        for i in range(P):
            r[idx_n(i, j)] = T[i]
        r[it] = -1
        A.append(r); lo.append(-np.inf); hi.append(0)
    for e, (s, d, D) in enumerate(edges):                # III.6 linearised
        for k in range(G):
            for h in range(G):
                r = row(); r[idx_e(e, k, h)] = 1; r[idx_n(s, k)] = -1
                A.append(r); lo.append(-np.inf); hi.append(0)
                r = row(); r[idx_e(e, k, h)] = 1; r[idx_n(d, h)] = -1
                A.append(r); lo.append(-np.inf); hi.append(0)
                r = row(); r[idx_e(e, k, h)] = 1; r[idx_n(s, k)] = -1; r[idx_n(d, h)] = -1
                A.append(r); lo.append(-1); hi.append(np.inf)
    for l in range(L):                                   # III.2 + III.3 + III.7
        r = row()
        for e, (s, d, D) in enumerate(edges):
            for k in range(G):
                for h in range(G):
                    if dt[l, k, h]:
                        r[idx_e(e, k, h)] = D / bw
        r[it] = -1
        A.append(r); lo.append(-np.inf); hi.append(-lat)
    integrality = np.ones(nv)
    integrality[it] = 0
    bounds = Bounds(np.zeros(nv), np.concatenate([np.ones(nv - 1), [np.inf]]))
    res = milp(c, constraints=LinearConstraint(np.array(A), lo, hi), integrality=integrality, bounds=bounds)
    assert res.success
    return res.fun


@pytest.mark.parametrize("seed", range(6))
@pytest.mark.parametrize("G,topo", [(2, 0), (4, 0), (4, 1)])
def test_ilp_matches_highs(sg, seed, G, topo):
    P = 7
    T, edges = _rand_instance(100 + seed, P, G)
    lat, bw = 0.2, 8.0
    dt = np.array(sg.topology_dtlist(topo, G))
    _, tmax, opt = sg.map_ilp(T, edges, G, topo, lat, bw)
    assert opt
    ref = _milp_tmax(T, edges, G, dt, lat, bw)
    assert abs(tmax - ref) <= 1e-6 * max(1.0, ref)


def test_ilp_single_gpu_and_no_edges(sg):
    a, t, opt = sg.map_ilp([3.0, 4.0, 5.0], [], 1, 0, 0.0, 1.0)
    assert a == [0, 0, 0] and abs(t - 12.0) < 1e-12 and opt
    a, t, opt = sg.map_ilp([3.0, 4.0, 5.0], [], 3, 0, 0.0, 1.0)
    assert sorted(a) == [0, 1, 2] and abs(t - 5.0) < 1e-12


# ------------------------------------------------------------- paper model
def test_paper_model_closed_form(sg):
    """Eq. III.8-III.12 with the paper's constants C1 = 38.4, C2 = 11.2."""
    t, f = [10.0, 4.0, 6.0], [1.0, 8.0, 3.0]
    S, W, F, D = 4, 16, 32, 1000.0
    T, tc, tdt, tdb = sg.paper_model(t, f, S, W, F, D)
    assert tc == pytest.approx(10 / 1 + 4 / 4 + 6 / 3)
    assert tdt == pytest.approx(38.4 * 1000 / 32)
    assert tdb == pytest.approx(11.2 * 1000 / (32 + 16 * 4))
    assert T == pytest.approx((max(tc, tdt) + tdb) / W)


# ------------------------------------------------------------ Algorithm 1
def _edges(prog):
    from test_oracle import _edge_list
    return [(u, v) for (u, _, v, _) in _edge_list(prog)]


def _convex(n, edges, part):
    succ = [[] for _ in range(n)]
    for u, v in edges:
        succ[u].append(v)
    inside = set(part)
    seen, st = set(), [w for u in part for w in succ[u] if w not in inside]
    while st:
        x = st.pop()
        if x in seen:
            continue
        seen.add(x)
        for w in succ[x]:
            if w in inside:
                return False
            st.append(w)
    return True


@pytest.mark.parametrize("name,G", [("fmradio10", 1), ("fmradio10", 2), ("filterbank64", 4), ("bitonic32", 2),
                                    ("beamformer12x4", 2), ("fft64", 1)])
def test_algorithm1_invariants(sg, name, G):
    prog = apps.CONFIGS[name]()
    with sg.plan(prog, G, plan_only=1) as p:
        i = p.info()
        n = i["n_nodes"]
        parts = {}
        for v, q in enumerate(i["node_partition"]):
            parts.setdefault(q, []).append(v)
        assert sorted(parts) == list(range(i["n_partitions"]))       # every node in exactly one partition
        E = _edges(prog)
        for q, nodes in parts.items():
            assert _convex(n, E, nodes), f"partition {q} not convex"
        assert all(0 <= g < G for g in i["partition_gpu"])
        loads = [0.0] * G
        for q, g in enumerate(i["partition_gpu"]):
            loads[g] += i["partition_time"][q]
        assert i["est_tmax"] >= max(loads) - 1e-9
        pdg = p.pdg()
        for (a, b, D) in pdg:
            assert a != b and D > 0
        if G == 1:
            assert i["n_partitions"] == 1    # phase 4(2): never worse than the single partition


def test_user_and_per_filter_partitions(sg):
    prog = apps.fmradio(3)
    with sg.plan(prog, 1, partitioner="per_filter", plan_only=1) as p:
        assert p.info()["n_partitions"] == p.info()["n_nodes"]
    n = 0
    with sg.plan(prog, 1, partitioner="single", plan_only=1) as p:
        n = p.info()["n_nodes"]
    with pytest.raises(sg.SgError) as e:    # non-convex: nodes 0 and 2 without 1
        sg.plan(prog, 1, node_partition=[0, 1, 0] + [2] * (n - 3), plan_only=1)
    assert e.value.code == sg.SG_E_PLAN


# ------------------------------------------------------------- codegen/NVRTC
@pytest.mark.parametrize("seed", range(10))
def test_random_graph_compiles(sg, seed):
    prog = apps.random_program(1000 + seed, "f32" if seed % 2 else "i32")
    with sg.plan(prog, 1, partitioner="single") as p:
        src = p.source(0)
        assert "extern \"C\" __global__" in src
    with sg.plan(prog, 1, partitioner="per_filter") as p:
        assert p.info()["n_partitions"] >= 1


def test_benchmark_kernels_are_blackwell_native(sg, tmp_path, monkeypatch):
    """The register-mode BitonicSort kernel streams with TMA (UTMALDG/UTMASTG); the FFT kernel with
    bulk copies (UBLKCP); both are sm_100a cubins from NVRTC."""
    import glob
    import subprocess
    monkeypatch.setenv("SG_CACHE_DIR", str(tmp_path))
    with sg.plan(apps.bitonic(32), 1) as p:
        assert "sg_tma_load_2d" in p.source(0)
    with sg.plan(apps.fft(64), 1) as p:
        assert "sg_bulk_g2s" in p.source(0)
    sass = ""
    for c in glob.glob(str(tmp_path / "*.cubin")):
        sass += subprocess.run(["cuobjdump", "-sass", c], capture_output=True, text=True).stdout
        assert "sm_100a" in subprocess.run(["cuobjdump", "--list-elf", c], capture_output=True, text=True).stdout
    assert "UTMALDG" in sass and "UTMASTG" in sass and "UBLKCP" in sass


@pytest.mark.parametrize("name", ["bitonic8", "fmradio3"])
@pytest.mark.parametrize("part", ["single", "per_filter"])
def test_kernel_entry_points_exist(sg, name, part):
    prog = apps.bitonic(8) if name == "bitonic8" else apps.fmradio(3)
    with sg.plan(prog, 1, partitioner=part) as p:
        for q in range(p.info()["n_partitions"]):
            src = p.source(q)
            assert re.search(r'__global__ void __launch_bounds__\([^)]*\) sg_part%d(_sync)?\(' % q, src), q


# ------------------------------------------------------------------- DES kinds
def test_des_kind_parameters_validated(sg):
    gi = sg.Graph("i32")
    for kind, iv in (("PERMUTE", [4, 0, 4]), ("PERMUTE", [4]), ("XOR_CONST", [3, 1, 0]), ("SBOX", [0] * 63),
                     ("SBOX", [16] + [0] * 63), ("XOR", [0])):
        with pytest.raises(sg.SgError) as e:
            gi.add_filter(kind, iv, [])
        assert e.value.code == sg.SG_E_ARG, (kind, iv)
    gf = sg.Graph("f32")
    for kind, iv in (("XOR", [2]), ("SBOX", [0] * 64), ("INTO_BITS", []), ("BITS_TO_INT", []), ("XOR_CONST", [1, 1])):
        with pytest.raises(sg.SgError) as e:
            gf.add_filter(kind, iv, [])
        assert e.value.code == sg.SG_E_UNSUPPORTED, kind
    gf.add_filter("PERMUTE", [3, 2, 1, 0], [])     # PERMUTE is dtype-agnostic


def test_des_compiles_register_and_staged(sg):
    """DES: every PERMUTE / splitter / joiner resolves at compile time (no data-movement code), the
    key bits are folded into the code, and the general staged path compiles the same graph.  The
    default plan is the bitsliced kernel (32 iterations per thread, S-boxes as LOP3 circuits)."""
    with sg.plan(apps.des(16), 1) as p:
        info = p.info()
        assert info["n_partitions"] == 1 and info["partition_mode"] == [1]
        assert info["intops_per_iter"] == 16 * (48 + 32 + 8) + 64 + 64
        src = p.source(0)
        assert "(bitslice, rolled rounds mode)" in src and "sg_transpose32(w0)" in src and "sg_transpose32(o1)" in src
        assert "16 identical rounds" in src and "SG_BSKEY" in src      # one round's circuit, per-round key table
        assert 8 * 30 < src.count("sg_lop3<") < 8 * 64                # <= 64 gates per S-box
        assert "sg_work_sbox(" not in src and "SG_PI" not in src
    with sg.plan(apps.des(16), 1, codegen_mode="register") as p:
        src = p.source(0)
        assert src.count("sg_work_sbox(") == 16 * 8 and "SG_PI" not in src
    with sg.plan(apps.des(2), 1) as p:                                  # too few rounds to roll
        src = p.source(0)
        assert "(bitslice mode)" in src and 2 * 8 * 30 < src.count("sg_lop3<") < 2 * 8 * 64
    with sg.plan(apps.des(2), 1, partitioner="per_filter") as p:
        assert p.info()["n_partitions"] > 1
        assert any("sg_work_xor<32>" in p.source(q) for q in range(p.info()["n_partitions"]))


# ------------------------------------------------ hybrid replica x pipeline plans
def test_hybrid_replicas_options(sg):
    """R replica groups of G/R GPUs.  R must divide G; the paper's mapping (R = 1)
    is the default; the auto model (-1) replicates compute-bound graphs whose input/output streams
    are thin (FilterBank: 64 B/iteration against ~1 ns of compute) and keeps HBM-bound graphs whose
    input would have to cross NVLink (BitonicSort: 256 B/iteration) on the input GPU."""
    with sg.plan(apps.filterbank(64), 8, plan_only=1, virtual_gpus=1) as p:
        assert p.info()["replicas"] == 1
    with sg.plan(apps.filterbank(64), 8, plan_only=1, virtual_gpus=1, replicas=-1) as p:
        i = p.info()
        assert i["replicas"] == 8 and i["n_partitions"] == 1
    with sg.plan(apps.bitonic(32), 8, plan_only=1, virtual_gpus=1, replicas=-1) as p:
        assert p.info()["replicas"] == 1
    with sg.plan(apps.filterbank(64), 8, plan_only=1, virtual_gpus=1, replicas=2) as p:
        i = p.info()
        assert i["replicas"] == 2 and max(i["partition_gpu"]) < 4
    with pytest.raises(sg.SgError) as e:
        sg.plan(apps.filterbank(8), 4, plan_only=1, virtual_gpus=1, replicas=3)
    assert e.value.code == sg.SG_E_ARG


def test_hybrid_estimate_scales(sg):
    """Group-local ILP + 1/R of the fragments: with thin streams the estimate falls ~1/R until the
    input distribution over the input GPU's NVLink uplink binds (large fragments: Lat amortised)."""
    t = {}
    for R in (1, 2, 4, 8):
        with sg.plan(apps.filterbank(64), 8, plan_only=1, virtual_gpus=1, replicas=R, partitioner="single",
                     iters_per_fragment=1 << 20) as p:
            t[R] = p.info()["est_tmax"]
    assert t[2] < t[1] * 0.6 and t[4] < t[2] * 0.6 and t[8] < t[4]


# ----------------------------------------------------------------- feedback loops
@pytest.mark.parametrize("name", list(apps.FEEDBACK))
def test_feedback_rates_and_input_items_match_oracle(sg, oracle_lib, name):
    prog = apps.FEEDBACK[name]()
    r = oracle_lib.rates(prog)
    with sg.plan(prog, 1, plan_only=1) as p:
        i = p.info()
        assert (i["in_per_iter"], i["out_per_iter"]) == (r["in_per_iter"], r["out_per_iter"])
        for n in (1, 2, 7, 100, 1000):
            assert p.input_items(n) == oracle_lib.in_items(prog, n), n
        # every loop is a partition of its own (mode 4: sequential)
        loops = [q for q, m in enumerate(i["partition_mode"]) if m == 4]
        assert loops and all(sum(1 for v in i["node_partition"] if v == q) == 1 for q in loops)


def test_feedback_loop_rejections(sg):
    from workloads.spec import FeedbackLoop, Filter, Pipeline, Program
    def plan(fb, **kw):
        return sg.plan(Program("x", "f32", Pipeline([fb])), kw.pop("G", 1), plan_only=1, **kw)
    with pytest.raises(sg.SgError) as e:      # peeking filter inside the loop
        plan(FeedbackLoop(Pipeline([Filter("ADD", [2]), Filter("FIR", [3, 1], [1.0, 1.0, 1.0])]), Filter("IDENTITY"),
                          enqueue=[0.0]))
    assert e.value.code == sg.SG_E_UNSUPPORTED
    with pytest.raises(sg.SgError) as e:      # no enqueued item: the joiner waits forever
        plan(FeedbackLoop(Filter("ADD", [2]), Filter("IDENTITY")))
    assert e.value.code == sg.SG_E_RATE
    with pytest.raises(sg.SgError) as e:      # rate-inconsistent loop
        plan(FeedbackLoop(Filter("ADD", [2]), Filter("EXPAND", [2]), enqueue=[0.0]))
    assert e.value.code == sg.SG_E_RATE
    with pytest.raises(sg.SgError) as e:      # nested loops
        plan(FeedbackLoop(Pipeline([Filter("ADD", [2]), FeedbackLoop(Filter("ADD", [2]), Filter("IDENTITY"),
                                                                     enqueue=[0.0])]),
                          Filter("IDENTITY"), enqueue=[0.0]))
    assert e.value.code == sg.SG_E_UNSUPPORTED
    with pytest.raises(sg.SgError) as e:      # replicas would split the loop's sequential state
        plan(FeedbackLoop(Filter("ADD", [2]), Filter("IDENTITY"), enqueue=[0.0]), G=2, virtual_gpus=1, replicas=2)
    assert e.value.code == sg.SG_E_UNSUPPORTED


def test_feedback_kernel_source(sg):
    with sg.plan(apps.echo(8), 1) as p:
        i = p.info()
        q = i["partition_mode"].index(4)
        src = p.source(q)
        assert "(feedback loop mode)" in src and "SG_STATE" in src and "sg_work_amplify" in src


@pytest.mark.parametrize("delay,lane_local", [(64, True), (96, False), (100, False), (300, False)])
def test_feedback_lane_local_only_when_slots_are_lane_private(sg, delay, lane_local):
    """Barrier-free lane-local chains need every ring and the history to be a multiple of the items
    one wavefront step writes (else lanes of different warps share slots and race); other wavefronts
    keep the per-step __syncthreads."""
    with sg.plan(apps.echo(delay, 0.5, 8), 1) as p:
        i = p.info()
        src = p.source(i["partition_mode"].index(4))
        assert ("no barrier" in src) == lane_local
        assert ("    __syncthreads();\n   }" in src) == (not lane_local)


def test_demand_ordered_register_kernels(sg):
    """Wide single-component rows (2-D DCT, MatMul): demand-ordered register kernels -- inputs re-read
    (volatile) from the shared-memory row, outputs stored straight to global memory, no TMA variant;
    FFT (two independent 64-point components) keeps the in-place component kernel.  The row-width
    threshold (384 items) is lowered so small shapes compile quickly (read once per process: run in a
    subprocess)."""
    import subprocess
    import sys
    code = ("import sys; sys.path.insert(0, %r)\n"
            "from paper_conf_cgo_nguyenl16_b200 import sg\nfrom workloads import apps\n"
            "for prog in (apps.dct2d(8), apps.matmul(8, 8, 8)):\n"
            "    with sg.plan(prog, 1) as p:\n"
            "        src = p.source(0)\n"
            "        assert p.info()['partition_mode'] == [1]\n"
            "        assert '(register, demand-ordered mode)' in src and 'SG_LDV(' in src and 'sg_tma' not in src\n"
            "        assert 'one demand run each' in src and 'if (q_ == 3)' in src   # four runs, four bodies\n"
            "        if prog.name.startswith('dct'):   # structurally identical output groups become loops\n"
            "            assert 'output groups, rolled' in src and 'SG_CT8_' in src\n"
            "print('ok')\n") % ROOT
    env = dict(os.environ, SG_DEMAND_MIN="100")
    r = subprocess.run([sys.executable, "-c", code], env=env, capture_output=True, text=True, timeout=600)
    assert r.returncode == 0 and "ok" in r.stdout, r.stderr[-2000:]
    with sg.plan(apps.fft(64), 1) as p:
        src = p.source(0)
        assert "demand-ordered" not in src and "sg_bulk_g2s" in src


def test_bit_transpose_device_code_on_host(tmp_path):
    """sg_transpose32 (the bitslice kernels' word <-> bit-plane conversion) compiled for the host from
    sg_device.cuh, with __byte_perm emulated from its definition: bit j of a[i] must equal bit i of the
    original a[j] for random matrices."""
    import subprocess
    src = open(os.path.join(ROOT, "paper_conf_cgo_nguyenl16_b200", "csrc", "sg_device.cuh")).read()
    i = src.index("SG_DEV void sg_transpose32")
    j = src.index("\n}\n", i) + 3
    prog = ("#include <cstdio>\n#include <cstdlib>\n#define SG_DEV static inline\n"
            "static unsigned __byte_perm(unsigned x, unsigned y, unsigned s) {\n"
            "  unsigned long long v = ((unsigned long long)y << 32) | x; unsigned r = 0;\n"
            "  for (int k = 0; k < 4; k++) r |= (unsigned)((v >> (8 * ((s >> (4 * k)) & 7))) & 0xFF) << (8 * k);\n"
            "  return r; }\n" + src[i:j] +
            "int main() { unsigned a[32], b[32]; int bad = 0; srand(7);\n"
            "  for (int t = 0; t < 50; t++) { for (int i = 0; i < 32; i++) b[i] = a[i] = rand() ^ (rand() << 16);\n"
            "    sg_transpose32(a);\n"
            "    for (int i = 0; i < 32; i++) for (int j = 0; j < 32; j++) bad += ((a[i] >> j) & 1) != ((b[j] >> i) & 1); }\n"
            "  printf(\"%d\\n\", bad); return 0; }\n")
    c = tmp_path / "tr.cpp"
    c.write_text(prog)
    exe = tmp_path / "tr"
    subprocess.check_call(["g++", "-O1", "-o", str(exe), str(c)])
    assert subprocess.run([str(exe)], capture_output=True, text=True).stdout.strip() == "0"


# ------------------------------------------------------ chain fission
@pytest.mark.parametrize("name,m", [("filterbank64", 2), ("filterbank64", 8), ("fmradio10", 3), ("fmradio10", 10)])
def test_chain_fission_structure(sg, name, m):
    """The fissioned graph has the same rates at its boundary (in/out items for any n) and per-node
    repetition 1 relative to the original split-join; m - 1 extra splitters, joiners and ADDs; the
    chain groups become partitions whose PDG carries exactly the forward stream plus the accumulator
    (FilterBank 8 + 8 f32 = 64 B per iteration and hop, FMRadio 1 + 1 f32 = 8 B)."""
    prog = apps.CONFIGS[name]()
    with sg.plan(prog, 1, plan_only=1, partitioner="single") as p0:
        i0 = p0.info()
        io0 = [(p0.input_items(n), p0.output_items(n)) for n in (1, 7, 1000)]
    with sg.plan(prog, m, plan_only=1, virtual_gpus=1, chain_groups=m, partitioner="chain") as p:
        i = p.info()
        assert i["chain_fission"] and i["n_partitions"] == m
        assert i["n_nodes"] == i0["n_nodes"] + 3 * (m - 1)
        assert [(p.input_items(n), p.output_items(n)) for n in (1, 7, 1000)] == io0
        kinds = i["node_kind"]
        assert kinds.count(sg.KINDS["ADD"]) == i0["node_kind"].count(sg.KINDS["ADD"]) + m - 1
        hop = 64.0 if name == "filterbank64" else 8.0
        per_pair = {}
        for a, b, nbytes in p.pdg():      # the forward stream (a duplicate splitter's data) and the accumulator
            per_pair[(a, b)] = per_pair.get((a, b), 0.0) + nbytes
        assert sorted(per_pair) == [(g, g + 1) for g in range(m - 1)]
        assert all(v == hop for v in per_pair.values())


def test_chain_fission_rejections(sg):
    with pytest.raises(sg.SgError) as e:      # BitonicSort: roundrobin splitters, no ADD
        sg.plan(apps.bitonic(8), 2, plan_only=1, virtual_gpus=1, chain_groups=2)
    assert e.value.code == sg.SG_E_PLAN
    with pytest.raises(sg.SgError) as e:
        sg.plan(apps.filterbank(8), 1, plan_only=1, partitioner="chain")
    assert e.value.code == sg.SG_E_ARG
    with pytest.raises(sg.SgError) as e:
        sg.plan(apps.filterbank(8), 1, plan_only=1, chain_groups=1)
    assert e.value.code == sg.SG_E_ARG


@pytest.mark.parametrize("G", [2, 4, 8])
def test_planner_picks_chain_for_filterbank(sg, G):
    """Algorithm 1 + ILP against the fissioned candidates: the largest graph maps to G balanced chain
    groups on G GPUs, 64 B per iteration and hop, the ILP proven optimal (naive
    branch splits ship the duplicated input once per branch)."""
    with sg.plan(apps.filterbank(64), G, plan_only=1, virtual_gpus=1, replicas=1) as p:
        i = p.info()
        assert i["chain_fission"] and i["n_partitions"] == G and i["ilp_optimal"]
        assert sorted(i["partition_gpu"]) == list(range(G))
        t = i["partition_time"]
        assert max(t) < 1.2 * min(t)          # equal branch work; the first group has one input stream fewer
        per_pair = {}
        for a, b, nbytes in p.pdg():
            per_pair[(a, b)] = per_pair.get((a, b), 0.0) + nbytes
        assert len(per_pair) == G - 1 and all(v == 64.0 for v in per_pair.values())


# ------------------------------------------------------------ PEE work
@pytest.mark.parametrize("name,flops", [("filterbank64", 8704), ("fmradio10", 1567), ("beamformer12x4", 13550592),
                                        ("fft64", 3840)])
def test_pee_prices_the_code_generators_pruned_work(sg, name, flops):
    """The PEE counts what the generated kernel executes: FilterBank 66 048 flop as written -> 8 704
    (dead FIR_H firings after Decimate(8), EXPAND zero taps of FIR_F); FMRadio 2 719 -> 1 567 (the 20
    band-pass LPFs share 11 cut-off filters: CSE); BeamFormer's zero-history triangles; FFT nothing to
    prune.  The same numbers the code generator reports (flops_per_iter_pruned)."""
    with sg.plan(apps.CONFIGS[name](), 1, plan_only=1, partitioner="single") as p:
        f = p.pee_features(0)
    assert f["flops"] == flops


def test_pee_counts_dead_firings_and_zero_taps_by_hand(sg):
    """Small pins computed by hand: FIR(4 taps) -> Decimate(2): half the FIR firings are live
    (4 * 2 flops per iteration of 2 inputs -> 1 output); Expand(3) -> FIR(3 taps): one non-zero tap per
    output (3 outputs per iteration, 2 flops each); a FIR split-joined twice with the same
    coefficients is computed once (CSE)."""
    from workloads.spec import Filter, Pipeline, Program, SplitJoin
    dec = Program("d", "f32", Pipeline([Filter("FIR", [4, 1], [1.0, 2.0, 3.0, 4.0]), Filter("DECIMATE", [2])]))
    with sg.plan(dec, 1, plan_only=1, partitioner="single") as p:
        assert p.pee_features(0)["flops"] == 8 and p.pee_features(0)["firings"] == 1
    exp = Program("e", "f32", Pipeline([Filter("EXPAND", [3]), Filter("FIR", [3, 1], [1.0, 2.0, 3.0])]))
    with sg.plan(exp, 1, plan_only=1, partitioner="single") as p:
        assert p.pee_features(0)["flops"] == 6
    c = [0.5, -1.0, 0.25]
    cse = Program("c", "f32", Pipeline([SplitJoin("dup", [Filter("FIR", [3, 1], c), Filter("FIR", [3, 1], c)]),
                                        Filter("ADD", [2])]))
    with sg.plan(cse, 1, plan_only=1, partitioner="single") as p:
        f = p.pee_features(0)
        assert f["cse_nodes"] == 1 and f["flops"] == 6 + 2


def test_pdg_counts_duplicated_stream_once_per_gpu(sg):
    """PDG reading 15: the branches of a duplicate splitter placed on another GPU
    receive its stream once.  FilterBank 8 with the splitter on GPU 0 and all branches on GPU 1: the
    4-byte x 8 items/iteration input crosses once (32 B), not once per branch (8 x 32 B); the rank
    schedule sends one message per fragment for the whole split."""
    prog = apps.filterbank(8)
    with sg.plan(prog, 1, plan_only=1, partitioner="single") as p0:
        n_nodes = p0.info()["n_nodes"]
    part = [1] * n_nodes
    part[0] = 0                                   # the duplicate splitter alone in partition 0
    with sg.plan(prog, 2, plan_only=1, virtual_gpus=1, node_partition=part, link_gbps=1e6,
                 link_latency_us=0.001, iters_per_fragment=1000) as p:
        i = p.info()
        assert i["partition_gpu"][0] != i["partition_gpu"][1]
        dup = [e for e in p.pdg() if e[0] == 0]
        assert len(dup) == 1 and dup[0][2] == 32.0
        src_rank, dst_rank = i["partition_gpu"][0], i["partition_gpu"][1]
        recvs = [o for o in p.rank_schedule(dst_rank, 3000) if o["op"] == sg.SG_OP_RECV]
        assert len(recvs) == 3 and all(o["items"] >= 8 * 1000 for o in recvs)
        sends = [o for o in p.rank_schedule(src_rank, 3000) if o["op"] == sg.SG_OP_SEND]
        assert len(sends) == 3                    # one message per fragment (3 fragments of 1000)


@pytest.mark.parametrize("name", list(apps.CONFIGS))
@pytest.mark.parametrize("G", [2, 4, 8])
def test_ilp_exact_for_every_config(sg, name, G):
    """The branch and bound (Eq. III.1-III.7) proves optimality for every BASELINE
    config at G = 2/4/8 within its deterministic node budget (the paper: Gurobi within 10 s,
    PAPER.md:651-652); HBM-bound graphs stay one partition (any NVLink cut is slower than one GPU,
    SURVEY.md 8(e)); FMRadio takes the 8 B/iteration chain cut at G = 2."""
    with sg.plan(apps.CONFIGS[name](), G, plan_only=1, virtual_gpus=1, replicas=1) as p:
        i = p.info()
        assert i["ilp_optimal"]
        if name in ("fft64", "bitonic32"):
            assert i["n_partitions"] == 1
        if name == "fmradio10" and G == 2:
            assert i["chain_fission"] and i["n_partitions"] == 2
            assert sum(b for _, _, b in p.pdg()) == 8.0


@pytest.mark.parametrize("name,G", [("beamformer12x4", 2), ("beamformer12x4", 4), ("dct16", 2)])
def test_planner_never_keeps_a_cut_worse_than_one_partition(sg, name, G):
    """After code generation the PEE is refined with the kernels' own decisions; a
    candidate the code generator cannot fit (shared memory) or whose refined Tmax is not better than one
    partition yields to the next candidate: the plan's refined estimate never exceeds one partition's."""
    prog = {**apps.CONFIGS, **apps.EXTRA}[name]()
    with sg.plan(prog, 1, partitioner="single") as p1:
        t1 = p1.info()["est_tmax"]
    with sg.plan(prog, G, virtual_gpus=1, replicas=1) as p:
        i = p.info()
        assert i["est_tmax"] <= t1 * 1.0001
        assert all(t > 0 for t in i["partition_time"])


def test_level_split_of_a_frame_fir_kernel(sg, monkeypatch):
    """One GPU: the code generator reports BeamFormer's matched-filter level as unable to fill the CTA
    (parallel efficiency), and the planner cuts the fused partition at that level boundary -- channel
    FIRs + beamforming | matched filters + magnitude -- when the refined estimate says so; the cut is
    convex and every node is covered once.  SG_NO_LEVEL_SPLIT=1 keeps one partition; one-GPU replica
    groups split the same way."""
    prog = apps.beamformer()
    with sg.plan(prog, 1) as p:
        i = p.info()
        assert i["n_partitions"] == 2
        kinds = i["node_kind"]
        part = i["node_partition"]
        # BEAM_FIR (12) nodes of the channel stage and BEAMFORM (13) in partition 0; the matched filters
        # (BEAM_FIR 512 taps) and MAGNITUDE (14) in partition 1
        assert all(part[v] == 0 for v in range(len(kinds)) if kinds[v] == 13)
        assert all(part[v] == 1 for v in range(len(kinds)) if kinds[v] == 14)
        assert sorted(set(part)) == [0, 1]
        f0, f1 = p.pee_features(0), p.pee_features(1)
        assert 0 < f0["par_eff"] <= 1 and 0 < f1["par_eff"] <= 1
        assert i["est_tmax"] > 0
    monkeypatch.setenv("SG_NO_LEVEL_SPLIT", "1")
    with sg.plan(prog, 1) as p:
        assert p.info()["n_partitions"] == 1
        assert p.pee_features(0)["par_eff"] < 0.8
    monkeypatch.delenv("SG_NO_LEVEL_SPLIT")
    with sg.plan(prog, 2, replicas=2, virtual_gpus=1) as p:
        assert p.info()["n_partitions"] == 2 and p.info()["replicas"] == 2
    # graphs without frame FIRs are not affected
    with sg.plan(apps.CONFIGS["filterbank64"](), 1) as p:
        assert p.info()["n_partitions"] == 1 and p.pee_features(0)["par_eff"] == 1.0


def test_frame_fir_sliding_window_source(sg):
    """The frame FIRs are emitted in the sliding-window form: warp-uniform tap groups (the trip count is
    the warp's largest triangle limit), uniform coefficient tables in constant memory, warp-uniform guard
    decisions; SG_BEAM_NOSLIDE=1 would restore the chunked form."""
    with sg.plan(apps.beamformer(), 1) as p:
        src = p.source(0) + p.source(1)
    assert "sliding window: B = " in src and "__reduce_max_sync(0xffffffffu" in src
    assert "__constant__ float2 SG_CTS" in src and "__all_sync(0xffffffffu, sb - " in src


def test_one_gpu_multi_partition_plan_is_one_fragment(sg):
    """A one-GPU plan of several partitions runs every partition once over the whole range (its partitions
    are sequential on one stream: fragments would only add waves); several GPUs keep
    about eight fragments per GPU so the pipeline fills."""
    with sg.plan(apps.beamformer(), 1) as p:
        assert p.info()["n_partitions"] == 2
        launches = [o for o in p.rank_schedule(0, 4096) if o["op"] == 0]
        assert len(launches) == 2 and {(o["k_begin"], o["k_end"]) for o in launches} == {(0, 4096)}
    with sg.plan(apps.CONFIGS["filterbank64"](), 2, virtual_gpus=1, replicas=1) as p:
        frags = {o["fragment"] for o in p.rank_schedule(0, 1 << 20) if o["op"] == 0}
        assert len(frags) >= 4   # 2^20 / (8 G) iterations, at least two waves of the largest tile each
