// dock_sparse.cuh -- sparse-ligand direct correlation engine.
//
// The paper's direct correlation sums "all the voxel-voxel interactions for each translation"
// over the whole m^3 probe box, but an FTMap probe grid is almost empty: a probe has a few
// atoms ("probes are never bigger than 4^3"), so at most n_atoms of the m^3 voxels carry
// weight, in every channel at once.  With the weights folded (Eq. 2) the score is
//   S_r[t] = sum_p sum_v w_p L_{r,p}[v] R_p[t+v] = sum_{occupied v} C_v[t+v],
//   C_v[x] = sum_p W_{r,p}[v] R_p[x],  W_{r,p}[v] = w_p * sum_{atoms a in v} coef[a][p].
// A voxel holding exactly one atom a has C_v = G_a with G_a[x] = sum_p (w_p coef[a][p]) R_p[x], which does
// not depend on the rotation: G_a is computed once per probe and call (k_atom_grids, the "desolvation
// accumulation" of the channels, done once instead of per rotation), and a rotation costs one
// gathered value per occupied voxel and translation.  A voxel holding several atoms (rare: 9 of the 8000
// production units) is correlated directly over the P channels from the receptor with the summed weights,
// exactly as the dense engines do, so no cancellation between atoms' coefficients is amplified.
//
// Arithmetic is FP32: G_a and the direct terms are P-term FMA chains in channel order; the score is the sum
// of the single-atom voxels' gathered values in voxel order of first occurrence, then the multi-atom voxels'
// direct terms -- |err| <= (P + n_terms) * 2^-24 * A (reading Q16), the same order as the FFMA engine;
// integer inputs are exact.
//
// k_corr_sparse: one CTA = (group of RB rotations of one probe, range of columns of TX x TY x nz translations).
// The producer warp streams z-planes of every atom grid G_a (TMA, one box [TY+m-1][TX+m-1] per atom and
// plane) through a ring of NPL plane slots; 16 consumer warps = TY rows x 2 plane groups of ZT planes per
// step (ZT = 2 for 64-translation rows, else 1) x 2 halves of the item's rotations (4 per warp: 4 warps per
// scheduler hide the gather latency); lane j owns the translations x0 + j + 32 i (i < XTS) of
// its row in each of its planes, so every shared-memory read of a warp is 32 consecutive words
// (conflict-free for any voxel offset).  Per rotation the occupied voxels' terms are gathered from the
// ring, then the per-warp top-32 key lists of the FFMA engine take the scores (no score grid in HBM);
// item end publishes bound / mu / candidates for k_merge exactly like the other engines.
#pragma once
#include "dock_kernels.cuh"

namespace sp {

using dk::FULL;
using dk::KEY_MAX;

constexpr int RB = 8;                     // rotations per item (accumulated side by side: independent chains)
constexpr int TY = 4;                     // translation rows per column
constexpr int NPG = 2;                    // plane groups per step (warps = TY rows x NPG groups)
constexpr int RSPLIT = 2;                 // rotation halves: two warps share a (row, plane group), RB/2 rotations each
constexpr int RBW = RB / RSPLIT;          // rotations per warp
constexpr int NWC = TY * NPG * RSPLIT;    // consumer warps (16: 4 per scheduler)
// ZT = planes per warp and step (a template parameter): 2 for the narrow 64-translation rows when the plane
// ring fits (more values per term decode and per gate), else 1; a step advances NPG * ZT planes
constexpr int NTHREADS = (NWC + 1) * 32;  // + 1 TMA producer warp
constexpr int TMAX = 32;                  // occupied voxels per rotation (= atoms) handled by the engine
constexpr int NPLMAX = 16;                // plane-ring depth limit
constexpr int DIRECT = -1;                // term source of a multi-atom voxel
constexpr int NULL_TERM = -1;             // shared-memory term code: no term (rotation has fewer occupied voxels)

// Rotation group of one probe: slots [slot0, slot0 + n) of the call, the probe's atom grids start at
// G[atom0], n_atoms of them.
struct Group {
    int slot0, n, atom0, n_atoms;
};

struct SpArgs {
    int nx, ny, nz;
    int m;                      // probe grid edge
    int TX, ntx, nty;           // column: TX = 32 * XTS translations along x, TY rows
    int TXB, TYB;               // plane box (floats): round4(TX + m - 1) x (TY + m - 1)
    int slot_words;             // plane slot stride (floats, 128-B aligned)
    int npl;                    // plane-ring depth (slots per atom)
    int cols_per_item;          // columns (TX x TY x all nz translations) per item; lists persist across them
    int bound_every;            // columns between refreshes of the lists' global pruning bound (0: never)
    int G;                      // items per group = ceil(ntx * nty / cols_per_item)
    int box_bytes;              // TXB * TYB * 4
    const Group* groups;        // [n_groups]
    const int* term_v;          // [slot][TMAX]: vz << 16 | vy << 8 | vx
    const int* term_src;        // [slot][TMAX]: local atom index (gather) or DIRECT
    const int* n_terms;         // [slot]
    const float* dw;            // [slot][TMAX][P] weights of direct terms
    int P;
    const float* rec;           // padded FP32 receptor [P][rZp][rYp][rXp] (direct terms)
    int rXp, rYp, rZp;
    // top-k mode
    int k, rho, cap;
    unsigned long long* T;
    unsigned long long* mu;
    unsigned int* cnt;
    unsigned long long* cand;
    // grid mode (single-rotation groups): grid[group][nz][ny][nx]
    float* grid;
    const unsigned* n_live;     // optional (device): groups >= *n_live are dead (device-driven fallback)
};

// Voxelization of the sparse engine: the same FP64 grid assignment as dk::k_voxelize (reading Q3/Q18,
// explicit IEEE roundings in the oracle's operation order), emitted as a list of occupied voxels.
struct SpVoxArgs {
    const double* xyz;
    const float* coef;
    const int* atom_off;
    const double* rot;
    const float* w;
    long long unit_begin;
    int n_rot, n_slots, P, m;
    double spacing;
    int* term_v;
    int* term_src;
    int* n_terms;
    float* dw;
    int* status;
    int* slot_atoms;            // [slot][2]: (first atom grid of the unit's probe, its atom count) -- fallback groups
    int atom_lo;                // atom index of the first atom grid
};

#ifndef DOCK_LAUNCHER_TU   // defined once, in dock.cu
__global__ void k_voxelize_sparse(SpVoxArgs a)
{
    const int slot = blockIdx.x * blockDim.x + threadIdx.x;
    if (slot >= a.n_slots) return;
    const long long unit = a.unit_begin + slot;
    const int probe = static_cast<int>(unit / a.n_rot), r = static_cast<int>(unit % a.n_rot);
    const double* q = a.rot + 9 * static_cast<size_t>(r);
    {   // rotation check: |Q^T Q - I| <= 1e-9 and det > 0 (reading Q5)
        bool ok = true;
        for (int i = 0; i < 3; i++)
            for (int j = 0; j < 3; j++) {
                double s = __dmul_rn(q[i], q[j]);
                s = __dadd_rn(s, __dmul_rn(q[3 + i], q[3 + j]));
                s = __dadd_rn(s, __dmul_rn(q[6 + i], q[6 + j]));
                const double want = (i == j) ? 1.0 : 0.0;
                if (!(fabs(s - want) <= 1e-9)) ok = false;
            }
        const double det = q[0] * (q[4] * q[8] - q[5] * q[7]) - q[1] * (q[3] * q[8] - q[5] * q[6]) +
                           q[2] * (q[3] * q[7] - q[4] * q[6]);
        if (!(det > 0.0)) ok = false;
        if (!ok) atomicOr(a.status, dk::ST_BAD_ROTATION);
    }
    const int m = a.m;
    const double c = (m - 1) / 2.0;
    const int a0 = a.atom_off[probe], na = a.atom_off[probe + 1] - a0;
    a.slot_atoms[2 * slot] = a0 - a.atom_lo;
    a.slot_atoms[2 * slot + 1] = na;
    int lin[TMAX], code[TMAX];
    bool outside = false;
    for (int at = 0; at < na && at < TMAX; at++) {
        const double* x = a.xyz + 3 * static_cast<size_t>(a0 + at);
        int v[3];
        bool in = true;
#pragma unroll
        for (int i = 0; i < 3; i++) {
            double rx = __dmul_rn(q[3 * i + 0], x[0]);
            rx = __dadd_rn(rx, __dmul_rn(q[3 * i + 1], x[1]));
            rx = __dadd_rn(rx, __dmul_rn(q[3 * i + 2], x[2]));
            const double g = __dadd_rn(__ddiv_rn(rx, a.spacing), c);
            const double f = floor(__dadd_rn(g, 0.5));
            in = in && (f >= 0.0 && f < static_cast<double>(m));
            v[i] = in ? static_cast<int>(f) : 0;
        }
        outside = outside || !in;
        lin[at] = (v[2] * m + v[1]) * m + v[0];
        code[at] = (v[2] << 16) | (v[1] << 8) | v[0];
    }
    int* tv = a.term_v + static_cast<size_t>(slot) * TMAX;
    int* ts = a.term_src + static_cast<size_t>(slot) * TMAX;
    if (outside || na > TMAX) {
        if (outside) atomicOr(a.status, dk::ST_OUTSIDE);
        a.n_terms[slot] = 0;
        return;
    }
    int nt = 0;
    for (int at = 0; at < na; at++) {
        bool first = true, multi = false;
        for (int b = 0; b < at; b++) first = first && lin[b] != lin[at];
        if (!first) continue;
        for (int b = at + 1; b < na; b++) multi = multi || lin[b] == lin[at];
        tv[nt] = code[at];
        if (!multi) {
            ts[nt] = at;
        } else {
            // several atoms share the voxel: summed coefficients (atom order), then the weight -- the
            // dense engines' L_p[v] * w_p (dk::k_voxelize)
            ts[nt] = DIRECT;
            float* dst = a.dw + (static_cast<size_t>(slot) * TMAX + nt) * a.P;
            for (int p = 0; p < a.P; p++) {
                float s = 0.0f;
                for (int b = at; b < na; b++)
                    if (lin[b] == lin[at]) s += a.coef[static_cast<size_t>(a0 + b) * a.P + p];
                dst[p] = s * a.w[p];
            }
        }
        nt++;
    }
    a.n_terms[slot] = nt;
}

// G_a[Z][Y][X] = sum_p (w_p coef[a][p]) R_p[Z mod nz][Y mod ny][X mod nx] for the atoms [atom_lo,
// atom_lo + n_atoms) of the call (cyclic halo materialised, like the padded receptor); FMA chain in channel
// order starting from 0 (the direct terms use the same chain).
__global__ void k_atom_grids(const float* __restrict__ rec, int rXp, int rYp, int rZp, int nx, int ny, int nz,
                             int P, const float* __restrict__ coef, const float* __restrict__ w, int atom_lo,
                             int n_atoms, float* __restrict__ G, int GXp, int GYp, int GZp)
{
    const int nx4 = GXp / 4;
    const size_t total = static_cast<size_t>(n_atoms) * GZp * GYp * nx4;
    for (size_t i = blockIdx.x * static_cast<size_t>(blockDim.x) + threadIdx.x; i < total;
         i += static_cast<size_t>(gridDim.x) * blockDim.x) {
        const int X4 = static_cast<int>(i % nx4);
        size_t rr = i / nx4;
        const int Y = static_cast<int>(rr % GYp);
        rr /= GYp;
        const int Z = static_cast<int>(rr % GZp);
        const int at = static_cast<int>(rr / GZp);
        const float* cf = coef + static_cast<size_t>(atom_lo + at) * P;
        const int zs = Z % nz, ys = Y % ny;
        float o[4];
#pragma unroll
        for (int j = 0; j < 4; j++) {
            const int xs = (4 * X4 + j) % nx;
            float acc = 0.0f;
            for (int p = 0; p < P; p++)
                acc = fmaf(cf[p] * w[p], rec[((static_cast<size_t>(p) * rZp + zs) * rYp + ys) * rXp + xs], acc);
            o[j] = acc;
        }
        reinterpret_cast<float4*>(G)[i] = make_float4(o[0], o[1], o[2], o[3]);
    }
}

// Fallback groups: one single-rotation group per live flagged slot (grid row = group index).
__global__ void k_sparse_fb_groups(const int* slots, const unsigned* n_live, const int* slot_probe_atoms,
                                   Group* groups, int ch)
{
    const int i = blockIdx.x * blockDim.x + threadIdx.x;
    if (i >= ch) return;
    const int n = static_cast<int>(*n_live);
    Group gr{};
    if (i < n) {
        const int s = slots[i];
        gr.slot0 = s;
        gr.n = 1;
        gr.atom0 = slot_probe_atoms[2 * s];
        gr.n_atoms = slot_probe_atoms[2 * s + 1];
    }
    groups[i] = gr;
}
#endif

// ------------------------------------------------------------------ the correlation kernel

// Slow path of the top-k gate (out of line: keeps the hot loop small for the instruction cache): insert the
// warp's keys below the list's 32nd key into the warp-distributed sorted list L (shared memory, lane i holds
// the i-th smallest), exactly as dk::k_corr does with its register lists.
template <int N>
struct Vec {   // passed by value to the out-of-line helpers (a pointer would force the accumulators to the stack)
    float v[N];
};

// tg: the unit's pruning bound T as last read (keys above it can never be picks): the gate key is
// min(list's 32nd key, tg).
template <int XTS, int ZT>
__device__ __noinline__ void sp_insert(unsigned long long* L, float2* th_rec, const Vec<XTS * ZT> acc, unsigned vmask,
                                       uint32_t tbase, uint32_t plane_stride, int lane, unsigned long long tg)
{
    unsigned long long lst = L[lane];
    unsigned long long thk = dk::shfl_u64(lst, 31);
    thk = thk < tg ? thk : tg;
#pragma unroll
    for (int v = 0; v < XTS * ZT; v++) {
        const uint32_t t = tbase + static_cast<uint32_t>(v / XTS) * plane_stride + 32u * static_cast<uint32_t>(v % XTS);
        const unsigned long long key = ((vmask >> v) & 1u) ? dk::make_key(acc.v[v], t) : KEY_MAX;
        unsigned mm = __ballot_sync(FULL, key < thk);
        while (mm) {
            const int src = __ffs(mm) - 1;
            dk::warp_list_insert(lst, dk::shfl_u64(key, src), lane);
            thk = dk::shfl_u64(lst, 31);
            thk = thk < tg ? thk : tg;
            mm &= ~(1u << src);
            mm &= __ballot_sync(FULL, key < thk);
        }
    }
    L[lane] = lst;
    if (lane == 31) {   // gate record of the list: score bound and t_lin of min(its 32nd key, tg)
        const unsigned long long g = lst < tg ? lst : tg;
        *th_rec = make_float2(dk::key_score_bound(static_cast<uint32_t>(g >> 32)),
                              __uint_as_float(static_cast<uint32_t>(g & 0xffffffffu)));
    }
    __syncwarp();
}

// T_w of a warp list (lane i holds its i-th smallest key): the key of the k-th entry of a greedy pick with
// pairwise cyclic Chebyshev distance > 2 rho; KEY_MAX if there are fewer.  Warp-uniform result.
__device__ __forceinline__ unsigned long long sp_list_bound(unsigned long long key, int k, int rho, int nx, int ny,
                                                            int nz)
{
    const uint32_t t = static_cast<uint32_t>(key & 0xffffffffu);
    bool excl = (key == KEY_MAX);
    unsigned long long Tw = KEY_MAX;
    for (int j = 0; j < k; j++) {
        const unsigned b = __ballot_sync(FULL, !excl);
        if (!b) break;
        const int f = __ffs(b) - 1;
        const unsigned long long kf = dk::shfl_u64(key, f);
        const uint32_t tf = static_cast<uint32_t>(kf & 0xffffffffu);
        excl = excl || (dk::cheb_cyc(t, tf, nx, ny, nz) <= 2 * rho);
        if (j == k - 1) Tw = kf;
    }
    return Tw;
}

// mbarrier wait on a 32-bit shared address (no generic-to-shared conversion in the loop)
__device__ __forceinline__ void mbar_wait_s(uint32_t bar, unsigned parity)
{
    uint32_t ok;
    asm volatile(
        "{\n\t.reg .pred p;\n\tmbarrier.try_wait.parity.shared::cta.b64 p, [%1], %2;\n\tselp.u32 %0, 1, 0, p;\n}\n"
        : "=r"(ok)
        : "r"(bar), "r"(parity)
        : "memory");
    if (ok) return;
    const long long t0 = clock64();
    do {
        asm volatile(
            "{\n\t.reg .pred p;\n\tmbarrier.try_wait.parity.shared::cta.b64 p, [%1], %2;\n\tselp.u32 %0, 1, 0, p;\n}\n"
            : "=r"(ok)
            : "r"(bar), "r"(parity)
            : "memory");
        if (clock64() - t0 > (1ll << 35)) __trap();
    } while (!ok);
}
__device__ __forceinline__ void mbar_arrive_s(uint32_t bar)
{
    asm volatile("mbarrier.arrive.shared::cta.b64 _, [%0];" ::"r"(bar) : "memory");
}

__device__ __forceinline__ float lds_f32(uint32_t addr)
{
    float v;
    asm volatile("ld.shared.f32 %0, [%1];" : "=f"(v) : "r"(addr));
    return v;
}

// A voxel holding several atoms: direct P-channel correlation from the padded receptor with the summed
// weights (rare; out of line).
template <int XTS>
__device__ __noinline__ Vec<XTS> sp_direct(const float* wv, int P, const float* rec, int rXp, int rYp, int rZp,
                                           int z, int y, int x, unsigned vmask)
{
    Vec<XTS> d;
#pragma unroll
    for (int i = 0; i < XTS; i++) {
        d.v[i] = 0.0f;
        if ((vmask >> i) & 1u)
            for (int p = 0; p < P; p++)
                d.v[i] = fmaf(wv[p], rec[((static_cast<size_t>(p) * rZp + z) * rYp + y) * rXp + x + 32 * i], d.v[i]);
    }
    return d;
}

template <int XTS, int ZT, bool GRID>
__global__ void __launch_bounds__(NTHREADS, 1) k_corr_sparse(const __grid_constant__ CUtensorMap gmap, const SpArgs a)
{
    constexpr int PZ = NPG * ZT, V = XTS * ZT;   // planes per step; values per lane and rotation
    extern __shared__ __align__(128) unsigned char smem[];
    __shared__ uint64_t full[NPLMAX], empty[NPLMAX];
    __shared__ int4 s_term[TMAX * RB];   // [term][rotation]: (byte offset (atom ring + (vy * TXB + vx) * 4),
                                         // vz * slot bytes, weight 1.0f, 0); absent or direct terms: weight 0.0f
                                         // (branch-free loop)
    __shared__ int s_dterm[TMAX * RB];   // [term][rotation]: direct term (vx | vy << 8 | vz << 16 | term << 24) or -1
    __shared__ int s_tmax, s_ndirect;    // most occupied voxels of a rotation of the group; direct terms in the group
    __shared__ unsigned long long s_lst[NWC][RBW][32];   // per warp and rotation: sorted top-32 keys (one per lane)
    __shared__ float2 s_th[NWC][RBW];                     // per list: score bound and t_lin of the gate key
    __shared__ unsigned long long s_tg[NWC][RBW];         // per list: the unit's pruning bound T as last read

    const int warp = threadIdx.x >> 5, lane = threadIdx.x & 31;
    const int grp = blockIdx.x / a.G, reg = blockIdx.x % a.G;
    if (a.n_live && grp >= static_cast<int>(*a.n_live)) return;   // uniform: dead fallback group
    const Group gr = a.groups[grp];
    const int ncol = a.ntx * a.nty;
    const int c0 = reg * a.cols_per_item, c1 = min(ncol, c0 + a.cols_per_item);
    if (c0 >= c1 || gr.n <= 0) return;                                // uniform
    const int nrot = min(gr.n, RB);
    const int M = a.m;
    const int n_planes = a.nz + M - 1;                                // z-planes streamed per column
    const int npl = a.npl;
    float* ring = reinterpret_cast<float*>(smem);                     // [atom][npl][slot_words]

    if (threadIdx.x == 0) {
        for (int s = 0; s < npl; s++) {
            dk::mbar_init(&full[s], 1);
            dk::mbar_init(&empty[s], NWC);
        }
        dk::fence_mbar_init();
    }
    // term tables of the group's rotations -> shared memory, [term][rotation] so that one term index serves
    // the RB rotations side by side
    const int slot_bytes = a.slot_words * 4;
    if (threadIdx.x == 0) {
        s_tmax = 0;
        s_ndirect = 0;
    }
    __syncthreads();
    for (int i = threadIdx.x; i < RB * TMAX; i += blockDim.x) {
        const int t = i / RB, r = i % RB;
        int4 term = make_int4(0, 0, 0, 0);   // weight 0: adds 0 x (a finite value of the current plane of atom 0)
        int dterm = -1;
        if (r < nrot) {
            const int slot = gr.slot0 + r;
            const int nt = a.n_terms[slot];
            if (t < nt) {
                const int code = a.term_v[static_cast<size_t>(slot) * TMAX + t];
                const int src = a.term_src[static_cast<size_t>(slot) * TMAX + t];
                const int vz = code >> 16, vy = (code >> 8) & 0xff, vx = code & 0xff;
                if (src >= 0) {
                    term = make_int4(src * npl * slot_bytes + (vy * a.TXB + vx) * 4, vz * slot_bytes,
                                     __float_as_int(1.0f), 0);
                } else {
                    dterm = (t << 24) | code;
                    atomicAdd(&s_ndirect, 1);
                }
            }
            if (t == 0) atomicMax(&s_tmax, nt);
        }
        s_term[i] = term;
        s_dterm[i] = dterm;
    }
    __syncthreads();
    const int tmax = s_tmax;
    const bool has_direct = s_ndirect > 0;

    if (warp == NWC) {
        // ---------------- producer: for each column of the item, z-planes 0 .. nz + m - 2 of every atom grid
        // into the ring (one plane sequence across the columns)
        if (lane == 0) {
            dk::prefetch_tmap(&gmap);
            const unsigned bytes = static_cast<unsigned>(gr.n_atoms) * a.box_bytes;
            int gp = 0;
            for (int c = c0; c < c1; c++) {
                const int tx = c % a.ntx, ty = c / a.ntx;
                for (int j = 0; j < n_planes; j++, gp++) {
                    const int s = gp % npl, use = gp / npl;
                    if (use > 0) dk::mbar_wait(&empty[s], (use - 1) & 1);
                    dk::mbar_arrive_expect_tx(&full[s], bytes);
                    for (int at = 0; at < gr.n_atoms; at++)
                        dk::tma_load_4d(ring + (static_cast<size_t>(at) * npl + s) * a.slot_words, &gmap, tx * a.TX,
                                        ty * TY, j, gr.atom0 + at, &full[s]);
                }
            }
        }
        return;
    }

    // ---------------- consumers: warp = (row ry, plane group pg: planes pg * ZT .. pg * ZT + ZT - 1 of a step)
    const int ry = warp % TY, pg = (warp / TY) % NPG, rbase = (warp / (TY * NPG)) * RBW;   // rotations rbase..+RBW-1
    unsigned long long(*lists)[32] = s_lst[warp];
#pragma unroll
    for (int r = 0; r < RBW; r++) lists[r][lane] = KEY_MAX;
    if (lane < RBW) {
        s_th[warp][lane] = make_float2(__int_as_float(0x7f800000), __uint_as_float(0xffffffffu));
        s_tg[warp][lane] = KEY_MAX;
    }
    __syncwarp();
    const uint32_t lane_base = dk::smem_u32(ring) + 4u * static_cast<uint32_t>(ry * a.TXB + lane);
    const uint32_t ring_bytes = static_cast<uint32_t>(npl * slot_bytes);
    const uint32_t plane_stride = static_cast<uint32_t>(a.nx * a.ny);
    const uint32_t full_s = dk::smem_u32(full), empty_s = dk::smem_u32(empty);
    int waited = 0, cbase = 0, wslot = 0, rslot = 0;   // next plane to wait for (slot), next plane to release
    unsigned wphase = 0;
    int pslot = (pg * ZT) % npl;   // ring slot of this warp's first plane, maintained incrementally
    for (int c = c0; c < c1; c++, cbase += n_planes) {
        if constexpr (!GRID) {
            if (a.bound_every > 0 && c > c0 && (c - c0) % a.bound_every == 0) {
                // publish each list's bound T_w and read back the unit's T: keys above T can never be picks
                // (DESIGN.md §8), so the gate also skips them (fewer insertions, same poses)
#pragma unroll 1
                for (int r = 0; r < RBW && rbase + r < nrot; r++) {
                    const int slot = gr.slot0 + rbase + r;
                    const unsigned long long key = lists[r][lane];
                    const unsigned long long tw = sp_list_bound(key, a.k, a.rho, a.nx, a.ny, a.nz);
                    unsigned long long tg = 0;
                    if (lane == 0) {
                        const unsigned long long old = tw != KEY_MAX ? atomicMin(&a.T[slot], tw)
                                                                     : *reinterpret_cast<volatile unsigned long long*>(&a.T[slot]);
                        tg = old < tw ? old : tw;
                        s_tg[warp][r] = tg;
                    }
                    const unsigned long long k31 = dk::shfl_u64(key, 31);
                    if (lane == 0) {
                        const unsigned long long gk = k31 < tg ? k31 : tg;
                        s_th[warp][r] = make_float2(dk::key_score_bound(static_cast<uint32_t>(gk >> 32)),
                                                    __uint_as_float(static_cast<uint32_t>(gk & 0xffffffffu)));
                    }
                }
                __syncwarp();
            }
        }
        const int tx = c % a.ntx, ty = c / a.ntx;
        const int y = ty * TY + ry;
        const int xb = tx * a.TX + lane;
        unsigned xmask = 0;
#pragma unroll
        for (int i = 0; i < XTS; i++) xmask |= (xb + 32 * i < a.nx) ? (1u << i) : 0u;
        int zz = 0;
        for (; zz < a.nz; zz += PZ) {
            const int need = cbase + min(zz + PZ - 1 + M - 1, n_planes - 1);
            while (waited <= need) {   // ring slot / phase of plane `waited` tracked without divisions
                mbar_wait_s(full_s + 8u * wslot, wphase);
                waited++;
                if (++wslot == npl) {
                    wslot = 0;
                    wphase ^= 1u;
                }
            }
            const int z0w = zz + pg * ZT;   // this warp's first plane
            // a warp whose first plane or row lies outside the grid skips the step (its ring slots may already
            // hold later planes); the condition is warp-uniform.  A later plane beyond the grid reads the first
            // plane's slot (masked out).
            if (z0w < a.nz && y < a.ny) {
                unsigned vmask = 0;
                uint32_t zoff[ZT];
#pragma unroll
                for (int j = 0; j < ZT; j++) {
                    const bool pj = z0w + j < a.nz;
                    int sj = pslot + j;
                    sj = sj >= npl ? sj - npl : sj;
                    zoff[j] = static_cast<uint32_t>((pj ? sj : pslot) * slot_bytes);
                    vmask |= pj ? (xmask << (j * XTS)) : 0u;
                }
                const bool vfull = __all_sync(FULL, vmask == (1u << V) - 1u);   // nothing masked (uniform)
                const uint32_t tbase = static_cast<uint32_t>((z0w * a.ny + y) * a.nx + xb);
                // term-outer, rotation-inner, branch-free: the RB rotations' gathers are independent (weight 1 for
                // a single-atom voxel, 0 for an absent or multi-atom term: fma(1, g, acc) == acc + g exactly);
                // term 0 initialises the accumulators
                float acc[RBW][V];
                if (tmax > 0) {
#pragma unroll
                    for (int r = 0; r < RBW; r++) {
                        const int4 term = s_term[rbase + r];
                        const float wt = __int_as_float(term.z);
#pragma unroll
                        for (int j = 0; j < ZT; j++) {
                            uint32_t zo = zoff[j] + static_cast<uint32_t>(term.y);
                            zo = zo >= ring_bytes ? zo - ring_bytes : zo;
                            const uint32_t ad = lane_base + zo + static_cast<uint32_t>(term.x);
#pragma unroll
                            for (int i = 0; i < XTS; i++) acc[r][j * XTS + i] = wt * lds_f32(ad + 128u * i);
                        }
                    }
                } else {   // a probe without atoms scores 0 everywhere
#pragma unroll
                    for (int r = 0; r < RBW; r++)
#pragma unroll
                        for (int v = 0; v < V; v++) acc[r][v] = 0.0f;
                }
#pragma unroll 1
                for (int t = 1; t < tmax; t++) {
#pragma unroll
                    for (int r = 0; r < RBW; r++) {
                        const int4 term = s_term[t * RB + rbase + r];
                        const float wt = __int_as_float(term.z);
#pragma unroll
                        for (int j = 0; j < ZT; j++) {
                            uint32_t zo = zoff[j] + static_cast<uint32_t>(term.y);
                            zo = zo >= ring_bytes ? zo - ring_bytes : zo;
                            const uint32_t ad = lane_base + zo + static_cast<uint32_t>(term.x);
#pragma unroll
                            for (int i = 0; i < XTS; i++)
                                acc[r][j * XTS + i] = fmaf(wt, lds_f32(ad + 128u * i), acc[r][j * XTS + i]);
                        }
                    }
                }
                if (has_direct) {
                    // voxels holding several atoms: direct P-channel correlation (rare), after the gathered terms
#pragma unroll 1
                    for (int t = 0; t < tmax; t++) {
#pragma unroll
                        for (int r = 0; r < RBW; r++) {
                            const int code = s_dterm[t * RB + rbase + r];
                            if (code >= 0) {
#pragma unroll
                                for (int j = 0; j < ZT; j++) {
                                    const Vec<XTS> d = sp_direct<XTS>(
                                        a.dw + (static_cast<size_t>(gr.slot0 + rbase + r) * TMAX + (code >> 24)) * a.P, a.P,
                                        a.rec, a.rXp, a.rYp, a.rZp, z0w + j + ((code >> 16) & 0xff),
                                        y + ((code >> 8) & 0xff), xb + (code & 0xff), (vmask >> (j * XTS)) & xmask);
#pragma unroll
                                    for (int i = 0; i < XTS; i++) acc[r][j * XTS + i] += d.v[i];
                                }
                            }
                        }
                    }
                }
                if constexpr (GRID) {
#pragma unroll
                    for (int r = 0; r < RBW; r++) {
                        if (rbase + r < nrot) {
                            float* out = a.grid + static_cast<size_t>(grp + rbase + r) * a.nx * a.ny * a.nz + tbase;
#pragma unroll
                            for (int v = 0; v < V; v++)
                                if ((vmask >> v) & 1u) out[(v / XTS) * plane_stride + 32 * (v % XTS)] = acc[r][v];
                        }
                    }
                } else {
                    // exact gate of every rotation at once: a strictly better score, or a tie whose t_lin could
                    // precede the list's 32nd key (tbase is the smallest t_lin of the lane); one warp vote for all
                    unsigned pass = 0;
#pragma unroll
                    for (int r = 0; r < RBW; r++) {
                        const float2 thr = s_th[warp][r];
                        float mn;
                        if (vfull) {
                            mn = acc[r][0];
#pragma unroll
                            for (int v = 1; v < V; v++) mn = fminf(mn, acc[r][v]);
                        } else {
                            mn = __int_as_float(0x7f800000);
#pragma unroll
                            for (int v = 0; v < V; v++) mn = ((vmask >> v) & 1u) ? fminf(mn, acc[r][v]) : mn;
                        }
                        const bool any = mn < thr.x || (mn == thr.x && tbase < __float_as_uint(thr.y));
                        pass |= (any && rbase + r < nrot) ? (1u << r) : 0u;
                    }
                    pass = __reduce_or_sync(FULL, pass);
                    if (pass) {
#pragma unroll
                        for (int r = 0; r < RBW; r++) {
                            if ((pass >> r) & 1u) {
                                Vec<V> av;
#pragma unroll
                                for (int v = 0; v < V; v++) av.v[v] = acc[r][v];
                                sp_insert<XTS, ZT>(lists[r], &s_th[warp][r], av, vmask, tbase, plane_stride, lane,
                                                   s_tg[warp][r]);
                            }
                        }
                    }
                }
            }
            __syncwarp();
#pragma unroll
            for (int q = 0; q < PZ; q++) {
                if (zz + q < n_planes) {
                    if (lane == 0) mbar_arrive_s(empty_s + 8u * rslot);
                    rslot = rslot + 1 == npl ? 0 : rslot + 1;
                }
            }
            pslot += PZ;
            pslot = pslot >= npl ? pslot - npl : pslot;
        }
        // column end: release its remaining halo planes; the next column's planes follow in the ring
        for (int j = zz; j < n_planes; j++) {
            if (lane == 0) mbar_arrive_s(empty_s + 8u * rslot);
            rslot = rslot + 1 == npl ? 0 : rslot + 1;
        }
        __syncwarp();
        pslot = rslot + pg * ZT;   // the next column's first plane is the next one to be released
        pslot = pslot >= npl ? pslot - npl : pslot;
    }

    if constexpr (!GRID) {
        // ---------------- item end: publish bound + surviving keys of each warp list (as dk::k_corr)
        const int nx = a.nx, ny = a.ny, nz = a.nz;
#pragma unroll 1
        for (int rr = 0; rr < RBW && rbase + rr < nrot; rr++) {
            {
                const int slot = gr.slot0 + rbase + rr;
                const unsigned long long key = lists[rr][lane];
                const uint32_t t = static_cast<uint32_t>(key & 0xffffffffu);
                const unsigned long long k31 = dk::shfl_u64(key, 31);
                bool excl = (key == KEY_MAX);
                unsigned long long Tw = KEY_MAX;
                for (int j = 0; j < a.k; j++) {
                    const unsigned b = __ballot_sync(FULL, !excl);
                    if (!b) break;
                    const int f = __ffs(b) - 1;
                    const unsigned long long kf = dk::shfl_u64(key, f);
                    const uint32_t tf = static_cast<uint32_t>(kf & 0xffffffffu);
                    excl = excl || (dk::cheb_cyc(t, tf, nx, ny, nz) <= 2 * a.rho);
                    if (j == a.k - 1) Tw = kf;
                }
                unsigned long long Tn = 0;
                if (lane == 0) {
                    const unsigned long long old = atomicMin(&a.T[slot], Tw);
                    Tn = old < Tw ? old : Tw;
                    atomicMin(&a.mu[slot], k31);
                }
                Tn = dk::shfl_u64(Tn, 0);
                const bool wr = (key != KEY_MAX) && (key <= Tn);
                const unsigned bal = __ballot_sync(FULL, wr);
                unsigned base = 0;
                if (lane == 0 && bal) base = atomicAdd(&a.cnt[slot], static_cast<unsigned>(__popc(bal)));
                base = __shfl_sync(FULL, base, 0);
                if (wr) {
                    const unsigned pos = base + __popc(bal & ((1u << lane) - 1u));
                    if (pos < static_cast<unsigned>(a.cap)) a.cand[static_cast<size_t>(slot) * a.cap + pos] = key;
                }
            }
        }
    }
}

}  // namespace sp
