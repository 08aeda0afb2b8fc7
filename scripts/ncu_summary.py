"""Summarise an .ncu-rep: key metrics, top stall reasons, dynamic opcode mix and
the hottest SASS lines, per profiled kernel.

    python scripts/ncu_summary.py gpurun_out/prof.ncu-rep [kernel-regex ...]
"""
import collections
import csv
import io
import subprocess
import sys

WANT = ['gpu__time_duration.sum', 'dram__bytes_read.sum', 'dram__bytes_write.sum',
        'gpu__dram_throughput.avg.pct_of_peak_sustained_elapsed', 'sm__warps_active.avg.pct_of_peak_sustained_active',
        'launch__registers_per_thread', 'launch__occupancy_limit_registers', 'launch__occupancy_limit_shared_mem',
        'launch__grid_size', 'launch__block_size', 'launch__cluster_dim_x',
        'sm__throughput.avg.pct_of_peak_sustained_elapsed', 'smsp__issue_active.avg.pct_of_peak_sustained_active',
        'l1tex__data_bank_conflicts_pipe_lsu_mem_shared_op_ld.sum', 'l1tex__data_bank_conflicts_pipe_lsu_mem_shared_op_st.sum',
        'smsp__inst_executed.sum', 'sm__pipe_fma_cycles_active.avg.pct_of_peak_sustained_active',
        'sm__inst_executed_pipe_xu.avg.pct_of_peak_sustained_active', 'launch__waves_per_multiprocessor',
        'lts__t_sectors_op_write.sum', 'l1tex__t_bytes_pipe_lsu_mem_local_op_ld.sum', 'l1tex__t_bytes_pipe_lsu_mem_local_op_st.sum']


def ncu(path, page, kfilter, *extra):
    cmd = ['ncu', '-i', path, '--page', page, '--csv', *extra]
    if kfilter:
        cmd += ['-k', 'regex:' + kfilter]
    return list(csv.reader(io.StringIO(subprocess.run(cmd, capture_output=True, text=True).stdout)))


def summarise(path, kfilter, nsrc=20):
    rows = ncu(path, 'raw', kfilter)
    if len(rows) < 3:
        print(f'== {path} [{kfilter}]: no kernel')
        return
    hdr, units, vals = rows[0], rows[1], rows[2]
    print(f'== {path}: {vals[hdr.index("Kernel Name")][:100]}')
    for w in WANT:
        if w in hdr:
            i = hdr.index(w)
            print(f'  {w:62s} {vals[i]:>18s} {units[i]}')
    st = []
    for i, h in enumerate(hdr):
        if h.startswith('smsp__pcsamp_warps_issue_stalled') and not h.endswith('not_issued'):
            try:
                st.append((float(vals[i]), h.replace('smsp__pcsamp_warps_issue_stalled_', '')))
            except ValueError:
                pass
    tot = sum(v for v, _ in st) or 1
    print('  stalls: ' + ', '.join(f'{h} {v / tot * 100:.0f}%' for v, h in sorted(st, reverse=True)[:9]))
    srows = ncu(path, 'source', kfilter, '--print-source', 'sass')
    hi = [i for i, r in enumerate(srows) if r and r[0] == 'Address']
    if not hi:
        return
    h = srows[hi[0]]
    body = []
    for r in srows[hi[0] + 1:]:
        if r and r[0] == 'Kernel Name':
            break
        body.append(r)
    si, ci, ei = h.index('Warp Stall Sampling (All Samples)'), h.index('Source'), h.index('Instructions Executed')
    body = [r for r in body if len(r) > ei and r[si].isdigit() and r[ei].isdigit()]
    mix = collections.Counter()
    for r in body:
        op = [o for o in r[ci].split() if not o.startswith('@')]
        mix[op[0].split('.')[0] if op else '?'] += int(r[ei])
    itot = sum(mix.values()) or 1
    print('  opcode mix: ' + ', '.join(f'{k} {v / itot * 100:.1f}%' for k, v in mix.most_common(16)))
    tot = sum(int(r[si]) for r in body) or 1
    print('  hottest SASS (stall samples):')
    for r in sorted(body, key=lambda r: -int(r[si]))[:nsrc]:
        print(f'    {int(r[si]) / tot * 100:5.1f}%  {r[ci].strip()[:90]}')


if __name__ == '__main__':
    path = sys.argv[1]
    for kf in (sys.argv[2:] or ['']):
        summarise(path, kf)
