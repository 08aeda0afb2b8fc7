"""Summarise an .ncu-rep: key metrics + top stall reasons + hottest source lines."""
import csv, subprocess, sys, io

WANT = ['gpu__time_duration.sum', 'dram__bytes_read.sum', 'dram__bytes_write.sum',
        'gpu__dram_throughput.avg.pct_of_peak_sustained_elapsed', 'sm__warps_active.avg.pct_of_peak_sustained_active',
        'launch__registers_per_thread', 'launch__occupancy_limit_registers', 'launch__occupancy_limit_shared_mem',
        'launch__grid_size', 'launch__block_size', 'launch__cluster_size' if False else 'launch__cluster_dim_x',
        'sm__throughput.avg.pct_of_peak_sustained_elapsed', 'smsp__issue_active.avg.pct_of_peak_sustained_active',
        'l1tex__data_bank_conflicts_pipe_lsu_mem_shared_op_ld.sum', 'l1tex__data_bank_conflicts_pipe_lsu_mem_shared_op_st.sum',
        'smsp__inst_executed.sum', 'sm__pipe_fma_cycles_active.avg.pct_of_peak_sustained_active',
        'sm__inst_executed_pipe_xu.avg.pct_of_peak_sustained_active', 'launch__waves_per_multiprocessor',
        'lts__t_sectors_op_write.sum', 'l1tex__t_bytes_pipe_lsu_mem_local_op_ld.sum', 'l1tex__t_bytes_pipe_lsu_mem_local_op_st.sum']

def main(path, nsrc=25):
    raw = subprocess.run(['ncu', '-i', path, '--page', 'raw', '--csv'], capture_output=True, text=True).stdout
    rows = list(csv.reader(io.StringIO(raw)))
    hdr, units, vals = rows[0], rows[1], rows[2]
    name = vals[hdr.index('Kernel Name')] if 'Kernel Name' in hdr else '?'
    print(f'== {path}: {name[:100]}')
    for w in WANT:
        if w in hdr:
            i = hdr.index(w); print(f'  {w:62s} {vals[i]:>18s} {units[i]}')
    st = []
    for i, h in enumerate(hdr):
        if h.startswith('smsp__pcsamp_warps_issue_stalled') and not h.endswith('not_issued'):
            try: st.append((float(vals[i]), h.replace('smsp__pcsamp_warps_issue_stalled_', '')))
            except ValueError: pass
    tot = sum(v for v, _ in st) or 1
    print('  stalls: ' + ', '.join(f'{h} {v/tot*100:.0f}%' for v, h in sorted(st, reverse=True)[:8]))
    src = subprocess.run(['ncu', '-i', path, '--page', 'source', '--csv', '--print-source', 'sass'], capture_output=True, text=True).stdout
    srows = list(csv.reader(io.StringIO(src)))
    hi = [i for i, r in enumerate(srows) if r and r[0] == 'Address']
    if hi:
        h = srows[hi[0]]; body = srows[hi[0] + 1:]
        si = h.index('Warp Stall Sampling (All Samples)'); ci = h.index('Source')
        body = [r for r in body if len(r) > si and r[si].isdigit()]
        tot = sum(int(r[si]) for r in body) or 1
        print('  hottest SASS:')
        for r in sorted(body, key=lambda r: -int(r[si]))[:nsrc]:
            print(f'    {int(r[si])/tot*100:5.1f}%  {r[ci].strip()[:90]}')

if __name__ == '__main__':
    for p in sys.argv[1:]:
        main(p)
