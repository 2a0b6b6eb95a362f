"""Summarise an .ncu-rep: key metrics + top stall reasons per kernel launch."""
import csv, subprocess, sys
KEYS = ['gpu__time_duration.sum', 'dram__bytes_read.sum', 'dram__bytes_write.sum',
        'dram__throughput.avg.pct_of_peak_sustained_elapsed', 'lts__t_sector_hit_rate.pct',
        'sm__warps_active.avg.pct_of_peak_sustained_active', 'launch__registers_per_thread',
        'launch__occupancy_limit_registers', 'smsp__inst_executed.sum',
        'smsp__issue_active.avg.pct_of_peak_sustained_active', 'lts__t_sectors.sum',
        'lts__t_sectors_op_atom.sum', 'lts__t_sectors_op_red.sum', 'lts__throughput.avg.pct_of_peak_sustained_elapsed',
        'l1tex__t_requests_pipe_lsu_mem_global_op_atom.sum', 'sm__throughput.avg.pct_of_peak_sustained_elapsed']
def main(path, top=8):
    out = subprocess.run(['ncu', '-i', path, '--page', 'raw', '--csv'], capture_output=True, text=True).stdout
    r = list(csv.reader(out.splitlines()))
    hdr, units, rows = r[0], r[1], r[2:]
    for row in rows:
        print(row[hdr.index('Kernel Name')], 'grid', row[hdr.index('launch__grid_size')] if 'launch__grid_size' in hdr else '')
        for k in KEYS:
            if k in hdr:
                print(f'   {k:60s} {row[hdr.index(k)]} {units[hdr.index(k)]}')
        st = [(h.replace('smsp__average_warps_issue_stalled_', '').replace('_per_issue_active.ratio', ''), row[i])
              for i, h in enumerate(hdr) if h.startswith('smsp__average_warps_issue_stalled_') and h.endswith('per_issue_active.ratio')]
        st = sorted([(a, float(b)) for a, b in st if b not in ('', 'n/a')], key=lambda x: -x[1])[:top]
        print('   stalls/issue:', ', '.join(f'{a}={b:.2f}' for a, b in st))
if __name__ == '__main__':
    main(sys.argv[1])
