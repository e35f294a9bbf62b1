"""Print the key metrics of an ncu report (raw page) — used to write profiles/*.md."""
import csv, io, subprocess, sys

KEYS = ['gpu__time_duration.sum', 'dram__bytes_read.sum', 'dram__bytes_write.sum',
        'dram__throughput.avg.pct_of_peak_sustained_elapsed', 'sm__throughput.avg.pct_of_peak_sustained_elapsed',
        'sm__warps_active.avg.pct_of_peak_sustained_active', 'sm__maximum_warps_per_active_cycle_pct',
        'launch__registers_per_thread', 'launch__grid_size', 'launch__block_size',
        'l1tex__data_bank_conflicts_pipe_lsu_mem_shared_op_ld.sum', 'l1tex__data_bank_conflicts_pipe_lsu_mem_shared_op_st.sum',
        'sm__inst_executed_pipe_alu.avg.pct_of_peak_sustained_active', 'sm__inst_executed_pipe_fma.avg.pct_of_peak_sustained_active',
        'sm__inst_executed_pipe_lsu.avg.pct_of_peak_sustained_active', 'smsp__issue_active.avg.pct_of_peak_sustained_active',
        'smsp__inst_executed.sum', 'sm__cycles_elapsed.avg', 'sm__cycles_elapsed.avg.per_second',
        'l1tex__data_pipe_lsu_wavefronts_mem_shared.sum', 'smsp__inst_executed_op_shfl.sum',
        'sm__pipe_shared_cycles_active.avg.pct_of_peak_sustained_active']
def main(path):
    raw = subprocess.run(['ncu', '-i', path, '--page', 'raw', '--csv'], capture_output=True, text=True).stdout
    rows = list(csv.reader(io.StringIO(raw)))
    h, u = rows[0], rows[1]
    for v in rows[2:]:
        print('--', v[h.index('Kernel Name')][:90])
        for i, name in enumerate(h):
            if name in KEYS or name.startswith('smsp__average_warps_issue_stalled_') and name.endswith('per_issue_active.ratio'):
                try:
                    if name.startswith('smsp__average_warps_issue_stalled_') and float(v[i]) < 0.05: continue
                except ValueError: pass
                print(f'{name:75s} {u[i]:>12s} {v[i]}')
if __name__ == '__main__':
    main(sys.argv[1])
